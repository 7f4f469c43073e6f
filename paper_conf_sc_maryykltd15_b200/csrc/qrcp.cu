// Truncated QRCP of the small sample B (l x n): Step 2 of random sampling (Fig. 2(b)
// line 6, "truncated QP3 on a GPU").  k sequential Householder steps, each choosing the
// remaining column with the largest residual 2-norm (Sec. 2).
//
// B200 design: one persistent cooperative kernel.  The columns of B are distributed over NB CTAs
// and stay resident in shared memory for all k steps; per step each CTA (A) recomputes the
// residual norms of its active columns with warp-shuffle reductions (reading R5: exact
// recomputation instead of downdating, P:L189-192/L212-217 -- every column is touched by the
// trailing update anyway, so the recompute is free) and publishes its best candidate column,
// (grid barrier), (B) every CTA picks the same global pivot (largest norm, ties -> lowest original
// index), forms the dlarfg reflector from the published column and applies it to its own
// columns.  One grid barrier per step; pivots and R̂ rows are final as soon as they are produced.
#include <algorithm>
#include <cstdio>

#include "common.cuh"
#include "internal.h"

namespace rs {

constexpr int QR_THREADS = 256;
constexpr int QR_WARPS = QR_THREADS / 32;

struct QrCand {
  double best;    // squared residual norm of the CTA's best active column (-1 if none)
  double second;  // second best squared norm in the CTA (-1 if none)
  long long idx;  // original column index of the best
  long long pad;
};

struct QrWork {
  GridBarrier bar;
  unsigned int pad[2];
  // followed by: QrCand cand[2][NB]; double candcol[2][NB][ell]; int64 inv[n]
};

RS_DEVINL bool better(double a, long long ia, double b, long long ib) {
  return a > b || (a == b && ia < ib);
}

__global__ void __launch_bounds__(QR_THREADS, 1)
    qrcp_kernel(const double* __restrict__ B, int ldb, int ell, long long n, int k, QrWork* work, int NB,
                int cols_per, int64_t* __restrict__ perm, double* __restrict__ Rho, int ldr,
                double* __restrict__ gaps, int* info) {
  extern __shared__ double sh[];
  const int blk = blockIdx.x;
  const long long c0 = static_cast<long long>(blk) * cols_per;
  const long long c1 = (c0 + cols_per < n) ? c0 + cols_per : n;
  const int nc = c1 > c0 ? static_cast<int>(c1 - c0) : 0;
  double* W = sh;                                   // nc x ell, column c at W + c*ell
  double* v = W + static_cast<size_t>(cols_per) * ell;  // Householder vector (ell)
  __shared__ unsigned char active[1024];
  __shared__ double s_wbest[QR_WARPS], s_wsecond[QR_WARPS];
  __shared__ long long s_widx[QR_WARPS];
  __shared__ int s_wloc[QR_WARPS];
  __shared__ double s_tau, s_beta, s_gbest, s_gsecond;
  __shared__ long long s_gidx;
  __shared__ int s_gblk, s_bloc;

  QrCand* cand = reinterpret_cast<QrCand*>(work + 1);
  double* candcol = reinterpret_cast<double*>(cand + 2 * NB);
  int64_t* inv = reinterpret_cast<int64_t*>(candcol + 2 * static_cast<size_t>(NB) * ell);

  const int tid = threadIdx.x, warp = tid >> 5, lane = tid & 31;
  for (int idx = tid; idx < nc * ell; idx += QR_THREADS) {
    const int c = idx / ell, i = idx % ell;
    W[c * ell + i] = B[i + (c0 + c) * static_cast<long long>(ldb)];
  }
  for (int c = tid; c < nc; c += QR_THREADS) active[c] = 1;
  if (blk == 0)
    for (long long c = tid; c < n; c += QR_THREADS) perm[c] = c, inv[c] = c;
  __syncthreads();

  for (int j = 0; j < k; ++j) {
    const int par = j & 1;
    // ---- (A) residual norms of active local columns, local top-2 ----
    double wb = -1.0, ws = -1.0;
    long long wi = -1;
    int wl = -1;
    for (int c = warp; c < nc; c += QR_WARPS) {
      if (!active[c]) continue;
      double s = 0.0;
      for (int i = j + lane; i < ell; i += 32) {
        const double x = W[c * ell + i];
        s = fma(x, x, s);
      }
#pragma unroll
      for (int o = 16; o > 0; o >>= 1) s += __shfl_xor_sync(0xffffffffu, s, o);
      const long long gi = c0 + c;
      if (better(s, gi, wb, wi)) {
        ws = wb;
        wb = s;
        wi = gi;
        wl = c;
      } else if (s > ws) {
        ws = s;
      }
    }
    if (lane == 0) {
      s_wbest[warp] = wb;
      s_wsecond[warp] = ws;
      s_widx[warp] = wi;
      s_wloc[warp] = wl;
    }
    __syncthreads();
    if (tid == 0) {
      double bb = -1.0, bs = -1.0;
      long long bi = -1;
      int bl = -1;
      for (int w = 0; w < QR_WARPS; ++w) {
        if (s_widx[w] < 0) continue;
        if (better(s_wbest[w], s_widx[w], bb, bi)) {
          bs = fmax(bb, bs);
          bb = s_wbest[w];
          bi = s_widx[w];
          bl = s_wloc[w];
        } else {
          bs = fmax(bs, s_wbest[w]);
        }
        bs = fmax(bs, s_wsecond[w]);
      }
      // the second-best of the winning warp may be larger than another warp's best
      cand[par * NB + blk].best = bb;
      cand[par * NB + blk].second = bs;
      cand[par * NB + blk].idx = bi;
      s_bloc = bl;
    }
    __syncthreads();
    if (s_bloc >= 0)
      for (int i = j + tid; i < ell; i += QR_THREADS)
        candcol[(static_cast<size_t>(par) * NB + blk) * ell + i] = W[s_bloc * ell + i];
    grid_sync(&work->bar, NB);

    // ---- (B) global pivot (every CTA computes the same answer) ----
    if (warp == 0) {
      double bb = -1.0;
      long long bi = -1;
      int bk = -1;
      for (int b = lane; b < NB; b += 32) {
        const long long ci = __ldcg(&cand[par * NB + b].idx);
        const double cb = __ldcg(&cand[par * NB + b].best);
        if (ci >= 0 && better(cb, ci, bb, bi)) {
          bb = cb;
          bi = ci;
          bk = b;
        }
      }
#pragma unroll
      for (int o = 16; o > 0; o >>= 1) {
        const double ob = __shfl_xor_sync(0xffffffffu, bb, o);
        const long long oi = __shfl_xor_sync(0xffffffffu, bi, o);
        const int ok = __shfl_xor_sync(0xffffffffu, bk, o);
        if (oi >= 0 && (bi < 0 || better(ob, oi, bb, bi))) {
          bb = ob;
          bi = oi;
          bk = ok;
        }
      }
      // global second best: the winner CTA's runner-up and every other CTA's best
      double bs = -1.0;
      for (int b = lane; b < NB; b += 32) {
        const long long ci = __ldcg(&cand[par * NB + b].idx);
        const double val = (b == bk) ? __ldcg(&cand[par * NB + b].second)
                                     : (ci >= 0 ? __ldcg(&cand[par * NB + b].best) : -1.0);
        bs = fmax(bs, val);
      }
#pragma unroll
      for (int o = 16; o > 0; o >>= 1) bs = fmax(bs, __shfl_xor_sync(0xffffffffu, bs, o));
      if (lane == 0) {
        s_gbest = bb;
        s_gsecond = bs;
        s_gidx = bi;
        s_gblk = bk;
      }
    }
    __syncthreads();
    const int gblk = s_gblk;
    const long long gidx = s_gidx;
    const int len = ell - j;
    for (int i = tid; i < len; i += QR_THREADS)
      v[i] = __ldcg(&candcol[(static_cast<size_t>(par) * NB + (gblk < 0 ? 0 : gblk)) * ell + j + i]);
    __syncthreads();
    if (warp == 0) {  // dlarfg on x = v[0..len)
      double xs = 0.0;
      for (int i = 1 + lane; i < len; i += 32) xs = fma(v[i], v[i], xs);
#pragma unroll
      for (int o = 16; o > 0; o >>= 1) xs += __shfl_xor_sync(0xffffffffu, xs, o);
      const double alpha = v[0];
      double tau = 0.0, beta = alpha;
      if (gblk >= 0 && xs > 0.0) {
        const double h = sqrt(fma(alpha, alpha, xs));
        beta = alpha >= 0.0 ? -h : h;
        tau = (beta - alpha) / beta;
      }
      __syncwarp();
      if (tau != 0.0) {
        const double den = alpha - beta;
        for (int i = 1 + lane; i < len; i += 32) v[i] = v[i] / den;
      }
      __syncwarp();
      if (lane == 0) {
        v[0] = 1.0;
        s_tau = tau;
        s_beta = beta;
        if (gblk < 0 || !(s_gbest > 0.0)) {
          if (info && blk == 0) atomicCAS(info, 0, 6 /* RS_ERR_RANK_DEFICIENT */), atomicCAS(info + 1, 0, j + 1);
        }
      }
    }
    __syncthreads();
    const double tau = s_tau, beta = s_beta;
    // ---- apply H = I - tau v v^T to local active columns; retire the pivot column ----
    for (int c = warp; c < nc; c += QR_WARPS) {
      if (!active[c]) continue;
      const long long gi = c0 + c;
      double* col = W + c * ell;
      if (gi == gidx) {
        for (int i = lane; i < k; i += 32) {
          const double val = (i < j) ? col[i] : (i == j ? beta : 0.0);
          Rho[i + gi * static_cast<long long>(ldr)] = val;
        }
        __syncwarp();
        if (lane == 0) active[c] = 0;
        continue;
      }
      if (tau == 0.0) continue;
      double w = 0.0;
      for (int i = lane; i < len; i += 32) w = fma(v[i], col[j + i], w);
#pragma unroll
      for (int o = 16; o > 0; o >>= 1) w += __shfl_xor_sync(0xffffffffu, w, o);
      const double tw = tau * w;
      for (int i = lane; i < len; i += 32) col[j + i] = fma(-tw, v[i], col[j + i]);
    }
    if (blk == 0 && tid == 0 && gidx >= 0) {
      const long long pw = inv[gidx];
      const long long oj = perm[j];
      perm[j] = gidx;
      perm[pw] = oj;
      inv[gidx] = j;
      inv[oj] = pw;
      const double nb = sqrt(fmax(s_gbest, 0.0)), ns = sqrt(fmax(s_gsecond, 0.0));
      if (gaps) gaps[j] = nb > 0.0 ? (nb - ns) / nb : 0.0;
    }
    __syncthreads();
  }
  // rows 0..k-1 of the never-pivoted columns
  for (int c = warp; c < nc; c += QR_WARPS) {
    if (!active[c]) continue;
    const long long gi = c0 + c;
    for (int i = lane; i < k; i += 32) Rho[i + gi * static_cast<long long>(ldr)] = W[c * ell + i];
  }
}

namespace {
int qr_blocks(int ell, long long n, int num_sms) {
  long long nb = std::min<long long>(num_sms, (n + 31) / 32);
  if (nb < 1) nb = 1;
  return static_cast<int>(nb);
}
}  // namespace

size_t qrcp_workspace_bytes(int ell, long long n) {
  const int NB = 1024;  // upper bound on blocks
  return sizeof(QrWork) + 2 * NB * sizeof(QrCand) + 2 * static_cast<size_t>(NB) * ell * 8 + n * 8 + 256;
}

cudaError_t qrcp_truncated(cudaStream_t st, const double* B, int ldb, int ell, long long n, int k, void* work,
                           int64_t* perm, double* Rho, int ldr, double* gaps, int* info, int num_sms) {
  int NB = qr_blocks(ell, n, num_sms);
  int cols_per = static_cast<int>((n + NB - 1) / NB);
  size_t smem = (static_cast<size_t>(cols_per) * ell + ell) * 8;
  while (smem > 200 * 1024 && NB < 2 * num_sms) {
    ++NB;
    cols_per = static_cast<int>((n + NB - 1) / NB);
    smem = (static_cast<size_t>(cols_per) * ell + ell) * 8;
  }
  if (smem > 200 * 1024 || cols_per > 1024) return cudaErrorInvalidValue;
  static bool attr = false;
  if (!attr) {
    cudaError_t e = cudaFuncSetAttribute(qrcp_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, 200 * 1024);
    if (e != cudaSuccess) return e;
    attr = true;
  }
  cudaError_t e = cudaMemsetAsync(work, 0, sizeof(QrWork), st);
  if (e != cudaSuccess) return e;
  QrWork* w = static_cast<QrWork*>(work);
  void* args[] = {(void*)&B, (void*)&ldb, (void*)&ell, (void*)&n, (void*)&k, (void*)&w, (void*)&NB, (void*)&cols_per,
                  (void*)&perm, (void*)&Rho, (void*)&ldr, (void*)&gaps, (void*)&info};
  count_launch();
  return cudaLaunchCooperativeKernel(reinterpret_cast<void*>(qrcp_kernel), dim3(NB), dim3(QR_THREADS), args, smem, st);
}

}  // namespace rs
