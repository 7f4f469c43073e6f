// Truncated QRCP of the small sample B (l x n): Step 2 of random sampling (Fig. 2(b)
// line 6, "truncated QP3 on a GPU").  k sequential Householder steps, each choosing the
// remaining column with the largest residual 2-norm (Sec. 2).
//
// B200 design: one persistent cooperative kernel.  The columns of B are distributed over NB CTAs
// and stay resident in shared memory for all k steps; per step each CTA (A) recomputes the
// residual norms of its active columns with warp-shuffle reductions (reading R5: exact
// recomputation instead of downdating, P:L189-192/L212-217 -- every column is touched by the
// trailing update anyway, so the recompute costs no extra pass) and publishes its best candidate
// column, (grid barrier), (B) every CTA reads all candidates in parallel, picks the same global
// pivot (largest norm, ties -> lowest original index), forms the dlarfg reflector from the
// published column and applies it to its own columns.  One grid barrier and two dependent L2
// round trips per step; pivots and R̂ rows are final as soon as they are produced.
#include <algorithm>
#include <cstdio>

#include "common.cuh"
#include "internal.h"

namespace rs {

constexpr int QR_THREADS = 512;
constexpr int QR_WARPS = QR_THREADS / 32;
constexpr int QR_MAX_COLS = 1024;    // columns per CTA (smem flags)
constexpr int QR_COLS_TARGET = 160;  // preferred columns per CTA: few CTAs -> cheap grid barrier

struct QrCand {
  double best;    // squared residual norm of the CTA's best active column (-1 if none)
  double second;  // second best squared norm in the CTA (-1 if none)
  long long idx;  // original column index of the best (-1 if none)
  long long pad;
};

struct QrWork {
  unsigned int count;  // monotone grid-barrier counter
  unsigned int pad[3];
  // followed by: QrCand cand[2][NB]; double candcol[2][NB][ell]; int64 inv[n]
};

RS_DEVINL bool better(double a, long long ia, double b, long long ib) {
  return ia >= 0 && (ib < 0 || a > b || (a == b && ia < ib));
}

RS_DEVINL unsigned int ld_acquire_u32(const unsigned int* p) {
  unsigned int v;
  asm volatile("ld.acquire.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}

// all NB CTAs: arrive once, wait until `target` arrivals have been counted
RS_DEVINL void grid_sync_count(unsigned int* count, unsigned int target) {
  __syncthreads();
  if (threadIdx.x == 0) {
    asm volatile("red.release.gpu.global.add.u32 [%0], 1;" ::"l"(count) : "memory");
    while (ld_acquire_u32(count) < target) {
    }
  }
  __syncthreads();
}

// (value, index, owner) argmax with ties to the lowest index, across the CTA
struct Arg {
  double v;
  long long i;
  int b;
};
RS_DEVINL Arg warp_argmax(Arg a) {
#pragma unroll
  for (int o = 16; o > 0; o >>= 1) {
    Arg x{__shfl_xor_sync(0xffffffffu, a.v, o), __shfl_xor_sync(0xffffffffu, a.i, o),
          __shfl_xor_sync(0xffffffffu, a.b, o)};
    if (better(x.v, x.i, a.v, a.i)) a = x;
  }
  return a;
}
RS_DEVINL double warp_max(double v) {
#pragma unroll
  for (int o = 16; o > 0; o >>= 1) v = fmax(v, __shfl_xor_sync(0xffffffffu, v, o));
  return v;
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
  double* W = sh;                                       // nc x ell, column c at W + c*ell
  double* v = W + static_cast<size_t>(cols_per) * ell;  // Householder vector (ell)
  __shared__ unsigned char active[QR_MAX_COLS];
  __shared__ Arg s_warg[QR_WARPS];
  __shared__ double s_wsec[QR_WARPS];
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
  __syncthreads();

  for (int j = 0; j < k; ++j) {
    const int par = j & 1;
    // ---- (A) residual norms of the local active columns; local best and runner-up ----
    Arg wb{-1.0, -1, -1};
    double ws = -1.0;
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
      if (better(s, gi, wb.v, wb.i)) {
        ws = fmax(ws, wb.v);
        wb = Arg{s, gi, c};
      } else {
        ws = fmax(ws, s);
      }
    }
    if (lane == 0) {
      s_warg[warp] = wb;
      s_wsec[warp] = ws;
    }
    __syncthreads();
    if (warp == 0) {
      Arg a = lane < QR_WARPS ? s_warg[lane] : Arg{-1.0, -1, -1};
      const Arg best = warp_argmax(a);
      double sec = lane < QR_WARPS ? s_wsec[lane] : -1.0;
      if (lane < QR_WARPS && a.i != best.i) sec = fmax(sec, a.v);
      sec = warp_max(sec);
      if (lane == 0) {
        QrCand cd;
        cd.best = best.v;
        cd.second = sec;
        cd.idx = best.i;
        cd.pad = 0;
        cand[par * NB + blk] = cd;
        s_bloc = best.i >= 0 ? best.b : -1;
      }
    }
    __syncthreads();
    if (s_bloc >= 0)
      for (int i = j + tid; i < ell; i += QR_THREADS)
        candcol[(static_cast<size_t>(par) * NB + blk) * ell + i] = W[s_bloc * ell + i];
    grid_sync_count(&work->count, static_cast<unsigned int>(j + 1) * NB);

    // ---- (B) global pivot: every CTA reads all candidates in parallel ----
    {
      Arg a{-1.0, -1, -1};
      double sec = -1.0;
      for (int b = tid; b < NB; b += QR_THREADS) {
        const long long ci = __ldcg(&cand[par * NB + b].idx);
        const double cb = __ldcg(&cand[par * NB + b].best);
        const double cs = __ldcg(&cand[par * NB + b].second);
        sec = fmax(sec, cs);
        if (better(cb, ci, a.v, a.i)) {
          if (a.i >= 0) sec = fmax(sec, a.v);
          a = Arg{cb, ci, b};
        } else if (ci >= 0) {
          sec = fmax(sec, cb);
        }
      }
      const Arg wbest = warp_argmax(a);
      if (a.i >= 0 && a.i != wbest.i) sec = fmax(sec, a.v);
      sec = warp_max(sec);
      if (lane == 0) {
        s_warg[warp] = wbest;
        s_wsec[warp] = sec;
      }
      __syncthreads();
      if (warp == 0) {
        Arg x = lane < QR_WARPS ? s_warg[lane] : Arg{-1.0, -1, -1};
        const Arg g = warp_argmax(x);
        double s2 = lane < QR_WARPS ? s_wsec[lane] : -1.0;
        if (lane < QR_WARPS && x.i >= 0 && x.i != g.i) s2 = fmax(s2, x.v);
        s2 = warp_max(s2);
        if (lane == 0) {
          s_gbest = g.v;
          s_gsecond = s2;
          s_gidx = g.i;
          s_gblk = g.b;
        }
      }
      __syncthreads();
    }
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
    // ---- apply H = I - tau v v^T to the local active columns; retire the pivot column ----
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
    if (blk == 0 && tid == 0) {  // pivot sequence (perm is assembled afterwards) and the gap
      inv[j] = gidx;              // `inv` holds the pivot sequence piv[0..k)
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

// perm from the pivot sequence with LAPACK swap semantics: step j exchanges positions j and
// pos(piv[j]).  One CTA; permutation and its inverse in shared memory (int32) when they fit.
__global__ void qrcp_perm_kernel(const int64_t* __restrict__ piv, int k, long long n, int64_t* __restrict__ perm,
                                 int64_t* __restrict__ gpos, bool use_smem) {
  extern __shared__ int sp[];
  __shared__ long long s_piv[512];
  for (int j = threadIdx.x; j < k && j < 512; j += blockDim.x) s_piv[j] = piv[j];
  if (use_smem) {
    int* P = sp;
    int* pos = sp + n;
    for (long long i = threadIdx.x; i < n; i += blockDim.x) P[i] = static_cast<int>(i), pos[i] = static_cast<int>(i);
    __syncthreads();
    if (threadIdx.x == 0) {
      for (int j = 0; j < k; ++j) {
        const long long g = j < 512 ? s_piv[j] : piv[j];
        if (g < 0) break;
        const int p = pos[g], o = P[j];
        P[j] = static_cast<int>(g);
        P[p] = o;
        pos[g] = j;
        pos[o] = p;
      }
    }
    __syncthreads();
    for (long long i = threadIdx.x; i < n; i += blockDim.x) perm[i] = P[i];
  } else {
    for (long long i = threadIdx.x; i < n; i += blockDim.x) perm[i] = i, gpos[i] = i;
    __syncthreads();
    if (threadIdx.x == 0) {
      for (int j = 0; j < k; ++j) {
        const long long g = j < 512 ? s_piv[j] : piv[j];
        if (g < 0) break;
        const long long p = gpos[g], o = perm[j];
        perm[j] = g;
        perm[p] = o;
        gpos[g] = j;
        gpos[o] = p;
      }
    }
  }
}

size_t qrcp_workspace_bytes(int ell, long long n) {
  const int NB = 1024;  // upper bound on blocks
  return sizeof(QrWork) + 2 * NB * sizeof(QrCand) + 2 * static_cast<size_t>(NB) * ell * 8 + 2 * n * 8 + 256;
}

cudaError_t qrcp_truncated(cudaStream_t st, const double* B, int ldb, int ell, long long n, int k, void* work,
                           int64_t* perm, double* Rho, int ldr, double* gaps, int* info, int num_sms) {
  constexpr size_t kSmemMax = 200 * 1024;
  int NB = static_cast<int>(std::max<long long>(1, std::min<long long>(num_sms, (n + QR_COLS_TARGET - 1) / QR_COLS_TARGET)));
  int cols_per = static_cast<int>((n + NB - 1) / NB);
  auto smem_of = [&](int cp) { return (static_cast<size_t>(cp) * ell + ell) * 8; };
  while ((smem_of(cols_per) > kSmemMax || cols_per > QR_MAX_COLS) && NB < num_sms) {
    ++NB;
    cols_per = static_cast<int>((n + NB - 1) / NB);
  }
  if (smem_of(cols_per) > kSmemMax || cols_per > QR_MAX_COLS) return cudaErrorInvalidValue;
  const size_t smem = smem_of(cols_per);
  static bool attr = false;
  if (!attr) {
    cudaError_t e = cudaFuncSetAttribute(qrcp_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                         static_cast<int>(kSmemMax));
    if (e != cudaSuccess) return e;
    attr = true;
  }
  cudaError_t e = cudaMemsetAsync(work, 0, sizeof(QrWork), st);
  if (e != cudaSuccess) return e;
  QrWork* w = static_cast<QrWork*>(work);
  void* args[] = {(void*)&B, (void*)&ldb, (void*)&ell, (void*)&n, (void*)&k, (void*)&w, (void*)&NB, (void*)&cols_per,
                  (void*)&perm, (void*)&Rho, (void*)&ldr, (void*)&gaps, (void*)&info};
  count_launch();
  e = cudaLaunchCooperativeKernel(reinterpret_cast<void*>(qrcp_kernel), dim3(NB), dim3(QR_THREADS), args, smem, st);
  if (e != cudaSuccess) return e;
  // assemble perm from the pivot sequence (stored by the kernel where `inv` lives)
  QrCand* cand = reinterpret_cast<QrCand*>(w + 1);
  double* candcol = reinterpret_cast<double*>(cand + 2 * NB);
  int64_t* piv = reinterpret_cast<int64_t*>(candcol + 2 * static_cast<size_t>(NB) * ell);
  int64_t* gpos = piv + n;
  const size_t psmem = static_cast<size_t>(n) * 8;
  const bool use_smem = psmem <= kSmemMax;
  static bool pattr = false;
  if (!pattr) {
    e = cudaFuncSetAttribute(qrcp_perm_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, static_cast<int>(kSmemMax));
    if (e != cudaSuccess) return e;
    pattr = true;
  }
  qrcp_perm_kernel<<<1, 1024, use_smem ? psmem : 0, st>>>(piv, k, n, perm, gpos, use_smem);
  count_launch();
  return cudaGetLastError();
}

}  // namespace rs
