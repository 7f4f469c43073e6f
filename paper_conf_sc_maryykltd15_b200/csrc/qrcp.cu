// Truncated QRCP of the small sample B (l x n): Step 2 of random sampling (Fig. 2(b)
// line 6, "truncated QP3 on a GPU").  k sequential Householder steps, each choosing the
// remaining column with the largest residual 2-norm (Sec. 2).
//
// B200 design: one persistent cooperative kernel.  The columns of B are distributed over NB CTAs
// (<= 256 columns each) and stay resident in shared memory for all k steps.  Four lanes own one
// column (rows i = q mod 4), so residual norms and reflector dot products are short independent
// chains plus two shuffles.  Per step each CTA (A) recomputes the residual norms of its active
// columns (reading R5: exact recomputation instead of downdating, P:L189-192/L212-217 -- every
// column is touched by the trailing update anyway) and publishes its best candidate column,
// (grid barrier), (B) every CTA reads all candidates in parallel, picks the same global pivot
// (largest norm, ties -> lowest original index), forms the dlarfg reflector from the published
// column and applies it to its own columns.  Pivots and R̂ rows are final as soon as they are
// produced; perm (LAPACK swap order) is assembled from the pivot sequence afterwards.
#include <algorithm>
#include <cstdio>
#include <cstdlib>

#include "common.cuh"
#include "internal.h"

namespace rs {

constexpr int QR_THREADS = 1024;
constexpr int QR_WARPS = QR_THREADS / 32;
constexpr int QR_LANES = 4;                            // lanes per column
constexpr int QR_MAX_COLS = QR_THREADS / QR_LANES;     // 256 columns per CTA
constexpr size_t QR_SMEM_MAX = 200 * 1024;

struct QrCand {
  double best;    // squared residual norm of the CTA's best active column (-1 if none)
  double second;  // second best squared norm in the CTA (-1 if none)
  long long idx;  // original column index of the best (-1 if none)
  long long pad;
};

struct QrWork {
  unsigned int count;  // monotone grid-barrier counter
  unsigned int pad[3];
  // followed by: QrCand cand[2][NB]; double candcol[2][NB][ell]; int64 piv[n]; int64 pos[n]
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

// (value, index, owner) argmax with ties to the lowest index
struct Arg {
  double v;
  long long i;
  int b;
};
RS_DEVINL Arg shfl_arg(const Arg& a, int o) {
  return Arg{__shfl_xor_sync(0xffffffffu, a.v, o), __shfl_xor_sync(0xffffffffu, a.i, o),
             __shfl_xor_sync(0xffffffffu, a.b, o)};
}
// warp-wide best and runner-up (value only) of per-lane (best a, runner-up sec), on REDUX.SYNC:
// squared norms are >= 0, and non-negative doubles order like their bit patterns, so the argmax
// is a 64-bit unsigned max taken as (hi word, then lo word among the hi winners), then the lowest
// original index among the lanes holding that key (ties -> lowest index, as `better`).  Keys are
// bits + 1 so a valid 0.0 beats "none" (i < 0 / sec < 0, key 0).  7 warp-wide ops instead of 5
// dependent levels of 7 shuffles plus divergent compares.
RS_DEVINL unsigned long long top2_key(bool has, double v) {
  return has ? static_cast<unsigned long long>(__double_as_longlong(v + 0.0)) + 1ull : 0ull;  // -0 -> +0
}
RS_DEVINL unsigned long long warp_max_u64(unsigned long long k) {
  const unsigned hi = static_cast<unsigned>(k >> 32), lo = static_cast<unsigned>(k);
  const unsigned mhi = __reduce_max_sync(0xffffffffu, hi);
  const unsigned mlo = __reduce_max_sync(0xffffffffu, hi == mhi ? lo : 0u);
  return (static_cast<unsigned long long>(mhi) << 32) | mlo;
}
RS_DEVINL void warp_top2(Arg& a, double& sec) {
  const bool has = a.i >= 0;
  const unsigned long long key = top2_key(has, a.v);
  const unsigned long long mk = warp_max_u64(key);
  const bool top = has && key == mk;
  const unsigned mi = __reduce_min_sync(0xffffffffu, top ? static_cast<unsigned>(a.i) : 0xffffffffu);
  const unsigned win = __ballot_sync(0xffffffffu, top && static_cast<unsigned>(a.i) == mi);
  const bool me = (win >> (threadIdx.x & 31)) & 1u;
  // runner-up: every lane's own runner-up and every non-winning lane's best
  const unsigned long long k2 = max(top2_key(sec >= 0.0, sec), me ? 0ull : key);
  const unsigned long long m2 = warp_max_u64(k2);
  sec = m2 ? __longlong_as_double(static_cast<long long>(m2 - 1ull)) : -1.0;
  if (win) {
    const int src = __ffs(win) - 1;
    a.b = __shfl_sync(0xffffffffu, a.b, src);
    a.v = __longlong_as_double(static_cast<long long>(mk - 1ull));
    a.i = static_cast<long long>(mi);
  } else {
    a = Arg{-1.0, -1, -1};
  }
}

__global__ void __launch_bounds__(QR_THREADS, 1)
    qrcp_kernel(const double* __restrict__ B, int ldb, int ell, long long n, int k, QrWork* work, int NB,
                int cols_per, int ldw, int64_t* __restrict__ Rho_piv, double* __restrict__ Rho, int ldr,
                double* __restrict__ gaps, int* info, long long* tbuf) {
  extern __shared__ double sh[];
  const int blk = blockIdx.x;
  const int tid = threadIdx.x, warp = tid >> 5, lane = tid & 31;
  const long long c0 = static_cast<long long>(blk) * cols_per;
  const long long c1 = (c0 + cols_per < n) ? c0 + cols_per : n;
  const int nc = c1 > c0 ? static_cast<int>(c1 - c0) : 0;
  double* W = sh;                                       // column c at W + c*ldw (ldw = 4 mod 16)
  double* v = W + static_cast<size_t>(cols_per) * ldw;  // Householder vector (ell)
  __shared__ Arg s_warg[QR_WARPS];
  __shared__ double s_wsec[QR_WARPS];
  __shared__ double s_tau, s_beta, s_gbest, s_gsecond, s_den;
  __shared__ long long s_gidx;
  __shared__ int s_gblk, s_bloc;

  QrCand* cand = reinterpret_cast<QrCand*>(work + 1);
  double* candcol = reinterpret_cast<double*>(cand + 2 * NB);
  int64_t* piv = Rho_piv;

  for (int idx = tid; idx < nc * ell; idx += QR_THREADS) {
    const int c = idx / ell, i = idx % ell;
    W[c * ldw + i] = B[i + (c0 + c) * static_cast<long long>(ldb)];
  }
  const int mc = tid / QR_LANES, q = tid % QR_LANES;  // my column and row phase
  bool active = mc < nc;
  double* col = W + mc * ldw;
  __syncthreads();

#define QT(ph) \
  if (tbuf && blk == 0 && tid == 0) tbuf[j * 8 + (ph)] = clock64();
  for (int j = 0; j < k; ++j) {
    const int par = j & 1;
    QT(0)
    // ---- (A) residual norms of the local active columns; CTA best and runner-up ----
    double s = 0.0;
    if (active)
      for (int i = j + q; i < ell; i += QR_LANES) s = fma(col[i], col[i], s);
    s += __shfl_xor_sync(0xffffffffu, s, 1);
    s += __shfl_xor_sync(0xffffffffu, s, 2);
    {
      Arg a = (active && q == 0) ? Arg{s, c0 + mc, mc} : Arg{-1.0, -1, -1};
      double sec = -1.0;
      warp_top2(a, sec);
      if (lane == 0) {
        s_warg[warp] = a;
        s_wsec[warp] = sec;
      }
      __syncthreads();
      if (warp == 0) {
        Arg x = s_warg[lane];
        double xs = s_wsec[lane];
        warp_top2(x, xs);
        if (lane == 0) {
          QrCand cd;
          cd.best = x.v;
          cd.second = xs;
          cd.idx = x.i;
          cd.pad = 0;
          cand[par * NB + blk] = cd;
          s_bloc = x.i >= 0 ? x.b : -1;
        }
      }
      __syncthreads();
    }
    QT(1)
    if (s_bloc >= 0)
      for (int i = j + tid; i < ell; i += QR_THREADS)
        candcol[(static_cast<size_t>(par) * NB + blk) * ell + i] = W[s_bloc * ldw + i];
    grid_sync_count(&work->count, static_cast<unsigned int>(j + 1) * NB);
    QT(2)

    // ---- (B) global pivot: every CTA reads all candidates in parallel ----
    if (warp == 0) {
      Arg a{-1.0, -1, -1};
      double sec = -1.0;
      for (int b = lane; b < NB; b += 32) {
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
      warp_top2(a, sec);
      if (lane == 0) {
        s_gbest = a.v;
        s_gsecond = sec;
        s_gidx = a.i;
        s_gblk = a.b;
      }
    }
    __syncthreads();
    QT(3)
    const int gblk = s_gblk;
    const long long gidx = s_gidx;
    const int len = ell - j;
    for (int i = tid; i < len; i += QR_THREADS)
      v[i] = __ldcg(&candcol[(static_cast<size_t>(par) * NB + (gblk < 0 ? 0 : gblk)) * ell + j + i]);
    __syncthreads();
    QT(4)
    if (warp == 0) {  // dlarfg on x = v[0..len)
      double xs = 0.0;
      for (int i = 1 + lane; i < len; i += 32) xs = fma(v[i], v[i], xs);
#pragma unroll
      for (int o = 16; o > 0; o >>= 1) xs += __shfl_xor_sync(0xffffffffu, xs, o);
      if (lane == 0) {
        const double alpha = v[0];
        double tau = 0.0, beta = alpha;
        if (gblk >= 0 && xs > 0.0) {
          const double h = sqrt(fma(alpha, alpha, xs));
          beta = alpha >= 0.0 ? -h : h;
          tau = (beta - alpha) / beta;
        }
        s_tau = tau;
        s_beta = beta;
        s_den = alpha - beta;
        if (gblk < 0 || !(s_gbest > 0.0)) {
          if (info && blk == 0) atomicCAS(info, 0, 6 /* RS_ERR_RANK_DEFICIENT */), atomicCAS(info + 1, 0, j + 1);
        }
      }
    }
    __syncthreads();
    const double tau = s_tau, beta = s_beta;
    if (tau != 0.0)
      for (int i = 1 + tid; i < len; i += QR_THREADS) v[i] = v[i] / s_den;
    __syncthreads();
    QT(5)
    // ---- apply H = I - tau v v^T to the local active columns; retire the pivot column ----
    {
      const long long gi = c0 + mc;
      const bool is_piv = active && gi == gidx;
      const bool upd = active && !is_piv && tau != 0.0;
      double w = 0.0;
      if (upd)
        for (int i = j + q; i < ell; i += QR_LANES) w = fma(i == j ? 1.0 : v[i - j], col[i], w);
      w += __shfl_xor_sync(0xffffffffu, w, 1);  // all lanes participate; groups of 4 are aligned
      w += __shfl_xor_sync(0xffffffffu, w, 2);
      if (upd) {
        const double tw = tau * w;
        for (int i = j + q; i < ell; i += QR_LANES) col[i] = fma(-tw, i == j ? 1.0 : v[i - j], col[i]);
      }
      if (is_piv) {
        for (int i = q; i < k; i += QR_LANES) {
          const double val = (i < j) ? col[i] : (i == j ? beta : 0.0);
          Rho[i + gi * static_cast<long long>(ldr)] = val;
        }
        active = false;
      }
    }
    QT(6)
    if (blk == 0 && tid == 0) {  // pivot sequence and the relative gap of this step
      piv[j] = gidx;
      const double nb = sqrt(fmax(s_gbest, 0.0)), ns = sqrt(fmax(s_gsecond, 0.0));
      if (gaps) gaps[j] = nb > 0.0 ? (nb - ns) / nb : 0.0;
    }
    __syncthreads();
  }
#undef QT
  // rows 0..k-1 of the never-pivoted columns
  if (active)
    for (int i = q; i < k; i += QR_LANES) Rho[i + (c0 + mc) * static_cast<long long>(ldr)] = col[i];
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

// ------------------------------------------------------------------------------------------
// Register-resident variant for l <= 128 (the paper-shaped configs): each column of B lives in
// the registers of 4 lanes (rows q + 4t, t < 32) for all k steps, so residual norms, reflector
// dot products and updates never touch shared memory; the next step's residual norm is fused
// into the update.  Every warp scans the candidates itself (no CTA broadcast), loads its rows
// of the winning column straight from L2 and forms the dlarfg reflector redundantly.
// ------------------------------------------------------------------------------------------
constexpr int QRR_THREADS = 512;
constexpr int QRR_COLS = QRR_THREADS / 4;  // 128 columns per CTA
constexpr int QRR_ROWS = 32;               // rows per lane: l <= 128

__global__ void __launch_bounds__(QRR_THREADS, 1)
    qrcp_reg_kernel(const double* __restrict__ B, int ldb, int ell, long long n, int k, QrWork* work, int NB,
                    int64_t* __restrict__ piv, double* __restrict__ Rho, int ldr, double* __restrict__ gaps,
                    int* info, long long* tbuf) {
  const int blk = blockIdx.x;
  const int tid = threadIdx.x, warp = tid >> 5, lane = tid & 31;
  const int mc = tid >> 2, q = tid & 3;
  const long long c0 = static_cast<long long>(blk) * QRR_COLS;
  const long long gi = c0 + mc;  // my column (original index)
  bool active = gi < n;
  __shared__ Arg s_warg[QRR_THREADS / 32];
  __shared__ double s_wsec[QRR_THREADS / 32];
  __shared__ double s_v[QRR_THREADS / 32][4 * QRR_ROWS];
  // every CTA's candidate and its column (rows j..ell-1), staged after the barrier in ONE round
  // trip: the pivot column no longer waits for the argmax
  extern __shared__ double s_dyn[];
  QrCand* s_cand = reinterpret_cast<QrCand*>(s_dyn);
  double* s_col = s_dyn + 4 * NB;  // s_col[b * ell + (i - j)]
  QrCand* cand = reinterpret_cast<QrCand*>(work + 1);
  double* candcol = reinterpret_cast<double*>(cand + 2 * NB);

  double x[QRR_ROWS];
#pragma unroll
  for (int t = 0; t < QRR_ROWS; ++t) {
    const int i = q + 4 * t;
    x[t] = (active && i < ell) ? B[i + gi * static_cast<long long>(ldb)] : 0.0;
  }
  // residual norm^2 over rows >= 0
  double s = 0.0;
#pragma unroll
  for (int t = 0; t < QRR_ROWS; ++t) s = fma(x[t], x[t], s);

#define QT(ph) \
  if (tbuf && blk == 0 && tid == 0) tbuf[j * 8 + (ph)] = clock64();
  for (int j = 0; j < k; ++j) {
    const int par = j & 1;
    QT(0)
    // ---- (A) CTA best / runner-up of the residual norms (s holds rows >= j) ----
    double sc = s;
    sc += __shfl_xor_sync(0xffffffffu, sc, 1);
    sc += __shfl_xor_sync(0xffffffffu, sc, 2);
    {
      Arg a = (active && q == 0) ? Arg{sc, gi, mc} : Arg{-1.0, -1, -1};
      double sec = -1.0;
      warp_top2(a, sec);
      if (lane == 0) {
        s_warg[warp] = a;
        s_wsec[warp] = sec;
      }
      __syncthreads();
      if (warp == 0) {
        Arg xx = lane < QRR_THREADS / 32 ? s_warg[lane] : Arg{-1.0, -1, -1};
        double xs = lane < QRR_THREADS / 32 ? s_wsec[lane] : -1.0;
        warp_top2(xx, xs);
        if (lane == 0) {
          QrCand cd;
          cd.best = xx.v;
          cd.second = xs;
          cd.idx = xx.i;
          cd.pad = 0;
          cand[par * NB + blk] = cd;
          s_warg[0] = xx;  // this CTA's winner (read by its owner lanes below)
        }
      }
      __syncthreads();
    }
    // the owner of this CTA's best column publishes rows j..ell-1
    if (active && s_warg[0].i == gi) {
      double* dst = candcol + (static_cast<size_t>(par) * NB + blk) * ell;
#pragma unroll
      for (int t = 0; t < QRR_ROWS; ++t) {
        const int i = q + 4 * t;
        if (i >= j && i < ell) dst[i] = x[t];
      }
    }
    QT(1)
    grid_sync_count(&work->count, static_cast<unsigned int>(j + 1) * NB);
    QT(2)

    // ---- (B) stage all candidates + columns, then every warp scans them in shared memory ----
    // one flat copy of the NB published columns (rows < j are stale and never read), issued as
    // batches of independent loads so the step pays about one L2 round trip, not one per element
    {
      constexpr int U = 12;
      const double* cc = candcol + static_cast<size_t>(par) * NB * ell;
      const int tot = NB * ell;
      QrCand cd;
      const bool mine = tid < NB;
      if (mine) {
        cd.best = __ldcg(&cand[par * NB + tid].best);
        cd.second = __ldcg(&cand[par * NB + tid].second);
        cd.idx = __ldcg(&cand[par * NB + tid].idx);
        cd.pad = 0;
      }
      for (int e0 = 0; e0 < tot; e0 += U * QRR_THREADS) {
        double v[U];
#pragma unroll
        for (int u = 0; u < U; ++u) {
          const int e = e0 + u * QRR_THREADS + tid;
          v[u] = e < tot ? __ldcg(cc + e) : 0.0;
        }
#pragma unroll
        for (int u = 0; u < U; ++u) {
          const int e = e0 + u * QRR_THREADS + tid;
          if (e < tot) s_col[e] = v[u];
        }
      }
      if (mine) s_cand[tid] = cd;
      for (int b = tid + QRR_THREADS; b < NB; b += QRR_THREADS) {  // NB <= 148 < QRR_THREADS: unused
        cd.best = __ldcg(&cand[par * NB + b].best);
        cd.second = __ldcg(&cand[par * NB + b].second);
        cd.idx = __ldcg(&cand[par * NB + b].idx);
        cd.pad = 0;
        s_cand[b] = cd;
      }
    }
    __syncthreads();
    Arg g{-1.0, -1, -1};
    double g2 = -1.0;
    for (int b = lane; b < NB; b += 32) {
      const long long ci = s_cand[b].idx;
      const double cb = s_cand[b].best;
      const double cs = s_cand[b].second;
      g2 = fmax(g2, cs);
      if (better(cb, ci, g.v, g.i)) {
        if (g.i >= 0) g2 = fmax(g2, g.v);
        g = Arg{cb, ci, b};
      } else if (ci >= 0) {
        g2 = fmax(g2, cb);
      }
    }
    warp_top2(g, g2);
    QT(3)
    const long long gidx = g.i;
    const int gblk = g.b < 0 ? 0 : g.b;
    // this warp's copy of the pivot column (rows >= j) in shared memory; alpha and
    // xs = ||x_p[j+1:]||^2 by a warp reduction, reflector formed redundantly per warp
    const double* src = s_col + gblk * ell;  // src[i] = row i of the pivot column, i >= j
    double* vw = s_v[warp];
    double pv[QRR_ROWS / 8];
    double xs = 0.0, alpha = 0.0;
#pragma unroll
    for (int u = 0; u < QRR_ROWS / 8; ++u) {
      const int i = lane + 32 * u;
      pv[u] = (i >= j && i < ell) ? src[i] : 0.0;
      if (i > j) xs = fma(pv[u], pv[u], xs);
      if (i == j) alpha = pv[u];
    }
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) {
      xs += __shfl_xor_sync(0xffffffffu, xs, o);
      alpha += __shfl_xor_sync(0xffffffffu, alpha, o);  // only lane j%32 holds a nonzero term
    }
    double tau = 0.0, beta = alpha;
    if (g.i >= 0 && xs > 0.0) {
      const double h = sqrt(fma(alpha, alpha, xs));
      beta = alpha >= 0.0 ? -h : h;
      tau = (beta - alpha) / beta;
    }
    // v = x / (alpha - beta) as x * (1 / (alpha - beta)): one division on the step's critical path
    // instead of QRR_ROWS / 8 (differs from the quotient by <= 1 ulp per entry)
    const double rden = tau != 0.0 ? 1.0 / (alpha - beta) : 0.0;
#pragma unroll
    for (int u = 0; u < QRR_ROWS / 8; ++u) {
      const int i = lane + 32 * u;
      vw[i] = (i < j) ? 0.0 : (i == j ? 1.0 : pv[u] * rden);
    }
    __syncwarp();
    QT(4)
    if (blk == 0 && tid == 0) {
      if (g.i < 0 || !(g.v > 0.0)) {
        if (info) atomicCAS(info, 0, 6 /* RS_ERR_RANK_DEFICIENT */), atomicCAS(info + 1, 0, j + 1);
      }
      piv[j] = gidx;
      const double nb = sqrt(fmax(g.v, 0.0)), ns = sqrt(fmax(g2, 0.0));
      if (gaps) gaps[j] = nb > 0.0 ? (nb - ns) / nb : 0.0;
    }
    // ---- apply H = I - tau v v^T; retire the pivot column; fuse the next residual norm ----
    const bool is_piv = active && gi == gidx;
    const bool upd = active && !is_piv && tau != 0.0;
    double w = 0.0;
    if (upd) {  // four partial sums: a 32-term FMA chain is latency-bound
      double w4[4] = {0.0, 0.0, 0.0, 0.0};
#pragma unroll
      for (int t = 0; t < QRR_ROWS; ++t) w4[t & 3] = fma(vw[q + 4 * t], x[t], w4[t & 3]);  // v = 0 outside rows >= j
      w = (w4[0] + w4[1]) + (w4[2] + w4[3]);
    }
    w += __shfl_xor_sync(0xffffffffu, w, 1);
    w += __shfl_xor_sync(0xffffffffu, w, 2);
    s = 0.0;
    {
      double s4[4] = {0.0, 0.0, 0.0, 0.0};
      if (upd) {
        const double tw = tau * w;
#pragma unroll
        for (int t = 0; t < QRR_ROWS; ++t) {
          x[t] = fma(-tw, vw[q + 4 * t], x[t]);
          const int i = q + 4 * t;
          if (i > j) s4[t & 3] = fma(x[t], x[t], s4[t & 3]);
        }
      } else if (active && !is_piv) {
#pragma unroll
        for (int t = 0; t < QRR_ROWS; ++t) {
          const int i = q + 4 * t;
          if (i > j) s4[t & 3] = fma(x[t], x[t], s4[t & 3]);
        }
      }
      s = (s4[0] + s4[1]) + (s4[2] + s4[3]);
    }
    if (is_piv) {
#pragma unroll
      for (int t = 0; t < QRR_ROWS; ++t) {
        const int i = q + 4 * t;
        if (i < k) Rho[i + gi * static_cast<long long>(ldr)] = (i < j) ? x[t] : (i == j ? beta : 0.0);
      }
      active = false;
    }
    QT(5)
    __syncthreads();  // s_warg reuse and candidate buffers of parity `par`
    QT(6)
  }
#undef QT
  if (active) {
#pragma unroll
    for (int t = 0; t < QRR_ROWS; ++t) {
      const int i = q + 4 * t;
      if (i < k) Rho[i + gi * static_cast<long long>(ldr)] = x[t];
    }
  }
}

// ------------------------------------------------------------------------------------------
// Flag-synchronised variant of the register kernel (the default for l <= 128, n <= 148 x COLS).
// No grid barrier and no bulk staging: per step each CTA publishes ONE record -- its best column's
// squared norm, the runner-up, the index, and the dlarfg reflector of that column (beta, tau,
// 1 / (alpha - beta), formed by the column's owner lanes BEFORE the exchange, off the critical
// path of every other CTA) -- written with a release store of the sequence number j + 1 last.
// Every CTA acquires the NB records (one L2 round trip after the last publication), picks the
// same global pivot (largest norm, ties -> lowest original index), and each warp reads only the
// winning column and its reflector (a second, small round trip).  LPC lanes own one column (rows
// q + LPC t): LPC = 8 halves the FP64 FMA work per SM of the trailing update when n <= 148 x 64.
// Records and columns are double-buffered by step parity: a CTA can only overwrite slot `par`
// at step j + 2 after every CTA has published step j + 1, i.e. finished reading step j.
// ------------------------------------------------------------------------------------------
struct QrRec {
  double best;             // squared residual norm of the CTA's best active column (-1 if none)
  double second;           // runner-up in the CTA (-1 if none)
  long long idx;           // original column index (-1 if none)
  unsigned long long seq;  // j + 1 once the record of step j (and its column) is published
};
constexpr int QRF_CST = 132;  // published column stride: rows 0..127, then beta, tau, 1/(alpha - beta)
constexpr int QRF_MAXNB = 148;

RS_DEVINL unsigned long long ld_acquire_u64(const unsigned long long* p) {
  unsigned long long v;
  asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}
RS_DEVINL void st_release_u64(unsigned long long* p, unsigned long long v) {
  asm volatile("st.release.gpu.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}

template <int LPC>
__global__ void __launch_bounds__(QRR_THREADS, 1)
    qrcp_flag_kernel(const double* __restrict__ B, int ldb, int ell, long long n, int k, QrRec* rec,
                     double* candcol, int NB, int64_t* __restrict__ piv, double* __restrict__ Rho, int ldr,
                     double* __restrict__ gaps, int* info, long long* tbuf, unsigned int* counter) {
  constexpr int COLS = QRR_THREADS / LPC;
  constexpr int RPL = 128 / LPC;  // rows per lane (l <= 128)
  constexpr int NW = QRR_THREADS / 32;
  const int blk = blockIdx.x;
  const int tid = threadIdx.x, warp = tid >> 5, lane = tid & 31;
  const int mc = tid / LPC, q = tid % LPC;
  const unsigned gmask = ((1u << LPC) - 1u) << (lane & ~(LPC - 1));  // my column's lanes
  const long long gi = static_cast<long long>(blk) * COLS + mc;
  bool active = gi < n;
  __shared__ Arg s_warg[NW];
  __shared__ double s_wsec[NW];
  __shared__ QrRec s_rec[QRF_MAXNB];
  __shared__ double s_v[NW][128];

  double x[RPL];
#pragma unroll
  for (int t = 0; t < RPL; ++t) {
    const int i = q + LPC * t;
    x[t] = (active && i < ell) ? B[i + gi * static_cast<long long>(ldb)] : 0.0;
  }
  double s = 0.0;  // residual norm^2 (my rows) over rows >= j
#pragma unroll
  for (int t = 0; t < RPL; ++t) s = fma(x[t], x[t], s);

#define QT(ph) \
  if (tbuf && blk == 0 && tid == 0) tbuf[j * 8 + (ph)] = clock64();
  for (int j = 0; j < k; ++j) {
    const int par = j & 1;
    QT(0)
    // ---- (A) CTA best / runner-up, the winner's owner lanes publish column + reflector ----
    double sc = s;
#pragma unroll
    for (int o = 1; o < LPC; o <<= 1) sc += __shfl_xor_sync(0xffffffffu, sc, o);
    {
      Arg a = (active && q == 0) ? Arg{sc, gi, mc} : Arg{-1.0, -1, -1};
      double sec = -1.0;
      warp_top2(a, sec);
      if (lane == 0) {
        s_warg[warp] = a;
        s_wsec[warp] = sec;
      }
    }
    __syncthreads();
    if (warp == 0) {
      Arg xx = lane < NW ? s_warg[lane] : Arg{-1.0, -1, -1};
      double xs = lane < NW ? s_wsec[lane] : -1.0;
      warp_top2(xx, xs);
      __syncwarp();
      if (lane == 0) {
        s_warg[0] = xx;
        s_wsec[0] = xs;
      }
    }
    __syncthreads();
    QT(1)
    {
      const Arg cw = s_warg[0];
      QrRec* myrec = rec + par * NB + blk;
      if (cw.i < 0) {  // nothing left in this CTA: publish an empty record
        if (tid == 0) {
          myrec->best = -1.0;
          myrec->second = s_wsec[0];
          myrec->idx = -1;
          if (!counter) st_release_u64(&myrec->seq, static_cast<unsigned long long>(j + 1));
        }
      } else if (active && cw.i == gi) {
        double* dst = candcol + (static_cast<size_t>(par) * NB + blk) * QRF_CST;
        double ap = 0.0, xp = 0.0;
#pragma unroll
        for (int t = 0; t < RPL; ++t) {
          const int i = q + LPC * t;
          if (i >= j && i < ell) dst[i] = x[t];
          if (i == j) ap = x[t];
          if (i > j) xp = fma(x[t], x[t], xp);
        }
#pragma unroll
        for (int o = 1; o < LPC; o <<= 1) {
          ap += __shfl_xor_sync(gmask, ap, o);  // one nonzero term
          xp += __shfl_xor_sync(gmask, xp, o);
        }
        __syncwarp(gmask);  // the group's column stores are ordered before the release below
        if (q == 0) {
          double beta = ap, tau = 0.0, rden = 0.0;
          if (xp > 0.0) {  // dlarfg: H = I when the part below the diagonal is zero
            const double h = sqrt(fma(ap, ap, xp));
            beta = ap >= 0.0 ? -h : h;
            tau = (beta - ap) / beta;
            rden = 1.0 / (ap - beta);
          }
          dst[128] = beta;
          dst[129] = tau;
          dst[130] = rden;
          myrec->best = cw.v;
          myrec->second = s_wsec[0];
          myrec->idx = cw.i;
          if (!counter) st_release_u64(&myrec->seq, static_cast<unsigned long long>(j + 1));
        }
      }
    }
    // ---- (B) acquire every CTA's record of step j, pick the global pivot ----
    // counter != NULL: one grid barrier (one poller per CTA) instead of NB pollers per CTA
    if (counter) grid_sync_count(counter, static_cast<unsigned int>(j + 1) * NB);
    if (tid < NB) {
      const QrRec* r = rec + par * NB + tid;
      if (!counter)
        while (ld_acquire_u64(&r->seq) < static_cast<unsigned long long>(j + 1)) {
        }
      QrRec cd;
      cd.best = __ldcg(&r->best);
      cd.second = __ldcg(&r->second);
      cd.idx = __ldcg(&r->idx);
      cd.seq = 0;
      s_rec[tid] = cd;
    }
    __syncthreads();
    QT(2)
    Arg g{-1.0, -1, -1};
    double g2 = -1.0;
    for (int b = lane; b < NB; b += 32) {
      const long long ci = s_rec[b].idx;
      const double cb = s_rec[b].best;
      g2 = fmax(g2, s_rec[b].second);
      if (better(cb, ci, g.v, g.i)) {
        if (g.i >= 0) g2 = fmax(g2, g.v);
        g = Arg{cb, ci, b};
      } else if (ci >= 0) {
        g2 = fmax(g2, cb);
      }
    }
    warp_top2(g, g2);
    QT(3)
    // ---- the winner's column (rows >= j) and reflector, straight from L2, per warp ----
    const double* src = candcol + (static_cast<size_t>(par) * NB + (g.b < 0 ? 0 : g.b)) * QRF_CST;
    double pv[4];
#pragma unroll
    for (int u = 0; u < 4; ++u) {
      const int i = lane + 32 * u;
      pv[u] = (g.i >= 0 && i >= j && i < ell) ? __ldcg(src + i) : 0.0;
    }
    const double beta = g.i >= 0 ? __ldcg(src + 128) : 0.0;
    const double tau = g.i >= 0 ? __ldcg(src + 129) : 0.0;
    const double rden = g.i >= 0 ? __ldcg(src + 130) : 0.0;
    double* vw = s_v[warp];
#pragma unroll
    for (int u = 0; u < 4; ++u) {
      const int i = lane + 32 * u;
      vw[i] = (i < j) ? 0.0 : (i == j ? 1.0 : pv[u] * rden);
    }
    __syncwarp();
    QT(4)
    const long long gidx = g.i;
    if (blk == 0 && tid == 0) {
      if (g.i < 0 || !(g.v > 0.0)) {
        if (info) atomicCAS(info, 0, 6 /* RS_ERR_RANK_DEFICIENT */), atomicCAS(info + 1, 0, j + 1);
      }
      piv[j] = gidx;
      const double nb = sqrt(fmax(g.v, 0.0)), ns = sqrt(fmax(g2, 0.0));
      if (gaps) gaps[j] = nb > 0.0 ? (nb - ns) / nb : 0.0;
    }
    // ---- apply H = I - tau v v^T; retire the pivot column; fuse the next residual norm ----
    const bool is_piv = active && gi == gidx;
    const bool upd = active && !is_piv && tau != 0.0;
    double w = 0.0;
    if (upd) {
      double w4[4] = {0.0, 0.0, 0.0, 0.0};
#pragma unroll
      for (int t = 0; t < RPL; ++t) w4[t & 3] = fma(vw[q + LPC * t], x[t], w4[t & 3]);
      w = (w4[0] + w4[1]) + (w4[2] + w4[3]);
    }
#pragma unroll
    for (int o = 1; o < LPC; o <<= 1) w += __shfl_xor_sync(0xffffffffu, w, o);
    {
      double s4[4] = {0.0, 0.0, 0.0, 0.0};
      if (upd) {
        const double tw = tau * w;
#pragma unroll
        for (int t = 0; t < RPL; ++t) {
          x[t] = fma(-tw, vw[q + LPC * t], x[t]);
          if (q + LPC * t > j) s4[t & 3] = fma(x[t], x[t], s4[t & 3]);
        }
      } else if (active && !is_piv) {
#pragma unroll
        for (int t = 0; t < RPL; ++t)
          if (q + LPC * t > j) s4[t & 3] = fma(x[t], x[t], s4[t & 3]);
      }
      s = (s4[0] + s4[1]) + (s4[2] + s4[3]);
    }
    if (is_piv) {
#pragma unroll
      for (int t = 0; t < RPL; ++t) {
        const int i = q + LPC * t;
        if (i < k) Rho[i + gi * static_cast<long long>(ldr)] = (i < j) ? x[t] : (i == j ? beta : 0.0);
      }
      active = false;
    }
    QT(5)
    QT(6)
  }
#undef QT
  if (active) {
#pragma unroll
    for (int t = 0; t < RPL; ++t) {
      const int i = q + LPC * t;
      if (i < k) Rho[i + gi * static_cast<long long>(ldr)] = x[t];
    }
  }
}

// ------------------------------------------------------------------------------------------
// Cluster variant (n <= 16 CTAs x COLS columns, l <= 4 ROWS): the CTAs of ONE thread-block
// cluster hold the columns in registers as above, and each step's exchange runs through
// distributed shared memory: every CTA pushes its candidate and candidate column (rows j..l-1)
// into every peer's shared memory (st.shared::cluster), one cluster barrier, then every CTA
// scans the NB candidates and forms the reflector from local shared memory.  No global-memory
// round trips in the step at all (the grid-barrier kernel above pays several per step).
// ------------------------------------------------------------------------------------------
constexpr int QRC_MAXNB = 16;

template <int ROWS, int THREADS>
__global__ void __launch_bounds__(THREADS, 1)
    qrcp_cluster_kernel(const double* __restrict__ B, int ldb, int ell, long long n, int k, int cols_per,
                        int64_t* __restrict__ piv, double* __restrict__ Rho, int ldr, double* __restrict__ gaps,
                        int* info) {
  constexpr int WARPS = THREADS / 32;
  const uint32_t blk = cluster_ctarank();
  const int NB = static_cast<int>(gridDim.x);
  const int tid = threadIdx.x, warp = tid >> 5, lane = tid & 31;
  const int mc = tid >> 2, q = tid & 3;
  const long long c0 = static_cast<long long>(blk) * cols_per;
  const long long gi = c0 + mc;
  bool active = mc < cols_per && gi < n;
  __shared__ Arg s_warg[WARPS];
  __shared__ double s_wsec[WARPS];
  __shared__ __align__(16) double s_v[WARPS][4 * ROWS];
  __shared__ __align__(16) QrCand s_cand[2][QRC_MAXNB];
  __shared__ __align__(16) double s_stage[4 * ROWS];
  extern __shared__ __align__(16) double s_dynq[];  // s_col[2][QRC_MAXNB][4 ROWS]
  double (*s_col)[QRC_MAXNB][4 * ROWS] = reinterpret_cast<double (*)[QRC_MAXNB][4 * ROWS]>(s_dynq);

  double x[ROWS];
#pragma unroll
  for (int t = 0; t < ROWS; ++t) {
    const int i = q + 4 * t;
    x[t] = (active && i < ell) ? B[i + gi * static_cast<long long>(ldb)] : 0.0;
  }
  double s = 0.0;
  {
    double s4[4] = {0.0, 0.0, 0.0, 0.0};
#pragma unroll
    for (int t = 0; t < ROWS; ++t) s4[t & 3] = fma(x[t], x[t], s4[t & 3]);
    s = (s4[0] + s4[1]) + (s4[2] + s4[3]);
  }
  cluster_sync_all();  // peers' shared memory exists before anyone writes into it

  for (int j = 0; j < k; ++j) {
    const int par = j & 1;
    // ---- (A) CTA best / runner-up ----
    double sc = s;
    sc += __shfl_xor_sync(0xffffffffu, sc, 1);
    sc += __shfl_xor_sync(0xffffffffu, sc, 2);
    {
      Arg a = (active && q == 0) ? Arg{sc, gi, mc} : Arg{-1.0, -1, -1};
      double sec = -1.0;
      warp_top2(a, sec);
      if (lane == 0) {
        s_warg[warp] = a;
        s_wsec[warp] = sec;
      }
      __syncthreads();
      if (warp == 0) {
        Arg xx = lane < WARPS ? s_warg[lane] : Arg{-1.0, -1, -1};
        double xs = lane < WARPS ? s_wsec[lane] : -1.0;
        warp_top2(xx, xs);
        if (lane == 0) {
          s_warg[0] = xx;
          s_wsec[0] = xs;
        }
      }
      __syncthreads();
    }
    // the owner stages its rows j..ell-1 locally, then everyone pushes candidate + column to all peers
    const Arg mine = s_warg[0];
    if (active && mine.i == gi) {
#pragma unroll
      for (int t = 0; t < ROWS; ++t) {
        const int i = q + 4 * t;
        if (i >= j && i < ell) s_stage[i] = x[t];
      }
    }
    __syncthreads();
    {
      const int len = ell - j;
      const uint32_t col_base = smem_u32(&s_col[par][blk][0]);
      for (int e = tid; e < NB * len; e += THREADS) {
        const int pc = e / len, i = j + (e - pc * len);
        const uint32_t ra = mapa_shared(col_base + 8u * i, static_cast<uint32_t>(pc));
        asm volatile("st.shared::cluster.f64 [%0], %1;" ::"r"(ra), "d"(s_stage[i]) : "memory");
      }
      if (tid < NB) {
        const uint32_t cb = mapa_shared(smem_u32(&s_cand[par][blk]), static_cast<uint32_t>(tid));
        const long long idx = mine.i;
        asm volatile("st.shared::cluster.v2.f64 [%0], {%1, %2};" ::"r"(cb), "d"(mine.v), "d"(s_wsec[0]) : "memory");
        asm volatile("st.shared::cluster.s64 [%0], %1;" ::"r"(cb + 16u), "l"(idx) : "memory");
      }
    }
    cluster_sync_all();

    // ---- (B) every warp scans the NB candidates in local shared memory ----
    Arg g{-1.0, -1, -1};
    double g2 = -1.0;
    for (int b = lane; b < NB; b += 32) {
      const long long ci = s_cand[par][b].idx;
      const double cb = s_cand[par][b].best;
      const double cs = s_cand[par][b].second;
      g2 = fmax(g2, cs);
      if (better(cb, ci, g.v, g.i)) {
        if (g.i >= 0) g2 = fmax(g2, g.v);
        g = Arg{cb, ci, b};
      } else if (ci >= 0) {
        g2 = fmax(g2, cb);
      }
    }
    warp_top2(g, g2);
    const long long gidx = g.i;
    const int gblk = g.b < 0 ? 0 : g.b;
    const double* src = &s_col[par][gblk][0];
    double* vw = s_v[warp];
    double pv[ROWS / 8];
    double xs = 0.0, alpha = 0.0;
#pragma unroll
    for (int u = 0; u < ROWS / 8; ++u) {
      const int i = lane + 32 * u;
      pv[u] = (i >= j && i < ell) ? src[i] : 0.0;
      if (i > j) xs = fma(pv[u], pv[u], xs);
      if (i == j) alpha = pv[u];
    }
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) {
      xs += __shfl_xor_sync(0xffffffffu, xs, o);
      alpha += __shfl_xor_sync(0xffffffffu, alpha, o);
    }
    double tau = 0.0, beta = alpha;
    if (g.i >= 0 && xs > 0.0) {
      const double h = sqrt(fma(alpha, alpha, xs));
      beta = alpha >= 0.0 ? -h : h;
      tau = (beta - alpha) / beta;
    }
    const double den = alpha - beta;
#pragma unroll
    for (int u = 0; u < ROWS / 8; ++u) {
      const int i = lane + 32 * u;
      vw[i] = (i < j) ? 0.0 : (i == j ? 1.0 : (tau != 0.0 ? pv[u] / den : 0.0));
    }
    __syncwarp();
    if (blk == 0 && tid == 0) {
      if (g.i < 0 || !(g.v > 0.0)) {
        if (info) atomicCAS(info, 0, 6 /* RS_ERR_RANK_DEFICIENT */), atomicCAS(info + 1, 0, j + 1);
      }
      piv[j] = gidx;
      const double nb = sqrt(fmax(g.v, 0.0)), ns = sqrt(fmax(g2, 0.0));
      if (gaps) gaps[j] = nb > 0.0 ? (nb - ns) / nb : 0.0;
    }
    // ---- apply H = I - tau v v^T; retire the pivot column; fuse the next residual norm ----
    const bool is_piv = active && gi == gidx;
    const bool upd = active && !is_piv && tau != 0.0;
    double w = 0.0;
    if (upd) {
      double w4[4] = {0.0, 0.0, 0.0, 0.0};
#pragma unroll
      for (int t = 0; t < ROWS; ++t) w4[t & 3] = fma(vw[q + 4 * t], x[t], w4[t & 3]);
      w = (w4[0] + w4[1]) + (w4[2] + w4[3]);
    }
    w += __shfl_xor_sync(0xffffffffu, w, 1);
    w += __shfl_xor_sync(0xffffffffu, w, 2);
    {
      double s4[4] = {0.0, 0.0, 0.0, 0.0};
      if (upd) {
        const double tw = tau * w;
#pragma unroll
        for (int t = 0; t < ROWS; ++t) {
          x[t] = fma(-tw, vw[q + 4 * t], x[t]);
          const int i = q + 4 * t;
          if (i > j) s4[t & 3] = fma(x[t], x[t], s4[t & 3]);
        }
      } else if (active && !is_piv) {
#pragma unroll
        for (int t = 0; t < ROWS; ++t) {
          const int i = q + 4 * t;
          if (i > j) s4[t & 3] = fma(x[t], x[t], s4[t & 3]);
        }
      }
      s = (s4[0] + s4[1]) + (s4[2] + s4[3]);
    }
    if (is_piv) {
#pragma unroll
      for (int t = 0; t < ROWS; ++t) {
        const int i = q + 4 * t;
        if (i < k) Rho[i + gi * static_cast<long long>(ldr)] = (i < j) ? x[t] : (i == j ? beta : 0.0);
      }
      active = false;
    }
    __syncthreads();  // s_warg / s_stage reuse
  }
  if (active) {
#pragma unroll
    for (int t = 0; t < ROWS; ++t) {
      const int i = q + 4 * t;
      if (i < k) Rho[i + gi * static_cast<long long>(ldr)] = x[t];
    }
  }
  cluster_sync_all();  // no CTA leaves while peers may still write its shared memory
}

template <int ROWS, int THREADS>
cudaError_t launch_qrcp_cluster(cudaStream_t st, int NB, const double* B, int ldb, int ell, long long n, int k,
                                int cols_per, int64_t* piv, double* Rho, int ldr, double* gaps, int* info) {
  constexpr int dsmem = 2 * QRC_MAXNB * 4 * ROWS * 8;
  {
    cudaError_t e = ensure_func_attr(reinterpret_cast<const void*>(qrcp_cluster_kernel<ROWS, THREADS>),
                                     cudaFuncAttributeNonPortableClusterSizeAllowed, 1);
    if (e != cudaSuccess) return e;
    e = ensure_smem(qrcp_cluster_kernel<ROWS, THREADS>, dsmem);
    if (e != cudaSuccess) return e;
  }
  cudaLaunchConfig_t cfg{};
  cfg.gridDim = dim3(NB, 1, 1);
  cfg.blockDim = dim3(THREADS, 1, 1);
  cfg.dynamicSmemBytes = dsmem;
  cfg.stream = st;
  cudaLaunchAttribute at[1];
  at[0].id = cudaLaunchAttributeClusterDimension;
  at[0].val.clusterDim.x = NB;
  at[0].val.clusterDim.y = 1;
  at[0].val.clusterDim.z = 1;
  cfg.attrs = at;
  cfg.numAttrs = 1;
  int nclusters = 0;
  cudaError_t e = cudaOccupancyMaxActiveClusters(&nclusters, qrcp_cluster_kernel<ROWS, THREADS>, &cfg);
  if (e != cudaSuccess || nclusters < 1) {
    cudaGetLastError();
    return cudaErrorNotSupported;
  }
  return cudaLaunchKernelEx(&cfg, qrcp_cluster_kernel<ROWS, THREADS>, B, ldb, ell, n, k, cols_per, piv, Rho, ldr,
                            gaps, info);
}

namespace {
int qr_ldw(int ell) { return (ell + 11) / 16 * 16 + 4; }  // >= ell, = 4 mod 16 doubles
size_t qr_smem(int cols, int ell) { return (static_cast<size_t>(cols) * qr_ldw(ell) + ell) * 8; }
}  // namespace

size_t qrcp_workspace_bytes(int ell, long long n) {
  const int NB = 1024;  // upper bound on blocks
  // the flag kernel uses QrRec records and QRF_CST-strided columns in the same region
  return sizeof(QrWork) + 2 * NB * sizeof(QrCand) + 2 * static_cast<size_t>(NB) * std::max(ell, QRF_CST) * 8 +
         2 * n * 8 + 256;
}

cudaError_t qrcp_truncated(cudaStream_t st, const double* B, int ldb, int ell, long long n, int k, void* work,
                           int64_t* perm, double* Rho, int ldr, double* gaps, int* info, int num_sms) {
  if (n >= (1LL << 31)) return cudaErrorInvalidValue;  // column indices ride in 32-bit REDUX keys
  // compile-time development switches: -DRS_DEV_QRCP_SMEM (shared-memory kernel), _NO_CLUSTER,
  // _TIMING (per-phase cycle counts of CTA 0 to stderr), _BARRIER, _LPC4, _POLL
#ifdef RS_DEV_QRCP_SMEM
  constexpr bool force_smem = true;
#else
  constexpr bool force_smem = false;
#endif
  const bool use_reg = !force_smem && ell <= 4 * QRR_ROWS && (n + QRR_COLS - 1) / QRR_COLS <= num_sms;
  int cols_per = use_reg ? QRR_COLS : QR_MAX_COLS;
  while (!use_reg && cols_per > 1 && qr_smem(cols_per, ell) > QR_SMEM_MAX) --cols_per;
  int NB = static_cast<int>((n + cols_per - 1) / cols_per);
  if (NB > num_sms || (!use_reg && qr_smem(cols_per, ell) > QR_SMEM_MAX)) return cudaErrorInvalidValue;
  if (!use_reg) cols_per = static_cast<int>((n + NB - 1) / NB);  // balance
  const size_t smem = use_reg ? 0 : qr_smem(cols_per, ell);
  const int ldw = qr_ldw(ell);
  {
    cudaError_t e = ensure_smem(qrcp_kernel, static_cast<int>(QR_SMEM_MAX));
    if (e != cudaSuccess) return e;
    e = ensure_smem(qrcp_perm_kernel, static_cast<int>(QR_SMEM_MAX));
    if (e != cudaSuccess) return e;
  }
  QrWork* w = static_cast<QrWork*>(work);
  {
    // cluster path: l <= 64 with <= 160 columns per CTA, or l <= 128 with <= 128, over <= 16 CTAs
#ifdef RS_DEV_QRCP_NO_CLUSTER
    constexpr bool no_cluster = true;
#else
    constexpr bool no_cluster = false;
#endif
    const int rows = ell <= 64 ? 16 : 32;
    const int maxc = rows == 16 ? 160 : 128;
    const int nbc = static_cast<int>((n + maxc - 1) / maxc);
    if (!no_cluster && !force_smem && ell <= 128 && nbc <= QRC_MAXNB) {
      const int cp = static_cast<int>((n + nbc - 1) / nbc);
      int64_t* pv = reinterpret_cast<int64_t*>(reinterpret_cast<double*>(reinterpret_cast<QrCand*>(w + 1) + 2 * nbc) +
                                               2 * static_cast<size_t>(nbc) * ell);
      cudaError_t ec = rows == 16
                           ? launch_qrcp_cluster<16, 640>(st, nbc, B, ldb, ell, n, k, cp, pv, Rho, ldr, gaps, info)
                           : launch_qrcp_cluster<32, 512>(st, nbc, B, ldb, ell, n, k, cp, pv, Rho, ldr, gaps, info);
      if (ec == cudaSuccess) {
        count_launch();
        const size_t psmem = static_cast<size_t>(n) * 8;
        const bool use_smem = psmem <= QR_SMEM_MAX;
        qrcp_perm_kernel<<<1, 1024, use_smem ? psmem : 0, st>>>(pv, k, n, perm, pv + n, use_smem);
        count_launch();
        return cudaGetLastError();
      }
      if (ec != cudaErrorNotSupported) return ec;
    }
  }
  // -DRS_DEV_QRCP_TIMING: per-phase cycle counts of CTA 0 printed to stderr (development aid)
#ifdef RS_DEV_QRCP_TIMING
  static long long* tbuf = nullptr;
  if (!tbuf && cudaMalloc(&tbuf, 8 * 8 * 1024) != cudaSuccess) tbuf = nullptr;
  long long* tb = k <= 1024 ? tbuf : nullptr;
#else
  long long* tb = nullptr;
#endif
  auto report = [&](const char* what, int nb, int cols) {
#ifndef RS_DEV_QRCP_TIMING
    (void)what, (void)nb, (void)cols;
    return;
#else
    if (!tb) return;
    static long long h[8 * 1024];
    cudaStreamSynchronize(st);
    cudaMemcpy(h, tb, 8 * 8 * static_cast<size_t>(k), cudaMemcpyDeviceToHost);
    double acc[7] = {0};
    for (int j = 1; j < k; ++j)
      for (int p = 0; p < 6; ++p) acc[p] += static_cast<double>(h[j * 8 + p + 1] - h[j * 8 + p]);
    for (int j = 1; j < k; ++j) acc[6] += static_cast<double>(h[j * 8] - h[(j - 1) * 8 + 6]);
    fprintf(stderr,
            "QRCP %s NB=%d cols=%d cycles/step: p0-1=%.0f p1-2=%.0f p2-3=%.0f p3-4=%.0f p4-5=%.0f p5-6=%.0f "
            "tail=%.0f\n",
            what, nb, cols, acc[0] / (k - 1), acc[1] / (k - 1), acc[2] / (k - 1), acc[3] / (k - 1), acc[4] / (k - 1),
            acc[5] / (k - 1), acc[6] / (k - 1));
#endif
  };
  {
    // flag-synchronised register kernel: 8 lanes per column when n <= NBmax x 64, else 4
#ifdef RS_DEV_QRCP_BARRIER
    constexpr bool barrier_kernel = true;
#else
    constexpr bool barrier_kernel = false;
#endif
    const int nbmax = std::min(num_sms, QRF_MAXNB);
    const int nb8 = static_cast<int>((n + 63) / 64), nb4 = static_cast<int>((n + 127) / 128);
#ifdef RS_DEV_QRCP_LPC4
    constexpr bool force4 = true;
#else
    constexpr bool force4 = false;
#endif
    const int lpc = (nb8 <= nbmax && !force4) ? 8 : (nb4 <= nbmax ? 4 : 0);
    if (!barrier_kernel && !force_smem && ell <= 128 && lpc) {
      const int nbf = lpc == 8 ? nb8 : nb4;
      QrRec* rec = reinterpret_cast<QrRec*>(w + 1);
      double* ccol = reinterpret_cast<double*>(rec + 2 * nbf);
      int64_t* pv = reinterpret_cast<int64_t*>(ccol + 2 * static_cast<size_t>(nbf) * QRF_CST);
      cudaError_t e = cudaMemsetAsync(work, 0, sizeof(QrWork) + 2 * static_cast<size_t>(nbf) * sizeof(QrRec), st);
      if (e != cudaSuccess) return e;
#ifdef RS_DEV_QRCP_POLL
      constexpr bool poll_records = true;
#else
      constexpr bool poll_records = false;
#endif
      unsigned int* counter = poll_records ? nullptr : &w->count;
      void* fargs[] = {(void*)&B,   (void*)&ldb, (void*)&ell, (void*)&n,   (void*)&k,    (void*)&rec,
                       (void*)&ccol, (void*)&nbf, (void*)&pv, (void*)&Rho, (void*)&ldr, (void*)&gaps,
                       (void*)&info, (void*)&tb, (void*)&counter};
      e = lpc == 8 ? cudaLaunchCooperativeKernel(reinterpret_cast<void*>(qrcp_flag_kernel<8>), dim3(nbf),
                                                 dim3(QRR_THREADS), fargs, 0, st)
                   : cudaLaunchCooperativeKernel(reinterpret_cast<void*>(qrcp_flag_kernel<4>), dim3(nbf),
                                                 dim3(QRR_THREADS), fargs, 0, st);
      if (e != cudaSuccess) return e;
      count_launch();
      const size_t psmem = static_cast<size_t>(n) * 8;
      const bool use_smem = psmem <= QR_SMEM_MAX;
      qrcp_perm_kernel<<<1, 1024, use_smem ? psmem : 0, st>>>(pv, k, n, perm, pv + n, use_smem);
      count_launch();
      report(poll_records ? "poll" : "flag", nbf, QRR_THREADS / lpc);
      return cudaGetLastError();
    }
  }
  cudaError_t e = cudaMemsetAsync(work, 0, sizeof(QrWork), st);
  if (e != cudaSuccess) return e;
  QrCand* cand = reinterpret_cast<QrCand*>(w + 1);
  double* candcol = reinterpret_cast<double*>(cand + 2 * NB);
  int64_t* piv = reinterpret_cast<int64_t*>(candcol + 2 * static_cast<size_t>(NB) * ell);
  int64_t* gpos = piv + n;
  void* args[] = {(void*)&B,   (void*)&ldb, (void*)&ell, (void*)&n,    (void*)&k,  (void*)&w,
                  (void*)&NB,  (void*)&cols_per, (void*)&ldw, (void*)&piv, (void*)&Rho, (void*)&ldr,
                  (void*)&gaps, (void*)&info, (void*)&tb};
  count_launch();
  if (use_reg) {
    void* rargs[] = {(void*)&B,   (void*)&ldb, (void*)&ell, (void*)&n,    (void*)&k,    (void*)&w, (void*)&NB,
                     (void*)&piv, (void*)&Rho, (void*)&ldr, (void*)&gaps, (void*)&info, (void*)&tb};
    const size_t rsmem = (4 * static_cast<size_t>(NB) + static_cast<size_t>(NB) * ell) * 8;
    e = ensure_smem(qrcp_reg_kernel, static_cast<int>(rsmem));
    if (e != cudaSuccess) return e;
    e = cudaLaunchCooperativeKernel(reinterpret_cast<void*>(qrcp_reg_kernel), dim3(NB), dim3(QRR_THREADS), rargs,
                                    rsmem, st);
  } else {
    e = cudaLaunchCooperativeKernel(reinterpret_cast<void*>(qrcp_kernel), dim3(NB), dim3(QR_THREADS), args, smem, st);
  }
  if (e != cudaSuccess) return e;
  const size_t psmem = static_cast<size_t>(n) * 8;
  const bool use_smem = psmem <= QR_SMEM_MAX;
  qrcp_perm_kernel<<<1, 1024, use_smem ? psmem : 0, st>>>(piv, k, n, perm, gpos, use_smem);
  count_launch();
  report(use_reg ? "barrier" : "smem", NB, cols_per);
  return cudaGetLastError();
}

}  // namespace rs
