// Truncated QP3 of the full A: the paper's deterministic baseline (Sec. 2; "QP3" in
// Figs. 7, 10-14).  Householder QR with column pivoting stopped after k columns,
// blocked as LAPACK's QP3: a panel of NB columns is factored with the trailing
// updates delayed (accumulated in F, n x NB), only the current row of the trailing matrix is
// updated per step, and the trailing submatrix gets one rank-NB update per panel.  Pivots use
// downdated column norms with LAPACK's cancellation test.
//
// B200 design (memory-bound: every step streams the trailing matrix once through the GEMV that
// forms F(:, j), "about half of its flops using BLAS-2"):
//  * per step four kernels and no host synchronisation -- the pivot index, the reflector and
//    the list of norms to recompute live in device memory;
//  * the trailing GEMV reads A column-major with 16-byte loads, the reflector staged in shared
//    memory, deterministic two-stage reduction;
//  * a column whose downdated norm failed the cancellation test is recomputed exactly on the
//    device from the delayed update A(:, c) - A(:, panel) F(c, :)^T (one column, no panel break):
//    the paper's "trailing submatrix is immediately updated ... and the column norms are
//    recomputed" without ending the panel early;
//  * the per-panel trailing update (rank NB, ~4 flop/byte: HBM-bound) is a DFMA tile kernel that
//    also recomputes every trailing column norm exactly while the tile is in registers.
#include <algorithm>
#include <cmath>

#include "common.cuh"
#include "internal.h"

namespace rs {

constexpr int QP3_NB = 32;             // panel width
constexpr int QP3_T = 256;             // threads of the grid kernels
constexpr int QP3_A_CTAS = 296;        // pivot-column kernel grid (2 x 148)
constexpr int QP3_GV_ROWS = 2048;      // GEMV: rows per CTA (reflector chunk in smem)
constexpr int QP3_GV_CPW = 2;          // GEMV: columns per warp
constexpr int QP3_GV_COLS = 8 * QP3_GV_CPW;
constexpr int QP3_UP_ROWS = 128;       // trailing update: rows per sub-tile (4 per lane)
constexpr int QP3_UP_SUB = 8;          // sub-tiles per CTA (1024 rows)
constexpr int QP3_UP_COLS = 32;        // columns per CTA (4 per warp)

struct Qp3Scalars {
  double beta, tau, scale, res;
  long long pvt;
  int nflag;
  unsigned int done;  // CTAs of the pivot kernel that finished (last one forms the reflector)
};

struct Qp3Work {
  Qp3Scalars* sc;
  double* vn1;     // n
  double* vn2;     // n
  double* F;       // n x NB, row-major: F(c, t) at F[c * NB + t]
  double* parts_a; // QP3_A_CTAS
  double* parts;   // nch x n (GEMV / trailing-update partial sums)
  int* flags;      // n
  long long nch;
};

static long long qp3_nch(long long m) { return (m + 1 + 1023) / 1024 + 1; }

static size_t align256(size_t b) { return (b + 255) & ~static_cast<size_t>(255); }

size_t qp3_workspace_bytes(long long m, long long n) {
  size_t b = align256(sizeof(Qp3Scalars));
  b += 2 * align256(n * 8);
  b += align256(static_cast<size_t>(n) * QP3_NB * 8);
  b += align256(QP3_A_CTAS * 8);
  b += align256(static_cast<size_t>(qp3_nch(m)) * n * 8);
  b += align256(n * 4);
  return b;
}

static Qp3Work qp3_carve(void* work, long long m, long long n) {
  char* p = static_cast<char*>(work);
  Qp3Work w;
  w.sc = reinterpret_cast<Qp3Scalars*>(p);
  p += align256(sizeof(Qp3Scalars));
  w.vn1 = reinterpret_cast<double*>(p);
  p += align256(n * 8);
  w.vn2 = reinterpret_cast<double*>(p);
  p += align256(n * 8);
  w.F = reinterpret_cast<double*>(p);
  p += align256(static_cast<size_t>(n) * QP3_NB * 8);
  w.parts_a = reinterpret_cast<double*>(p);
  p += align256(QP3_A_CTAS * 8);
  w.nch = qp3_nch(m);
  w.parts = reinterpret_cast<double*>(p);
  p += align256(static_cast<size_t>(w.nch) * n * 8);
  w.flags = reinterpret_cast<int*>(p);
  return w;
}

RS_DEVINL double warp_sum(double v) {
#pragma unroll
  for (int o = 16; o > 0; o >>= 1) v += __shfl_xor_sync(0xffffffffu, v, o);
  return v;
}

// block-wide deterministic sum (blockDim.x multiple of 32, <= 1024); result valid in all threads
RS_DEVINL double block_sum(double v, double* red) {
  v = warp_sum(v);
  const int w = threadIdx.x >> 5, nw = blockDim.x >> 5;
  __syncthreads();
  if ((threadIdx.x & 31) == 0) red[w] = v;
  __syncthreads();
  double s = 0.0;
  for (int i = 0; i < nw; ++i) s += red[i];
  return s;
}

// ---- initial column norms, perm = identity ----------------------------------------------
__global__ void __launch_bounds__(QP3_T) qp3_init_kernel(const double* __restrict__ A, long long lda, long long m,
                                                         long long n, double* vn1, double* vn2, int64_t* perm,
                                                         Qp3Scalars* sc) {
  const long long c = static_cast<long long>(blockIdx.x) * 8 + (threadIdx.x >> 5);
  const int lane = threadIdx.x & 31;
  if (blockIdx.x == 0 && threadIdx.x == 0) {
    sc->nflag = 0;
    sc->done = 0;
  }
  if (c >= n) return;
  const double* col = A + c * lda;
  double s = 0.0, s4[4] = {0.0, 0.0, 0.0, 0.0};
  const long long m2 = m & ~1LL;
  long long i = 2 * lane;
  for (; i + 192 < m2; i += 256) {  // four independent 16-byte loads in flight per lane
    double2 x[4];
#pragma unroll
    for (int u = 0; u < 4; ++u) x[u] = *reinterpret_cast<const double2*>(col + i + 64 * u);
#pragma unroll
    for (int u = 0; u < 4; ++u) s4[u] = fma(x[u].y, x[u].y, fma(x[u].x, x[u].x, s4[u]));
  }
  for (; i < m2; i += 64) {
    const double2 x = *reinterpret_cast<const double2*>(col + i);
    s = fma(x.y, x.y, fma(x.x, x.x, s));
  }
  s += (s4[0] + s4[1]) + (s4[2] + s4[3]);
  if ((m & 1) && lane == 0) s = fma(col[m - 1], col[m - 1], s);
  s = warp_sum(s);
  if (lane == 0) {
    vn1[c] = sqrt(s);
    vn2[c] = vn1[c];
    perm[c] = c;
  }
}

// ---- steps (a)+(b): pivot choice, column swap, delayed update of the pivot column, reflector -----
// A(rk:m, j) := A(rk:m, pvt) - A(rk:m, j0:j) F(pvt, 0:kk)^T, A(:, pvt) := old A(:, j);
// parts_a[cta] = partial sum of squares of the new A(rk+1:m, j); the last CTA to finish sums the
// partials in index order, forms the dlarfg reflector and swaps perm / vn / F rows.
__global__ void __launch_bounds__(QP3_T) qp3_pivot_kernel(double* __restrict__ A, long long lda, long long m,
                                                          long long n, long long j, long long j0, int kk,
                                                          double* vn1, double* vn2, int64_t* perm, double* F,
                                                          double* parts_a, double* tau_out, Qp3Scalars* sc) {
  __shared__ double s_best[QP3_T / 32];
  __shared__ long long s_idx[QP3_T / 32], s_org[QP3_T / 32];
  __shared__ double s_f[QP3_NB];
  __shared__ double red[QP3_T / 32];
  __shared__ long long s_pvt;
  // largest residual norm, ties -> lowest original column index (reading R5 / oracle rule)
  double best = -1.0;
  long long bi = -1, bo = 0;
  long long c = j + threadIdx.x;
  for (; c + 7 * blockDim.x < n; c += 8 * blockDim.x) {  // eight independent loads in flight
    double v[8];
    long long o[8];
#pragma unroll
    for (int u = 0; u < 8; ++u) {
      v[u] = vn1[c + u * blockDim.x];
      o[u] = perm[c + u * blockDim.x];
    }
#pragma unroll
    for (int u = 0; u < 8; ++u) {
      if (v[u] > best || (v[u] == best && o[u] < bo)) {
        best = v[u];
        bi = c + u * blockDim.x;
        bo = o[u];
      }
    }
  }
  for (; c < n; c += blockDim.x) {
    const double v = vn1[c];
    const long long o = perm[c];
    if (v > best || (v == best && o < bo)) {
      best = v;
      bi = c;
      bo = o;
    }
  }
#pragma unroll
  for (int off = 16; off > 0; off >>= 1) {
    const double ov = __shfl_xor_sync(0xffffffffu, best, off);
    const long long oi = __shfl_xor_sync(0xffffffffu, bi, off);
    const long long oo = __shfl_xor_sync(0xffffffffu, bo, off);
    if (oi >= 0 && (bi < 0 || ov > best || (ov == best && oo < bo))) {
      best = ov;
      bi = oi;
      bo = oo;
    }
  }
  const int w = threadIdx.x >> 5;
  if ((threadIdx.x & 31) == 0) {
    s_best[w] = best;
    s_idx[w] = bi;
    s_org[w] = bo;
  }
  __syncthreads();
  if (threadIdx.x == 0) {
    double b = -1.0;
    long long i = -1, o = 0;
    for (int q = 0; q < QP3_T / 32; ++q) {
      if (s_idx[q] >= 0 && (i < 0 || s_best[q] > b || (s_best[q] == b && s_org[q] < o))) {
        b = s_best[q];
        i = s_idx[q];
        o = s_org[q];
      }
    }
    s_pvt = i < 0 ? j : i;
    if (blockIdx.x == 0) sc->pvt = s_pvt;
  }
  __syncthreads();
  const long long pvt = s_pvt;
  if (threadIdx.x < kk) s_f[threadIdx.x] = F[pvt * QP3_NB + threadIdx.x];
  __syncthreads();
  const long long rk = j;
  double ss = 0.0;
  double* colj = A + j * lda;
  double* colp = A + pvt * lda;
  for (long long i = static_cast<long long>(blockIdx.x) * blockDim.x + threadIdx.x; i < m;
       i += static_cast<long long>(gridDim.x) * blockDim.x) {
    double a = colp[i];
    if (pvt != j) colp[i] = colj[i];
    if (i >= rk) {
#pragma unroll 8
      for (int t = 0; t < kk; ++t) a = fma(-A[i + (j0 + t) * lda], s_f[t], a);
      if (i > rk) ss = fma(a, a, ss);
    }
    colj[i] = a;
  }
  ss = block_sum(ss, red);
  __shared__ bool s_last;
  if (threadIdx.x == 0) {
    parts_a[blockIdx.x] = ss;
    __threadfence();
    s_last = atomicAdd(&sc->done, 1u) == gridDim.x - 1;
  }
  __syncthreads();
  if (!s_last) return;
  // ---- step (b), last CTA: reflector (dlarfg) and bookkeeping ----
  __threadfence();
  double v = 0.0;
  for (int i = threadIdx.x; i < static_cast<int>(gridDim.x); i += blockDim.x) v += __ldcg(parts_a + i);
  const double xnorm2 = block_sum(v, red);
  if (threadIdx.x == 0) {
    const double alpha = __ldcg(colj + rk);
    const double xnorm = sqrt(xnorm2);
    double beta = alpha, tau = 0.0, scale = 0.0;
    if (xnorm != 0.0) {
      const double h = hypot(alpha, xnorm);
      beta = alpha >= 0.0 ? -h : h;
      tau = (beta - alpha) / beta;
      scale = 1.0 / (alpha - beta);
    }
    sc->beta = beta;
    sc->tau = tau;
    sc->scale = scale;
    sc->nflag = 0;
    sc->done = 0;
    tau_out[j] = tau;
    if (pvt != j) {
      const int64_t tp = perm[j];
      perm[j] = perm[pvt];
      perm[pvt] = tp;
      vn1[pvt] = vn1[j];
      vn2[pvt] = vn2[j];
    }
  }
  if (pvt != j && threadIdx.x < kk) {  // swap rows j and pvt of F(:, 0:kk)
    const long long t = threadIdx.x;
    const double a = F[j * QP3_NB + t];
    F[j * QP3_NB + t] = F[pvt * QP3_NB + t];
    F[pvt * QP3_NB + t] = a;
  }
}

// ---- step (c): z(c) = A(rk:m, c)^T v, c in [j0, n), v = (1, scale * A(rk+1:m, j)) ------------
// CTA (x, y): 16 columns x rows [rs + y * rows_per_cta, ...), in sub-chunks of QP3_GV_ROWS whose
// reflector slice is staged in shared memory; one partial sum per (y, column).
__global__ void __launch_bounds__(QP3_T) qp3_gemv_kernel(const double* __restrict__ A, long long lda, long long m,
                                                         long long n, long long j, long long j0,
                                                         long long rows_per_cta, const Qp3Scalars* __restrict__ sc,
                                                         double* parts) {
  __shared__ __align__(16) double sv[QP3_GV_ROWS];
  const long long rk = j;
  const long long rbeg = (rk & ~1LL) + static_cast<long long>(blockIdx.y) * rows_per_cta;
  const long long rend = rbeg + rows_per_cta < m ? rbeg + rows_per_cta : m;
  const double scale = sc->scale;
  const double* colj = A + j * lda;
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const long long c0 = j0 + static_cast<long long>(blockIdx.x) * QP3_GV_COLS + warp * QP3_GV_CPW;
  const bool active = c0 < n;
  double acc[QP3_GV_CPW];
#pragma unroll
  for (int q = 0; q < QP3_GV_CPW; ++q) acc[q] = 0.0;
  for (long long rs = rbeg; rs < rend; rs += QP3_GV_ROWS) {
    const long long re = rs + QP3_GV_ROWS < rend ? rs + QP3_GV_ROWS : rend;
    __syncthreads();
    for (int r = threadIdx.x; r < QP3_GV_ROWS; r += blockDim.x) {
      const long long i = rs + r;
      double v = 0.0;
      if (i < re && i >= rk) v = i == rk ? 1.0 : colj[i] * scale;
      sv[r] = v;
    }
    __syncthreads();
    if (!active) continue;
    const long long nrow = re - rs;
    const long long npair = nrow >> 1;
    const double* cols[QP3_GV_CPW];
#pragma unroll
    for (int q = 0; q < QP3_GV_CPW; ++q) cols[q] = A + (c0 + q < n ? c0 + q : c0) * lda + rs;
    long long p = lane;
    for (; p + 96 < npair; p += 128) {
      double2 x[4][QP3_GV_CPW];
#pragma unroll
      for (int u = 0; u < 4; ++u)
#pragma unroll
        for (int q = 0; q < QP3_GV_CPW; ++q)
          x[u][q] = *reinterpret_cast<const double2*>(cols[q] + 2 * (p + 32 * u));
#pragma unroll
      for (int u = 0; u < 4; ++u) {
        const double2 v = *reinterpret_cast<const double2*>(sv + 2 * (p + 32 * u));
#pragma unroll
        for (int q = 0; q < QP3_GV_CPW; ++q) acc[q] = fma(x[u][q].y, v.y, fma(x[u][q].x, v.x, acc[q]));
      }
    }
    for (; p < npair; p += 32) {
      const double2 v = *reinterpret_cast<const double2*>(sv + 2 * p);
#pragma unroll
      for (int q = 0; q < QP3_GV_CPW; ++q) {
        const double2 x = *reinterpret_cast<const double2*>(cols[q] + 2 * p);
        acc[q] = fma(x.y, v.y, fma(x.x, v.x, acc[q]));
      }
    }
    if ((nrow & 1) && lane == 0) {
#pragma unroll
      for (int q = 0; q < QP3_GV_CPW; ++q) acc[q] = fma(cols[q][nrow - 1], sv[nrow - 1], acc[q]);
    }
  }
  if (!active) return;
#pragma unroll
  for (int q = 0; q < QP3_GV_CPW; ++q) {
    const double s = warp_sum(acc[q]);
    if (lane == 0 && c0 + q < n) parts[static_cast<long long>(blockIdx.y) * n + c0 + q] = s;
  }
}

// ---- steps (d)+(e), one warp per column c in [j0, n):
//   F(c, kk) = [c > j] tau z(c) - tau sum_t F(c, t) z(j0 + t)                       (F column kk)
//   c > j:  A(rk, c) -= sum_{t<kk} A(rk, j0+t) F(c, t) + F(c, kk);  downdate vn1(c)   (row rk)
// plus the reflector scaled into A(rk+1:m, j) and A(rk, j) := beta.  Lane t holds F(c, t) (one
// 256-byte row of F); the z partial sums are split over lanes; fixed-tree warp sums.
__global__ void __launch_bounds__(QP3_T) qp3_fcol_row_kernel(double* __restrict__ A, long long lda, long long m,
                                                             long long n, long long j, long long j0, int kk, int nch,
                                                             const double* __restrict__ parts, double* F, double* vn1,
                                                             double* vn2, int* flags, Qp3Scalars* sc, int downdate) {
  __shared__ double s_aux8[QP3_NB][8];
  __shared__ double s_aux[QP3_NB];
  __shared__ double s_r[QP3_NB];
  const long long rk = j;
  const double tau = sc->tau;
  {  // aux(t) = -tau z(j0 + t), t < kk: thread (t, g) sums partials q = g, g+8, ...
    const int t = threadIdx.x >> 3, g = threadIdx.x & 7;
    double z = 0.0;
    if (t < kk)
      for (int q = g; q < nch; q += 8) z += parts[static_cast<long long>(q) * n + j0 + t];
    s_aux8[t][g] = z;
    if (threadIdx.x < kk) s_r[threadIdx.x] = A[rk + (j0 + threadIdx.x) * lda];
  }
  __syncthreads();
  if (threadIdx.x < kk) {
    const double* z8 = s_aux8[threadIdx.x];
    s_aux[threadIdx.x] = -tau * (((z8[0] + z8[1]) + (z8[2] + z8[3])) + ((z8[4] + z8[5]) + (z8[6] + z8[7])));
  }
  __syncthreads();
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const long long c = j0 + static_cast<long long>(blockIdx.x) * (QP3_T / 32) + warp;
  if (c < n) {
    double z = 0.0;
    if (c > j)
      for (int q = lane; q < nch; q += 32) z += parts[static_cast<long long>(q) * n + c];
    const double fct = lane < kk ? F[c * QP3_NB + lane] : 0.0;
    double fsum = lane < kk ? fct * s_aux[lane] : 0.0;
    double asum = lane < kk ? s_r[lane] * fct : 0.0;
    z = warp_sum(z);
    fsum = warp_sum(fsum);
    asum = warp_sum(asum);
    if (lane == 0) {
      const double f = (c > j ? tau * z : 0.0) + fsum;
      F[c * QP3_NB + kk] = f;
      if (c > j) {
        const double a = A[rk + c * lda] - asum - f;  // v(rk) = 1
        A[rk + c * lda] = a;
        const double v1 = vn1[c];
        if (downdate && v1 != 0.0) {  // LAPACK dlaqps: tol3z = sqrt(eps)
          double temp = fabs(a) / v1;
          temp = fmax(0.0, (1.0 + temp) * (1.0 - temp));
          const double r = v1 / vn2[c];
          const double temp2 = temp * r * r;
          if (temp2 <= 1.0536712127723509e-08) {
            const int slot = atomicAdd(&sc->nflag, 1);
            flags[slot] = static_cast<int>(c);
          } else {
            vn1[c] = v1 * sqrt(temp);
          }
        }
      }
    }
  }
  const double scale = sc->scale;
  double* colj = A + j * lda;
  for (long long i = j + 1 + static_cast<long long>(blockIdx.x) * blockDim.x + threadIdx.x; i < m;
       i += static_cast<long long>(gridDim.x) * blockDim.x)
    colj[i] *= scale;
  if (blockIdx.x == 0 && threadIdx.x == 0) colj[j] = sc->beta;
}

// ---- step (f): exact norms of flagged columns from the delayed update ------------------------
__global__ void __launch_bounds__(QP3_T) qp3_recompute_kernel(const double* __restrict__ A, long long lda, long long m,
                                                              long long n, long long j, long long j0, int kk,
                                                              const double* __restrict__ F, double* vn1, double* vn2,
                                                              const int* flags, const Qp3Scalars* __restrict__ sc) {
  __shared__ double s_f[QP3_NB];
  __shared__ double red[QP3_T / 32];
  const int nflag = sc->nflag;
  for (int f = blockIdx.x; f < nflag; f += gridDim.x) {
    const long long c = flags[f];
    __syncthreads();
    if (threadIdx.x <= kk) s_f[threadIdx.x] = F[c * QP3_NB + threadIdx.x];
    __syncthreads();
    double ss = 0.0;
    for (long long i = j + 1 + threadIdx.x; i < m; i += blockDim.x) {
      double a = A[i + c * lda];
      for (int t = 0; t <= kk; ++t) a = fma(-A[i + (j0 + t) * lda], s_f[t], a);
      ss = fma(a, a, ss);
    }
    ss = block_sum(ss, red);
    if (threadIdx.x == 0) {
      vn1[c] = sqrt(ss);
      vn2[c] = vn1[c];
    }
  }
}

// ---- panel end: A(r0:m, c0:n) -= A(r0:m, j0:j0+kb) F(c0:n, 0:kb)^T, fused exact column norms --
// CTA: 32 columns (4 per warp) x 1024 rows in sub-tiles of 128 (two row pairs per lane).  The thread's
// 4 x 4 block of A is loaded before the panel slice is staged, so the HBM reads overlap the
// shared-memory staging; F(tile, :) and the panel slice are broadcast / conflict-free LDS.128.
__global__ void __launch_bounds__(QP3_T, 2) qp3_trailing_kernel(double* __restrict__ A, long long lda, long long m,
                                                                long long n, long long j0, int kb, long long r0,
                                                                long long c0, const double* __restrict__ F,
                                                                double* parts) {
  __shared__ __align__(16) double Ls[QP3_NB][QP3_UP_ROWS];
  __shared__ __align__(16) double Fs[QP3_NB][QP3_UP_COLS];
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const long long cb = c0 + static_cast<long long>(blockIdx.x) * QP3_UP_COLS;
  for (int e = threadIdx.x; e < QP3_NB * QP3_UP_COLS; e += blockDim.x) {
    const int t = e / QP3_UP_COLS, cc = e % QP3_UP_COLS;
    Fs[t][cc] = (t < kb && cb + cc < n) ? F[(cb + cc) * QP3_NB + t] : 0.0;
  }
  const long long cw = cb + warp * 4;  // this warp's 4 columns
  double ssq[4] = {0.0, 0.0, 0.0, 0.0};
  const long long rbase = (r0 & ~1LL) + static_cast<long long>(blockIdx.y) * (QP3_UP_ROWS * QP3_UP_SUB);
  for (int sub = 0; sub < QP3_UP_SUB; ++sub) {
    const long long rs = rbase + sub * QP3_UP_ROWS;
    if (rs >= m) break;
    // lane rows: pair h = 0, 1 at rs + 64 h + 2 lane (+0, +1): conflict-free LDS.128 of the slice
    long long ih[2];
    bool full[2];
#pragma unroll
    for (int hh = 0; hh < 2; ++hh) {
      ih[hh] = rs + 64 * hh + 2 * lane;
      full[hh] = ih[hh] + 1 < m;
    }
    double2 a[4][2];
#pragma unroll
    for (int q = 0; q < 4; ++q)
#pragma unroll
      for (int hh = 0; hh < 2; ++hh) {
        a[q][hh] = make_double2(0.0, 0.0);
        if (full[hh] && cw + q < n) a[q][hh] = *reinterpret_cast<const double2*>(A + (cw + q) * lda + ih[hh]);
      }
    __syncthreads();
    for (int e = threadIdx.x; e < QP3_NB * (QP3_UP_ROWS / 2); e += blockDim.x) {
      const int t = e / (QP3_UP_ROWS / 2), rp = e % (QP3_UP_ROWS / 2);
      const long long i = rs + 2 * rp;
      double2 x = make_double2(0.0, 0.0);
      if (t < kb) {
        const double* col = A + (j0 + t) * lda;
        if (i + 1 < m) {
          x = *reinterpret_cast<const double2*>(col + i);
        } else if (i < m) {
          x.x = col[i];
        }
        if (i < r0) x.x = 0.0;
        if (i + 1 < r0) x.y = 0.0;
      }
      *reinterpret_cast<double2*>(&Ls[t][2 * rp]) = x;
    }
    __syncthreads();
    if (ih[0] >= m) continue;
    double acc[4][4];  // [column][row: pair 0 (.x, .y), pair 1 (.x, .y)]
#pragma unroll
    for (int q = 0; q < 4; ++q)
#pragma unroll
      for (int r = 0; r < 4; ++r) acc[q][r] = 0.0;
#pragma unroll 8
    for (int t = 0; t < QP3_NB; ++t) {
      if (t >= kb) break;
      const double2 l01 = *reinterpret_cast<const double2*>(&Ls[t][2 * lane]);
      const double2 l23 = *reinterpret_cast<const double2*>(&Ls[t][64 + 2 * lane]);
      const double2 f01 = *reinterpret_cast<const double2*>(&Fs[t][warp * 4]);
      const double2 f23 = *reinterpret_cast<const double2*>(&Fs[t][warp * 4 + 2]);
      const double l[4] = {l01.x, l01.y, l23.x, l23.y};
      const double f[4] = {f01.x, f01.y, f23.x, f23.y};
#pragma unroll
      for (int q = 0; q < 4; ++q)
#pragma unroll
        for (int r = 0; r < 4; ++r) acc[q][r] = fma(l[r], f[q], acc[q][r]);
    }
#pragma unroll
    for (int q = 0; q < 4; ++q) {
      const long long c = cw + q;
      if (c >= n) continue;
      double* col = A + c * lda;
#pragma unroll
      for (int hh = 0; hh < 2; ++hh) {
        const long long i = ih[hh];
        if (full[hh]) {  // rows < r0 have acc = 0 (masked slice): the store leaves them unchanged
          double2 v = a[q][hh];
          v.x -= acc[q][2 * hh];
          v.y -= acc[q][2 * hh + 1];
          *reinterpret_cast<double2*>(col + i) = v;
          if (i >= r0) ssq[q] = fma(v.x, v.x, ssq[q]);
          ssq[q] = fma(v.y, v.y, ssq[q]);  // i + 1 >= r0 always (r0 - rbase <= 1)
        } else if (i < m && i >= r0) {
          const double v = col[i] - acc[q][2 * hh];
          col[i] = v;
          ssq[q] = fma(v, v, ssq[q]);
        }
      }
    }
  }
#pragma unroll
  for (int q = 0; q < 4; ++q) {
    const double s = warp_sum(ssq[q]);
    if (lane == 0 && cw + q < n) parts[static_cast<long long>(blockIdx.y) * n + cw + q] = s;
  }
}

__global__ void __launch_bounds__(QP3_T) qp3_norms_kernel(long long n, long long c0, int nrb,
                                                          const double* __restrict__ parts, double* vn1, double* vn2) {
  const long long c = c0 + static_cast<long long>(blockIdx.x) * blockDim.x + threadIdx.x;
  if (c >= n) return;
  double s = 0.0;
  for (int q = 0; q < nrb; ++q) s += parts[static_cast<long long>(q) * n + c];
  vn1[c] = sqrt(s);
  vn2[c] = vn1[c];
}

__global__ void __launch_bounds__(1024) qp3_residual_kernel(long long n, long long c0, const double* __restrict__ vn1,
                                                            Qp3Scalars* sc) {
  __shared__ double red[32];
  double s = 0.0;
  for (long long c = c0 + threadIdx.x; c < n; c += blockDim.x) s = fma(vn1[c], vn1[c], s);
  s = block_sum(s, red);
  if (threadIdx.x == 0) sc->res = sqrt(s);
}

#define QP3_LAUNCHED()               \
  do {                               \
    count_launch();                  \
    cudaError_t e_ = cudaGetLastError(); \
    if (e_ != cudaSuccess) return e_; \
  } while (0)

cudaError_t qp3_truncated_large(cudaStream_t st, double* A, long long lda, long long m, long long n, int k,
                                void* work, int64_t* perm, double* tau, bool want_residual, double* residual) {
  const Qp3Work w = qp3_carve(work, m, n);
  qp3_init_kernel<<<static_cast<unsigned>((n + 7) / 8), QP3_T, 0, st>>>(A, lda, m, n, w.vn1, w.vn2, perm, w.sc);
  QP3_LAUNCHED();
  const long long lastrk = m < n ? m : n;
  for (long long j0 = 0; j0 < k; j0 += QP3_NB) {
    const int kb = static_cast<int>(k - j0 < QP3_NB ? k - j0 : QP3_NB);
    for (int kk = 0; kk < kb; ++kk) {
      const long long j = j0 + kk;
      qp3_pivot_kernel<<<QP3_A_CTAS, QP3_T, 0, st>>>(A, lda, m, n, j, j0, kk, w.vn1, w.vn2, perm, w.F, w.parts_a,
                                                     tau, w.sc);
      QP3_LAUNCHED();
      const long long rows = m - (j & ~1LL);
      const long long ncg = (n - j0 + QP3_GV_COLS - 1) / QP3_GV_COLS;
      const long long rpc = QP3_GV_ROWS;
      const unsigned nchg = static_cast<unsigned>((rows + rpc - 1) / rpc);
      qp3_gemv_kernel<<<dim3(static_cast<unsigned>(ncg), nchg), QP3_T, 0, st>>>(A, lda, m, n, j, j0, rpc, w.sc,
                                                                               w.parts);
      QP3_LAUNCHED();
      const unsigned nfb = static_cast<unsigned>((n - j0 + QP3_T / 32 - 1) / (QP3_T / 32));
      const int downdate = j + 1 < lastrk && j + 1 < k ? 1 : 0;  // norms are not needed after step k
      qp3_fcol_row_kernel<<<nfb < 64 ? 64 : nfb, QP3_T, 0, st>>>(A, lda, m, n, j, j0, kk, static_cast<int>(nchg),
                                                                w.parts, w.F, w.vn1, w.vn2, w.flags, w.sc, downdate);
      QP3_LAUNCHED();
      if (downdate) {
        qp3_recompute_kernel<<<148, QP3_T, 0, st>>>(A, lda, m, n, j, j0, kk, w.F, w.vn1, w.vn2, w.flags, w.sc);
        QP3_LAUNCHED();
      }
    }
    const long long r0 = j0 + kb, c0 = j0 + kb;
    const bool last = j0 + kb >= k;
    if ((!last || want_residual) && r0 < m && c0 < n) {
      const long long rows = m - (r0 & ~1LL);
      const unsigned nrb = static_cast<unsigned>((rows + QP3_UP_ROWS * QP3_UP_SUB - 1) / (QP3_UP_ROWS * QP3_UP_SUB));
      const unsigned ncb = static_cast<unsigned>((n - c0 + QP3_UP_COLS - 1) / QP3_UP_COLS);
      qp3_trailing_kernel<<<dim3(ncb, nrb), QP3_T, 0, st>>>(A, lda, m, n, j0, kb, r0, c0, w.F, w.parts);
      QP3_LAUNCHED();
      qp3_norms_kernel<<<static_cast<unsigned>((n - c0 + QP3_T - 1) / QP3_T), QP3_T, 0, st>>>(n, c0, nrb, w.parts,
                                                                                           w.vn1, w.vn2);
      QP3_LAUNCHED();
    }
  }
  if (want_residual) {
    if (k < m && k < n) {
      qp3_residual_kernel<<<1, 1024, 0, st>>>(n, k, w.vn1, w.sc);
      QP3_LAUNCHED();
      cudaError_t e = cudaMemcpyAsync(residual, &w.sc->res, sizeof(double), cudaMemcpyDeviceToHost, st);
      if (e != cudaSuccess) return e;
      return cudaStreamSynchronize(st);
    }
    *residual = 0.0;
  }
  return cudaSuccess;
}

}  // namespace rs
