// Cholesky factor of a Gram matrix and its inverse: CholQR steps (ii)-(iii)
// ("R^T R := G, R upper-triangular with non-negative diagonal; Q = R^{-T} B").
//
// n <= 128: blocked (16 x 16) right-looking Cholesky in one CTA, then a blocked forward solve
// R^T X = I for X = R^{-T} (= Linv), all in shared memory.  Per 16-wide block:
//   (1) one warp factors the diagonal block in registers (shuffles, rsqrt per pivot),
//   (2) every thread solves one column of the panel R12 = R11^{-T} A12,
//   (3) the trailing update A22 -= R12^T R12 is spread over all threads,
// so a block costs 2 __syncthreads instead of 16 (one per pivot).  The inverse proceeds by block
// rows of X: a parallel update from the finished block rows, then a 16-step in-block solve per
// column.  R (upper part of M) and X (strict lower part of M, its diagonal 1/R_ii kept apart)
// share one padded n x n array.
// n > 128: chol_cluster_kernel below (8-CTA cluster, L2-resident matrix, smem-staged rank-16
// updates on 4 x 4 register tiles).
// A pivot d_k <= 0 or NaN is a CholQR breakdown: reported through *info (LAPACK potrf-style
// 1-based column) and replaced by 1 so no NaN propagates.
#include <cstdio>
#include <cstdlib>

#include "common.cuh"
#include "internal.h"

namespace rs {

constexpr int CB = 16;              // block size
constexpr int CH_BLK_THREADS = 512;
constexpr int CH_SMEM_MAX_N = 128;

// ------------------------------------------------------------------------------------------
// blocked kernel (n <= 128)
// ------------------------------------------------------------------------------------------
template <bool SMEM>
__global__ void __launch_bounds__(CH_BLK_THREADS, 1)
    chol_blocked_kernel(const double* __restrict__ G, int ldg, int n, double* __restrict__ R, int ldr,
                        double* __restrict__ Linv, int ldl, double* __restrict__ gwork, int* info, int code,
                        int npad) {
  extern __shared__ double sm[];
  double* M = SMEM ? sm : gwork;  // np x (np+1), column-major: M[i + j*LM]
  __shared__ double rdinv[512];   // 1 / R_ii
  const int np = (n + CB - 1) / CB * CB;
  const int LM = np + 1;
  const int tid = threadIdx.x, warp = tid >> 5, lane = tid & 31;
  const int nb = np / CB;

  // load the upper triangle of G; identity on the padding
  for (int idx = tid; idx < np * np; idx += CH_BLK_THREADS) {
    const int i = idx % np, j = idx / np;
    double v = 0.0;
    if (i <= j) v = (j < n) ? G[i + static_cast<long long>(j) * ldg] : (i == j ? 1.0 : 0.0);
    M[i + j * LM] = v;
  }
  __syncthreads();

  for (int b = 0; b < nb; ++b) {
    const int b0 = b * CB;
    // (1) diagonal block: lane j < 16 owns column b0+j (rows b0..b0+15) in registers
    if (warp == 0) {
      double col[CB];
#pragma unroll
      for (int i = 0; i < CB; ++i) col[i] = (lane < CB && i <= lane) ? M[(b0 + i) + (b0 + lane) * LM] : 0.0;
#pragma unroll
      for (int kk = 0; kk < CB; ++kk) {
        double d = __shfl_sync(0xffffffffu, col[kk], kk);
        if (!(d > 0.0)) {
          if (lane == 0 && info && b0 + kk < n) atomicCAS(info, 0, code), atomicCAS(info + 1, 0, b0 + kk + 1);
          d = 1.0;
        }
        const double ri = rsqrt(d);  // 1 / R_kk
        if (lane == kk) {
          col[kk] = d * ri;           // R_kk = sqrt(d)
          rdinv[b0 + kk] = ri;
        } else if (lane > kk) {
          col[kk] *= ri;              // R[kk][lane]
        }
        const double rkj = col[kk];
#pragma unroll
        for (int i = kk + 1; i < CB; ++i) {
          const double rki = __shfl_sync(0xffffffffu, col[kk], i);  // R[kk][i] from lane i
          if (lane >= i && lane < CB) col[i] = fma(-rki, rkj, col[i]);
        }
      }
      if (lane < CB) {
#pragma unroll
        for (int i = 0; i < CB; ++i)
          if (i <= lane) M[(b0 + i) + (b0 + lane) * LM] = col[i];
      }
    }
    __syncthreads();
    // (2) panel: R12 = R11^{-T} A12, one thread per trailing column
    const int t2 = np - b0 - CB;
    if (tid < t2) {
      const int c = b0 + CB + tid;
      double x[CB];
#pragma unroll
      for (int i = 0; i < CB; ++i) x[i] = M[(b0 + i) + c * LM];
#pragma unroll
      for (int kk = 0; kk < CB; ++kk) {
        x[kk] *= rdinv[b0 + kk];
#pragma unroll
        for (int i = kk + 1; i < CB; ++i) x[i] = fma(-M[(b0 + kk) + (b0 + i) * LM], x[kk], x[i]);
      }
#pragma unroll
      for (int i = 0; i < CB; ++i) M[(b0 + i) + c * LM] = x[i];
    }
    __syncthreads();
    // (3) trailing update A22 -= R12^T R12 (upper part); 1 x 2 micro-tiles
    if (t2 > 0) {
      const int half = (t2 + 1) / 2;
      for (int idx = tid; idx < t2 * half; idx += CH_BLK_THREADS) {
        const int i = b0 + CB + idx % t2;
        const int j0 = b0 + CB + 2 * (idx / t2);
        if (i > j0 + 1) continue;
        const double* pi = M + b0 + i * LM;
        const double* pj0 = M + b0 + j0 * LM;
        const double* pj1 = pj0 + LM;
        double s0 = 0.0, s1 = 0.0;
#pragma unroll
        for (int kk = 0; kk < CB; ++kk) {
          const double a = pi[kk];
          s0 = fma(a, pj0[kk], s0);
          if (j0 + 1 < np) s1 = fma(a, pj1[kk], s1);
        }
        if (i <= j0) M[i + j0 * LM] -= s0;
        if (j0 + 1 < np && i <= j0 + 1) M[i + (j0 + 1) * LM] -= s1;
      }
    }
    __syncthreads();
  }

  // ---- X = R^{-T} (lower), block row by block row; X[l][c] (l > c) stored at M[l + c*LM] ----
  for (int bi = 0; bi < nb; ++bi) {
    const int I0 = bi * CB;
    // (a) X[i][c] = delta_ic - sum_{l=c}^{I0-1} R[l][i] X[l][c],  i in block, c < I0 + 16, c < i
    //     (the c == i diagonal is handled in (b))
    for (int idx = tid; idx < CB * I0; idx += CH_BLK_THREADS) {
      const int i = I0 + idx % CB, c = idx / CB;  // c < I0
      double s = M[c + i * LM] * rdinv[c];        // l = c term: R[c][i] * X[c][c]
      for (int l = c + 1; l < I0; ++l) s = fma(M[l + i * LM], M[l + c * LM], s);
      M[i + c * LM] = -s;
    }
    __syncthreads();
    // (b) in-block forward solve, one thread per column c < I0 + 16
    if (tid < I0 + CB) {
      const int c = tid;
      double x[CB];
#pragma unroll
      for (int ii = 0; ii < CB; ++ii) {
        const int i = I0 + ii;
        x[ii] = (i > c) ? M[i + c * LM] : 0.0;  // rhs from (a) (zero for c inside the block)
      }
#pragma unroll
      for (int ii = 0; ii < CB; ++ii) {
        const int i = I0 + ii;
        if (i < c) continue;
        double v;
        if (i == c) {
          v = rdinv[i];                          // X[c][c] = 1 / R_cc
        } else {
          double s = x[ii];
#pragma unroll
          for (int jj = 0; jj < ii; ++jj) {
            const int l = I0 + jj;
            if (l >= c) s = fma(-M[l + i * LM], x[jj], s);  // R[l][i] * X[l][c]
          }
          v = s * rdinv[i];
        }
        x[ii] = v;
      }
#pragma unroll
      for (int ii = 0; ii < CB; ++ii) {
        const int i = I0 + ii;
        if (i > c) M[i + c * LM] = x[ii];
      }
    }
    __syncthreads();
  }

  // outputs, zero-padded to npad x npad
  for (int idx = tid; idx < npad * npad; idx += CH_BLK_THREADS) {
    const int i = idx % npad, j = idx / npad;
    double rv = 0.0, lv = 0.0;
    if (i < n && j < n) {
      if (i <= j) rv = M[i + j * LM];
      if (i == j) lv = rdinv[i];
      else if (i > j) lv = M[i + j * LM];
    }
    R[i + static_cast<long long>(j) * ldr] = rv;
    Linv[i + static_cast<long long>(j) * ldl] = lv;
  }
}

// ------------------------------------------------------------------------------------------
// large kernel (128 < n <= 512): one 8-CTA thread-block cluster.  The matrix lives in an
// L2-resident work array (every CTA reads it with ld.global.cg: other CTAs write it); each step's
// rank-16 operands are staged in every CTA's shared memory and the work of each phase is split
// over the 2048 threads of the cluster, phases separated by cluster barriers.
//   factor  block b: (1) CTA 0 warp 0 factors the diagonal block in registers; (2) panel
//           P = R11^{-T} A12, one thread per trailing column; (3) A22 -= P^T P on 4 x 4
//           register tiles of the upper triangle, P from shared memory (LDS.128).
//   inverse X = R^{-T} (strict lower part of M, diagonal 1/R_ii apart), right-looking by block
//           row: (a) in-block forward solve of block row b, one thread per column c < b0+16;
//           (b) X(i, c) -= sum_kk R(b0+kk, i) X(b0+kk, c) for the later rows, 4 x 4 tiles.
// ------------------------------------------------------------------------------------------
constexpr int CHL_THREADS = 256;
constexpr int CHL_MAXN = 512;
constexpr int CHL_CLUSTER = 8;

__global__ void __launch_bounds__(CHL_THREADS, 1)
    chol_cluster_kernel(const double* __restrict__ G, int ldg, int n, double* __restrict__ R, int ldr,
                        double* __restrict__ Linv, int ldl, double* M, double* rdg, int* info, int code,
                        int npad) {
  extern __shared__ double P_dyn[];  // 2 x CB x CHL_MAXN: panel / X block row, and Rs
  double (*P)[CHL_MAXN] = reinterpret_cast<double (*)[CHL_MAXN]>(P_dyn);
  double (*Rs)[CHL_MAXN] = reinterpret_cast<double (*)[CHL_MAXN]>(P_dyn + CB * CHL_MAXN);
  __shared__ double D[CB][CB + 1];  // diagonal block: D[kk][j] = R[b0+kk][b0+j]
  // volatile view for the per-column solves: keeps the block values from being hoisted into
  // registers across the column loop (they spill otherwise)
  volatile double (*Dv)[CB + 1] = D;
  __shared__ double rdl[CHL_MAXN];  // 1 / R_ii
  const int np = (n + CB - 1) / CB * CB;
  const int LM = np + 1;
  const int nb = np / CB;
  const int tid = threadIdx.x, warp = tid >> 5, lane = tid & 31;
  const int crank = static_cast<int>(cluster_ctarank());
  constexpr int GT = CHL_THREADS * CHL_CLUSTER;
  const int gt = crank * CHL_THREADS + tid;

  // upper triangle of G, identity on the padding, zero strict lower part (X's right-hand side);
  // eight elements per thread per round so the loads overlap
  for (int base = 0; base < np * np; base += 8 * GT) {
    double v[8];
#pragma unroll
    for (int u = 0; u < 8; ++u) {
      const int idx = base + u * GT + gt;
      const int i = idx % np, j = idx / np;
      v[u] = 0.0;
      if (idx < np * np && i <= j) v[u] = (j < n) ? G[i + static_cast<long long>(j) * ldg] : (i == j ? 1.0 : 0.0);
    }
#pragma unroll
    for (int u = 0; u < 8; ++u) {
      const int idx = base + u * GT + gt;
      if (idx < np * np) M[idx % np + (idx / np) * LM] = v[u];
    }
  }
  cluster_sync_all();

  for (int b = 0; b < nb; ++b) {
    const int b0 = b * CB;
    const int t2 = np - b0 - CB;
    // (1) diagonal block (CTA 0, warp 0; lane j owns column b0+j)
    if (crank == 0 && warp == 0) {
      double col[CB];
#pragma unroll
      for (int i = 0; i < CB; ++i) col[i] = (lane < CB && i <= lane) ? __ldcg(&M[(b0 + i) + (b0 + lane) * LM]) : 0.0;
#pragma unroll
      for (int kk = 0; kk < CB; ++kk) {
        double d = __shfl_sync(0xffffffffu, col[kk], kk);
        if (!(d > 0.0)) {
          if (lane == 0 && info && b0 + kk < n) atomicCAS(info, 0, code), atomicCAS(info + 1, 0, b0 + kk + 1);
          d = 1.0;
        }
        const double ri = rsqrt(d);
        if (lane == kk) {
          col[kk] = d * ri;
          rdg[b0 + kk] = ri;
        } else if (lane > kk) {
          col[kk] *= ri;
        }
        const double rkj = col[kk];
#pragma unroll
        for (int i = kk + 1; i < CB; ++i) {
          const double rki = __shfl_sync(0xffffffffu, col[kk], i);
          if (lane >= i && lane < CB) col[i] = fma(-rki, rkj, col[i]);
        }
      }
      if (lane < CB) {
#pragma unroll
        for (int i = 0; i <= lane && i < CB; ++i) M[(b0 + i) + (b0 + lane) * LM] = col[i];
      }
    }
    cluster_sync_all();
    for (int e = tid; e < CB * CB; e += CHL_THREADS) {
      const int kk = e / CB, j = e % CB;
      D[kk][j] = kk <= j ? __ldcg(&M[(b0 + kk) + (b0 + j) * LM]) : 0.0;
    }
    if (tid < CB) rdl[b0 + tid] = __ldcg(&rdg[b0 + tid]);
    __syncthreads();
    // (2) panel: one thread per trailing column c, x = R11^{-T} A12(:, c)
    for (int cc = gt; cc < t2; cc += GT) {
      const int c = b0 + CB + cc;
      double x[CB];
#pragma unroll
      for (int i = 0; i < CB; ++i) x[i] = __ldcg(&M[(b0 + i) + c * LM]);
#pragma unroll
      for (int kk = 0; kk < CB; ++kk) {
        x[kk] *= rdl[b0 + kk];
#pragma unroll
        for (int i = kk + 1; i < CB; ++i) x[i] = fma(-Dv[kk][i], x[kk], x[i]);
      }
#pragma unroll
      for (int i = 0; i < CB; ++i) M[(b0 + i) + c * LM] = x[i];
    }
    cluster_sync_all();
    if (t2 == 0) continue;
    for (int e = tid; e < CB * t2; e += CHL_THREADS) {
      const int cc = e / CB, kk = e % CB;
      P[kk][cc] = __ldcg(&M[(b0 + kk) + (b0 + CB + cc) * LM]);
    }
    __syncthreads();
    // (3) trailing update, 4 x 4 tiles (I, J), I <= J, over the upper triangle
    {
      const int nt = t2 / 4;
      const int ntiles = nt * (nt + 1) / 2;
      for (int t = gt; t < ntiles; t += GT) {
        int J = static_cast<int>((sqrt(8.0 * t + 1.0) - 1.0) * 0.5);
        while (J * (J + 1) / 2 > t) --J;
        while ((J + 1) * (J + 2) / 2 <= t) ++J;
        const int I = t - J * (J + 1) / 2;
        const int r0 = b0 + CB + 4 * I, c0 = b0 + CB + 4 * J;
        double a[4][4];
#pragma unroll
        for (int q = 0; q < 4; ++q)
#pragma unroll
          for (int r = 0; r < 4; ++r) a[q][r] = __ldcg(&M[(r0 + r) + (c0 + q) * LM]);
#pragma unroll
        for (int kk = 0; kk < CB; ++kk) {
          const double2 p01 = *reinterpret_cast<const double2*>(&P[kk][4 * I]);
          const double2 p23 = *reinterpret_cast<const double2*>(&P[kk][4 * I + 2]);
          const double2 q01 = *reinterpret_cast<const double2*>(&P[kk][4 * J]);
          const double2 q23 = *reinterpret_cast<const double2*>(&P[kk][4 * J + 2]);
          const double pr[4] = {p01.x, p01.y, p23.x, p23.y};
          const double pc[4] = {q01.x, q01.y, q23.x, q23.y};
#pragma unroll
          for (int q = 0; q < 4; ++q)
#pragma unroll
            for (int r = 0; r < 4; ++r) a[q][r] = fma(-pr[r], pc[q], a[q][r]);
        }
#pragma unroll
        for (int q = 0; q < 4; ++q)
#pragma unroll
          for (int r = 0; r < 4; ++r)
            if (I < J || r <= q) M[(r0 + r) + (c0 + q) * LM] = a[q][r];
      }
    }
    cluster_sync_all();
  }

  // ---- inverse: X = R^{-T}, X(i, c) (i > c) at M[i + c*LM] (zero-initialised above) ----
  for (int b = 0; b < nb; ++b) {
    const int b0 = b * CB;
    const int ncol = b0 + CB;
    for (int e = tid; e < CB * CB; e += CHL_THREADS) {
      const int kk = e / CB, j = e % CB;
      D[kk][j] = kk <= j ? __ldcg(&M[(b0 + kk) + (b0 + j) * LM]) : 0.0;
    }
    __syncthreads();
    // (a) in-block forward solve R_bb^T X(b, c) = rhs, one thread per column c < ncol
    for (int c = gt; c < ncol; c += GT) {
      double x[CB];
#pragma unroll
      for (int ii = 0; ii < CB; ++ii) {
        const int i = b0 + ii;
        x[ii] = i > c ? __ldcg(&M[i + c * LM]) : 0.0;
      }
#pragma unroll
      for (int ii = 0; ii < CB; ++ii) {
        const int i = b0 + ii;
        double v;
        if (i < c) {
          v = 0.0;
        } else if (i == c) {
          v = rdl[i];
        } else {
          double s = x[ii];
#pragma unroll
          for (int jj = 0; jj < ii; ++jj) s = fma(-Dv[jj][ii], x[jj], s);
          v = s * rdl[i];
        }
        x[ii] = v;
      }
#pragma unroll
      for (int ii = 0; ii < CB; ++ii) {
        const int i = b0 + ii;
        if (i > c) M[i + c * LM] = x[ii];
      }
    }
    cluster_sync_all();
    const int nrow = np - ncol;
    if (nrow == 0) continue;
    // stage X(b rows, c < ncol) (with its diagonal and zeros above) and R(b rows, later rows)
    for (int e = tid; e < CB * ncol; e += CHL_THREADS) {
      const int c = e / CB, ii = e % CB;
      const int i = b0 + ii;
      P[ii][c] = i > c ? __ldcg(&M[i + c * LM]) : (i == c ? rdl[i] : 0.0);
    }
    for (int e = tid; e < CB * nrow; e += CHL_THREADS) {
      const int ii = e / CB, kk = e % CB;
      Rs[kk][ii] = __ldcg(&M[(b0 + kk) + (ncol + ii) * LM]);
    }
    __syncthreads();
    // (b) later rows: (nrow x 16) x (16 x ncol), 4 x 4 tiles
    const int ntr = nrow / 4, ntc = ncol / 4;
    for (int t = gt; t < ntr * ntc; t += GT) {
      const int I = t % ntr, J = t / ntr;
      const int r0 = ncol + 4 * I, c0 = 4 * J;
      double a[4][4];
#pragma unroll
      for (int q = 0; q < 4; ++q)
#pragma unroll
        for (int r = 0; r < 4; ++r) a[q][r] = __ldcg(&M[(r0 + r) + (c0 + q) * LM]);
#pragma unroll
      for (int kk = 0; kk < CB; ++kk) {
        const double2 p01 = *reinterpret_cast<const double2*>(&Rs[kk][4 * I]);
        const double2 p23 = *reinterpret_cast<const double2*>(&Rs[kk][4 * I + 2]);
        const double2 q01 = *reinterpret_cast<const double2*>(&P[kk][c0]);
        const double2 q23 = *reinterpret_cast<const double2*>(&P[kk][c0 + 2]);
        const double pr[4] = {p01.x, p01.y, p23.x, p23.y};
        const double pc[4] = {q01.x, q01.y, q23.x, q23.y};
#pragma unroll
        for (int q = 0; q < 4; ++q)
#pragma unroll
          for (int r = 0; r < 4; ++r) a[q][r] = fma(-pr[r], pc[q], a[q][r]);
      }
#pragma unroll
      for (int q = 0; q < 4; ++q)
#pragma unroll
        for (int r = 0; r < 4; ++r) M[(r0 + r) + (c0 + q) * LM] = a[q][r];
    }
    cluster_sync_all();
  }

  // outputs, zero-padded to npad x npad
  for (int base = 0; base < npad * npad; base += 8 * GT) {
    double mv[8];
#pragma unroll
    for (int u = 0; u < 8; ++u) {
      const int idx = base + u * GT + gt;
      const int i = idx % npad, j = idx / npad;
      mv[u] = (idx < npad * npad && i < n && j < n) ? __ldcg(&M[i + j * LM]) : 0.0;
    }
#pragma unroll
    for (int u = 0; u < 8; ++u) {
      const int idx = base + u * GT + gt;
      if (idx >= npad * npad) continue;
      const int i = idx % npad, j = idx / npad;
      double rv = 0.0, lv = 0.0;
      if (i < n && j < n) {
        if (i <= j) rv = mv[u];
        if (i > j) lv = mv[u];
        else if (i == j) lv = rdl[i];
      }
      R[i + static_cast<long long>(j) * ldr] = rv;
      Linv[i + static_cast<long long>(j) * ldl] = lv;
    }
  }
}

// ------------------------------------------------------------------------------------------
// register-tile kernel (n <= 128): right-looking Cholesky and forward substitution for
// X = R^{-T} advanced together, ONE barrier per pivot.  The upper triangle of G and the lower
// triangle of the right-hand-side accumulators of X live in 4 x 4 register tiles (TPT per
// thread).  At step k every thread reads the published row k of G and of X's accumulators and
// forms 1/d_k = rsqrt(d_k)^2 itself (all threads see the same d_k, so all get the same value);
// the rank-1 updates are G(i, j) -= G(k, i) G(k, j) / d_k (= R(k, i) R(k, j)) and
// acc(i, c) -= G(k, i) acc(k, c) / d_k (= R(k, i) X(k, c)); the owners of row k + 1 publish it
// into the other buffer.  The step loop is unrolled by 4 so the tile row being published is a
// compile-time register index.  Rows <= k of a tile are dead after step k (already written out),
// so the updates need no predicates.  Tiles are ordered by row block, descending, so whole warps
// retire as k grows.
// ------------------------------------------------------------------------------------------
constexpr int CT_MAXN = 128;

template <int TPT, int NTHR>
struct CholTile {
  double v[TPT][4][4];
  int kind[TPT], TI[TPT], TJ[TPT];
  bool has[TPT];
};

// Published rows are kept for the whole factorisation in shared memory, packed: row k of G from
// column 4(k/4) on (the columns any live tile can read), row k of X's accumulators up to column
// 4(k/4) + 3.  Nothing is written to global memory inside the pivot loop; R and Linv are written
// once at the end from the packed rows and the per-pivot 1/sqrt(d_k) (coalesced, all threads).
RS_DEVINL int ct_gofs(int k, int np) {
  const int b = k >> 2, r = k & 3;
  return 4 * np * b - 8 * b * (b - 1) + r * (np - 4 * b);
}
RS_DEVINL int ct_xofs(int k) {
  const int b = k >> 2, r = k & 3;
  return 8 * b * (b + 1) + r * 4 * (b + 1);
}
// packed shared memory (doubles) for an np x np problem
__host__ __device__ constexpr int ct_smem_doubles(int np) {
  return (4 * np * (np / 4) - 8 * (np / 4) * (np / 4 - 1)) + 8 * (np / 4) * (np / 4 + 1) + np + 8;
}

// one pivot step k with (k + 1) % 4 == A1 (the tile row that holds row k + 1)
template <int A1, int TPT, int NTHR>
RS_DEVINL void chol_tile_step(CholTile<TPT, NTHR>& T, int k, int n, int np, double* Gs, double* Xs, double* s_ri,
                              int* info, int code, int col0) {
  const int tid = threadIdx.x;
  const int k4 = 4 * (k >> 2);
  const double* Gk = Gs + ct_gofs(k, np) - k4;  // Gk[c] = G(k, c), c >= 4 (k / 4)
  const double* Xk = Xs + ct_xofs(k);           // Xk[c] = acc(k, c), c < 4 (k / 4) + 4
  // 1 / sqrt(d_k) was formed once by the thread that published row k (below / at the start)
  const double ri = s_ri[k];
  const double dinv = ri * ri;
  const int ipub = (k + 1) >> 2;  // tile row block holding row k + 1
  double* Gn = Gs + ct_gofs(k + 1, np) - 4 * ipub;
  double* Xn = Xs + ct_xofs(k + 1);
#pragma unroll
  for (int s2 = 0; s2 < TPT; ++s2) {
    if (!T.has[s2] || 4 * T.TI[s2] + 3 <= k) continue;  // rows of the tile all finished
    if (T.kind[s2] == 0 || 4 * T.TJ[s2] <= k) {          // (X(k, c) = 0 for c > k: nothing to add)
      const double2* gpi = reinterpret_cast<const double2*>(&Gk[4 * T.TI[s2]]);
      const double2 gi0 = gpi[0], gi1 = gpi[1];
      const double ra[4] = {gi0.x * dinv, gi0.y * dinv, gi1.x * dinv, gi1.y * dinv};
      const double2* src = T.kind[s2] == 0 ? reinterpret_cast<const double2*>(&Gk[4 * T.TJ[s2]])
                                           : reinterpret_cast<const double2*>(&Xk[4 * T.TJ[s2]]);
      const double2 c0 = src[0], c1 = src[1];
      const double cb[4] = {c0.x, c0.y, c1.x, c1.y};
#pragma unroll
      for (int a = 0; a < 4; ++a)
#pragma unroll
        for (int bb = 0; bb < 4; ++bb) T.v[s2][a][bb] = fma(-ra[a], cb[bb], T.v[s2][a][bb]);
    }
    if (T.TI[s2] == ipub && k + 1 < np) {  // publish row k + 1 = tile row A1
      const int c = 4 * T.TJ[s2];
      if (T.kind[s2] == 0) {
        reinterpret_cast<double2*>(&Gn[c])[0] = make_double2(T.v[s2][A1][0], T.v[s2][A1][1]);
        reinterpret_cast<double2*>(&Gn[c])[1] = make_double2(T.v[s2][A1][2], T.v[s2][A1][3]);
        if (T.TJ[s2] == ipub) {  // the diagonal tile: d_{k+1} = G(k+1, k+1), checked and inverted once
          double dn = T.v[s2][A1][A1];
          if (!(dn > 0.0)) {
            if (info && k + 1 < n) atomicCAS(info, 0, code), atomicCAS(info + 1, 0, col0 + k + 2);
            dn = 1.0;
          }
          s_ri[k + 1] = rsqrt(dn);
        }
      } else {
        const int lim = k + 1 - c;  // X(k + 1, c + bb) = 0 for c + bb > k + 1
        reinterpret_cast<double2*>(&Xn[c])[0] =
            make_double2(lim >= 0 ? T.v[s2][A1][0] : 0.0, lim >= 1 ? T.v[s2][A1][1] : 0.0);
        reinterpret_cast<double2*>(&Xn[c])[1] =
            make_double2(lim >= 2 ? T.v[s2][A1][2] : 0.0, lim >= 3 ? T.v[s2][A1][3] : 0.0);
      }
    }
  }
  __syncthreads();
}

template <int TPT, int NTHR>
__global__ void __launch_bounds__(NTHR, 1)
    chol_tile_kernel(const double* __restrict__ G, int ldg, int n, double* __restrict__ R, int ldr,
                     double* __restrict__ Linv, int ldl, int* info, int code, int npad, int col0) {
  extern __shared__ __align__(16) double ct_smem[];
  const int tid = threadIdx.x;
  const int np = (n + 3) / 4 * 4;
  const int nt = np / 4;  // tile blocks per dimension
  double* Gs = ct_smem;
  double* Xs = Gs + ct_gofs(np, np);
  double* s_ri = Xs + ct_xofs(np);
  CholTile<TPT, NTHR> T;
#pragma unroll
  for (int s2 = 0; s2 < TPT; ++s2) {
    const int t = tid + s2 * NTHR;
    T.has[s2] = t < nt * (nt + 1);
    T.kind[s2] = 0, T.TI[s2] = 0, T.TJ[s2] = 0;
    if (T.has[s2]) {
      // row block I (from nt-1 down) holds (nt - I) G tiles (J = I..nt-1), then I + 1 X tiles
      const int q = t / (nt + 1), rr = t - q * (nt + 1);
      const int I = nt - 1 - q;
      T.TI[s2] = I;
      if (rr < nt - I) {
        T.TJ[s2] = I + rr;
      } else {
        T.kind[s2] = 1;
        T.TJ[s2] = rr - (nt - I);
      }
    }
#pragma unroll
    for (int a = 0; a < 4; ++a)
#pragma unroll
      for (int bb = 0; bb < 4; ++bb) {
        const int i = 4 * T.TI[s2] + a, j = 4 * T.TJ[s2] + bb;
        double x = 0.0;
        if (T.has[s2]) {
          if (T.kind[s2] == 0) {
            const int lo = i < j ? i : j, hi = i < j ? j : i;
            x = (hi < n) ? G[lo + static_cast<long long>(hi) * ldg] : (i == j ? 1.0 : 0.0);
          } else {
            x = (i == j) ? 1.0 : 0.0;
          }
        }
        T.v[s2][a][bb] = x;
      }
  }
  // row 0 of G (identity-padded past n) and of X's accumulators (e_0)
  for (int j = tid; j < np; j += NTHR) Gs[j] = (j < n) ? G[static_cast<long long>(j) * ldg] : (j == 0 ? 1.0 : 0.0);
  if (tid < 4) Xs[tid] = tid == 0 ? 1.0 : 0.0;
  if (tid == 0) {
    double d0 = n > 0 ? G[0] : 1.0;
    if (!(d0 > 0.0)) {
      if (info) atomicCAS(info, 0, code), atomicCAS(info + 1, 0, col0 + 1);
      d0 = 1.0;
    }
    s_ri[0] = rsqrt(d0);
  }
  __syncthreads();
  for (int k = 0; k < np; k += 4) {  // np is a multiple of 4
    chol_tile_step<1>(T, k, n, np, Gs, Xs, s_ri, info, code, col0);
    chol_tile_step<2>(T, k + 1, n, np, Gs, Xs, s_ri, info, code, col0);
    chol_tile_step<3>(T, k + 2, n, np, Gs, Xs, s_ri, info, code, col0);
    chol_tile_step<0>(T, k + 3, n, np, Gs, Xs, s_ri, info, code, col0);
  }
  // R(k, t) = G(k, t) / sqrt(d_k) (t >= k), Linv(k, t) = acc(k, t) / sqrt(d_k) (t <= k), zero
  // elsewhere and in the padding; consecutive threads take consecutive rows (column-major)
  for (int idx = tid; idx < npad * npad; idx += NTHR) {
    const int kk = idx % npad, t = idx / npad;
    double rv = 0.0, lv = 0.0;
    if (kk < n && t < n) {
      const double ri = s_ri[kk];
      if (t >= kk) rv = Gs[ct_gofs(kk, np) - 4 * (kk >> 2) + t] * ri;
      if (t <= kk) lv = Xs[ct_xofs(kk) + t] * ri;
    }
    R[kk + static_cast<long long>(t) * ldr] = rv;
    Linv[kk + static_cast<long long>(t) * ldl] = lv;
  }
}

cudaError_t chol_inv_at(cudaStream_t st, const double* G, int ldg, int n, int npad, double* R, int ldr, double* Linv,
                        int ldl, double* gwork, int* info, int info_code, int col0);

// 128 < n <= 256: 2 x 2 blocks on the register-tile kernel.  G = R^T R with R = [R11 R12; 0 R22]:
// R11 = chol(G11), R12 = R11^{-T} G12 = L11^{-1} G12, R22 = chol(G22 - R12^T R12), and
// L^{-1} = R^{-T} = [L11^{-1} 0; -L22^{-1} R12^T L11^{-1}  L22^{-1}] -- two one-CTA factorisations and
// four small GEMMs instead of the 8-CTA cluster kernel's one barrier per pivot (cfg3's l = 220).
static cudaError_t chol_inv_2x2(cudaStream_t st, const double* G, int ldg, int n, int npad, double* R, int ldr,
                                double* Linv, int ldl, double* gwork, int* info, int info_code, int col0) {
  const int n1 = 16 * ((n + 31) / 32), n2 = n - n1;
  double* S = gwork;                                   // n2 x n2: G22 - R12^T R12
  double* Tm = gwork + static_cast<size_t>(n2) * n2;   // n2 x n1: R12^T L11^{-1}
  cudaError_t e = cudaMemset2DAsync(R, static_cast<size_t>(ldr) * 8, 0, static_cast<size_t>(npad) * 8, npad, st);
  if (e == cudaSuccess)
    e = cudaMemset2DAsync(Linv, static_cast<size_t>(ldl) * 8, 0, static_cast<size_t>(npad) * 8, npad, st);
  if (e == cudaSuccess) e = chol_inv_at(st, G, ldg, n1, n1, R, ldr, Linv, ldl, nullptr, info, info_code, col0);
  double* R12 = R + static_cast<long long>(n1) * ldr;
  if (e == cudaSuccess)  // R12 = L11^{-1} G12
    e = small_gemm(st, n1, n2, n1, Linv, 1, ldl, G + static_cast<long long>(n1) * ldg, 1, ldg, R12, 1, ldr, false);
  if (e == cudaSuccess) e = copy_2d(st, G + n1 + static_cast<long long>(n1) * ldg, ldg, S, n2, n2, n2);
  if (e == cudaSuccess)  // S = G22 - R12^T R12 (full, both triangles)
    e = small_gemm(st, n2, n2, n1, R12, ldr, 1, R12, 1, ldr, S, 1, n2, true, -1.0);
  double* R22 = R + n1 + static_cast<long long>(n1) * ldr;
  double* L22 = Linv + n1 + static_cast<long long>(n1) * ldl;
  if (e == cudaSuccess) e = chol_inv_at(st, S, n2, n2, n2, R22, ldr, L22, ldl, nullptr, info, info_code, col0 + n1);
  if (e == cudaSuccess)  // T = R12^T L11^{-1}
    e = small_gemm(st, n2, n1, n1, R12, ldr, 1, Linv, 1, ldl, Tm, 1, n2, false);
  if (e == cudaSuccess)  // L21^{-1} block = -L22^{-1} T
    e = small_gemm(st, n2, n1, n2, L22, 1, ldl, Tm, 1, n2, Linv + n1, 1, ldl, false, -1.0);
  return e;
}

cudaError_t chol_inv(cudaStream_t st, const double* G, int ldg, int n, int npad, double* R, int ldr, double* Linv,
                     int ldl, double* gwork, int* info, int info_code) {
  return chol_inv_at(st, G, ldg, n, npad, R, ldr, Linv, ldl, gwork, info, info_code, 0);
}

cudaError_t chol_inv_at(cudaStream_t st, const double* G, int ldg, int n, int npad, double* R, int ldr, double* Linv,
                        int ldl, double* gwork, int* info, int info_code, int col0) {
  if (n <= 0) return cudaSuccess;
  if (n > 512) return cudaErrorInvalidValue;
#ifndef RS_DEV_CHOL_CLUSTER_256
  if (n > CT_MAXN && n <= 2 * CT_MAXN && gwork)
    return chol_inv_2x2(st, G, ldg, n, npad, R, ldr, Linv, ldl, gwork, info, info_code, col0);
#endif
  // compile-time development switches: -DRS_DEV_CHOL_SMEM_MAX_N=<n> (crossover experiments),
  // -DRS_DEV_CHOL_BLOCKED (the blocked kernel for n <= 128), -DRS_DEV_CHOL_TPT=2 (two tiles per thread)
#ifdef RS_DEV_CHOL_SMEM_MAX_N
  constexpr int smem_max_n = RS_DEV_CHOL_SMEM_MAX_N;
#else
  constexpr int smem_max_n = CH_SMEM_MAX_N;
#endif
#ifdef RS_DEV_CHOL_BLOCKED
  constexpr bool use_tile = false;
#else
  constexpr bool use_tile = true;
#endif
  if (use_tile && n <= CT_MAXN) {
    const int nt = (n + 3) / 4;
#ifdef RS_DEV_CHOL_TPT
    constexpr int tpt = RS_DEV_CHOL_TPT;
#else
    constexpr int tpt = 1;
#endif
    constexpr int ct_max_smem = ct_smem_doubles(CT_MAXN) * 8;
    for (auto fn : {chol_tile_kernel<1, 256>, chol_tile_kernel<1, 512>, chol_tile_kernel<1, 832>,
                    chol_tile_kernel<1, 1024>, chol_tile_kernel<2, 576>}) {
      cudaError_t e = ensure_smem(fn, ct_max_smem);
      if (e != cudaSuccess) return e;
    }
    const size_t ct_smem = static_cast<size_t>(ct_smem_doubles(4 * nt)) * 8;
    // one tile per thread, in the smallest CTA that holds all nt (nt + 1) tiles: idle warps would
    // still take part in every pivot's barrier
    const int tiles = nt * (nt + 1);
    if (tpt == 1 && tiles <= 256)  // n <= 60 (adaptive blocks, Fig. 7's k = 54)
      chol_tile_kernel<1, 256><<<1, 256, ct_smem, st>>>(G, ldg, n, R, ldr, Linv, ldl, info, info_code, npad, col0);
    else if (tpt == 1 && tiles <= 512)  // n <= 88 (l = 64)
      chol_tile_kernel<1, 512><<<1, 512, ct_smem, st>>>(G, ldg, n, R, ldr, Linv, ldl, info, info_code, npad, col0);
    else if (tpt == 1 && tiles <= 832)  // n <= 112 (l = 110: 72 registers per thread instead of 64)
      chol_tile_kernel<1, 832><<<1, 832, ct_smem, st>>>(G, ldg, n, R, ldr, Linv, ldl, info, info_code, npad, col0);
    else if (tpt == 1 && tiles <= 1024)  // n <= 124
      chol_tile_kernel<1, 1024><<<1, 1024, ct_smem, st>>>(G, ldg, n, R, ldr, Linv, ldl, info, info_code, npad, col0);
    else
      chol_tile_kernel<2, 576><<<1, 576, ct_smem, st>>>(G, ldg, n, R, ldr, Linv, ldl, info, info_code, npad, col0);
  } else if (n <= smem_max_n && n <= CH_SMEM_MAX_N) {
    const int np = (n + CB - 1) / CB * CB;
    const size_t smem = static_cast<size_t>(np) * (np + 1) * 8;
    {
      cudaError_t e = ensure_smem(chol_blocked_kernel<true>, CH_SMEM_MAX_N * (CH_SMEM_MAX_N + 1) * 8);
      if (e != cudaSuccess) return e;
    }
    chol_blocked_kernel<true><<<1, CH_BLK_THREADS, smem, st>>>(G, ldg, n, R, ldr, Linv, ldl, gwork, info, info_code,
                                                                npad);
  } else {  // one 8-CTA cluster on an L2-resident copy in the workspace (np x (np+1) + np doubles)
    const size_t smem = 2 * static_cast<size_t>(CB) * CHL_MAXN * 8;
    {
      cudaError_t e = ensure_smem(chol_cluster_kernel, static_cast<int>(smem));
      if (e != cudaSuccess) return e;
      if (CHL_CLUSTER > 8) {
        e = ensure_func_attr(reinterpret_cast<const void*>(chol_cluster_kernel),
                             cudaFuncAttributeNonPortableClusterSizeAllowed, 1);
        if (e != cudaSuccess) return e;
      }
    }
    const int np = (n + CB - 1) / CB * CB;
    cudaLaunchConfig_t cfg{};
    cfg.gridDim = dim3(CHL_CLUSTER, 1, 1);
    cfg.blockDim = dim3(CHL_THREADS, 1, 1);
    cfg.dynamicSmemBytes = smem;
    cfg.stream = st;
    cudaLaunchAttribute attr[1];
    attr[0].id = cudaLaunchAttributeClusterDimension;
    attr[0].val.clusterDim.x = CHL_CLUSTER;
    attr[0].val.clusterDim.y = 1;
    attr[0].val.clusterDim.z = 1;
    cfg.attrs = attr;
    cfg.numAttrs = 1;
    double* rdg = gwork + static_cast<size_t>(np) * (np + 1);
    cudaError_t e = cudaLaunchKernelEx(&cfg, chol_cluster_kernel, G, ldg, n, R, ldr, Linv, ldl, gwork, rdg, info,
                                       info_code, npad);
    if (e != cudaSuccess) return e;
  }
  count_launch();
  return cudaGetLastError();
}

}  // namespace rs
