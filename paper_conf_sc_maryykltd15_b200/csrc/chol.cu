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
// n > 128: the same blocked schedule on an L2-resident copy in the workspace.
// A pivot d_k <= 0 or NaN is a CholQR breakdown: reported through *info (LAPACK potrf-style
// 1-based column) and replaced by 1 so no NaN propagates.
#include <cstdio>

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

cudaError_t chol_inv(cudaStream_t st, const double* G, int ldg, int n, int npad, double* R, int ldr, double* Linv,
                     int ldl, double* gwork, int* info, int info_code) {
  if (n <= 0) return cudaSuccess;
  if (n > 512) return cudaErrorInvalidValue;
  if (n <= CH_SMEM_MAX_N) {
    const int np = (n + CB - 1) / CB * CB;
    const size_t smem = static_cast<size_t>(np) * (np + 1) * 8;
    static bool attr = false;
    if (!attr) {
      cudaError_t e = cudaFuncSetAttribute(chol_blocked_kernel<true>, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                           CH_SMEM_MAX_N * (CH_SMEM_MAX_N + 1) * 8);
      if (e != cudaSuccess) return e;
      attr = true;
    }
    chol_blocked_kernel<true><<<1, CH_BLK_THREADS, smem, st>>>(G, ldg, n, R, ldr, Linv, ldl, gwork, info, info_code,
                                                                npad);
  } else {  // same schedule on an L2-resident copy in the workspace (np x (np+1) doubles)
    chol_blocked_kernel<false><<<1, CH_BLK_THREADS, 0, st>>>(G, ldg, n, R, ldr, Linv, ldl, gwork, info, info_code,
                                                             npad);
  }
  count_launch();
  return cudaGetLastError();
}

}  // namespace rs
