// Cholesky factor of a Gram matrix and its inverse in one pass: CholQR steps (ii)-(iii)
// ("R^T R := G, R upper-triangular with non-negative diagonal; Q = R^{-T} B").
//
// Right-looking LDL^T elimination of G with the same row operations applied to an identity E,
// which becomes L_unit^{-1}:   at pivot k, for every row i > k,
//     S[i][j] -= S[k][i] S[k][j] / d_k          (j >= i)
//     E[i][c] -= S[k][i] / d_k * E[k][c]         (c <= k, E[k][k] = 1)
// Then R[i][j] = S[i][j] / sqrt(d_i) and Linv = R^{-T} = D^{-1/2} E.  S (upper) and E (strict
// lower; its unit diagonal is implicit) share one n x n array M.
//
// One CTA of 1024 threads.  Each thread owns strips of 8 consecutive columns of a row and keeps
// them in registers (n <= 128); row k is published to shared memory by its owners right after
// step k-1, so each pivot costs one __syncthreads and every active thread does ~16 FMAs per step
// on registers with row k read as broadcast LDS.128.  For n > 128 the same schedule runs on an
// L2-resident copy in the workspace.  A pivot d_k <= 0 or NaN is a CholQR breakdown: reported
// through *info (LAPACK potrf-style 1-based column) and replaced by 1 so no NaN propagates.
#include <cstdio>

#include "common.cuh"
#include "internal.h"

namespace rs {

constexpr int CH_THREADS = 1024;
constexpr int CH_SMEM_MAX_N = 128;
constexpr int CH_SW = 8;                                                          // strip width
constexpr int CH_MAXS = (CH_SMEM_MAX_N * (CH_SMEM_MAX_N / CH_SW) + CH_THREADS - 1) / CH_THREADS;  // 2

template <bool SMALL>
__global__ void __launch_bounds__(CH_THREADS, 1) chol_inv_kernel(const double* __restrict__ G, int ldg, int n,
                                                                  double* __restrict__ R, int ldr,
                                                                  double* __restrict__ Linv, int ldl,
                                                                  double* __restrict__ gwork, int* info, int code,
                                                                  int npad) {
  extern __shared__ double sm[];
  __shared__ double s_inv[CH_SMEM_MAX_N > 512 ? CH_SMEM_MAX_N : 512];
  const int tid = threadIdx.x;
  const int ns = (n + CH_SW - 1) / CH_SW;  // strips per row
  const int ldm = ns * CH_SW;              // row pitch of M (multiple of 8 -> 64-byte aligned strips)
  double* M = SMALL ? sm : gwork;
  const int nstrips = n * ns;

  auto pivot_inv = [&](int k, double d) {  // by the owner of M[k][k]
    if (!(d > 0.0)) {
      if (info) atomicCAS(info, 0, code), atomicCAS(info + 1, 0, k + 1);
      d = 1.0;
    }
    s_inv[k] = 1.0 / d;
  };

  if (SMALL) {
    double reg[CH_MAXS][CH_SW];
    int ri[CH_MAXS], rj[CH_MAXS];
#pragma unroll
    for (int u = 0; u < CH_MAXS; ++u) {
      const int id = tid + u * CH_THREADS;
      ri[u] = id < nstrips ? id / ns : n;  // n = no strip
      rj[u] = id < nstrips ? (id % ns) * CH_SW : 0;
#pragma unroll
      for (int e = 0; e < CH_SW; ++e) {
        const int j = rj[u] + e;
        reg[u][e] = (ri[u] < n && j < n) ? (j >= ri[u] ? G[ri[u] + static_cast<long long>(j) * ldg] : 0.0) : 0.0;
      }
      if (ri[u] == 0) {  // publish row 0
#pragma unroll
        for (int e = 0; e < CH_SW; ++e) M[rj[u] + e] = reg[u][e];
        if (rj[u] == 0) pivot_inv(0, reg[u][0]);
      }
    }
    __syncthreads();
    for (int k = 0; k < n - 1; ++k) {
      const double* Mk = M + static_cast<long long>(k) * ldm;
      const double inv = s_inv[k];
#pragma unroll
      for (int u = 0; u < CH_MAXS; ++u) {
        const int i = ri[u];
        if (i <= k || i >= n) continue;
        const double l = Mk[i] * inv;  // S[k][i] / d_k
        const double2* rk = reinterpret_cast<const double2*>(Mk + rj[u]);
#pragma unroll
        for (int e2 = 0; e2 < CH_SW / 2; ++e2) {
          const double2 m2 = rk[e2];
#pragma unroll
          for (int h = 0; h < 2; ++h) {
            const int e = 2 * e2 + h;
            const int j = rj[u] + e;
            const double mkj = h ? m2.y : m2.x;
            if (j >= i)
              reg[u][e] = fma(-l, mkj, reg[u][e]);                     // S part
            else if (j <= k)
              reg[u][e] = fma(-l, j == k ? 1.0 : mkj, reg[u][e]);      // E part (E[k][k] = 1)
          }
        }
        if (i == k + 1) {  // row k+1 is final: publish it and its pivot
          double* dst = M + static_cast<long long>(i) * ldm + rj[u];
#pragma unroll
          for (int e = 0; e < CH_SW; ++e) dst[e] = reg[u][e];
          if (rj[u] <= i && i < rj[u] + CH_SW) {
#pragma unroll
            for (int e = 0; e < CH_SW; ++e)
              if (rj[u] + e == i) pivot_inv(i, reg[u][e]);
          }
        }
      }
      __syncthreads();
    }
  } else {
    // large n: M lives in the L2-resident workspace, updated in place
    for (int id = tid; id < nstrips; id += CH_THREADS) {
      const int i = id / ns, j0 = (id % ns) * CH_SW;
      for (int e = 0; e < CH_SW; ++e) {
        const int j = j0 + e;
        M[static_cast<long long>(i) * ldm + j] = (j < n && j >= i) ? G[i + static_cast<long long>(j) * ldg] : 0.0;
      }
    }
    __syncthreads();
    if (tid == 0) pivot_inv(0, M[0]);
    __syncthreads();
    for (int k = 0; k < n - 1; ++k) {
      const double* Mk = M + static_cast<long long>(k) * ldm;
      const double inv = s_inv[k];
      for (int id = tid; id < nstrips; id += CH_THREADS) {
        const int i = id / ns, j0 = (id % ns) * CH_SW;
        if (i <= k) continue;
        const double l = Mk[i] * inv;
        double* row = M + static_cast<long long>(i) * ldm + j0;
        for (int e = 0; e < CH_SW; ++e) {
          const int j = j0 + e;
          if (j >= n) break;
          if (j >= i)
            row[e] = fma(-l, Mk[j], row[e]);
          else if (j <= k)
            row[e] = fma(-l, j == k ? 1.0 : Mk[j], row[e]);
        }
        if (i == k + 1 && j0 <= i && i < j0 + CH_SW) pivot_inv(i, row[i - j0]);
      }
      __syncthreads();
    }
  }
  // R (upper, zero below) and Linv = D^{-1/2} E (lower, unit diagonal scaled), zero-padded
  for (int idx = tid; idx < npad * npad; idx += CH_THREADS) {
    const int i = idx % npad, j = idx / npad;
    double rv = 0.0, lv = 0.0;
    if (i < n && j < n) {
      const double rs = sqrt(s_inv[i]);  // 1/sqrt(d_i)
      const double mij = M[static_cast<long long>(i) * ldm + j];
      if (i <= j) rv = mij * rs;
      if (j < i) lv = mij * rs;
      if (j == i) lv = rs;
    }
    R[i + static_cast<long long>(j) * ldr] = rv;
    Linv[i + static_cast<long long>(j) * ldl] = lv;
  }
}

cudaError_t chol_inv(cudaStream_t st, const double* G, int ldg, int n, int npad, double* R, int ldr, double* Linv,
                     int ldl, double* gwork, int* info, int info_code) {
  if (n <= 0) return cudaSuccess;
  if (n > 512) return cudaErrorInvalidValue;
  const int ldm = (n + CH_SW - 1) / CH_SW * CH_SW;
  const size_t work = static_cast<size_t>(n) * ldm * 8;
  if (n <= CH_SMEM_MAX_N) {
    static bool attr = false;
    if (!attr) {
      cudaError_t e = cudaFuncSetAttribute(chol_inv_kernel<true>, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                           CH_SMEM_MAX_N * CH_SMEM_MAX_N * 8);
      if (e != cudaSuccess) return e;
      attr = true;
    }
    chol_inv_kernel<true><<<1, CH_THREADS, work, st>>>(G, ldg, n, R, ldr, Linv, ldl, gwork, info, info_code, npad);
  } else {
    chol_inv_kernel<false><<<1, CH_THREADS, 0, st>>>(G, ldg, n, R, ldr, Linv, ldl, gwork, info, info_code, npad);
  }
  count_launch();
  return cudaGetLastError();
}

}  // namespace rs
