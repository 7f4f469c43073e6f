// Cholesky factor of a Gram matrix and its inverse in one pass: CholQR steps (ii)-(iii)
// ("R^T R := G, R upper-triangular with non-negative diagonal; Q = R^{-T} B").
//
// Right-looking elimination on the packed upper triangle S of G with the same row operations
// applied to an identity E (E becomes the unit-lower L^{-1} up to row scaling), one
// __syncthreads per pivot: at step k every thread updates the elements it owns,
//     S[i][j] -= S[k][i] S[k][j] / d_k          (k < i <= j)
//     E[i][c] -= S[k][i] / d_k * E[k][c]         (c <= k < i)
// then R[k][j] = S[k][j] / sqrt(d_k) and Linv = R^{-T} has rows E[i][:] / sqrt(d_i).
// Both triangles are stored ROW-packed so that row k (read by every thread at step k) is
// contiguous: consecutive lanes own consecutive elements of one row -> conflict-free LDS and
// broadcasts.  One CTA of 1024 threads; packed triangles in shared memory for n <= 128 (element
// coordinates kept in registers), in the L2-resident workspace otherwise.  A pivot d_k <= 0 or
// NaN is a CholQR breakdown: it is reported through *info (LAPACK potrf-style 1-based column) and
// replaced by 1 so no NaN propagates.
#include <cstdio>

#include "common.cuh"
#include "internal.h"

namespace rs {

constexpr int CH_THREADS = 1024;
constexpr int CH_SMEM_MAX_N = 128;
constexpr int CH_MAXE = (CH_SMEM_MAX_N * (CH_SMEM_MAX_N + 1) / 2 + CH_THREADS - 1) / CH_THREADS;  // 9

// upper triangle, row-packed: (i, j), i <= j < n, at up(i) + j - i,  up(i) = i*n - i*(i-1)/2
RS_DEVINL int up_off(int i, int n) { return i * n - i * (i - 1) / 2; }
RS_DEVINL void up_decode(int e, int n, int& i, int& j) {
  const double b = 2.0 * n + 1.0;
  int ii = static_cast<int>((b - sqrt(b * b - 8.0 * e)) * 0.5);
  if (ii < 0) ii = 0;
  while (ii > 0 && up_off(ii, n) > e) --ii;
  while (ii + 1 < n && up_off(ii + 1, n) <= e) ++ii;
  i = ii;
  j = ii + (e - up_off(ii, n));
}
// lower triangle, row-packed: (r, c), c <= r, at r(r+1)/2 + c
RS_DEVINL int lo_off(int r) { return r * (r + 1) / 2; }
RS_DEVINL void lo_decode(int e, int& r, int& c) {
  int rr = static_cast<int>((sqrt(8.0 * e + 1.0) - 1.0) * 0.5);
  while (lo_off(rr + 1) <= e) ++rr;
  while (lo_off(rr) > e) --rr;
  r = rr;
  c = e - lo_off(rr);
}

template <bool SMEM>
__global__ void __launch_bounds__(CH_THREADS) chol_inv_kernel(const double* __restrict__ G, int ldg, int n,
                                                               double* __restrict__ R, int ldr,
                                                               double* __restrict__ Linv, int ldl,
                                                               double* __restrict__ gwork, int* info, int code,
                                                               int npad) {
  extern __shared__ double sm[];
  const int T = n * (n + 1) / 2;
  double* S = SMEM ? sm : gwork;
  double* E = S + T;
  const int tid = threadIdx.x;

  constexpr int NE = SMEM ? CH_MAXE : 1;
  int si[NE], sj[NE], er[NE], ec[NE];
  if (SMEM) {
#pragma unroll
    for (int s = 0; s < NE; ++s) {
      const int e = tid + s * CH_THREADS;
      si[s] = sj[s] = er[s] = ec[s] = -1;
      if (e < T) {
        up_decode(e, n, si[s], sj[s]);
        lo_decode(e, er[s], ec[s]);
      }
    }
  }
  for (int e = tid; e < T; e += CH_THREADS) {
    int i, j, r, c;
    up_decode(e, n, i, j);
    lo_decode(e, r, c);
    S[e] = G[i + static_cast<long long>(j) * ldg];
    E[e] = (r == c) ? 1.0 : 0.0;
  }
  __syncthreads();

  for (int k = 0; k < n; ++k) {
    const double* Sk = S + up_off(k, n) - k;  // Sk[j] = S[k][j], j >= k
    const double* Ek = E + lo_off(k);         // Ek[c] = E[k][c], c <= k
    const double dk = Sk[k];
    const double inv = 1.0 / (dk > 0.0 ? dk : 1.0);
    if (tid == 0 && !(dk > 0.0) && info) atomicCAS(info, 0, code), atomicCAS(info + 1, 0, k + 1);
    if (SMEM) {
#pragma unroll
      for (int s = 0; s < NE; ++s) {
        const int e = tid + s * CH_THREADS;
        if (si[s] > k) S[e] -= Sk[si[s]] * Sk[sj[s]] * inv;
        if (er[s] > k && ec[s] <= k) E[e] -= Sk[er[s]] * inv * Ek[ec[s]];
      }
    } else {
      for (int e = tid; e < T; e += CH_THREADS) {
        int i, j, r, c;
        up_decode(e, n, i, j);
        lo_decode(e, r, c);
        if (i > k) S[e] -= Sk[i] * Sk[j] * inv;
        if (r > k && c <= k) E[e] -= Sk[r] * inv * Ek[c];
      }
    }
    __syncthreads();
  }
  // R (upper, zero below) and Linv = R^{-T} (lower, zero above), zero-padded to npad x npad
  for (int idx = tid; idx < npad * npad; idx += CH_THREADS) {
    const int i = idx % npad, j = idx / npad;
    double rv = 0.0, lv = 0.0;
    if (i < n && j < n) {
      const double di = S[up_off(i, n)];
      const double ri = sqrt(di > 0.0 ? di : 1.0);
      if (i <= j) rv = S[up_off(i, n) + j - i] / ri;
      if (j <= i) lv = E[lo_off(i) + j] / ri;
    }
    R[i + static_cast<long long>(j) * ldr] = rv;
    Linv[i + static_cast<long long>(j) * ldl] = lv;
  }
}

cudaError_t chol_inv(cudaStream_t st, const double* G, int ldg, int n, int npad, double* R, int ldr, double* Linv,
                     int ldl, double* gwork, int* info, int info_code) {
  if (n <= 0) return cudaSuccess;
  const size_t work = static_cast<size_t>(n) * (n + 1) * 8;  // both packed triangles
  if (n <= CH_SMEM_MAX_N) {
    static bool attr = false;
    if (!attr) {
      cudaError_t e = cudaFuncSetAttribute(chol_inv_kernel<true>, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                           CH_SMEM_MAX_N * (CH_SMEM_MAX_N + 1) * 8);
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
