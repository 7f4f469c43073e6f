// Small / memory-bound kernels of the pipeline: deterministic split-K reduction, Cholesky of a
// Gram matrix with the triangular inverse (CholQR steps (ii)-(iii)), small dense
// products (T, R = Rbar [I T], Linv * B), column gather A(:, P_{1:k}) and the back substitution
// T := R̂_{1:k}^{-1} R̂_{k+1:n} (Fig. 2(b) lines 8-10).
#include <algorithm>
#include <atomic>
#include <cstdio>

#include "common.cuh"
#include "internal.h"
#include "philox.cuh"

namespace rs {

namespace {
std::atomic<long long> g_launches{0};
}
void count_launch() { g_launches.fetch_add(1, std::memory_order_relaxed); }
long long launch_count() { return g_launches.load(); }

// ---------------------------------------------------------------------------------------------
// out[i] = sum_{s=0}^{nsplit-1} parts[s*stride + i], summed in increasing s (deterministic).
// ---------------------------------------------------------------------------------------------
__global__ void splitk_reduce_kernel(double* __restrict__ out, const double* __restrict__ parts, int nsplit,
                                     long long count, long long stride) {
  const long long n2 = count / 2;
  for (long long i = blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x; i < n2;
       i += static_cast<long long>(gridDim.x) * blockDim.x) {
    double2 acc = make_double2(0.0, 0.0);
    for (int s = 0; s < nsplit; ++s) {
      const double2 v = __ldcs(reinterpret_cast<const double2*>(parts + s * stride) + i);
      acc.x += v.x;
      acc.y += v.y;
    }
    reinterpret_cast<double2*>(out)[i] = acc;
  }
  if ((count & 1) && blockIdx.x == 0 && threadIdx.x == 0) {
    double acc = 0.0;
    for (int s = 0; s < nsplit; ++s) acc += parts[s * stride + count - 1];
    out[count - 1] = acc;
  }
}

cudaError_t splitk_reduce(cudaStream_t st, double* out, const double* parts, int nsplit, long long count,
                          long long stride) {
  if (count <= 0) return cudaSuccess;
  // stride and pointers are multiples of 2 doubles (planner guarantees 16-byte alignment)
  const long long n2 = count / 2 + 1;
  int blocks = static_cast<int>(std::min<long long>((n2 + 255) / 256, 148LL * 8));
  splitk_reduce_kernel<<<blocks, 256, 0, st>>>(out, parts, nsplit, count, stride);
  count_launch();
  return cudaGetLastError();
}

// ---------------------------------------------------------------------------------------------
// Small dense product C = A*B (+C), general element strides, 64x64 tiles, FP64 FMA.
// ---------------------------------------------------------------------------------------------
__global__ void __launch_bounds__(256) small_gemm_kernel(int M, int N, int K, const double* __restrict__ A,
                                                         long long a_rs, long long a_cs, const double* __restrict__ B,
                                                         long long b_rs, long long b_cs, double* __restrict__ C,
                                                         long long c_rs, long long c_cs, bool accumulate,
                                                         double alpha) {
  __shared__ double As[16][64 + 1];
  __shared__ double Bs[16][64 + 1];
  const int tx = threadIdx.x & 15, ty = threadIdx.x >> 4;
  const int m0 = blockIdx.y * 64, n0 = blockIdx.x * 64;
  double acc[4][4] = {};
  for (int k0 = 0; k0 < K; k0 += 16) {
    for (int idx = threadIdx.x; idx < 16 * 64; idx += 256) {
      const int kk = idx / 64, mm = idx % 64;
      const int gm = m0 + mm, gk = k0 + kk;
      As[kk][mm] = (gm < M && gk < K) ? A[gm * a_rs + gk * a_cs] : 0.0;
      const int gn = n0 + mm;
      Bs[kk][mm] = (gn < N && gk < K) ? B[gk * b_rs + gn * b_cs] : 0.0;
    }
    __syncthreads();
#pragma unroll
    for (int kk = 0; kk < 16; ++kk) {
      double av[4], bv[4];
#pragma unroll
      for (int i = 0; i < 4; ++i) av[i] = As[kk][ty + 16 * i];
#pragma unroll
      for (int j = 0; j < 4; ++j) bv[j] = Bs[kk][tx + 16 * j];
#pragma unroll
      for (int i = 0; i < 4; ++i)
#pragma unroll
        for (int j = 0; j < 4; ++j) acc[i][j] = fma(av[i], bv[j], acc[i][j]);
    }
    __syncthreads();
  }
#pragma unroll
  for (int i = 0; i < 4; ++i)
#pragma unroll
    for (int j = 0; j < 4; ++j) {
      const int gm = m0 + ty + 16 * i, gn = n0 + tx + 16 * j;
      if (gm < M && gn < N) {
        double* p = C + gm * c_rs + gn * c_cs;
        *p = accumulate ? fma(alpha, acc[i][j], *p) : alpha * acc[i][j];
      }
    }
}

cudaError_t small_gemm(cudaStream_t st, int M, int N, int K, const double* A, long long a_rs, long long a_cs,
                       const double* B, long long b_rs, long long b_cs, double* C, long long c_rs, long long c_cs,
                       bool accumulate, double alpha) {
  if (M <= 0 || N <= 0) return cudaSuccess;
  dim3 grid((N + 63) / 64, (M + 63) / 64);
  small_gemm_kernel<<<grid, 256, 0, st>>>(M, N, K, A, a_rs, a_cs, B, b_rs, b_cs, C, c_rs, c_cs, accumulate, alpha);
  count_launch();
  return cudaGetLastError();
}

// ---------------------------------------------------------------------------------------------
// Q(:, c) = A(:, perm[c]), c < k  (A P_{1:k}, Fig. 2(b) line 8)
// ---------------------------------------------------------------------------------------------
__global__ void gather_cols_kernel(const double* __restrict__ A, long long lda, long long m,
                                   const int64_t* __restrict__ perm, double* __restrict__ Q, long long ldq) {
  const int c = blockIdx.y;
  const double* src = A + perm[c] * lda;
  double* dst = Q + c * ldq;
  for (long long i = blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x; i < m;
       i += static_cast<long long>(gridDim.x) * blockDim.x)
    dst[i] = __ldcs(src + i);
}

cudaError_t gather_cols(cudaStream_t st, const double* A, long long lda, long long m, const int64_t* perm, int k,
                        double* Q, long long ldq) {
  if (m <= 0 || k <= 0) return cudaSuccess;
  const int bx = static_cast<int>(std::min<long long>((m + 255) / 256, 64));
  gather_cols_kernel<<<dim3(bx, k), 256, 0, st>>>(A, lda, m, perm, Q, ldq);
  count_launch();
  return cudaGetLastError();
}

// Rp(:, p) = Rorig(:, perm[p])  (R̂ in pivot order)
__global__ void permute_cols_kernel(const double* __restrict__ Ro, int ldro, int k, long long n,
                                    const int64_t* __restrict__ perm, double* __restrict__ Rp, int ldrp) {
  for (long long idx = blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x; idx < n * k;
       idx += static_cast<long long>(gridDim.x) * blockDim.x) {
    const long long p = idx / k;
    const int i = static_cast<int>(idx % k);
    Rp[i + p * ldrp] = Ro[i + perm[p] * ldro];
  }
}

cudaError_t permute_cols(cudaStream_t st, const double* Rorig, int ldro, int k, long long n, const int64_t* perm,
                         double* Rp, int ldrp) {
  const long long tot = n * k;
  const int blocks = static_cast<int>(std::min<long long>((tot + 255) / 256, 148LL * 8));
  permute_cols_kernel<<<blocks, 256, 0, st>>>(Rorig, ldro, k, n, perm, Rp, ldrp);
  count_launch();
  return cudaGetLastError();
}

// ---------------------------------------------------------------------------------------------
// X(:, c) = U^{-1} Y(:, c) for upper-triangular U (k x k): column-oriented back substitution,
// one warp per right-hand side (T := R̂_{1:k}^{-1} R̂_{k+1:n}, Fig. 2(b) line 9).
// ---------------------------------------------------------------------------------------------
constexpr int TRSM_WARPS = 8;
__global__ void __launch_bounds__(TRSM_WARPS * 32)
    trsm_upper_cols_kernel(const double* __restrict__ U, int ldu, int k, const double* __restrict__ Y, long long ldy,
                           long long ncols, double* __restrict__ X, long long ldx) {
  extern __shared__ double sb[];
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  double* b = sb + warp * k;
  for (long long c = blockIdx.x * static_cast<long long>(TRSM_WARPS) + warp; c < ncols;
       c += static_cast<long long>(gridDim.x) * TRSM_WARPS) {
    for (int i = lane; i < k; i += 32) b[i] = Y[i + c * ldy];
    __syncwarp();
    for (int i = k - 1; i >= 0; --i) {
      const double xi = b[i] / U[i + static_cast<long long>(i) * ldu];
      __syncwarp();
      if (lane == 0) b[i] = xi;
      const double* ucol = U + static_cast<long long>(i) * ldu;
      for (int i2 = lane; i2 < i; i2 += 32) b[i2] -= xi * ucol[i2];
      __syncwarp();
    }
    for (int i = lane; i < k; i += 32) X[i + c * ldx] = b[i];
    __syncwarp();
  }
}

// k <= 128: U and 1/U_ii staged once per CTA in shared memory (no division, no global reads in
// the dependent chain); one warp per right-hand side, every lane forms x_i itself from the
// broadcast b_i, then the lanes update b_0..b_{i-1}.
constexpr int TRSM2_WARPS = 32;
__global__ void __launch_bounds__(TRSM2_WARPS * 32, 1)
    trsm_upper_cols_smem_kernel(const double* __restrict__ U, int ldu, int k, const double* __restrict__ Y,
                                long long ldy, long long ncols, double* __restrict__ X, long long ldx) {
  extern __shared__ double sb[];
  double* Us = sb;               // k x k, column-major, ld k
  double* rd = Us + k * k;       // 1 / U_ii
  double* bw = rd + k;           // per-warp right-hand side
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  for (int idx = threadIdx.x; idx < k * k; idx += blockDim.x) {
    const int i = idx % k, j = idx / k;
    Us[idx] = i <= j ? U[i + static_cast<long long>(j) * ldu] : 0.0;
  }
  for (int i = threadIdx.x; i < k; i += blockDim.x) rd[i] = 1.0 / U[i + static_cast<long long>(i) * ldu];
  __syncthreads();
  double* b = bw + warp * k;
  for (long long c = blockIdx.x * static_cast<long long>(TRSM2_WARPS) + warp; c < ncols;
       c += static_cast<long long>(gridDim.x) * TRSM2_WARPS) {
    for (int i = lane; i < k; i += 32) b[i] = Y[i + c * ldy];
    __syncwarp();
    for (int i = k - 1; i >= 0; --i) {
      const double xi = b[i] * rd[i];
      const double* ucol = Us + i * k;
      for (int i2 = lane; i2 < i; i2 += 32) b[i2] = fma(-xi, ucol[i2], b[i2]);
      __syncwarp();                        // every lane has read b_i
      if (lane == (i & 31)) b[i] = xi;     // b_i is not read again before the final store
    }
    __syncwarp();
    for (int i = lane; i < k; i += 32) X[i + c * ldx] = b[i];
    __syncwarp();
  }
}

cudaError_t trsm_upper_cols(cudaStream_t st, const double* U, int ldu, int k, const double* Y, long long ldy,
                            long long ncols, double* X, long long ldx) {
  if (ncols <= 0) return cudaSuccess;
  if (k <= 128) {
    const size_t smem2 = (static_cast<size_t>(k) * k + k + static_cast<size_t>(TRSM2_WARPS) * k) * 8;
    {
      cudaError_t e = ensure_smem(trsm_upper_cols_smem_kernel, static_cast<int>((128 * 128 + 128 + TRSM2_WARPS * 128) * 8));
      if (e != cudaSuccess) return e;
    }
    const int blocks = static_cast<int>(std::min<long long>((ncols + TRSM2_WARPS - 1) / TRSM2_WARPS, 148LL));
    trsm_upper_cols_smem_kernel<<<blocks, TRSM2_WARPS * 32, smem2, st>>>(U, ldu, k, Y, ldy, ncols, X, ldx);
    count_launch();
    return cudaGetLastError();
  }
  const size_t smem = static_cast<size_t>(TRSM_WARPS) * k * 8;
  if (smem > 220 * 1024) return cudaErrorInvalidValue;
  {
    cudaError_t e = ensure_smem(trsm_upper_cols_kernel, 220 * 1024);
    if (e != cudaSuccess) return e;
  }
  const int blocks = static_cast<int>(std::min<long long>((ncols + TRSM_WARPS - 1) / TRSM_WARPS, 148LL * 16));
  trsm_upper_cols_kernel<<<blocks, TRSM_WARPS * 32, smem, st>>>(U, ldu, k, Y, ldy, ncols, X, ldx);
  count_launch();
  return cudaGetLastError();
}

__global__ void copy_2d_kernel(const double* __restrict__ src, long long lds, double* __restrict__ dst, long long ldd,
                               long long rows, long long cols) {
  for (long long idx = blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x; idx < rows * cols;
       idx += static_cast<long long>(gridDim.x) * blockDim.x) {
    const long long i = idx % rows, j = idx / rows;
    dst[i + j * ldd] = src[i + j * lds];
  }
}

cudaError_t copy_2d(cudaStream_t st, const double* src, long long lds, double* dst, long long ldd, long long rows,
                    long long cols) {
  const long long tot = rows * cols;
  if (tot <= 0) return cudaSuccess;
  const int blocks = static_cast<int>(std::min<long long>((tot + 255) / 256, 148LL * 8));
  copy_2d_kernel<<<blocks, 256, 0, st>>>(src, lds, dst, ldd, rows, cols);
  count_launch();
  return cudaGetLastError();
}

// Omega[i, j0 + jj] for i < ell, jj < ncols (test accessor: the same generator the GEMM fuses)
__global__ void omega_kernel(PhiloxKey key, uint32_t tag, int ell, long long j0, long long ncols, double* out,
                             long long ldo) {
  for (long long idx = blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x; idx < ncols * ell;
       idx += static_cast<long long>(gridDim.x) * blockDim.x) {
    const int i = static_cast<int>(idx % ell);
    const long long jj = idx / ell;
    const long long j = j0 + jj;
    double v[4];
    omega_block4(static_cast<uint32_t>(i), static_cast<uint64_t>(j >> 2), tag, key, v);
    out[i + jj * ldo] = v[j & 3];
  }
}

cudaError_t omega_materialize(cudaStream_t st, uint64_t seed, uint32_t tag, int ell, long long j0, long long ncols,
                              double* out, long long ldo) {
  const long long tot = ncols * ell;
  if (tot <= 0) return cudaSuccess;
  PhiloxKey key{static_cast<uint32_t>(seed), static_cast<uint32_t>(seed >> 32)};
  const int blocks = static_cast<int>(std::min<long long>((tot + 255) / 256, 148LL * 8));
  omega_kernel<<<blocks, 256, 0, st>>>(key, tag, ell, j0, ncols, out, ldo);
  count_launch();
  return cudaGetLastError();
}

// out[0] = max over rows of the row 2-norms of X (rows x ncols, column-major): the adaptive
// scheme's error estimate eps~ (Fig. 3 line 15, reading R18).  One CTA.
__global__ void rows_maxnorm_kernel(const double* __restrict__ X, long long ld, int rows, long long ncols,
                                    double* out) {
  __shared__ double red[1024 / 32];
  double best = 0.0;
  for (int i = 0; i < rows; ++i) {
    double s = 0.0;
    for (long long c = threadIdx.x; c < ncols; c += blockDim.x) {
      const double x = X[i + c * ld];
      s = fma(x, x, s);
    }
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) s += __shfl_xor_sync(0xffffffffu, s, o);
    if ((threadIdx.x & 31) == 0) red[threadIdx.x >> 5] = s;
    __syncthreads();
    if (threadIdx.x == 0) {
      double t = 0.0;
      for (int w = 0; w < static_cast<int>(blockDim.x >> 5); ++w) t += red[w];
      best = fmax(best, sqrt(t));
    }
    __syncthreads();
  }
  if (threadIdx.x == 0) out[0] = best;
}

cudaError_t rows_maxnorm(cudaStream_t st, const double* X, long long ld, int rows, long long ncols, double* out) {
  rows_maxnorm_kernel<<<1, 1024, 0, st>>>(X, ld, rows, ncols, out);
  count_launch();
  return cudaGetLastError();
}

}  // namespace rs

namespace rs {

// Shift for shifted CholeskyQR (breakdown-free first pass for ill-conditioned blocks):
// G[i][i] += c * trace(G).  One CTA.
__global__ void shift_diag_kernel(double* G, int ldg, int n, double c) {
  __shared__ double red[32];
  double s = 0.0;
  for (int i = threadIdx.x; i < n; i += blockDim.x) s += G[i + static_cast<long long>(i) * ldg];
#pragma unroll
  for (int o = 16; o > 0; o >>= 1) s += __shfl_xor_sync(0xffffffffu, s, o);
  if ((threadIdx.x & 31) == 0) red[threadIdx.x >> 5] = s;
  __syncthreads();
  __shared__ double tr;
  if (threadIdx.x == 0) {
    double t = 0.0;
    for (int w = 0; w < static_cast<int>(blockDim.x >> 5); ++w) t += red[w];
    tr = t;
  }
  __syncthreads();
  for (int i = threadIdx.x; i < n; i += blockDim.x) G[i + static_cast<long long>(i) * ldg] += c * tr;
}

cudaError_t shift_diag(cudaStream_t st, double* G, int ldg, int n, double c) {
  shift_diag_kernel<<<1, 256, 0, st>>>(G, ldg, n, c);
  count_launch();
  return cudaGetLastError();
}

}  // namespace rs
