// Internal host-side interfaces between the C-ABI orchestration and the kernel launchers.
#pragma once
#include <cstdint>
#include <cuda.h>
#include <cuda_runtime.h>

namespace rs {

// A 2-D FP64 view: element (i, j) at base[i + j*ld]  (i runs along the contiguous dim0).
struct View2D {
  const double* base;
  long long dim0, dim1, ld;
};

// Operand descriptions for the two GEMM families (see gemm_f64.cuh).
struct GemmOutDesc {
  double* ptr;
  long long ld_m, ld_n, split_stride;
  int m_store, n_store;
  int mode = 0;  // 0: store, 1: subtract from the existing output
  // KC tail fold (kc_tail_applies): workspace for the per-CTA tail partials (nullptr: no fold)
  double* tail_ws = nullptr;
  long long tail_cap = 0;  // doubles
};

// KC tail fold: when N % 128 is in [1, 16] (n = 5 000: 8; n = 10 000: 16) and the product is
// DMMA-bound (M tile >= 64 rows), the last N % 128 columns get no 128-wide N tile of their own
// (which would cost a whole tile's DMMAs for <= 16 useful columns: 2.4 % of the work at
// n = 5 000); the full N tiles of each K split compute them on every (N / 128)-th K stage instead.
bool kc_tail_applies(int M, int N);
long long kc_tail_elems(int M, int N, int splits);  // tail partial doubles for `splits` K splits

struct PhiloxDesc {
  bool enabled;
  uint64_t seed;
  uint32_t tag;
  long long row_offset;
  int ell;                   // Omega rows generated
  long long omega_row0 = 0;  // first Omega row (global sample index)
};

// Out[M x N] (+split partials) = L[M x K] * R[K x N]
//   KC: R = Rv with dim0 = K (contiguous), dim1 = N;  L = Lv with dim0 = K, dim1 = M  (or Philox)
//   MC: L = Lv with dim0 = M (contiguous), dim1 = K;  R = Rv with dim0 = N, dim1 = K
// splits: number of K splits (>= 1); out.split_stride must be set when splits > 1.
// `ns_kernel` (optional) receives the kernel's device time when events != nullptr.
cudaError_t gemm_kc(cudaStream_t st, int M, int N, long long K, const View2D& Lv, const View2D& Rv,
                    const PhiloxDesc& phx, const GemmOutDesc& out, int splits);
// tri (MC only): 0 dense; 1 L lower triangular; 2 R upper triangular -- structurally zero K
// blocks are skipped (exact: they only add zeros).
cudaError_t gemm_mc(cudaStream_t st, int M, int N, long long K, const View2D& Lv, const View2D& Rv,
                    const GemmOutDesc& out, int splits, int tri = 0);
// G (+split partials) = X X^T for the rows <= 128 rows of a K-contiguous X (Xv: dim0 = K, dim1 =
// rows); lower-triangle blocks only, stored to both triangles (out.ld_m must be 1).
// Y = X U for a tall X (Xv: dim0 = m rows, contiguous; dim1 = k <= 128 columns) and an upper-
// triangular k x k U with U[t][j] = W[j + t * ldw] (the transposed storage of a lower-triangular
// L^{-1}, or the row-major R^{-1}); Y column-major (ldy), columns < n_store written (n_store <=
// 16 ceil(k / 16); columns >= k are zero).  Returns cudaErrorNotSupported when k > 128.
cudaError_t gemm_tsa(cudaStream_t st, long long m, int k, const View2D& Xv, const double* W, long long ldw, double* Y,
                     long long ldy, int n_store);
// Sample GEMM B = Omega A with Omega generated once per K split into an L2 ring of chunks shared by
// all N tiles (sample_ring.cuh): split partials into `out` (split_stride), *nsplit_out splits.
// Returns cudaErrorNotSupported when the shape or the ring workspace does not fit (use gemm_kc).
struct SampleRingPlan {
  int ntn, S, rounds, ngroups;
  long long kspl;
};
SampleRingPlan sample_ring_plan(int N, long long K, int max_splits, int G);
size_t sample_ring_bytes(int M, int N, long long K, int max_splits, int G);
cudaError_t gemm_sample_ring(cudaStream_t st, int M, int N, long long K, const View2D& Av, const PhiloxDesc& phx,
                             const GemmOutDesc& out, int max_splits, void* ring_ws, size_t ring_bytes,
                             int* nsplit_out);
int num_sms_cached();
cudaError_t gemm_syrk(cudaStream_t st, int rows, long long K, const View2D& Xv, const GemmOutDesc& out, int splits);
// tail: the KC tail fold will be used (N tiles = N / 128)
int gemm_choose_splits(int M, int N, long long K, int max_splits, int num_sms, bool tail = false);
int gemm_nsplit(long long K, int splits);   // splits actually launched for a requested count
int gemm_mtile(int M);   // rows per CTA tile used for M

// cudaFuncSetAttribute(fn, attr, value) once per (device, kernel, attribute, value).  Function
// attributes belong to the device context, so a per-process "done" flag would skip them when a
// process drives a second GPU; a value above the one already set is applied again.
cudaError_t ensure_func_attr(const void* fn, cudaFuncAttribute attr, int value);
template <typename F>
inline cudaError_t ensure_smem(F* fn, int bytes) {
  return ensure_func_attr(reinterpret_cast<const void*>(fn), cudaFuncAttributeMaxDynamicSharedMemorySize, bytes);
}

// Development A/B switches are COMPILE-TIME only (RS_EXTRA_NVCC_FLAGS="-DRS_DEV_..."): the shipped
// library reads no environment variable.

// kernel launch accounting (every launcher calls count_launch once per kernel launch)
void count_launch();
long long launch_count();

// small kernels (small.cu)
cudaError_t splitk_reduce(cudaStream_t st, double* out, const double* parts, int nsplit, long long count,
                          long long stride);
// n x n factor of G; R and Linv are written (zero-padded) as npad x npad.
cudaError_t chol_inv(cudaStream_t st, const double* G, int ldg, int n, int npad, double* R, int ldr, double* Linv,
                     int ldl, double* gwork, int* info, int info_code);
// C[M x N] = A[M x K] * B[K x N] (+ C if accumulate); element strides (row, col) for each.
cudaError_t small_gemm(cudaStream_t st, int M, int N, int K, const double* A, long long a_rs, long long a_cs,
                       const double* B, long long b_rs, long long b_cs, double* C, long long c_rs, long long c_cs,
                       bool accumulate, double alpha = 1.0);
// out[0] = max_i ||X[i, :]||_2 over rows i < rows (X column-major, ld)
cudaError_t rows_maxnorm(cudaStream_t st, const double* X, long long ld, int rows, long long ncols, double* out);
// G[i][i] += c * trace(G), i < n  (shifted CholeskyQR: c = 11 (N n + n(n+1)) u, ||X||_2^2 <= trace(G))
cudaError_t shift_diag(cudaStream_t st, double* G, int ldg, int n, double c);
cudaError_t gather_cols(cudaStream_t st, const double* A, long long lda, long long m, const int64_t* perm, int k,
                        double* Q, long long ldq);
cudaError_t permute_cols(cudaStream_t st, const double* Rorig, int ldro, int k, long long n, const int64_t* perm,
                         double* Rp, int ldrp);
cudaError_t trsm_upper_cols(cudaStream_t st, const double* U, int ldu, int k, const double* Y, long long ldy,
                            long long ncols, double* X, long long ldx);
cudaError_t copy_2d(cudaStream_t st, const double* src, long long lds, double* dst, long long ldd, long long rows,
                    long long cols);
cudaError_t omega_materialize(cudaStream_t st, uint64_t seed, uint32_t tag, int ell, long long j0, long long ncols,
                              double* out, long long ldo);

// truncated QRCP (qrcp.cu)
size_t qrcp_workspace_bytes(int ell, long long n);
cudaError_t qrcp_truncated(cudaStream_t st, const double* B, int ldb, int ell, long long n, int k, void* work,
                           int64_t* perm, double* Rhat_orig, int ldr, double* gaps, int* info, int num_sms);

// truncated QP3 of the full A (qp3.cu): the paper's deterministic baseline
size_t qp3_workspace_bytes(long long m, long long n);
cudaError_t qp3_truncated_large(cudaStream_t st, double* A, long long lda, long long m, long long n, int k,
                                void* work, int64_t* perm, double* tau, bool want_residual, double* residual);

}  // namespace rs
