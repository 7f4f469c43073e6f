/*
 * rs_lowrank.h -- C ABI of the B200 (sm_100a) random-sampling rank-k approximation
 *
 *     A P ~= Q R,   A: m x n,  Q: m x k (orthonormal columns),  R: k x n,  P: column permutation
 *
 * following Mary, Yamazaki, Kurzak, Luszczek, Tomov, Dongarra, "Performance of random sampling
 * for computing low-rank approximations of a dense matrix on GPUs", SC15 (PAPER.md, cited as
 * P:L<lines>).  Eq. (1); the algorithm is Fig. 2:
 *
 *   Step 1  sample        B := Omega A,  Omega l x m Gaussian, l = k + p
 *           power_iterate q x { B := QR(B); C := B A^T; C := QR(C); B := C A }  (Fig. 2(a))
 *   Step 2  pivot         [Q^, R^, P] := truncated QRCP(B), T := R^_{1:k}^{-1} R^_{k+1:n}
 *   Step 3  factor        [Q, Rbar] := QR(A P_{1:k}),  R := Rbar [I_k T]
 *
 * QR(.) of the short-wide B (l x n) and C (l x m) and of the tall A P_{1:k} is CholQR with one
 * full re-orthogonalisation ("CholQR2").  Omega is generated on the
 * device by Philox4x32-10 + the RS-BM32 Gaussian transform inside the GEMM tile
 * loader and is never stored.
 *
 * CONVENTIONS
 *  - All matrices are FP64, column-major (LAPACK/MAGMA convention), 0-based indices.
 *  - All matrix pointers passed to sample/power_iterate/pivot/factor are DEVICE pointers on the
 *    device that was current at rs_lowrank_create; they must be 16-byte aligned and every
 *    leading dimension must be even (TMA: 16-byte row pitch).
 *  - Multi-GPU (1-D block-row distribution): rank r passes its row block A(r)
 *    (m_local rows starting at global row row_offset).  Omega is keyed by GLOBAL row index, so
 *    the result does not depend on the partition (up to summation order).  B and R are
 *    replicated on every rank, Q is row-distributed like A.
 *  - Every call enqueues work on the handle's CUDA stream.  sample and power_iterate never
 *    synchronise the host (a CholQR breakdown inside the power iteration is flagged on the device
 *    and handled by pivot, see there); pivot and factor synchronise the stream before returning
 *    so that device-side failures (Cholesky breakdown, zero pivot norm) can be reported
 *    (cuSOLVER devInfo style).  rs_lowrank_run does the whole step as one CUDA-graph replay with
 *    a single synchronisation.
 *  - Ownership: the caller owns A, Q, R, perm and the workspace (allocate them with any device
 *    allocator); the library never frees them.  A must stay unmodified from sample through
 *    factor (it is re-read by power_iterate and factor).  The handle owns only host state.
 *  - Call order: create -> sample -> power_iterate? -> pivot -> factor -> destroy.  sample may
 *    be called again at any time (fresh pipeline).  Out-of-order calls return RS_ERR_BAD_STATE.
 *  - No exceptions cross the ABI; rs_lowrank_last_error returns a static per-handle message.
 */
#ifndef RS_LOWRANK_H_
#define RS_LOWRANK_H_

#include <stddef.h>
#include <stdint.h>

#if defined(__GNUC__)
#define RS_API __attribute__((visibility("default")))
#else
#define RS_API
#endif

#ifdef __cplusplus
extern "C" {
#endif

typedef struct rs_lowrank_s* rs_lowrank_t;

typedef enum {
  RS_OK = 0,
  RS_ERR_INVALID_ARG = 1,    /* bad size / pointer alignment / leading dimension */
  RS_ERR_BAD_STATE = 2,      /* call out of order */
  RS_ERR_CUDA = 3,           /* CUDA runtime error (message in last_error) */
  RS_ERR_NCCL = 4,           /* NCCL error */
  RS_ERR_NOT_SPD = 5,        /* CholQR breakdown: Gram matrix not numerically SPD (see get_info) */
  RS_ERR_RANK_DEFICIENT = 6, /* QRCP found a zero residual norm before k steps (see get_info) */
  RS_ERR_WORKSPACE = 7,      /* workspace too small */
  RS_ERR_UNSUPPORTED = 8,    /* device is not sm_100 / size outside the supported range */
  RS_ERR_NOT_CONVERGED = 9   /* adaptive sampling reached l_max before eps~ <= eps */
} rs_status_t;

/* In-place sum over the ranks of `count` doubles at device pointer `buf`, ordered on
 * `cuda_stream` (cudaStream_t); returns 0 on success.  See rs_lowrank_set_allreduce_hook. */
typedef int (*rs_allreduce_fn)(void* ctx, double* buf, int64_t count, void* cuda_stream);

/* Bytes of device workspace rs_lowrank_create needs for these sizes (no device access): the
 * sample B and its copies, C and C1 (l x m_local), split-K partials (<= 1 GiB), the small factors,
 * QRCP work, Q1 (m_local x k), -- for l <= 128 and m_local >= 2048 -- the ring of Omega chunks
 * of the sample GEMM (~43 MB at m = 1e6, n = 5 000, l = 110) and -- when n mod 128 is 1..16 --
 * the per-tile partials of the KC tail fold (~36 MB at cfg4).  cfg4: 2.99 GB.                  */
RS_API size_t rs_lowrank_workspace_bytes(int64_t m_local, int64_t n, int32_t k, int32_t p, int32_t nranks);

/* Create a handle.
 *  m_global, m_local, row_offset : global rows, this rank's rows, first global row of this rank
 *  n, k, p                       : columns, target rank, oversampling (l = k + p);
 *                                  require 1 <= k <= l <= min(m_global, n), l <= 512
 *  seed                          : Philox key (64 bit) of Omega
 *  workspace, workspace_bytes    : device buffer of at least rs_lowrank_workspace_bytes(...)
 *  cuda_stream                   : cudaStream_t (NULL = legacy default stream)
 *  nccl_comm                     : ncclComm_t spanning all ranks, or NULL for a single GPU     */
RS_API rs_status_t rs_lowrank_create(rs_lowrank_t* h, int64_t m_global, int64_t m_local, int64_t row_offset, int64_t n,
                              int32_t k, int32_t p, uint64_t seed, void* workspace, size_t workspace_bytes,
                              void* cuda_stream, void* nccl_comm);

/* Step 1: B := Omega A  (l x n, summed over ranks; Fig. 2(b) lines 2-3).  A: m_local x n, lda. */
RS_API rs_status_t rs_lowrank_sample(rs_lowrank_t h, const double* A, int64_t lda);

/* q passes of the power method with CholQR2 re-orthonormalisation of B and C (Fig. 2(a)).
 * q = 0 is a no-op.  No orthonormalisation after the last B := C A.  Enqueues only: the sample
 * B is kept, and if a CholQR of some pass breaks down (kappa^2 u > 1, "unstable for an
 * ill-conditioned matrix") pivot redoes the iteration from it -- re-reading A, which
 * must still be valid -- with the shifted-CholQR fallback of DESIGN.md R20.  At most once per
 * sample (RS_ERR_BAD_STATE otherwise).                                                        */
RS_API rs_status_t rs_lowrank_power_iterate(rs_lowrank_t h, const double* A, int64_t lda, int32_t q);

/* Step 2: truncated QRCP of B (k steps, largest residual column norm, ties -> lowest index)
 * and T := R^_{1:k}^{-1} R^_{k+1:n}.  perm (device int64[n], may be NULL) receives P:
 * perm[0..k) are the pivot columns, perm[k..n) the rest in LAPACK swap order.  Synchronises;
 * reports (and recovers from) a breakdown of the preceding power_iterate as described there. */
RS_API rs_status_t rs_lowrank_pivot(rs_lowrank_t h, int64_t* perm);

/* Step 3: Q := orth(A(:, P_{1:k})) by CholQR2 (Q: m_local x k, ldq >= m_local, even) and
 * R := Rbar [I_k T] (k x n, ldr >= k, even, columns in pivot order; replicated).  Synchronises. */
RS_API rs_status_t rs_lowrank_factor(rs_lowrank_t h, const double* A, int64_t lda, double* Q, int64_t ldq, double* R,
                              int64_t ldr);

/* The whole step sample -> power_iterate(q) -> pivot -> factor (CholQR2) with the arguments of
 * those calls (perm: device int64[n] or NULL).  The first call with a given set of pointers and q
 * captures the step as a CUDA graph on the handle's stream (kernels and NCCL collectives); later
 * calls replay it: one launch and one synchronisation per step.  If the step saw a CholQR
 * breakdown it is redone through the phase calls with their fallbacks.  Not captured when an
 * allreduce hook is installed (the hook runs host code).  Synchronises; state as after factor. */
RS_API rs_status_t rs_lowrank_run(rs_lowrank_t h, const double* A, int64_t lda, int32_t q, int64_t* perm, double* Q,
                                  int64_t ldq, double* R, int64_t ldr);

/* End-to-end call with HOST buffers: copies A (m_local x n, lda, host) to the device buffer
 * A_dev (ld_dev), runs rs_lowrank_run (sample -> power_iterate(q) -> pivot -> factor), and copies perm (int64[n]),
 * Q (m_local x k, ldq) and R (k x n, ldr) back to host memory.  Host buffers should be pinned
 * for full PCIe bandwidth.  Q_dev (m_local x k, even ld_qdev) and R_dev (k x n, even ld_rdev)
 * are device scratch for the outputs.  Synchronises.                                          */
RS_API rs_status_t rs_lowrank_run_host(rs_lowrank_t h, const double* A_host, int64_t lda, double* A_dev, int64_t ld_dev,
                                int32_t q, int64_t* perm_host, double* Q_host, int64_t ldq, double* R_host,
                                int64_t ldr, double* Q_dev, int64_t ld_qdev, double* R_dev, int64_t ld_rdev);

/* Adaptive sample size for the fixed-accuracy problem (Fig. 3; Sec. 10):
 * grows l block by block -- new rows of the same Omega (Philox rows [l, l + l_inc)), q power
 * iterations of the new block, each BOrth + QR being block classical Gram-Schmidt in its two-pass
 * form (project against the previous blocks, CholQR; project, CholQR again: DESIGN.md R17) --
 * until the estimate eps~ = max_i ||b_i - b_i B^T B|| of the next block's rows is <= eps (bound
 * (4)).  l_inc (a multiple of 8) is the first block size; inc_policy chooses
 * f(l, l_inc) of line 11: RS_INC_STATIC keeps it (Figs. 16-18), RS_INC_INTERP extrapolates
 * log10 eps~ linearly from the previous two estimates (Fig. 17 "adapt. linc"),
 * rounded up to a multiple of 8.  The handle must be created with k = l_max and p = 0.  On
 * return B holds l orthonormal rows and pivot/factor run with k = l.  history (host, may be NULL)
 * receives up to history_len pairs (l, eps~).  Returns RS_ERR_NOT_CONVERGED (B still valid,
 * *ell_out = l reached) when the next block would not fit in l_max.  Synchronises once per round
 * (eps~ and the next increment are decided on the host).                                      */
#define RS_INC_STATIC 0
#define RS_INC_INTERP 1
RS_API rs_status_t rs_lowrank_sample_adaptive(rs_lowrank_t h, const double* A, int64_t lda, double eps,
                                              int32_t ell_inc, int32_t q, int32_t inc_policy, int32_t* ell_out,
                                              double* est_out, double* history, int32_t history_len);

/* Column sampling (Fig. 8(b)): B_c := Omega_c A^T, l x m_local, where Omega_c is the
 * l x n Gaussian of DESIGN.md §3 keyed by the COLUMN index of A with Philox tag 1 (independent of
 * the row-sampling Omega).  B_c (device, column-major, ldb >= l even) receives the columns of B_c
 * that belong to this rank's rows of A -- no communication.  Enqueues only; independent of the
 * sample/pivot/factor state (uses handle scratch only).                                        */
RS_API rs_status_t rs_lowrank_sample_columns(rs_lowrank_t h, const double* A, int64_t lda, double* Bc, int64_t ldb);

RS_API rs_status_t rs_lowrank_destroy(rs_lowrank_t h);

/* ---- accessors (tests / bench) ---- */
/* B (l x n, device, column-major, ldb >= l) after sample / power_iterate.                   */
RS_API rs_status_t rs_lowrank_get_sample(rs_lowrank_t h, double* B, int64_t ldb);
/* Replace B (l x n, device) -- e.g. the Omega = I special case (B := A, l = m).             */
RS_API rs_status_t rs_lowrank_set_sample(rs_lowrank_t h, const double* B, int64_t ldb);
/* After pivot: T (k x (n-k), ldt >= k) and R^ (k x n in pivot order, ldrh >= k), device;
 * gaps (host double[k], may be NULL): per-step relative gap (best - second)/best of norms.    */
RS_API rs_status_t rs_lowrank_get_pivot_data(rs_lowrank_t h, double* T, int64_t ldt, double* Rhat, int64_t ldrh,
                                      double* gaps_host);
/* Materialise Omega[0:l, j0:j0+ncols) (global columns) into out (device, l x ncols, ldo >= l):
 * the exact values the fused sampling GEMM generates.                                        */
RS_API rs_status_t rs_lowrank_omega(rs_lowrank_t h, int64_t j0, int64_t ncols, double* out, int64_t ldo);
/* info[0] = status code of the first device-detected failure (0 if none), info[1] = 1-based
 * failing Cholesky column / QRCP step.  Synchronises.                                        */
RS_API rs_status_t rs_lowrank_get_info(rs_lowrank_t h, int64_t* info);
/* CholQR breakdown fallbacks taken (R20), host-side, no sync:
 *  counts[0] = power iterations since the last sample redone with shifted CholQR on B and C
 *              (2 shifted + 2 plain passes each) after the plain CholQR2 broke down;
 *  counts[1] = shifted passes the last factor call put ahead of its two plain CholQR passes
 *              (0 = plain CholQR2 succeeded, 2 or 4 = shifted CholQR4 / CholQR6).            */
RS_API rs_status_t rs_lowrank_get_fallbacks(rs_lowrank_t h, int32_t* counts);
/* Per-kernel-class device time (ms, CUDA events on the handle's stream) accumulated while
 * profiling is enabled.  names: "gemm_sample", "gemm_power_c", "gemm_power_b", "gram",
 * "apply", "chol", "qrcp", "factor", "reduce", "comm", "other".                              */
RS_API rs_status_t rs_lowrank_set_profiling(rs_lowrank_t h, int32_t enable);
RS_API rs_status_t rs_lowrank_get_profile(rs_lowrank_t h, const char* name, double* ms, int64_t* launches,
                                   double* flops);
RS_API rs_status_t rs_lowrank_reset_profile(rs_lowrank_t h);
/* Number of CUDA kernels this library has launched in the process (all handles). */
RS_API int64_t rs_lowrank_kernel_launches(void);
RS_API const char* rs_lowrank_last_error(rs_lowrank_t h);
/* Replace NCCL by a caller-supplied allreduce for this handle (the reductions of the
 * 1-D row distribution are sums of B (l x n) and of the l x l / k x k Gram matrices).  Used to run
 * several ranks' handles in ONE process on ONE GPU (the multi-rank parity tests), or to plug in
 * another transport.  nranks / rank: this handle's place in the row partition (create's
 * m_local / row_offset must match it); fn is called from the pipeline calls, on the calling host
 * thread, every time the multi-GPU path reduces (same order on every rank); it must return after
 * the sum is enqueued on (or completed before) cuda_stream.  Only directly after create and only
 * on a handle created without an NCCL communicator; RS_ERR_BAD_STATE otherwise.  A nonzero
 * return from fn fails the pipeline call with RS_ERR_NCCL.                                    */
RS_API rs_status_t rs_lowrank_set_allreduce_hook(rs_lowrank_t h, int32_t nranks, int32_t rank, rs_allreduce_fn fn,
                                                 void* ctx);

/* ---- the paper's deterministic baseline: truncated QP3 of A itself (one GPU) ----
 * Householder QR with column pivoting stopped after k columns (Sec. 2; "QP3" of
 * Figs. 7, 10-14), blocked like LAPACK dgeqp3/dlaqps: panels of 32 columns, delayed trailing
 * updates, downdated column norms with LAPACK's cancellation test (a failing column's norm is
 * recomputed exactly on the device).  Pivot rule: largest residual column norm, ties -> lowest
 * original index; perm in LAPACK swap order.
 *  A (device, m x n, lda >= m even, 16-byte aligned) is overwritten LAPACK-style: rows 0..k-1
 *    hold R (upper trapezoidal, k x n, columns in perm order), the columns 0..k-1 below the
 *    diagonal hold the Householder vectors (unit leading entry implicit); the trailing block
 *    A(k:m, k:n) holds R22 if residual_host != NULL, else it is only partly updated.
 *  perm (device int64[n]), tau (device double[k]): outputs; caller-owned.
 *  residual_host (may be NULL): receives ||R22||_F (the error of Fig. 6's "QP3" column is
 *    ||R22||_F / ||A||_F); requesting it adds the last panel's trailing update and synchronises.
 *  workspace: device, 256-byte aligned, >= rs_qp3_workspace_bytes(m, n, k).
 *  cuda_stream: cudaStream_t (NULL = legacy default stream).  Enqueues only (no synchronisation)
 *    unless residual_host != NULL.  Errors: RS_ERR_INVALID_ARG, RS_ERR_WORKSPACE, RS_ERR_CUDA. */
RS_API size_t rs_qp3_workspace_bytes(int64_t m, int64_t n, int32_t k);
RS_API rs_status_t rs_qp3_truncated(int64_t m, int64_t n, int32_t k, double* A, int64_t lda, int64_t* perm,
                                    double* tau, double* residual_host, void* workspace, size_t workspace_bytes,
                                    void* cuda_stream);

/* ---- NCCL plumbing (the harness exchanges the id with torch.distributed) ---- */
RS_API rs_status_t rs_comm_get_unique_id(char id_out[128]);
RS_API rs_status_t rs_comm_init(void** comm, int32_t nranks, const char id[128], int32_t rank);
RS_API rs_status_t rs_comm_destroy(void* comm);
/* Number of ranks of a communicator (ncclCommCount) and this process's rank in it. */
RS_API rs_status_t rs_comm_info(void* comm, int32_t* nranks, int32_t* rank);

#ifdef __cplusplus
}
#endif
#endif /* RS_LOWRANK_H_ */
