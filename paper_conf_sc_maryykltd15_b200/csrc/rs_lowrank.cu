// C-ABI and host orchestration of the random-sampling pipeline (Fig. 2) on one
// B200 per process, with NCCL over NVLink for the reductions of the 1-D block-row distribution
// (P:L535-575).  See include/rs_lowrank.h for the contract and DESIGN.md for the design.
#include <nccl.h>

#include <algorithm>
#include <cstdarg>
#include <cmath>
#include <cstdio>
#include <cstring>
#include <map>
#include <string>
#include <vector>

#include "internal.h"
#include "rs_lowrank.h"

using namespace rs;

namespace {

enum State { ST_CREATED = 0, ST_SAMPLED = 1, ST_PIVOTED = 2, ST_FACTORED = 3 };

// internal device info code: CholQR breakdown in power-iteration pass (code - RS_INFO_POWER),
// never returned to the caller (pivot replays the iteration with the R20 fallback)
constexpr int RS_INFO_POWER = 100;

inline long long round_up(long long x, long long a) { return (x + a - 1) / a * a; }

struct ProfEntry {
  double ms = 0.0;
  long long launches = 0;
  double flops = 0.0;
};

struct Pending {
  std::string name;
  cudaEvent_t e0, e1;
  double flops;
};

// Workspace layout (byte offsets), shared by rs_lowrank_workspace_bytes and create.
struct Layout {
  int ell, lp, kp, lmax;
  long long ldc, ldq1;
  int smax;          // max split-K partial tiles of an l x n product
  long long part_elems;
  size_t off_B, off_B0, off_Bt, off_B1, off_C, off_C1, off_part, off_G, off_Rf, off_Linv, off_cholw, off_Rho, off_Rhat,
      off_T, off_Q1, off_R1, off_R2, off_Rbar, off_perm, off_info, off_qr, off_gaps, off_ring, off_tail;
  size_t ring_bytes;
  long long tail_elems;  // KC tail-fold partials of the l x n products (kc_tail_applies), smax splits  // Omega chunk ring of the sample GEMM (0: the cluster kernel generates in smem)
  size_t total;
};

Layout plan(long long m_local, long long n, int k, int p) {
  Layout L{};
  L.ell = k + p;
  L.lp = static_cast<int>(round_up(L.ell, 8));
  L.kp = static_cast<int>(round_up(k, 8));
  L.lmax = std::max(L.lp, L.kp);
  L.ldc = round_up(std::max<long long>(m_local, 1), 16);
  L.ldq1 = L.ldc;
  const long long lxn = static_cast<long long>(L.lp) * n;
  const long long cap = (1LL << 30) / 8;  // <= 1 GiB of partial tiles
  L.smax = static_cast<int>(std::max<long long>(8, std::min<long long>(64, cap / std::max<long long>(lxn, 1))));
  L.part_elems = std::max<long long>(static_cast<long long>(L.smax) * lxn,
                                     1024LL * L.lmax * L.lmax);  // Gram partials: up to 1024 splits
  size_t off = 0;
  auto take = [&](size_t bytes) {
    const size_t o = off;
    off = (off + bytes + 255) / 256 * 256;
    return o;
  };
  L.off_B = take(lxn * 8);
  L.off_B0 = take(lxn * 8);
  L.off_Bt = take(lxn * 8);
  L.off_B1 = take(lxn * 8);
  L.off_C = take(static_cast<size_t>(L.lp) * L.ldc * 8);
  L.off_C1 = take(static_cast<size_t>(L.lp) * L.ldc * 8);
  L.off_part = take(static_cast<size_t>(L.part_elems) * 8);
  const size_t sq = static_cast<size_t>(L.lmax) * L.lmax * 8;
  L.off_G = take(sq);
  L.off_Rf = take(sq);
  L.off_Linv = take(sq);
  const size_t np16 = static_cast<size_t>(round_up(L.lmax, 16));
  L.off_cholw = take(np16 * (np16 + 1) * 8 + np16 * 8);  // chol_inv work array + 1/R_ii (n > 128)
  L.off_Rho = take(static_cast<size_t>(L.kp) * n * 8);
  L.off_Rhat = take(static_cast<size_t>(L.kp) * n * 8);
  L.off_T = take(static_cast<size_t>(L.kp) * std::max<long long>(n - 1, 1) * 8);  // adaptive runs use k < k0
  L.off_Q1 = take(static_cast<size_t>(L.ldq1) * std::max(k, 1) * 8);
  L.off_R1 = take(static_cast<size_t>(L.kp) * L.kp * 8);
  L.off_R2 = take(static_cast<size_t>(L.kp) * L.kp * 8);
  L.off_Rbar = take(static_cast<size_t>(L.kp) * L.kp * 8);
  L.off_perm = take(static_cast<size_t>(n) * 8);
  L.off_info = take(64);
  L.off_qr = take(qrcp_workspace_bytes(L.ell, n));
  L.off_gaps = take(static_cast<size_t>(std::max(k, 1)) * 8);
  // sized for a 148-SM B200; a device with other SM counts re-plans at launch (and falls back to the
  // cluster kernel if the ring does not fit)
  L.ring_bytes = sample_ring_bytes(L.lp, static_cast<int>(n), m_local, L.smax, 148);
  L.off_ring = take(L.ring_bytes);
  L.tail_elems = kc_tail_elems(L.lp, static_cast<int>(n), L.smax);
  L.off_tail = take(static_cast<size_t>(L.tail_elems) * 8);
  L.total = off + 1024;
  return L;
}

}  // namespace

struct rs_lowrank_s {
  long long m_global, m_local, row_offset, n;
  int k, p, ell;
  int k0;                // k at create (fixed-rank runs); adaptive runs set k = ell = l found
  bool adaptive = false;
  int robust_iters = 0;   // power iterations redone with shifted CholQR since the last sample
  int factor_shifts = 0;  // shifted CholQR passes the last factor needed (0: plain CholQR2)
  uint64_t seed;
  cudaStream_t st;
  ncclComm_t comm;
  int nranks, rank, sms;
  rs_allreduce_fn ar_fn = nullptr;  // rs_lowrank_set_allreduce_hook: replaces NCCL for this handle
  void* ar_ctx = nullptr;
  Layout L;
  char* ws;
  void* ring;
  double* tailp;  // KC tail-fold partials (L.tail_elems doubles)
  double *B, *B0, *Bt, *B1, *C, *C1, *part, *G, *Rf, *Linv, *cholw, *Rho, *Rhat, *T, *Q1, *R1, *R2, *Rbar, *gaps;
  int64_t* perm;
  int* info;
  void* qr;
  int state;
  int powers;
  std::string err;
  bool prof = false;
  std::map<std::string, ProfEntry> profile;
  std::vector<Pending> pending;
  std::vector<cudaEvent_t> event_pool;
  std::vector<double> gaps_host;
  bool gaps_valid = false;
  // power_iterate enqueues only: its Cholesky factorisations report a breakdown with the
  // internal code RS_INFO_POWER + pass, and pivot replays the iteration from the stored sample
  int chol_code = RS_ERR_NOT_SPD;
  const double* pow_A = nullptr;
  long long pow_lda = 0;
  int pow_q = 0;
  // rs_lowrank_run: the whole step captured once as a CUDA graph and replayed
  bool capturing = false;
  bool graph_disabled = false;
  cudaGraphExec_t gexec = nullptr;
  // the graph is captured on and launched into an internal stream (the caller's stream may be the
  // legacy default stream, which cannot be captured), fenced with events on both sides
  cudaStream_t gstream = nullptr;
  cudaEvent_t gev_in = nullptr, gev_out = nullptr;
  std::vector<long long> gkey;
  std::vector<Pending> gscopes;  // profiling scopes baked into the graph (external event records)
};

namespace {

rs_status_t fail(rs_lowrank_t h, rs_status_t code, const char* fmt, ...) {
  if (h) {
    char buf[512];
    va_list ap;
    va_start(ap, fmt);
    vsnprintf(buf, sizeof(buf), fmt, ap);
    va_end(ap);
    h->err = buf;
  }
  return code;
}

#define RS_CUDA(h, call)                                                                      \
  do {                                                                                        \
    cudaError_t e_ = (call);                                                                  \
    if (e_ != cudaSuccess) return fail(h, RS_ERR_CUDA, "%s: %s (%s:%d)", #call, cudaGetErrorString(e_), __FILE__, __LINE__); \
  } while (0)

#define RS_NCCL(h, call)                                                                      \
  do {                                                                                        \
    ncclResult_t r_ = (call);                                                                 \
    if (r_ != ncclSuccess) return fail(h, RS_ERR_NCCL, "%s: %s", #call, ncclGetErrorString(r_)); \
  } while (0)

cudaEvent_t get_event(rs_lowrank_t h) {
  if (!h->event_pool.empty()) {
    cudaEvent_t e = h->event_pool.back();
    h->event_pool.pop_back();
    return e;
  }
  cudaEvent_t e = nullptr;
  if (cudaEventCreate(&e) != cudaSuccess) {
    cudaGetLastError();
    return nullptr;  // profiling of this scope is skipped (Scope checks)
  }
  return e;
}

// Times the enclosed launches on the handle's stream when profiling is on.
struct Scope {
  rs_lowrank_t h;
  const char* name;
  double flops;
  cudaEvent_t e0{};
  Scope(rs_lowrank_t hh, const char* nm, double fl) : h(hh), name(nm), flops(fl) {
    if (h->prof) {
      e0 = get_event(h);
      if (e0) record(e0);
    }
  }
  // inside a graph capture the events become external event-record nodes, re-recorded at every
  // replay and read back after each rs_lowrank_run (drain_graph_scopes)
  void record(cudaEvent_t e) {
    if (h->capturing)
      cudaEventRecordWithFlags(e, h->st, cudaEventRecordExternal);
    else
      cudaEventRecord(e, h->st);
  }
  ~Scope() {
    if (h->prof && e0) {
      cudaEvent_t e1 = get_event(h);
      if (!e1) {
        h->event_pool.push_back(e0);
        return;
      }
      record(e1);
      (h->capturing ? h->gscopes : h->pending).push_back(Pending{name, e0, e1, flops});
    }
  }
};

void drain_profile(rs_lowrank_t h) {
  for (auto& p : h->pending) {
    cudaEventSynchronize(p.e1);
    float ms = 0.f;
    cudaEventElapsedTime(&ms, p.e0, p.e1);
    auto& e = h->profile[p.name];
    e.ms += ms;
    e.launches += 1;
    e.flops += p.flops;
    h->event_pool.push_back(p.e0);
    h->event_pool.push_back(p.e1);
  }
  h->pending.clear();
}

void drain_graph_scopes(rs_lowrank_t h) {
  for (auto& p : h->gscopes) {
    float ms = 0.f;
    if (cudaEventElapsedTime(&ms, p.e0, p.e1) != cudaSuccess) {
      cudaGetLastError();
      continue;
    }
    auto& e = h->profile[p.name];
    e.ms += ms;
    e.launches += 1;
    e.flops += p.flops;
  }
}

rs_status_t allreduce(rs_lowrank_t h, double* buf, long long count) {
  if (h->ar_fn && h->nranks > 1 && count > 0) {
    Scope sc(h, "comm", 0.0);
    if (h->ar_fn(h->ar_ctx, buf, count, h->st) != 0) return fail(h, RS_ERR_NCCL, "allreduce hook failed");
    return RS_OK;
  }
  // NCCL whenever a communicator is attached -- also at world size 1, so that code path runs
  if (!h->comm || count <= 0) return RS_OK;
  Scope sc(h, "comm", 0.0);
  RS_NCCL(h, ncclAllReduce(buf, buf, static_cast<size_t>(count), ncclDouble, ncclSum, h->comm, h->st));
  return RS_OK;
}

int max_splits_for(rs_lowrank_t h, long long tile_elems) {
  const long long s = h->L.part_elems / std::max<long long>(tile_elems, 1);
  return static_cast<int>(std::max<long long>(1, std::min<long long>(s, 1024)));
}

// Gram of the rows of a row-major X (lp x ldx, K = m_local along the rows): G = X X^T  (KC)
rs_status_t gram_rows_kc(rs_lowrank_t h, const double* X, long long ldx, long long K, int rows, int ld_g) {
  const int splits = gemm_choose_splits(rows, rows, K, max_splits_for(h, static_cast<long long>(ld_g) * ld_g), h->sms);
  const int ns = gemm_nsplit(K, splits);
  {
    Scope sc(h, "gram", 2.0 * rows * rows * static_cast<double>(K));
    if (K > 0) {
      View2D Xv{X, K, rows, ldx};
      GemmOutDesc out{h->part, 1, ld_g, static_cast<long long>(ld_g) * ld_g, ld_g, ld_g};
      if (rows <= 128) {  // symmetric: lower-triangle blocks only
        RS_CUDA(h, gemm_syrk(h->st, rows, K, Xv, out, splits));
      } else {
        PhiloxDesc nophx{false, 0, 0, 0, 0};
        RS_CUDA(h, gemm_kc(h->st, rows, rows, K, Xv, Xv, nophx, out, splits));
      }
    } else {
      RS_CUDA(h, cudaMemsetAsync(h->part, 0, static_cast<size_t>(ld_g) * ld_g * 8, h->st));
    }
  }
  {
    Scope sc(h, "reduce", 0.0);
    RS_CUDA(h, splitk_reduce(h->st, h->G, h->part, K > 0 ? ns : 1, static_cast<long long>(ld_g) * ld_g,
                             static_cast<long long>(ld_g) * ld_g));
  }
  return RS_OK;
}

// dst := L^{-1} src for the rows [0, rp) of the row-major distributed C blocks (ld ldc; rows >= rr
// zero): C1^T = C^T L^{-T} on the tall-skinny triangular kernel (L^{-T}[t][j] = Linv[j + t rp], one
// pass over C); the MC family when rr > 128.
cudaError_t apply_rows_tri(rs_lowrank_t h, const double* src, int rr, int rp, double* dst) {
  const long long ml = h->m_local;
  View2D Xv{src, ml, rr, h->L.ldc};
  cudaError_t e = gemm_tsa(h->st, ml, rr, Xv, h->Linv, rp, dst, h->L.ldc, rp);
  if (e != cudaErrorNotSupported) return e;
  View2D Lv{h->Linv, rp, rp, rp};
  View2D Cv{src, ml, rp, h->L.ldc};
  GemmOutDesc out{dst, h->L.ldc, 1, 0, rp, static_cast<int>(ml)};
  return gemm_mc(h->st, rp, static_cast<int>(ml), rp, Lv, Cv, out, 1, 1);  // Linv lower
}

// One CholQR pass on a replicated short-wide block X (rp x n, column-major, ld rp; rows >= rr are
// zero): G = X X^T (+ s I when shift), R^T R = G, Y = R^{-T} X.  The shift
// s = 11 (n rr + rr (rr+1)) u ||X||_F^2 is shifted CholeskyQR's: breakdown-free for kappa(X) < ~1/u,
// the remedy for "unstable for an ill-conditioned matrix" the paper lists.
rs_status_t cholqr_small_pass(rs_lowrank_t h, const double* src, int rr, int rp, double* dst, bool shift) {
  const int splits = gemm_choose_splits(rp, rp, h->n, max_splits_for(h, static_cast<long long>(rp) * rp), h->sms);
  const int ns = gemm_nsplit(h->n, splits);
  {
    Scope sc(h, "gram", 2.0 * rp * rp * static_cast<double>(h->n));
    View2D Xv{src, rp, h->n, rp};
    GemmOutDesc out{h->part, 1, rp, static_cast<long long>(rp) * rp, rp, rp};
    RS_CUDA(h, gemm_mc(h->st, rp, rp, h->n, Xv, Xv, out, splits));
  }
  {
    Scope sc(h, "reduce", 0.0);
    RS_CUDA(h, splitk_reduce(h->st, h->G, h->part, ns, static_cast<long long>(rp) * rp,
                             static_cast<long long>(rp) * rp));
  }
  {
    Scope sc(h, "chol", rr * static_cast<double>(rr) * rr / 3.0);
    if (shift)
      RS_CUDA(h, shift_diag(h->st, h->G, rp, rr, 11.0 * (static_cast<double>(h->n) * rr + rr * (rr + 1.0)) * 0x1p-53));
    RS_CUDA(h, chol_inv(h->st, h->G, rp, rr, rp, h->Rf, rp, h->Linv, rp, h->cholw, h->info, h->chol_code));
  }
  {
    Scope sc(h, "apply", 2.0 * rr * rr * static_cast<double>(h->n));
    RS_CUDA(h, small_gemm(h->st, rp, static_cast<int>(h->n), rp, h->Linv, 1, rp, src, 1, rp, dst, 1, rp, false));
  }
  return RS_OK;
}

// CholQR of X into Y with nshift shifted passes followed by two plain ones: CholQR2 (nshift = 0),
// shifted CholQR3 (nshift = 1), ...  Each shifted pass is breakdown-free and cuts kappa by about
// 1 / sqrt(11 n rr u), so the plain passes see kappa^2 u < 1 (R20).
rs_status_t cholqr2_block(rs_lowrank_t h, const double* X, int rr, int rp, double* Y, int nshift = 0) {
  const double* src = X;
  const int npass = nshift + 2;
  for (int pass = 0; pass < npass; ++pass) {
    // X -> B1 (-> Rho -> B1 ...) -> Y: Y may alias X; Rho (k x n) is free outside pivot and holds
    // rp x n whenever shifted passes are used (adaptive runs, p = 0)
    double* dst = pass + 1 < npass ? (pass % 2 == 0 ? h->B1 : h->Rho) : Y;
    rs_status_t s = cholqr_small_pass(h, src, rr, rp, dst, pass < nshift);
    if (s != RS_OK) return s;
    src = dst;
  }
  return RS_OK;
}

// Distributed CholQR of the rows [Cn, Cn + rp) of C (row-major, ld ldc; rows >= rr are zero):
// npass passes (even: the result ends in Cn, C1 is the ping-pong buffer), the first nshift shifted.
rs_status_t cholqr_dist(rs_lowrank_t h, double* Cn, int rr, int rp, int npass, int nshift) {
  const Layout& L = h->L;
  const long long ml = h->m_local;
  rs_status_t s;
  for (int pass = 0; pass < npass; ++pass) {
    const double* src = pass % 2 == 0 ? Cn : h->C1;
    double* dst = pass % 2 == 0 ? h->C1 : Cn;
    if ((s = gram_rows_kc(h, src, L.ldc, ml, rp, rp)) != RS_OK) return s;
    if ((s = allreduce(h, h->G, static_cast<long long>(rp) * rp)) != RS_OK) return s;
    {
      Scope sc(h, "chol", rr * static_cast<double>(rr) * rr / 3.0);
      if (pass < nshift)
        RS_CUDA(h, shift_diag(h->st, h->G, rp, rr,
                              11.0 * (static_cast<double>(h->m_global) * rr + rr * (rr + 1.0)) * 0x1p-53));
      RS_CUDA(h, chol_inv(h->st, h->G, rp, rr, rp, h->Rf, rp, h->Linv, rp, h->cholw, h->info, h->chol_code));
    }
    if (ml > 0) {
      Scope sc(h, "apply", 2.0 * rr * static_cast<double>(rr) * ml);
      RS_CUDA(h, apply_rows_tri(h, src, rr, rp, dst));
    }
  }
  return RS_OK;
}

rs_status_t cholqr2_rows_small(rs_lowrank_t h, const double* X, double* Y) {
  return cholqr2_block(h, X, h->L.ell, h->L.lp, Y);
}

rs_status_t check_matrix(rs_lowrank_t h, const void* p, long long ld, long long rows, const char* name) {
  if (!p) return fail(h, RS_ERR_INVALID_ARG, "%s is NULL", name);
  if (reinterpret_cast<uintptr_t>(p) % 16 != 0) return fail(h, RS_ERR_INVALID_ARG, "%s not 16-byte aligned", name);
  if (ld < rows || ld % 2 != 0) return fail(h, RS_ERR_INVALID_ARG, "%s leading dimension %lld invalid (rows %lld, must be even)", name, ld, rows);
  return RS_OK;
}

// internal status: a power-iteration CholQR breakdown was flagged (info[0] >= RS_INFO_POWER)
constexpr rs_status_t RS_INFO_REPLAY = static_cast<rs_status_t>(1000);

rs_status_t sync_and_check(rs_lowrank_t h) {
  RS_CUDA(h, cudaStreamSynchronize(h->st));
  if (h->comm) {  // a failed peer or network error surfaces here rather than as a hang later
    ncclResult_t ar = ncclSuccess;
    RS_NCCL(h, ncclCommGetAsyncError(h->comm, &ar));
    if (ar != ncclSuccess) return fail(h, RS_ERR_NCCL, "NCCL asynchronous error: %s", ncclGetErrorString(ar));
  }
  int info[2] = {0, 0};
  RS_CUDA(h, cudaMemcpy(info, h->info, sizeof(info), cudaMemcpyDeviceToHost));
  if (info[0] >= RS_INFO_POWER) return RS_INFO_REPLAY;
  if (info[0] == RS_ERR_NOT_SPD)
    return fail(h, RS_ERR_NOT_SPD, "CholQR breakdown: Gram matrix not positive definite at column %d", info[1]);
  if (info[0] == RS_ERR_RANK_DEFICIENT)
    return fail(h, RS_ERR_RANK_DEFICIENT, "QRCP: zero residual norm at step %d (rank < k)", info[1]);
  return RS_OK;
}

// ---------------------------------------------------------------------------------------------
// The four steps of Fig. 2, enqueue-only (no host synchronisation), shared by the phase calls
// and by the graph-captured rs_lowrank_run.
// ---------------------------------------------------------------------------------------------

// Step 1: B := Omega A summed over ranks (Fig. 2(b) lines 2-3)
rs_status_t enqueue_sample(rs_lowrank_t h, const double* A, long long lda) {
  const Layout& L = h->L;
  RS_CUDA(h, cudaMemsetAsync(h->info, 0, 16, h->st));
  const long long lxn = static_cast<long long>(L.lp) * h->n;
  if (h->m_local > 0) {
    int ns = 0;
    {
      Scope sc(h, "gemm_sample", 2.0 * h->ell * static_cast<double>(h->m_local) * h->n);
      View2D Av{A, h->m_local, h->n, lda};
      GemmOutDesc out{h->part, 1, L.lp, lxn, L.lp, static_cast<int>(h->n)};
      out.tail_ws = h->tailp;
      out.tail_cap = L.tail_elems;
      PhiloxDesc phx{true, h->seed, 0u, h->row_offset, h->ell};
      // Omega generated once per K split into an L2 ring shared by all N tiles; the cluster kernel
      // (Omega generated in shared memory per pair of N tiles) when the ring does not apply
      cudaError_t e = gemm_sample_ring(h->st, L.lp, static_cast<int>(h->n), h->m_local, Av, phx, out,
                                       max_splits_for(h, lxn), h->ring, L.ring_bytes, &ns);
      if (e == cudaErrorNotSupported) {
        const int splits = gemm_choose_splits(L.lp, static_cast<int>(h->n), h->m_local, max_splits_for(h, lxn), h->sms);
        ns = gemm_nsplit(h->m_local, splits);
        e = gemm_kc(h->st, L.lp, static_cast<int>(h->n), h->m_local, Av, Av, phx, out, splits);
      }
      RS_CUDA(h, e);
    }
    {
      Scope sc(h, "reduce", 0.0);
      RS_CUDA(h, splitk_reduce(h->st, h->B, h->part, ns, lxn, lxn));
    }
  } else {
    RS_CUDA(h, cudaMemsetAsync(h->B, 0, lxn * 8, h->st));
  }
  return allreduce(h, h->B, lxn);
}

// line 12: dst := Csrc A summed over ranks
rs_status_t gemm_b(rs_lowrank_t h, const double* A, long long lda, const double* Csrc, double* dst) {
  const Layout& L = h->L;
  const long long ml = h->m_local, n = h->n;
  const long long lxn = static_cast<long long>(L.lp) * n;
  if (ml > 0) {
    const int splits = gemm_choose_splits(L.lp, static_cast<int>(n), ml, max_splits_for(h, lxn), h->sms, true);
    const int ns = gemm_nsplit(ml, splits);
    {
      Scope sc(h, "gemm_power_b", 2.0 * h->ell * static_cast<double>(ml) * n);
      View2D Cv{Csrc, ml, L.lp, L.ldc};
      View2D Av{A, ml, n, lda};
      GemmOutDesc out{h->part, 1, L.lp, lxn, L.lp, static_cast<int>(n)};
      out.tail_ws = h->tailp;
      out.tail_cap = L.tail_elems;
      PhiloxDesc nophx{false, 0, 0, 0, 0};
      RS_CUDA(h, gemm_kc(h->st, L.lp, static_cast<int>(n), ml, Cv, Av, nophx, out, splits));
    }
    Scope sc(h, "reduce", 0.0);
    RS_CUDA(h, splitk_reduce(h->st, dst, h->part, ns, lxn, lxn));
  } else {
    RS_CUDA(h, cudaMemsetAsync(dst, 0, lxn * 8, h->st));
  }
  return allreduce(h, dst, lxn);
}

// line 7: C := Bt A^T   (C row-major lp x ldc: C[i, j] at i*ldc + j)
rs_status_t gemm_c(rs_lowrank_t h, const double* A, long long lda) {
  const Layout& L = h->L;
  const long long ml = h->m_local, n = h->n;
  if (ml > 0) {
    Scope sc(h, "gemm_power_c", 2.0 * h->ell * static_cast<double>(ml) * n);
    View2D Bv{h->Bt, L.lp, n, L.lp};
    View2D Av{A, ml, n, lda};
    GemmOutDesc out{h->C, L.ldc, 1, 0, L.lp, static_cast<int>(ml)};
    RS_CUDA(h, gemm_mc(h->st, L.lp, static_cast<int>(ml), n, Bv, Av, out, 1));
  }
  return RS_OK;
}

// One plain pass of Fig. 2(a) lines 5-12 up to B1 = C1 A (allreduced): B := QR(B) (replicated
// CholQR2), C := B A^T, C := QR(C) (distributed CholQR2 whose second R^{-T} is applied to the
// l x n product instead of C -- exact re-association, R2 = I + O(kappa^2 u)).  The caller finishes
// with B := R2^{-T} B1 (power_apply).  Cholesky breakdowns are flagged with h->chol_code.
rs_status_t power_to_b1(rs_lowrank_t h, const double* A, long long lda) {
  const Layout& L = h->L;
  const long long ml = h->m_local;
  rs_status_t s = cholqr2_rows_small(h, h->B, h->Bt);  // line 5
  if (s != RS_OK) return s;
  if ((s = gemm_c(h, A, lda)) != RS_OK) return s;     // line 7
  // line 10
  if ((s = gram_rows_kc(h, h->C, L.ldc, ml, L.lp, L.lp)) != RS_OK) return s;
  if ((s = allreduce(h, h->G, static_cast<long long>(L.lp) * L.lp)) != RS_OK) return s;
  {
    Scope sc(h, "chol", L.ell * static_cast<double>(L.ell) * L.ell / 3.0);
    RS_CUDA(h, chol_inv(h->st, h->G, L.lp, L.ell, L.lp, h->Rf, L.lp, h->Linv, L.lp, h->cholw, h->info, h->chol_code));
  }
  if (ml > 0) {
    Scope sc(h, "apply", 2.0 * L.ell * static_cast<double>(L.ell) * ml);
    RS_CUDA(h, apply_rows_tri(h, h->C, L.ell, L.lp, h->C1));
  }
  if ((s = gram_rows_kc(h, h->C1, L.ldc, ml, L.lp, L.lp)) != RS_OK) return s;
  if ((s = allreduce(h, h->G, static_cast<long long>(L.lp) * L.lp)) != RS_OK) return s;
  {
    Scope sc(h, "chol", L.ell * static_cast<double>(L.ell) * L.ell / 3.0);
    RS_CUDA(h, chol_inv(h->st, h->G, L.lp, L.ell, L.lp, h->Rf, L.lp, h->Linv, L.lp, h->cholw, h->info, h->chol_code));
  }
  return gemm_b(h, A, lda, h->C1, h->B1);  // line 12 (B1 = C1 A)
}

rs_status_t power_apply(rs_lowrank_t h) {
  const Layout& L = h->L;
  Scope sc(h, "apply", 2.0 * L.ell * static_cast<double>(L.ell) * h->n);
  RS_CUDA(h, small_gemm(h->st, L.lp, static_cast<int>(h->n), L.lp, h->Linv, 1, L.lp, h->B1, 1, L.lp, h->B, 1, L.lp,
                        false));
  return RS_OK;
}

// The R20 fallback of one pass, from its input B: 2 shifted + 2 plain CholQR passes on B and on C.
rs_status_t power_robust(rs_lowrank_t h, const double* A, long long lda) {
  const Layout& L = h->L;
  rs_status_t s;
  const double* src = h->B;
  for (int pass = 0; pass < 4; ++pass) {  // B -> B1 -> Bt -> B1 -> Bt
    double* dst = pass % 2 == 0 ? h->B1 : h->Bt;
    if ((s = cholqr_small_pass(h, src, L.ell, L.lp, dst, pass < 2)) != RS_OK) return s;
    src = dst;
  }
  if ((s = gemm_c(h, A, lda)) != RS_OK) return s;
  if ((s = cholqr_dist(h, h->C, L.ell, L.lp, 4, 2)) != RS_OK) return s;
  return gemm_b(h, A, lda, h->C, h->B);
}

// q passes, enqueue only.  The sample is kept in B0; a breakdown in pass it sets info to
// RS_INFO_POWER + it, which pivot (or rs_lowrank_run) turns into replay_power_and_pivot.
rs_status_t enqueue_power(rs_lowrank_t h, const double* A, long long lda, int q) {
  const Layout& L = h->L;
  RS_CUDA(h, cudaMemcpyAsync(h->B0, h->B, static_cast<size_t>(L.lp) * h->n * 8, cudaMemcpyDeviceToDevice, h->st));
  h->pow_A = A;
  h->pow_lda = lda;
  h->pow_q = q;
  rs_status_t s = RS_OK;
  for (int it = 0; it < q && s == RS_OK; ++it) {
    h->chol_code = RS_INFO_POWER + it;
    s = power_to_b1(h, A, lda);
    if (s == RS_OK) s = power_apply(h);
  }
  h->chol_code = RS_ERR_NOT_SPD;
  if (s == RS_OK) h->powers = q;
  return s;
}

// The breakdown path: q passes from the stored sample with a host check after each pass; a pass
// whose CholQR broke down is redone from its input B with shifted CholQR (R20).
rs_status_t power_sync(rs_lowrank_t h, const double* A, long long lda, int q) {
  rs_status_t s;
  h->chol_code = RS_ERR_NOT_SPD;
  for (int it = 0; it < q; ++it) {
    if ((s = power_to_b1(h, A, lda)) != RS_OK) return s;
    int info[2] = {0, 0};
    RS_CUDA(h, cudaMemcpyAsync(info, h->info, sizeof(info), cudaMemcpyDeviceToHost, h->st));
    RS_CUDA(h, cudaStreamSynchronize(h->st));
    if (info[0] == RS_ERR_NOT_SPD) {
      RS_CUDA(h, cudaMemsetAsync(h->info, 0, 16, h->st));
      if ((s = power_robust(h, A, lda)) != RS_OK) return s;
      h->robust_iters++;
    } else if ((s = power_apply(h)) != RS_OK) {
      return s;
    }
  }
  h->powers = q;
  return RS_OK;
}

// Step 2: truncated QRCP of B (Fig. 2(b) line 6) and T = R^_11^{-1} R^_12 (line 9)
rs_status_t enqueue_pivot(rs_lowrank_t h, int64_t* perm) {
  const Layout& L = h->L;
  {
    Scope sc(h, "qrcp", 0.0);
    RS_CUDA(h, qrcp_truncated(h->st, h->B, L.lp, h->ell, h->n, h->k, h->qr, h->perm, h->Rho, L.kp, h->gaps, h->info,
                              h->sms));
  }
  {
    Scope sc(h, "other", static_cast<double>(h->k) * h->k * (h->n - h->k));
    RS_CUDA(h, permute_cols(h->st, h->Rho, L.kp, h->k, h->n, h->perm, h->Rhat, L.kp));
    RS_CUDA(h, trsm_upper_cols(h->st, h->Rhat, L.kp, h->k, h->Rhat + static_cast<long long>(h->k) * L.kp, L.kp,
                               h->n - h->k, h->T, L.kp));
  }
  if (perm) RS_CUDA(h, cudaMemcpyAsync(perm, h->perm, h->n * 8, cudaMemcpyDeviceToDevice, h->st));
  return RS_OK;
}

rs_status_t replay_power_and_pivot(rs_lowrank_t h, int64_t* perm) {
  const Layout& L = h->L;
  RS_CUDA(h, cudaMemsetAsync(h->info, 0, 16, h->st));
  RS_CUDA(h, cudaMemcpyAsync(h->B, h->B0, static_cast<size_t>(L.lp) * h->n * 8, cudaMemcpyDeviceToDevice, h->st));
  h->robust_iters = 0;
  rs_status_t s = power_sync(h, h->pow_A, h->pow_lda, h->pow_q);
  if (s != RS_OK) return s;
  if ((s = enqueue_pivot(h, perm)) != RS_OK) return s;
  s = sync_and_check(h);
  return s == RS_INFO_REPLAY ? fail(h, RS_ERR_NOT_SPD, "CholQR breakdown in the power iteration") : s;
}

rs_status_t check_factor_args(rs_lowrank_t h, const double* A, long long lda, const double* Q, long long ldq,
                              const double* R, long long ldr) {
  rs_status_t s;
  if (h->m_local > 0) {
    if ((s = check_matrix(h, A, lda, h->m_local, "A")) != RS_OK) return s;
    if ((s = check_matrix(h, Q, ldq, h->m_local, "Q")) != RS_OK) return s;
  }
  return check_matrix(h, R, ldr, h->k, "R");
}

// Step 3: [Q, Rbar] := QR(A P_{1:k}) by CholQR with npass passes (even, so the last lands in Q),
// the first nshift with the Gram shifted by 11 (m k + k(k+1)) u ||X||_F^2 (R20); R := Rbar [I_k T]
// (Fig. 2(b) lines 8 and 10).
rs_status_t enqueue_factor(rs_lowrank_t h, const double* A, long long lda, double* Q, long long ldq, double* R,
                           long long ldr, int npass, int nshift) {
  const Layout& L = h->L;
  const long long ml = h->m_local, n = h->n;
  const int k = h->k;
  // Q := A(:, P_{1:k})
  if (ml > 0) {
    Scope sc(h, "factor", 0.0);
    RS_CUDA(h, gather_cols(h->st, A, lda, ml, h->perm, k, Q, ldq));
  }
  const double* src = Q;
  long long ld_src = ldq;
  double* bufs[2] = {h->Rbar, h->R2};
  int which = -1;  // index of the running product Rbar = R_p ... R_1 (-1: identity)
  for (int pass = 0; pass < npass; ++pass) {
    double* dst = pass % 2 == 0 ? h->Q1 : Q;
    const long long ld_dst = pass % 2 == 0 ? L.ldq1 : ldq;
    // Gram G = X^T X (k x k) of the tall X = src (m_local x k column-major)
    rs_status_t st2 = gram_rows_kc(h, src, ld_src, ml, k, L.kp);
    if (st2 != RS_OK) return st2;
    st2 = allreduce(h, h->G, static_cast<long long>(L.kp) * L.kp);
    if (st2 != RS_OK) return st2;
    {
      Scope sc(h, "chol", k * static_cast<double>(k) * k / 3.0);
      if (pass < nshift)
        RS_CUDA(h, shift_diag(h->st, h->G, L.kp, k,
                              11.0 * (static_cast<double>(h->m_global) * k + k * (k + 1.0)) * 0x1p-53));
      RS_CUDA(h, chol_inv(h->st, h->G, L.kp, k, L.kp, h->R1, L.kp, h->Linv, L.kp, h->cholw, h->info,
                          RS_ERR_NOT_SPD));
    }
    // dst = src * R_p^{-1}  (R_p^{-1}[kk, c] = Linv[c + kk*kp]: N-contiguous operand)
    if (ml > 0) {
      Scope sc(h, "factor", 2.0 * k * static_cast<double>(k) * ml);
      View2D Xv{src, ml, k, ld_src};
      cudaError_t e = gemm_tsa(h->st, ml, k, Xv, h->Linv, L.kp, dst, ld_dst, k);  // R^-1 upper, resident
      if (e == cudaErrorNotSupported) {  // k > 128
        View2D Wv{h->Linv, k, k, L.kp};
        GemmOutDesc out{dst, 1, ld_dst, 0, static_cast<int>(ml), k};
        e = gemm_mc(h->st, static_cast<int>(ml), k, k, Xv, Wv, out, 1, 2);
      }
      RS_CUDA(h, e);
    }
    {
      Scope sc(h, "other", 2.0 * k * static_cast<double>(k) * k);
      if (which < 0) {
        which = 0;
        RS_CUDA(h, copy_2d(h->st, h->R1, L.kp, bufs[0], L.kp, L.kp, L.kp));
      } else {  // Rbar := R_p Rbar
        RS_CUDA(h, small_gemm(h->st, k, k, k, h->R1, 1, L.kp, bufs[which], 1, L.kp, bufs[1 - which], 1, L.kp,
                              false));
        which = 1 - which;
      }
    }
    src = dst;
    ld_src = ld_dst;
  }
  Scope sc(h, "other", 2.0 * k * static_cast<double>(k) * n);
  // R = Rbar [I_k T]
  RS_CUDA(h, copy_2d(h->st, bufs[which], L.kp, R, ldr, k, k));
  if (n > k)
    RS_CUDA(h, small_gemm(h->st, k, static_cast<int>(n - k), k, bufs[which], 1, L.kp, h->T, 1, L.kp,
                          R + static_cast<long long>(k) * ldr, 1, ldr, false));
  return RS_OK;
}

// CholQR2 broke down (kappa(A P_1)^2 u > 1, e.g. an adaptive l past the numerical rank): shifted
// CholQR with 2, then 4 shifted passes ahead of the two plain ones (R20)
rs_status_t factor_fallback(rs_lowrank_t h, const double* A, long long lda, double* Q, long long ldq, double* R,
                            long long ldr) {
  rs_status_t s = RS_ERR_NOT_SPD;
  for (int nshift = 2; s == RS_ERR_NOT_SPD && nshift <= 4; nshift += 2) {
    RS_CUDA(h, cudaMemsetAsync(h->info, 0, 16, h->st));
    s = enqueue_factor(h, A, lda, Q, ldq, R, ldr, nshift + 2, nshift);
    if (s == RS_OK) s = sync_and_check(h);
    h->factor_shifts = nshift;
  }
  return s;
}

void release_graph(rs_lowrank_t h) {
  if (h->gexec) cudaGraphExecDestroy(h->gexec);
  h->gexec = nullptr;
  h->gkey.clear();
  for (auto& p : h->gscopes) {
    h->event_pool.push_back(p.e0);
    h->event_pool.push_back(p.e1);
  }
  h->gscopes.clear();
}

// Capture sample -> power (q) -> pivot -> factor (CholQR2) on the handle's stream as one CUDA
// graph: replays launch the ~70 kernels and NCCL collectives of a step with one call
// and no host round trip.  Anything the capture cannot hold disables the graph for this handle
// (the phases then run directly).
rs_status_t capture_step(rs_lowrank_t h, const double* A, long long lda, int q, int64_t* perm, double* Q,
                         long long ldq, double* R, long long ldr) {
  release_graph(h);
  if (!h->gstream) {
    if (cudaStreamCreateWithFlags(&h->gstream, cudaStreamNonBlocking) != cudaSuccess ||
        cudaEventCreateWithFlags(&h->gev_in, cudaEventDisableTiming) != cudaSuccess ||
        cudaEventCreateWithFlags(&h->gev_out, cudaEventDisableTiming) != cudaSuccess) {
      cudaGetLastError();
      h->graph_disabled = true;
      return RS_OK;
    }
  }
  cudaGraph_t g = nullptr;
  if (cudaStreamBeginCapture(h->gstream, cudaStreamCaptureModeThreadLocal) != cudaSuccess) {
    cudaGetLastError();
    h->graph_disabled = true;
    return RS_OK;
  }
  cudaStream_t user = h->st;
  h->st = h->gstream;  // every enqueue below goes to the capturing stream
  h->capturing = true;
  rs_status_t s = enqueue_sample(h, A, lda);
  if (s == RS_OK && q > 0) s = enqueue_power(h, A, lda, q);
  if (s == RS_OK) s = enqueue_pivot(h, perm);
  if (s == RS_OK) s = enqueue_factor(h, A, lda, Q, ldq, R, ldr, 2, 0);
  h->capturing = false;
  h->st = user;
  const cudaError_t ec = cudaStreamEndCapture(h->gstream, &g);
  cudaError_t ei = cudaErrorUnknown;
  if (s == RS_OK && ec == cudaSuccess && g) ei = cudaGraphInstantiate(&h->gexec, g, 0);
  if (g) cudaGraphDestroy(g);
  if (ei != cudaSuccess) {
    cudaGetLastError();
    h->gexec = nullptr;
    h->graph_disabled = true;
    release_graph(h);
    h->err.clear();
  }
  return RS_OK;
}

// one replay, ordered after the work already on the handle's stream and before what follows it
cudaError_t launch_step(rs_lowrank_t h) {
  cudaError_t e = cudaEventRecord(h->gev_in, h->st);
  if (e == cudaSuccess) e = cudaStreamWaitEvent(h->gstream, h->gev_in, 0);
  if (e == cudaSuccess) e = cudaGraphLaunch(h->gexec, h->gstream);
  if (e == cudaSuccess) e = cudaEventRecord(h->gev_out, h->gstream);
  if (e == cudaSuccess) e = cudaStreamWaitEvent(h->st, h->gev_out, 0);
  return e;
}
}  // namespace

extern "C" {

size_t rs_lowrank_workspace_bytes(int64_t m_local, int64_t n, int32_t k, int32_t p, int32_t nranks) {
  (void)nranks;
  if (m_local < 0 || n < 1 || k < 1 || p < 0) return 0;
  return plan(m_local, n, k, p).total;
}

rs_status_t rs_lowrank_create(rs_lowrank_t* out, int64_t m_global, int64_t m_local, int64_t row_offset, int64_t n,
                              int32_t k, int32_t p, uint64_t seed, void* workspace, size_t workspace_bytes,
                              void* cuda_stream, void* nccl_comm) {
  if (!out) return RS_ERR_INVALID_ARG;
  *out = nullptr;
  const long long ell = static_cast<long long>(k) + p;
  if (k < 1 || p < 0 || ell > 512 || ell > m_global || ell > n || m_local < 0 || row_offset < 0 ||
      row_offset + m_local > m_global || m_global >= (1LL << 31) || n >= (1LL << 31))
    return RS_ERR_INVALID_ARG;
  int dev = 0, major = 0, sms = 0;
  if (cudaGetDevice(&dev) != cudaSuccess) return RS_ERR_CUDA;
  cudaDeviceGetAttribute(&major, cudaDevAttrComputeCapabilityMajor, dev);
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
  if (major != 10) return RS_ERR_UNSUPPORTED;
  Layout L = plan(m_local, n, k, p);
  if (!workspace || workspace_bytes < L.total) return RS_ERR_WORKSPACE;
  auto* h = new rs_lowrank_s();
  h->m_global = m_global;
  h->m_local = m_local;
  h->row_offset = row_offset;
  h->n = n;
  h->k = k;
  h->k0 = k;
  h->p = p;
  h->ell = static_cast<int>(ell);
  h->seed = seed;
  h->st = static_cast<cudaStream_t>(cuda_stream);
  h->comm = static_cast<ncclComm_t>(nccl_comm);
  h->nranks = 1;
  h->rank = 0;
  h->sms = sms;
  if (h->comm) {
    if (ncclCommCount(h->comm, &h->nranks) != ncclSuccess || ncclCommUserRank(h->comm, &h->rank) != ncclSuccess) {
      delete h;
      return RS_ERR_NCCL;
    }
  }
  h->L = L;
  char* base = reinterpret_cast<char*>((reinterpret_cast<uintptr_t>(workspace) + 255) & ~uintptr_t(255));
  h->ws = base;
  auto D = [&](size_t off) { return reinterpret_cast<double*>(base + off); };
  h->B = D(L.off_B);
  h->B0 = D(L.off_B0);
  h->ring = base + L.off_ring;
  h->tailp = reinterpret_cast<double*>(base + L.off_tail);
  h->Bt = D(L.off_Bt);
  h->B1 = D(L.off_B1);
  h->C = D(L.off_C);
  h->C1 = D(L.off_C1);
  h->part = D(L.off_part);
  h->G = D(L.off_G);
  h->Rf = D(L.off_Rf);
  h->Linv = D(L.off_Linv);
  h->cholw = D(L.off_cholw);
  h->Rho = D(L.off_Rho);
  h->Rhat = D(L.off_Rhat);
  h->T = D(L.off_T);
  h->Q1 = D(L.off_Q1);
  h->R1 = D(L.off_R1);
  h->R2 = D(L.off_R2);
  h->Rbar = D(L.off_Rbar);
  h->gaps = D(L.off_gaps);
  h->perm = reinterpret_cast<int64_t*>(base + L.off_perm);
  h->info = reinterpret_cast<int*>(base + L.off_info);
  h->qr = base + L.off_qr;
  h->state = ST_CREATED;
  h->powers = 0;
  // zero everything once: padding rows/columns of B, C, Linv, R stay zero forever
  if (cudaMemsetAsync(workspace, 0, L.total, h->st) != cudaSuccess) {
    delete h;
    return RS_ERR_CUDA;
  }
  *out = h;
  return RS_OK;
}

rs_status_t rs_lowrank_sample(rs_lowrank_t h, const double* A, int64_t lda) {
  if (!h) return RS_ERR_INVALID_ARG;
  if (h->m_local > 0) {
    rs_status_t s = check_matrix(h, A, lda, h->m_local, "A");
    if (s != RS_OK) return s;
  }
  rs_status_t s = enqueue_sample(h, A, lda);
  if (s != RS_OK) return s;
  h->state = ST_SAMPLED;
  h->powers = 0;
  h->robust_iters = 0;
  h->pow_q = 0;
  h->ell = h->L.ell;
  h->k = h->k0;
  h->adaptive = false;
  return RS_OK;
}

rs_status_t rs_lowrank_power_iterate(rs_lowrank_t h, const double* A, int64_t lda, int32_t q) {
  if (!h) return RS_ERR_INVALID_ARG;
  if (h->state != ST_SAMPLED) return fail(h, RS_ERR_BAD_STATE, "power_iterate needs a fresh sample");
  if (h->adaptive) return fail(h, RS_ERR_BAD_STATE, "the adaptive sample already includes its power iterations");
  if (h->pow_q > 0) return fail(h, RS_ERR_BAD_STATE, "power_iterate already ran on this sample");
  if (q < 0) return fail(h, RS_ERR_INVALID_ARG, "q < 0");
  if (q == 0) return RS_OK;
  if (h->m_local > 0) {
    rs_status_t s = check_matrix(h, A, lda, h->m_local, "A");
    if (s != RS_OK) return s;
  }
  return enqueue_power(h, A, lda, q);
}

rs_status_t rs_lowrank_pivot(rs_lowrank_t h, int64_t* perm) {
  if (!h) return RS_ERR_INVALID_ARG;
  if (h->state != ST_SAMPLED) return fail(h, RS_ERR_BAD_STATE, "pivot needs a sample");
  rs_status_t s = enqueue_pivot(h, perm);
  if (s != RS_OK) return s;
  s = sync_and_check(h);
  if (s == RS_INFO_REPLAY) s = replay_power_and_pivot(h, perm);
  if (s != RS_OK) return s;
  h->gaps_valid = false;
  h->state = ST_PIVOTED;
  return RS_OK;
}

rs_status_t rs_lowrank_factor(rs_lowrank_t h, const double* A, int64_t lda, double* Q, int64_t ldq, double* R,
                              int64_t ldr) {
  if (!h) return RS_ERR_INVALID_ARG;
  if (h->state != ST_PIVOTED && h->state != ST_FACTORED) return fail(h, RS_ERR_BAD_STATE, "factor needs pivot");
  rs_status_t s = check_factor_args(h, A, lda, Q, ldq, R, ldr);
  if (s != RS_OK) return s;
  s = enqueue_factor(h, A, lda, Q, ldq, R, ldr, 2, 0);
  if (s == RS_OK) s = sync_and_check(h);
  h->factor_shifts = 0;
  if (s == RS_ERR_NOT_SPD) s = factor_fallback(h, A, lda, Q, ldq, R, ldr);
  if (s != RS_OK) return s;
  h->state = ST_FACTORED;
  return RS_OK;
}

rs_status_t rs_lowrank_run(rs_lowrank_t h, const double* A, int64_t lda, int32_t q, int64_t* perm, double* Q,
                           int64_t ldq, double* R, int64_t ldr) {
  if (!h) return RS_ERR_INVALID_ARG;
  if (q < 0) return fail(h, RS_ERR_INVALID_ARG, "q < 0");
  rs_status_t s;
  if (h->m_local > 0 && (s = check_matrix(h, A, lda, h->m_local, "A")) != RS_OK) return s;
  if ((s = check_factor_args(h, A, lda, Q, ldq, R, ldr)) != RS_OK) return s;
  h->k = h->k0;  // a fixed-rank run (an earlier adaptive sample set k = l)
  h->ell = h->L.ell;
  h->adaptive = false;
  if (!h->ar_fn && !h->graph_disabled) {
    const std::vector<long long> key = {reinterpret_cast<long long>(A), lda, q, reinterpret_cast<long long>(perm),
                                        reinterpret_cast<long long>(Q), ldq, reinterpret_cast<long long>(R), ldr,
                                        h->prof ? 1 : 0};
    if (!h->gexec || key != h->gkey) {
      if ((s = capture_step(h, A, lda, q, perm, Q, ldq, R, ldr)) != RS_OK) return s;
      if (h->gexec) h->gkey = key;
    }
    if (h->gexec) {
      RS_CUDA(h, launch_step(h));
      s = sync_and_check(h);
      if (h->prof) drain_graph_scopes(h);
      if (s == RS_OK) {
        h->state = ST_FACTORED;
        h->powers = q;
        h->robust_iters = 0;
        h->factor_shifts = 0;
        h->pow_A = A;
        h->pow_lda = lda;
        h->pow_q = q;
        h->gaps_valid = false;
        return RS_OK;
      }
      if (s != RS_INFO_REPLAY && s != RS_ERR_NOT_SPD) return s;
      // a CholQR breakdown somewhere in the step: redo it through the phases, which apply the
      // shifted-CholQR fallbacks (R20) where the breakdown happened
      RS_CUDA(h, cudaMemsetAsync(h->info, 0, 16, h->st));
    }
  }
  if ((s = rs_lowrank_sample(h, A, lda)) != RS_OK) return s;
  if ((s = rs_lowrank_power_iterate(h, A, lda, q)) != RS_OK) return s;
  if ((s = rs_lowrank_pivot(h, perm)) != RS_OK) return s;
  return rs_lowrank_factor(h, A, lda, Q, ldq, R, ldr);
}

// ---------------------------------------------------------------------------------------------
// Adaptive sample-size scheme (Fig. 3; readings R16-R19 in DESIGN.md)
// ---------------------------------------------------------------------------------------------
}  // extern "C"

namespace {

// Bn (rp x n, ld rp) := Bn - (Bn Bold^T) Bold (one BCGS projection) -- replicated, no communication.
rs_status_t borth_small(rs_lowrank_t h, const double* Bold, int ldo, int lold, double* Bn, int rp) {
  if (lold <= 0) return RS_OK;
  const long long n = h->n;
  {
    const int splits = gemm_choose_splits(rp, lold, n, max_splits_for(h, static_cast<long long>(rp) * lold), h->sms);
    const int ns = gemm_nsplit(n, splits);
    {
      Scope sc(h, "borth", 2.0 * rp * lold * static_cast<double>(n));
      View2D Xv{Bn, rp, n, rp};
      View2D Ov{Bold, lold, n, ldo};
      GemmOutDesc out{h->part, 1, rp, static_cast<long long>(rp) * lold, rp, lold};
      RS_CUDA(h, gemm_mc(h->st, rp, lold, n, Xv, Ov, out, splits));
      RS_CUDA(h, splitk_reduce(h->st, h->G, h->part, ns, static_cast<long long>(rp) * lold,
                               static_cast<long long>(rp) * lold));
      RS_CUDA(h, small_gemm(h->st, rp, static_cast<int>(n), lold, h->G, 1, rp, Bold, 1, ldo, Bn, 1, rp, true, -1.0));
    }
  }
  return RS_OK;
}

// Cn (rr rows at Cn, row-major, ld ldc, distributed over ranks) := Cn - (Cn Cold^T) Cold (one pass).
rs_status_t borth_dist(rs_lowrank_t h, const double* Cold, int lold, double* Cn, int rr) {
  if (lold <= 0) return RS_OK;
  const Layout& L = h->L;
  const long long ml = h->m_local;
  {
    const int splits = gemm_choose_splits(rr, lold, ml, max_splits_for(h, static_cast<long long>(rr) * lold), h->sms);
    const int ns = gemm_nsplit(ml, splits);
    Scope sc(h, "borth", 4.0 * rr * lold * static_cast<double>(ml));
    if (ml > 0) {
      View2D Xv{Cn, ml, rr, L.ldc};
      View2D Ov{Cold, ml, lold, L.ldc};
      GemmOutDesc out{h->part, 1, rr, static_cast<long long>(rr) * lold, rr, lold};
      PhiloxDesc nophx{false, 0, 0, 0, 0};
      RS_CUDA(h, gemm_kc(h->st, rr, lold, ml, Xv, Ov, nophx, out, splits));
      RS_CUDA(h, splitk_reduce(h->st, h->G, h->part, ns, static_cast<long long>(rr) * lold,
                               static_cast<long long>(rr) * lold));
    } else {
      RS_CUDA(h, cudaMemsetAsync(h->G, 0, static_cast<size_t>(rr) * lold * 8, h->st));
    }
    rs_status_t s = allreduce(h, h->G, static_cast<long long>(rr) * lold);
    if (s != RS_OK) return s;
    if (ml > 0) {
      View2D Wv{h->G, rr, lold, rr};
      View2D Ov{Cold, ml, lold, L.ldc};
      GemmOutDesc out{Cn, L.ldc, 1, 0, rr, static_cast<int>(ml)};
      out.mode = 1;  // Cn -= W Cold
      RS_CUDA(h, gemm_mc(h->st, rr, static_cast<int>(ml), lold, Wv, Ov, out, 1));
    }
  }
  return RS_OK;
}

// BOrth + QR of a replicated block (R17): twice { project against B_{1:l}; block CholQR }.  The
// first CholQR has nshift shifted passes (the projected block may be ill-conditioned), the second
// acts on a block that is orthonormal to O(kappa u), where CholQR2 is exact to O(u).
rs_status_t borth_qr_small(rs_lowrank_t h, int lold, double* Bn, int rr, int nshift) {
  rs_status_t s;
  if (lold <= 0) return cholqr2_block(h, Bn, rr, rr, Bn, nshift);
  for (int pass = 0; pass < 2; ++pass) {
    if ((s = borth_small(h, h->B, h->L.lp, lold, Bn, rr)) != RS_OK) return s;
    if ((s = cholqr2_block(h, Bn, rr, rr, Bn, pass == 0 ? nshift : 0)) != RS_OK) return s;
  }
  return RS_OK;
}

// BOrth + QR of a distributed C block (R17), as borth_qr_small (pass counts rounded up to even).
rs_status_t borth_qr_dist(rs_lowrank_t h, int lold, double* Cn, int rr, int nshift) {
  rs_status_t s;
  const int npass = (nshift + 3) / 2 * 2;
  if (lold <= 0) return cholqr_dist(h, Cn, rr, rr, npass, nshift);
  for (int pass = 0; pass < 2; ++pass) {
    if ((s = borth_dist(h, h->C, lold, Cn, rr)) != RS_OK) return s;
    if ((s = cholqr_dist(h, Cn, rr, rr, pass == 0 ? npass : 2, pass == 0 ? nshift : 0)) != RS_OK) return s;
  }
  return RS_OK;
}

// Bn (rr x n, ld rr) := Omega[row0 : row0+rr] A, summed over ranks
rs_status_t sample_block(rs_lowrank_t h, const double* A, long long lda, int row0, int rr, double* Bn) {
  const long long ml = h->m_local, n = h->n;
  const long long cnt = static_cast<long long>(rr) * n;
  if (ml > 0) {
    const int splits = gemm_choose_splits(rr, static_cast<int>(n), ml, max_splits_for(h, cnt), h->sms);
    const int ns = gemm_nsplit(ml, splits);
    {
      Scope sc(h, "gemm_sample", 2.0 * rr * static_cast<double>(ml) * n);
      View2D Av{A, ml, n, lda};
      GemmOutDesc out{h->part, 1, rr, cnt, rr, static_cast<int>(n)};
      PhiloxDesc phx{true, h->seed, 0u, h->row_offset, rr};
      phx.omega_row0 = row0;
      RS_CUDA(h, gemm_kc(h->st, rr, static_cast<int>(n), ml, Av, Av, phx, out, splits));
    }
    Scope sc(h, "reduce", 0.0);
    RS_CUDA(h, splitk_reduce(h->st, Bn, h->part, ns, cnt, cnt));
  } else {
    RS_CUDA(h, cudaMemsetAsync(Bn, 0, cnt * 8, h->st));
  }
  return allreduce(h, Bn, cnt);
}

// POWER (Fig. 2(a)) on the new block (rows [l, l+rr)) with BOrth against rows [0, l)
rs_status_t power_block(rs_lowrank_t h, const double* A, long long lda, int l, int rr, int q, double* Bn,
                        int nshift) {
  const Layout& L = h->L;
  const long long ml = h->m_local, n = h->n;
  const long long cnt = static_cast<long long>(rr) * n;
  double* Cn = h->C + static_cast<long long>(l) * L.ldc;
  rs_status_t s;
  for (int it = 0; it < q; ++it) {
    if ((s = borth_qr_small(h, l, Bn, rr, nshift)) != RS_OK) return s;          // lines 4-5
    if (ml > 0) {                                                               // line 7: C := B A^T
      Scope sc(h, "gemm_power_c", 2.0 * rr * static_cast<double>(ml) * n);
      View2D Bv{Bn, rr, n, rr};
      View2D Av{A, ml, n, lda};
      GemmOutDesc out{Cn, L.ldc, 1, 0, rr, static_cast<int>(ml)};
      RS_CUDA(h, gemm_mc(h->st, rr, static_cast<int>(ml), n, Bv, Av, out, 1));
    }
    if ((s = borth_qr_dist(h, l, Cn, rr, nshift)) != RS_OK) return s;           // lines 9-10
    // line 12: B := C A
    if (ml > 0) {
      const int splits = gemm_choose_splits(rr, static_cast<int>(n), ml, max_splits_for(h, cnt), h->sms);
      const int ns = gemm_nsplit(ml, splits);
      {
        Scope sc(h, "gemm_power_b", 2.0 * rr * static_cast<double>(ml) * n);
        View2D Cv{Cn, ml, rr, L.ldc};
        View2D Av{A, ml, n, lda};
        GemmOutDesc out{h->part, 1, rr, cnt, rr, static_cast<int>(n)};
        PhiloxDesc nophx{false, 0, 0, 0, 0};
        RS_CUDA(h, gemm_kc(h->st, rr, static_cast<int>(n), ml, Cv, Av, nophx, out, splits));
      }
      Scope sc(h, "reduce", 0.0);
      RS_CUDA(h, splitk_reduce(h->st, Bn, h->part, ns, cnt, cnt));
    } else {
      RS_CUDA(h, cudaMemsetAsync(Bn, 0, cnt * 8, h->st));
    }
    if ((s = allreduce(h, Bn, cnt)) != RS_OK) return s;
  }
  return RS_OK;
}

// f(l, l_inc) of Fig. 3 line 11 (readings R19 / R19b): static, or the "simple linear
// interpolation of the previous two steps": extrapolate log10 eps~ linearly in l to
// where it reaches eps and round the increment up to a multiple of 8 (at least 8).
int next_inc(int policy, const std::vector<std::pair<int, double>>& hv, int l, int inc, double eps) {
  if (policy == RS_INC_STATIC || hv.size() < 2 || !(eps > 0.0)) return inc;
  const double l1 = hv[hv.size() - 2].first, e1 = hv[hv.size() - 2].second;
  const double l2 = hv.back().first, e2 = hv.back().second;
  if (!(e1 > 0.0 && e2 > 0.0 && e2 < e1)) return inc;
  const double slope = (std::log10(e2) - std::log10(e1)) / (l2 - l1);
  const double lstar = l2 + (std::log10(eps) - std::log10(e2)) / slope;
  const double steps = std::ceil((lstar - l) / 8.0);
  if (!(steps < 1e6)) return inc;
  return std::max(8, 8 * static_cast<int>(steps));
}

}  // namespace

extern "C" {

rs_status_t rs_lowrank_sample_adaptive(rs_lowrank_t h, const double* A, int64_t lda, double eps, int32_t ell_inc,
                                       int32_t q, int32_t inc_policy, int32_t* ell_out, double* est_out,
                                       double* history, int32_t history_len) {
  if (!h) return RS_ERR_INVALID_ARG;
  const Layout& L = h->L;
  if (h->p != 0) return fail(h, RS_ERR_INVALID_ARG, "adaptive sampling needs a handle created with p = 0 (k = l_max)");
  if (ell_inc < 8 || ell_inc % 8 != 0 || ell_inc > L.ell || q < 0 || !(eps >= 0.0))
    return fail(h, RS_ERR_INVALID_ARG, "need l_inc a positive multiple of 8, l_inc <= l_max, q >= 0, eps >= 0");
  if (inc_policy != RS_INC_STATIC && inc_policy != RS_INC_INTERP)
    return fail(h, RS_ERR_INVALID_ARG, "unknown l_inc policy %d", inc_policy);
  if (h->m_local > 0) {
    rs_status_t s = check_matrix(h, A, lda, h->m_local, "A");
    if (s != RS_OK) return s;
  }
  RS_CUDA(h, cudaMemsetAsync(h->info, 0, 16, h->st));
  RS_CUDA(h, cudaMemsetAsync(h->B, 0, static_cast<size_t>(L.lp) * h->n * 8, h->st));
  int rr = ell_inc;
  const long long n = h->n;
  std::vector<std::pair<int, double>> hv;  // (l, eps~) for f(l, l_inc)
  double* Bn = h->Bt;           // new block, rr x n, ld rr
  double* E = h->Rho;           // error block rr x n (Rho is free until pivot)
  double* dscal = h->gaps;      // device scalar for eps~
  rs_status_t s = sample_block(h, A, lda, 0, rr, Bn);  // lines 2-3
  if (s != RS_OK) return s;
  int l = 0, hist = 0;
  double est = -1.0;
  bool converged = false;
  h->robust_iters = 0;
  for (;;) {
    // lines 7-8 (R17) with one shifted CholQR pass; if a block CholQR still breaks down (a block
    // reaching far past the numerical rank, kappa ~ 1/u), redo the round from the saved sample
    // with three shifted passes (R20)
    RS_CUDA(h, copy_2d(h->st, Bn, rr, h->Rhat, rr, rr, n));
    for (int attempt = 0;; ++attempt) {
      const int nshift = attempt == 0 ? 1 : 3;
      if ((s = power_block(h, A, lda, l, rr, q, Bn, nshift)) != RS_OK) return s;   // line 7
      if ((s = borth_qr_small(h, l, Bn, rr, nshift)) != RS_OK) return s;          // line 8
      int info[2] = {0, 0};
      RS_CUDA(h, cudaMemcpyAsync(info, h->info, sizeof(info), cudaMemcpyDeviceToHost, h->st));
      RS_CUDA(h, cudaStreamSynchronize(h->st));
      if (info[0] != RS_ERR_NOT_SPD || attempt == 1) break;
      RS_CUDA(h, cudaMemsetAsync(h->info, 0, 16, h->st));
      RS_CUDA(h, copy_2d(h->st, h->Rhat, rr, Bn, rr, rr, n));
      h->robust_iters++;
    }
    RS_CUDA(h, copy_2d(h->st, Bn, rr, h->B + l, L.lp, rr, n));
    l += rr;                                                                  // line 9
    int inc = next_inc(inc_policy, hv, l, rr, eps);                          // line 11
    if (l + inc > L.ell) {
      if (inc_policy == RS_INC_STATIC) break;
      inc = (L.ell - l) / 8 * 8;
      if (inc < 8) break;
    }
    rr = inc;
    if ((s = sample_block(h, A, lda, l, rr, Bn)) != RS_OK) return s;          // lines 12-13
    // line 15: eps~ = max_i || b_i - b_i B_{1:l}^T B_{1:l} ||  (R18)
    RS_CUDA(h, copy_2d(h->st, Bn, rr, E, rr, rr, n));
    {
      const int splits = gemm_choose_splits(rr, l, n, max_splits_for(h, static_cast<long long>(rr) * l), h->sms);
      const int ns = gemm_nsplit(n, splits);
      Scope sc(h, "borth", 4.0 * rr * l * static_cast<double>(n));
      View2D Xv{Bn, rr, n, rr};
      View2D Ov{h->B, l, n, L.lp};
      GemmOutDesc out{h->part, 1, rr, static_cast<long long>(rr) * l, rr, l};
      RS_CUDA(h, gemm_mc(h->st, rr, l, n, Xv, Ov, out, splits));
      RS_CUDA(h, splitk_reduce(h->st, h->G, h->part, ns, static_cast<long long>(rr) * l,
                               static_cast<long long>(rr) * l));
      RS_CUDA(h, small_gemm(h->st, rr, static_cast<int>(n), l, h->G, 1, rr, h->B, 1, L.lp, E, 1, rr, true, -1.0));
      RS_CUDA(h, rows_maxnorm(h->st, E, rr, rr, n, dscal));
    }
    RS_CUDA(h, cudaMemcpyAsync(&est, dscal, sizeof(double), cudaMemcpyDeviceToHost, h->st));
    RS_CUDA(h, cudaStreamSynchronize(h->st));
    if (history && hist < history_len) {
      history[2 * hist] = l;
      history[2 * hist + 1] = est;
    }
    ++hist;
    hv.emplace_back(l, est);
    if (est <= eps) {                                                         // line 16
      converged = true;
      break;
    }
  }
  rs_status_t st = sync_and_check(h);
  if (st != RS_OK) return st;
  h->ell = l;
  h->k = l;
  h->adaptive = true;
  h->pow_q = 0;
  h->state = ST_SAMPLED;
  h->powers = q;
  if (ell_out) *ell_out = l;
  if (est_out) *est_out = est;
  return converged ? RS_OK : fail(h, RS_ERR_NOT_CONVERGED, "eps~ = %g > eps after l = %d (l_max = %d)", est, l, L.ell);
}

rs_status_t rs_lowrank_run_host(rs_lowrank_t h, const double* A_host, int64_t lda, double* A_dev, int64_t ld_dev,
                                int32_t q, int64_t* perm_host, double* Q_host, int64_t ldq, double* R_host,
                                int64_t ldr, double* Q_dev, int64_t ld_qdev, double* R_dev, int64_t ld_rdev) {
  if (!h || !A_host || lda < h->m_local) return RS_ERR_INVALID_ARG;
  const long long ml = h->m_local, n = h->n;
  if (ml > 0)
    RS_CUDA(h, cudaMemcpy2DAsync(A_dev, ld_dev * 8, A_host, lda * 8, ml * 8, n, cudaMemcpyHostToDevice, h->st));
  rs_status_t s = rs_lowrank_run(h, A_dev, ld_dev, q, nullptr, Q_dev, ld_qdev, R_dev, ld_rdev);
  if (s != RS_OK) return s;
  if (perm_host) RS_CUDA(h, cudaMemcpyAsync(perm_host, h->perm, n * 8, cudaMemcpyDeviceToHost, h->st));
  if (Q_host && ml > 0)
    RS_CUDA(h, cudaMemcpy2DAsync(Q_host, ldq * 8, Q_dev, ld_qdev * 8, ml * 8, h->k, cudaMemcpyDeviceToHost, h->st));
  if (R_host)
    RS_CUDA(h, cudaMemcpy2DAsync(R_host, ldr * 8, R_dev, ld_rdev * 8, static_cast<size_t>(h->k) * 8, n,
                                 cudaMemcpyDeviceToHost, h->st));
  RS_CUDA(h, cudaStreamSynchronize(h->st));
  return RS_OK;
}

rs_status_t rs_lowrank_destroy(rs_lowrank_t h) {
  if (!h) return RS_ERR_INVALID_ARG;
  for (auto& p : h->pending) {
    cudaEventDestroy(p.e0);
    cudaEventDestroy(p.e1);
  }
  release_graph(h);
  if (h->gstream) {
    cudaStreamSynchronize(h->gstream);
    cudaStreamDestroy(h->gstream);
    cudaEventDestroy(h->gev_in);
    cudaEventDestroy(h->gev_out);
  }
  for (auto e : h->event_pool) cudaEventDestroy(e);
  delete h;
  return RS_OK;
}

rs_status_t rs_lowrank_get_sample(rs_lowrank_t h, double* B, int64_t ldb) {
  if (!h || !B || ldb < h->ell) return RS_ERR_INVALID_ARG;
  RS_CUDA(h, cudaMemcpy2DAsync(B, ldb * 8, h->B, h->L.lp * 8, h->ell * 8, h->n, cudaMemcpyDeviceToDevice, h->st));
  RS_CUDA(h, cudaStreamSynchronize(h->st));
  return RS_OK;
}

rs_status_t rs_lowrank_set_sample(rs_lowrank_t h, const double* B, int64_t ldb) {
  if (!h || !B || ldb < h->ell) return RS_ERR_INVALID_ARG;
  // a fixed-rank sample of l = k0 + p rows: undo what an earlier adaptive run set
  h->ell = h->L.ell;
  h->k = h->k0;
  h->adaptive = false;
  h->robust_iters = 0;
  h->pow_q = 0;
  RS_CUDA(h, cudaMemcpy2DAsync(h->B, h->L.lp * 8, B, ldb * 8, h->ell * 8, h->n, cudaMemcpyDeviceToDevice, h->st));
  RS_CUDA(h, cudaMemsetAsync(h->info, 0, 16, h->st));
  h->state = ST_SAMPLED;
  h->powers = 0;
  return RS_OK;
}

rs_status_t rs_lowrank_get_pivot_data(rs_lowrank_t h, double* T, int64_t ldt, double* Rhat, int64_t ldrh,
                                      double* gaps_host) {
  if (!h) return RS_ERR_INVALID_ARG;
  if (h->state < ST_PIVOTED) return fail(h, RS_ERR_BAD_STATE, "no pivot data yet");
  const int k = h->k;
  if (T && h->n > k)
    RS_CUDA(h, cudaMemcpy2DAsync(T, ldt * 8, h->T, h->L.kp * 8, k * 8, h->n - k, cudaMemcpyDeviceToDevice, h->st));
  if (Rhat)
    RS_CUDA(h, cudaMemcpy2DAsync(Rhat, ldrh * 8, h->Rhat, h->L.kp * 8, k * 8, h->n, cudaMemcpyDeviceToDevice, h->st));
  RS_CUDA(h, cudaStreamSynchronize(h->st));
  if (!h->gaps_valid) {  // read lazily: pivot and rs_lowrank_run keep no host copy
    h->gaps_host.assign(k, 0.0);
    RS_CUDA(h, cudaMemcpy(h->gaps_host.data(), h->gaps, static_cast<size_t>(k) * 8, cudaMemcpyDeviceToHost));
    h->gaps_valid = true;
  }
  if (gaps_host) std::copy(h->gaps_host.begin(), h->gaps_host.end(), gaps_host);
  return RS_OK;
}

rs_status_t rs_lowrank_omega(rs_lowrank_t h, int64_t j0, int64_t ncols, double* out, int64_t ldo) {
  if (!h || !out || ldo < h->ell || j0 < 0 || ncols < 0) return RS_ERR_INVALID_ARG;
  RS_CUDA(h, omega_materialize(h->st, h->seed, 0u, h->ell, j0, ncols, out, ldo));
  RS_CUDA(h, cudaStreamSynchronize(h->st));
  return RS_OK;
}

// Column sampling B_c = Omega_c A^T (Fig. 8(b)).  Omega_c (l x n, keyed by the column
// index of A, Philox tag 1) is small -- n << m -- so it is materialised once into B1 and the
// product runs on the MC GEMM family (L = Omega_c M-contiguous, R = A with N = rows contiguous);
// every rank produces the columns of B_c that belong to its own rows of A (no communication).
rs_status_t rs_lowrank_sample_columns(rs_lowrank_t h, const double* A, int64_t lda, double* Bc, int64_t ldb) {
  if (!h) return RS_ERR_INVALID_ARG;
  const Layout& L = h->L;
  const long long ml = h->m_local, n = h->n;
  if (ml > 0) {
    rs_status_t s = check_matrix(h, A, lda, ml, "A");
    if (s != RS_OK) return s;
    if ((s = check_matrix(h, Bc, ldb, h->ell, "B_c")) != RS_OK) return s;
  }
  RS_CUDA(h, cudaMemsetAsync(h->B1, 0, static_cast<size_t>(L.lp) * n * 8, h->st));
  {
    Scope sc(h, "other", 0.0);
    RS_CUDA(h, omega_materialize(h->st, h->seed, 1u, h->ell, 0, n, h->B1, L.lp));
  }
  if (ml > 0) {
    Scope sc(h, "gemm_sample", 2.0 * h->ell * static_cast<double>(ml) * n);
    View2D Ov{h->B1, L.lp, n, L.lp};
    View2D Av{A, ml, n, lda};
    GemmOutDesc out{Bc, 1, ldb, 0, h->ell, static_cast<int>(ml)};
    RS_CUDA(h, gemm_mc(h->st, L.lp, static_cast<int>(ml), n, Ov, Av, out, 1));
  }
  return RS_OK;
}

rs_status_t rs_lowrank_get_info(rs_lowrank_t h, int64_t* info) {
  if (!h || !info) return RS_ERR_INVALID_ARG;
  RS_CUDA(h, cudaStreamSynchronize(h->st));
  int v[2];
  RS_CUDA(h, cudaMemcpy(v, h->info, sizeof(v), cudaMemcpyDeviceToHost));
  info[0] = v[0];
  info[1] = v[1];
  return RS_OK;
}

rs_status_t rs_lowrank_get_fallbacks(rs_lowrank_t h, int32_t* counts) {
  if (!h || !counts) return RS_ERR_INVALID_ARG;
  counts[0] = h->robust_iters;
  counts[1] = h->factor_shifts;
  return RS_OK;
}

rs_status_t rs_lowrank_set_profiling(rs_lowrank_t h, int32_t enable) {
  if (!h) return RS_ERR_INVALID_ARG;
  h->prof = enable != 0;
  return RS_OK;
}

rs_status_t rs_lowrank_get_profile(rs_lowrank_t h, const char* name, double* ms, int64_t* launches, double* flops) {
  if (!h || !name) return RS_ERR_INVALID_ARG;
  drain_profile(h);
  auto it = h->profile.find(name);
  const ProfEntry e = it == h->profile.end() ? ProfEntry{} : it->second;
  if (ms) *ms = e.ms;
  if (launches) *launches = e.launches;
  if (flops) *flops = e.flops;
  return RS_OK;
}

rs_status_t rs_lowrank_reset_profile(rs_lowrank_t h) {
  if (!h) return RS_ERR_INVALID_ARG;
  drain_profile(h);
  h->profile.clear();
  return RS_OK;
}

int64_t rs_lowrank_kernel_launches(void) { return rs::launch_count(); }

rs_status_t rs_lowrank_set_allreduce_hook(rs_lowrank_t h, int32_t nranks, int32_t rank, rs_allreduce_fn fn,
                                          void* ctx) {
  if (!h) return RS_ERR_INVALID_ARG;
  if (h->state != ST_CREATED) return fail(h, RS_ERR_BAD_STATE, "set_allreduce_hook must follow create");
  if (h->comm) return fail(h, RS_ERR_BAD_STATE, "handle already has an NCCL communicator");
  if (nranks < 1 || rank < 0 || rank >= nranks || (nranks > 1 && !fn)) return RS_ERR_INVALID_ARG;
  h->ar_fn = fn;
  h->ar_ctx = ctx;
  h->nranks = nranks;
  h->rank = rank;
  return RS_OK;
}

size_t rs_qp3_workspace_bytes(int64_t m, int64_t n, int32_t k) {
  (void)k;
  return m > 0 && n > 0 ? qp3_workspace_bytes(m, n) : 0;
}

rs_status_t rs_qp3_truncated(int64_t m, int64_t n, int32_t k, double* A, int64_t lda, int64_t* perm, double* tau,
                             double* residual_host, void* workspace, size_t workspace_bytes, void* cuda_stream) {
  if (m < 1 || n < 1 || k < 1 || k > std::min<int64_t>(m, n)) return RS_ERR_INVALID_ARG;
  if (!A || !perm || !tau || !workspace) return RS_ERR_INVALID_ARG;
  if (reinterpret_cast<uintptr_t>(A) % 16 != 0 || lda < m || lda % 2 != 0) return RS_ERR_INVALID_ARG;
  if (workspace_bytes < qp3_workspace_bytes(m, n)) return RS_ERR_WORKSPACE;
  if (reinterpret_cast<uintptr_t>(workspace) % 256 != 0) return RS_ERR_INVALID_ARG;
  cudaStream_t st = static_cast<cudaStream_t>(cuda_stream);
  const cudaError_t e = qp3_truncated_large(st, A, lda, m, n, k, workspace, perm, tau, residual_host != nullptr,
                                            residual_host);
  return e == cudaSuccess ? RS_OK : RS_ERR_CUDA;
}

const char* rs_lowrank_last_error(rs_lowrank_t h) { return h ? h->err.c_str() : "null handle"; }

rs_status_t rs_comm_get_unique_id(char id_out[128]) {
  ncclUniqueId id;
  if (ncclGetUniqueId(&id) != ncclSuccess) return RS_ERR_NCCL;
  static_assert(sizeof(ncclUniqueId) == 128, "ncclUniqueId size");
  std::memcpy(id_out, &id, 128);
  return RS_OK;
}

rs_status_t rs_comm_init(void** comm, int32_t nranks, const char id[128], int32_t rank) {
  if (!comm) return RS_ERR_INVALID_ARG;
  ncclUniqueId uid;
  std::memcpy(&uid, id, 128);
  ncclComm_t c;
  if (ncclCommInitRank(&c, nranks, uid, rank) != ncclSuccess) return RS_ERR_NCCL;
  *comm = c;
  return RS_OK;
}

rs_status_t rs_comm_info(void* comm, int32_t* nranks, int32_t* rank) {
  if (!comm || !nranks || !rank) return RS_ERR_INVALID_ARG;
  int n = 0, r = 0;
  if (ncclCommCount(static_cast<ncclComm_t>(comm), &n) != ncclSuccess ||
      ncclCommUserRank(static_cast<ncclComm_t>(comm), &r) != ncclSuccess)
    return RS_ERR_NCCL;
  *nranks = n;
  *rank = r;
  return RS_OK;
}

rs_status_t rs_comm_destroy(void* comm) {
  if (!comm) return RS_OK;
  return ncclCommDestroy(static_cast<ncclComm_t>(comm)) == ncclSuccess ? RS_OK : RS_ERR_NCCL;
}

}  // extern "C"
