// FP64 tensor-core GEMM tiles for the sampling / power-iteration contractions
// (Fig. 2(a) lines 7 and 12, Fig. 2(b) line 3) and the CholQR Gram products
// (P:L476).  sm_100a has no FP64 tcgen05 (no kind::f64), so the FP64 tensor path is the
// warp-level mma.sync.m8n8k4.f64 -> SASS DMMA.8x8x4 (measured 37.1 TF/s = 99.8 % of
// 148 SM x 64 FMA/clk x 2 x 1.965 GHz, profiles/r01_probe_fp64_peak.jsonl).  Operands are
// streamed by TMA (cp.async.bulk.tensor, 128B swizzle) through an NSTAGE mbarrier ring; 8 MMA
// warps hold the FP64 accumulators in registers, and one elected thread issues the TMA loads
// NSTAGE-1 stages ahead.  (A dedicated producer warp would put 3 warps on one SM sub-partition
// and cap registers at 168/thread, which spills the 56-double accumulator tile.)
//
// Every non-DMMA instruction issued on an SM sub-partition costs DMMA throughput
// (profiles/r01_probe_dmma_interference.jsonl: ~14 % at one extra instruction per DMMA), so the
// fragment loads are 16-byte (LDS.128) and bank-conflict-free by construction:
//
//  KC  "K-contiguous":  Out[MxN] = L[MxK] * R[KxN], R given as a column-major matrix whose
//      columns run along K (A itself for B = Omega A and B = C A); L either generated on the
//      fly (Philox, Omega never touches HBM) or a row-major matrix (rows along K).  A thread
//      loads the K pair (8p+2kk, 8p+2kk+1) of its row and feeds two MMA k-steps with it (any
//      permutation of K inside a tile is exact).  Fragment row r of fragment f in 16-row group g
//      is tile row 16g + 8f + r/2 + 4(r%2), so the two rows of a quarter-warp sit in opposite
//      halves of the 128B swizzle pattern.
//  MC  "M/N-contiguous": L column-major (M contiguous), R stored with N contiguous (A for
//      C = B A^T, C for Linv*C, Q for Q*R^-1).  A thread loads the M (or N) pair (2r, 2r+1) at
//      K row krow = 8(s/2) + 2kk + s%2 and feeds two fragments (even / odd rows) with it.
// Both support split-K (blockIdx.z = split; partial tiles are reduced in a fixed order later).
#pragma once
#include "common.cuh"
#include "philox.cuh"

namespace rs {

constexpr int KT = 16;             // K per pipeline stage (one 128-byte swizzle row of FP64)
constexpr int NT = 128;            // N per CTA
constexpr int NSTAGE = 4;          // TMA ring depth
constexpr int NCONS = 8;           // MMA warps; lane 0 of warp 0 also issues TMA
constexpr int GEMM_THREADS = NCONS * 32;  // 2 warps per SM sub-partition -> up to 255 regs/thread
constexpr int PHX_LD = KT + 8;     // padded Omega tile row (doubles): LDS.128 conflict-free

struct GemmOut {
  double* ptr;
  long long ld_m, ld_n;       // element (m, n) at ptr[m*ld_m + n*ld_n]
  long long split_stride;     // + blockIdx.z * split_stride
  int m_store, n_store;       // store only m < m_store, n < n_store
  int mode;                   // 0: out = acc, 1: out -= acc (block Gram-Schmidt updates)
};

RS_DEVINL void gemm_put(double* p, double v, int mode) {
  if (mode) *p -= v;
  else *p = v;
}

struct GemmArgs {
  int M, N;                   // rows / cols covered by the grid
  long long K;                // total K
  long long k_chunk;          // K per split (multiple of KT)
  GemmOut out;
  // Philox Omega (KC with generated L): Omega[i, row_offset + k] for i < ell, else 0
  PhiloxKey key;
  uint32_t tag;
  long long row_offset;
  long long omega_row0;  // first Omega row of this tile set (adaptive rounds draw rows [l, l + l_inc))
  int ell;               // number of Omega rows generated (rows >= ell of the tile are zero)
  int tri;       // MC: 0 dense, 1 L lower triangular, 2 R upper triangular (zero blocks skipped)
  // KC tail fold (kc_tail_applies): the last N % 128 <= 16 columns [tail_n0, N) get no N tile of
  // their own; the tail_ntn full N tiles of a split share them along K -- tile nt takes the K
  // stages it = nt, nt + tail_ntn, ... -- and write per-CTA partials (MT x 16 each, index
  // (split * mtiles + mtile) * tail_ntn + nt) that kc_tail_reduce sums in a fixed order
  double* tail_p;
  int tail_n0, tail_ntn;
  unsigned long long nmap;  // persistent MC: N box of warp column wn, slot nb = byte 2 wn + nb
  int l3d, r3d;  // MC: operand tensor map is the 3-D stacked-box form (one TMA per stage), see mc_load
};

// KC ring depths (compile-time; -DRS_PHX_NS / -DRS_KC_NS only for ring-depth experiments)
#ifndef RS_PHX_NS
#define RS_PHX_NS 4
#endif
#ifndef RS_KC_NS
#define RS_KC_NS 4
#endif
template <int MFW, bool PHILOX, bool TAIL = false>
struct KCSmem {
  static constexpr int MT = 16 * MFW;
  static constexpr int R_BYTES = NT * KT * 8;
  static constexpr int T_BYTES = TAIL ? 16 * KT * 8 : 0;  // tail-fold stage: 16 columns of A
  static constexpr int ACC_BYTES = TAIL ? 4 * MFW * 32 * 16 : 0;  // tail accumulators (MT x 16 doubles)
  static constexpr int L_BYTES_TMA = MT * KT * 8;
  static constexpr int L_BYTES_RAW = PHILOX ? MT * PHX_LD * 8 : L_BYTES_TMA;
  static constexpr int L_BYTES = (L_BYTES_RAW + 1023) / 1024 * 1024;
  // small M (l <= 32): little MMA work per stage, so a deeper ring keeps more of A in flight and
  // lets several generator groups work on different stages at once
  static constexpr int NS = MFW <= 2 ? 8 : (PHILOX ? RS_PHX_NS : RS_KC_NS);
  static constexpr int TOTAL = 1024 + NS * (R_BYTES + L_BYTES + T_BYTES) + ACC_BYTES + (TAIL ? 3 : 2) * NS * 8;
};

// Align the dynamic shared-memory base to 1024 bytes (128B-swizzle atoms) by pointer arithmetic
// on the __shared__ array itself, so the compiler keeps the shared address space and emits
// LDS.128 (a uintptr round trip would turn every fragment load into a generic LD).
RS_DEVINL unsigned char* align1024(unsigned char* p) {
  return p + ((1024u - (smem_u32(p) & 1023u)) & 1023u);
}

// KC: tile row of fragment row r in fragment f of 16-row group g
RS_DEVINL int kc_row(int g, int f, int r) { return 16 * g + 8 * f + (r >> 1) + 4 * (r & 1); }
// KC: byte offset of the K pair (8p + 2kk, +1) of `row` in a 128B-swizzled K-contiguous tile
RS_DEVINL uint32_t kc_pair_off(int row, int p, int kk) {
  return static_cast<uint32_t>(row) * 128u + ((((4 * p + kk) ^ row) & 7) << 4);
}

// KC accumulate one stage: af(mf, p) / bf(nf, p) return the double2 K pairs.
template <int MFW, typename LA, typename LB>
RS_DEVINL void kc_stage_mma(double (&acc)[MFW][4][2], LA&& la, LB&& lb) {
#pragma unroll
  for (int p = 0; p < 2; ++p) {
    double2 b2[4];
#pragma unroll
    for (int nf = 0; nf < 4; ++nf) b2[nf] = lb(nf, p);
#pragma unroll
    for (int mf = 0; mf < MFW; ++mf) {
      const double2 a2 = la(mf, p);
#pragma unroll
      for (int nf = 0; nf < 4; ++nf) {
        dmma_8x8x4(acc[mf][nf][0], acc[mf][nf][1], a2.x, b2[nf].x);
        dmma_8x8x4(acc[mf][nf][0], acc[mf][nf][1], a2.y, b2[nf].y);
      }
    }
  }
}

// KC epilogue: fragment (mf, nf) element (r, 2kk+e); rowL(mf) gives the tile row of fragment row r
template <int MFW, typename RL>
RS_DEVINL void kc_store(const double (&acc)[MFW][4][2], const GemmOut& ou, int m0, int n0, int wn, int kk,
                        RL&& rowL) {
  double* base = ou.ptr + static_cast<long long>(blockIdx.z) * ou.split_stride;
#pragma unroll
  for (int mf = 0; mf < MFW; ++mf) {
    const long long gm = m0 + rowL(mf);
    if (gm >= ou.m_store) continue;
#pragma unroll
    for (int nf = 0; nf < 4; ++nf) {
      const int ng = wn * 4 + nf;
#pragma unroll
      for (int e = 0; e < 2; ++e) {
        const long long gn = n0 + 16 * (ng >> 1) + 8 * (ng & 1) + kk + 4 * e;
        if (gn < ou.n_store) gemm_put(base + gm * ou.ld_m + gn * ou.ld_n, acc[mf][nf][e], ou.mode);
      }
    }
  }
}

// KC tail fold, run by the three otherwise idle warps of the producer warpgroup (warps 9-11;
// warp 8 lane 0 issues TMA): on the tail stages it = nt, nt + tail_ntn, ... of this CTA (N tile
// nt) they accumulate D[MT x 16] += L[MT x 16 K] T[16 K x 16], T = the stage's tail columns of A,
// and release the stage slot themselves (the producer pre-arrives their 3 arrivals on every other
// stage), so the MMA warps run the plain main loop.  The producer also arrives on tiss[s] when it
// has issued a tail stage into slot s; a tail warp sleeps on it before it waits on full[s].  That
// order matters: an mbarrier parity wait cannot tell phase p from p - 2, and a waiter that skips
// stages could otherwise take the slot's previous, still pending phase for the one it wants --
// once the stage is issued, its slot's previous phase has completed.  Warp t takes the fragments
// q = t, t + 3, ... of the 2 MFW x nj grid (M fragment q / nj, tail n8 block q % nj; nj = 1 when
// the tail is <= 8 columns wide); accumulators in shared memory, one double2 per lane per fragment
// (tail stages are 1 / tail_ntn of the stages).  The CTA's partial goes to tp: element (tile row,
// tail column c) at tp[row * 16 + c] (columns 8..15 only when nj = 2).
template <int MFW, int NS>
RS_DEVINL void kc_tail_warp(int t, int lane, int nt, int nk, int ntn, int nj, const unsigned char* sL, int l_bytes,
                            const unsigned char* sT, double2* acc, uint64_t* full, uint64_t* empty, uint64_t* tiss,
                            double* tp) {
  const int r = lane >> 2, kk = lane & 3;
  const int nq = 2 * MFW * nj;
#pragma unroll 1
  for (int q = t; q < nq; q += 3) acc[q * 32 + lane] = make_double2(0.0, 0.0);
  unsigned tpar = 0;  // per slot: parity of its next tiss phase
#pragma unroll 1
  for (int it = nt; it < nk; it += ntn) {
    const int s = it % NS;
    mbar_wait_sleep(&tiss[s], (tpar >> s) & 1u);
    tpar ^= 1u << s;
    mbar_wait_sleep(&full[s], (it / NS) & 1);
    const unsigned char* Ls = sL + s * l_bytes;
    const unsigned char* Ts = sT + s * (16 * KT * 8);
#pragma unroll 1
    for (int q = t; q < nq; q += 3) {
      const int mg = q / nj, j = q - mg * nj;
      double2 c = acc[q * 32 + lane];
#pragma unroll
      for (int p = 0; p < 2; ++p) {
        const double2 a2 = *reinterpret_cast<const double2*>(Ls + kc_pair_off(kc_row(mg >> 1, mg & 1, r), p, kk));
        const double2 b2 = *reinterpret_cast<const double2*>(Ts + kc_pair_off(kc_row(0, j, r), p, kk));
        dmma_8x8x4(c.x, c.y, a2.x, b2.x);
        dmma_8x8x4(c.x, c.y, a2.y, b2.y);
      }
      acc[q * 32 + lane] = c;
    }
    ring_release_fenced(empty, s, lane);
  }
  // fragment element (r, 2kk + e) of n8 block j: tail column 8j + kk + 4e (kc_row of the B column)
#pragma unroll 1
  for (int q = t; q < nq; q += 3) {
    const int mg = q / nj, j = q - mg * nj;
    const double2 c = acc[q * 32 + lane];
    double* row = tp + kc_row(mg >> 1, mg & 1, r) * 16 + 8 * j + kk;
    row[0] = c.x;
    row[4] = c.y;
  }
}

// ------------------------------------------------------------------------------------------
// KC family, both operands by TMA.  tmR: A-type tensor, dims {K (contiguous), N}, box {16, 128};
// tmL: dims {K (contiguous), M}, box {16, MT}.
// ------------------------------------------------------------------------------------------
template <int MFW>
__global__ void __launch_bounds__(GEMM_THREADS, 1)
    kc_gemm_kernel(const __grid_constant__ CUtensorMap tmR, const __grid_constant__ CUtensorMap tmL,
                   const GemmArgs a) {
  using SM = KCSmem<MFW, false>;
  constexpr int MT = SM::MT;
  extern __shared__ unsigned char smem_raw[];
  unsigned char* smem = align1024(smem_raw);
  unsigned char* sR = smem;
  unsigned char* sL = sR + SM::NS * SM::R_BYTES;
  uint64_t* full = reinterpret_cast<uint64_t*>(sL + SM::NS * SM::L_BYTES);
  uint64_t* empty = full + SM::NS;

  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int n0 = blockIdx.x * NT, m0 = blockIdx.y * MT;
  const long long kb = static_cast<long long>(blockIdx.z) * a.k_chunk;
  const long long ke = min(a.K, kb + a.k_chunk);
  const int nk = kb < ke ? static_cast<int>((ke - kb + KT - 1) / KT) : 0;

  if (threadIdx.x == 0) {
#pragma unroll
    for (int s = 0; s < SM::NS; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], NCONS);
    }
    fence_mbar_init();
  }
  __syncthreads();

  auto issue = [&](int it) {  // one thread: fill stage `it`
    const int s = it % SM::NS;
    if (it >= SM::NS) mbar_wait_sleep(&empty[s], ((it / SM::NS) - 1) & 1);
    mbar_arrive_expect_tx(&full[s], SM::R_BYTES + SM::L_BYTES_TMA);
    const int kc = static_cast<int>(kb + static_cast<long long>(it) * KT);
    tma_load_2d(sR + s * SM::R_BYTES, &tmR, &full[s], kc, n0);
    tma_load_2d(sL + s * SM::L_BYTES, &tmL, &full[s], kc, m0);
  };
  if (threadIdx.x == 0) {
    tma_prefetch_desc(&tmR);
    tma_prefetch_desc(&tmL);
    for (int it = 0; it < SM::NS - 1 && it < nk; ++it) issue(it);
  }

  const int wm = warp >> 2, wn = warp & 3;
  const int r = lane >> 2, kk = lane & 3;
  double acc[MFW][4][2];
#pragma unroll
  for (int mf = 0; mf < MFW; ++mf)
#pragma unroll
    for (int nf = 0; nf < 4; ++nf) acc[mf][nf][0] = acc[mf][nf][1] = 0.0;
  auto rowL = [&](int mf) {
    const int mg = wm * MFW + mf;
    return kc_row(mg >> 1, mg & 1, r);
  };
  auto rowR = [&](int nf) {
    const int ng = wn * 4 + nf;
    return kc_row(ng >> 1, ng & 1, r);
  };

  for (int it = 0; it < nk; ++it) {
    const int s = it % SM::NS;
    mbar_wait(&full[s], (it / SM::NS) & 1);
#ifndef RS_RELEASE_FENCE
    ring_release_prev(empty, it, SM::NS, lane);
#endif
    // refill the slot of stage it - 1 (waits until every warp has released it)
    if (threadIdx.x == 0 && it + SM::NS - 1 < nk) issue(it + SM::NS - 1);
    const unsigned char* Ls = sL + s * SM::L_BYTES;
    const unsigned char* Rs = sR + s * SM::R_BYTES;
    kc_stage_mma<MFW>(
        acc, [&](int mf, int p) { return *reinterpret_cast<const double2*>(Ls + kc_pair_off(rowL(mf), p, kk)); },
        [&](int nf, int p) { return *reinterpret_cast<const double2*>(Rs + kc_pair_off(rowR(nf), p, kk)); });
#ifdef RS_RELEASE_FENCE
    ring_release_fenced(empty, s, lane);
#endif
  }
  kc_store<MFW>(acc, a.out, m0, n0, wn, kk, rowL);
}

// KC with a dedicated producer warpgroup (warps 8-11; one thread issues, setmaxnreg moves their
// registers to the MMA warps): the MMA warps never wait on the ring's "empty" barriers, so no
// MMA warp is coupled to the slowest one at every stage.
constexpr int KCP_THREADS = GEMM_THREADS + 128;
constexpr int MCP_PROD_REGS = 40;
constexpr int MCP_MMA_REGS = 232;  // 4*32*40 + 8*32*232 = 64512 <= 65536
template <int MFW, bool TAIL = false>
__global__ void __launch_bounds__(KCP_THREADS, 1)
    kc_gemm_pwg_kernel(const __grid_constant__ CUtensorMap tmR, const __grid_constant__ CUtensorMap tmL,
                       const __grid_constant__ CUtensorMap tmT, const GemmArgs a) {
  using SM = KCSmem<MFW, false, TAIL>;
  constexpr int MT = SM::MT;
  constexpr int TAILW = TAIL ? 3 : 0;  // tail warps (kc_tail_warp), counted by every slot release
  extern __shared__ unsigned char smem_raw[];
  unsigned char* smem = align1024(smem_raw);
  unsigned char* sR = smem;
  unsigned char* sL = sR + SM::NS * SM::R_BYTES;
  unsigned char* sT = sL + SM::NS * SM::L_BYTES;  // tail-fold stages (TAIL only)
  double2* sAcc = reinterpret_cast<double2*>(sT + SM::NS * SM::T_BYTES);
  uint64_t* full = reinterpret_cast<uint64_t*>(sT + SM::NS * SM::T_BYTES + SM::ACC_BYTES);
  uint64_t* empty = full + SM::NS;
  uint64_t* tiss = empty + SM::NS;  // tail stage issued into slot s (TAIL only)

  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int n0 = blockIdx.x * NT, m0 = blockIdx.y * MT;
  const long long kb = static_cast<long long>(blockIdx.z) * a.k_chunk;
  const long long ke = min(a.K, kb + a.k_chunk);
  const int nk = kb < ke ? static_cast<int>((ke - kb + KT - 1) / KT) : 0;

  if (threadIdx.x == 0) {
#pragma unroll
    for (int s = 0; s < SM::NS; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], NCONS + TAILW);
      if constexpr (TAIL) mbar_init(&tiss[s], 1);
    }
    fence_mbar_init();
  }
  __syncthreads();
  if (warp >= NCONS) {
    asm volatile("setmaxnreg.dec.sync.aligned.u32 %0;\n" ::"n"(MCP_PROD_REGS));
    if (warp == NCONS && lane == 0) {
      tma_prefetch_desc(&tmR);
      tma_prefetch_desc(&tmL);
      if constexpr (TAIL) tma_prefetch_desc(&tmT);
      int nxt = blockIdx.x;  // next tail stage of this N tile
      for (int it = 0; it < nk; ++it) {
        const int s = it % SM::NS;
        if (it >= SM::NS) mbar_wait_sleep(&empty[s], ((it / SM::NS) - 1) & 1);
        const bool tl = TAIL && it == nxt;
        mbar_arrive_expect_tx(&full[s], SM::R_BYTES + SM::L_BYTES_TMA + (tl ? SM::T_BYTES : 0));
        const int kc = static_cast<int>(kb + static_cast<long long>(it) * KT);
        tma_load_2d(sR + s * SM::R_BYTES, &tmR, &full[s], kc, n0);
        tma_load_2d(sL + s * SM::L_BYTES, &tmL, &full[s], kc, m0);
        if constexpr (TAIL) {
          if (tl) {
            tma_load_2d(sT + s * SM::T_BYTES, &tmT, &full[s], kc, a.tail_n0);
            mbar_arrive(&tiss[s]);
            nxt += a.tail_ntn;
          } else {
            mbar_arrive_cnt(&empty[s], TAILW);  // on behalf of the tail warps, which skip this stage
          }
        }
      }
    } else if (TAIL && warp > NCONS) {
      const long long cta = (static_cast<long long>(blockIdx.z) * gridDim.y + blockIdx.y) * gridDim.x + blockIdx.x;
      const int nj = a.N - a.tail_n0 > 8 ? 2 : 1;
      kc_tail_warp<MFW, SM::NS>(warp - NCONS - 1, lane, blockIdx.x, nk, a.tail_ntn, nj, sL, SM::L_BYTES, sT, sAcc,
                                full, empty, tiss, a.tail_p + cta * MT * 16);
    }
    return;
  }
  asm volatile("setmaxnreg.inc.sync.aligned.u32 %0;\n" ::"n"(MCP_MMA_REGS));
  const int wm = warp >> 2, wn = warp & 3;
  const int r = lane >> 2, kk = lane & 3;
  double acc[MFW][4][2];
#pragma unroll
  for (int mf = 0; mf < MFW; ++mf)
#pragma unroll
    for (int nf = 0; nf < 4; ++nf) acc[mf][nf][0] = acc[mf][nf][1] = 0.0;
  auto rowL = [&](int mf) {
    const int mg = wm * MFW + mf;
    return kc_row(mg >> 1, mg & 1, r);
  };
  auto rowR = [&](int nf) {
    const int ng = wn * 4 + nf;
    return kc_row(ng >> 1, ng & 1, r);
  };
  for (int it = 0; it < nk; ++it) {
    const int s = it % SM::NS;
    mbar_wait(&full[s], (it / SM::NS) & 1);
#ifndef RS_RELEASE_FENCE
    ring_release_prev(empty, it, SM::NS, lane);
#endif
    const unsigned char* Ls = sL + s * SM::L_BYTES;
    const unsigned char* Rs = sR + s * SM::R_BYTES;
    kc_stage_mma<MFW>(
        acc, [&](int mf, int p) { return *reinterpret_cast<const double2*>(Ls + kc_pair_off(rowL(mf), p, kk)); },
        [&](int nf, int p) { return *reinterpret_cast<const double2*>(Rs + kc_pair_off(rowR(nf), p, kk)); });
#ifdef RS_RELEASE_FENCE
    ring_release_fenced(empty, s, lane);
#endif
  }
  kc_store<MFW>(acc, a.out, m0, n0, wn, kk, rowL);
}

// ------------------------------------------------------------------------------------------
// KC family with Omega generated in the tile loader, warp-specialised: warpgroup 0 (4 warps,
// one per SM sub-partition) runs Philox + RS-BM32 on the INT/FP32 pipes and issues the TMA
// loads of A; warpgroups 1-2 (8 warps) run the FP64 DMMA tiles.  setmaxnreg moves registers
// from the generator warps to the MMA warps.  Omega never leaves shared memory.
// CS > 1: a thread-block cluster of CS CTAs along N shares one Omega tile; CTA rank c generates
// rows [c*MT/CS, (c+1)*MT/CS) and stores them into every CTA's ring through distributed shared
// memory, so each Omega value is generated once per CS*128 columns of A.
// ------------------------------------------------------------------------------------------
// Two generator warpgroups (2 warps per SM sub-partition): Philox/RS-BM32 is a long dependent
// chain per Omega block, so generation is latency-bound; a second warp per sub-partition hides it.
constexpr int PHX_GEN_WARPS = 8;
constexpr int PHX_THREADS = (PHX_GEN_WARPS + NCONS) * 32;
constexpr int PHX_GEN_REGS = 56;
constexpr int PHX_MMA_REGS = 200;  // 8*32*56 + 8*32*200 = 65536

template <int MFW, int CS>
__global__ void __launch_bounds__(PHX_THREADS, 1)
    kc_philox_kernel(const __grid_constant__ CUtensorMap tmR, const GemmArgs a) {
  using SM = KCSmem<MFW, true>;
  constexpr int MT = SM::MT;
  constexpr int ROWS = MT / CS;
  // Generator groups: a stage needs ROWS*4 Philox blocks, i.e. ceil(ROWS*4/32) warps; the spare
  // warps form further groups that generate other stages concurrently (group g takes stages
  // it = g mod NGRP), since one stage's generation is a latency-bound dependent chain.
  constexpr int GEN_WARPS_NEEDED = (ROWS * 4 + 31) / 32;
  constexpr int NGRP_RAW = PHX_GEN_WARPS / GEN_WARPS_NEEDED;
  constexpr int NGRP = NGRP_RAW < 1 ? 1 : (NGRP_RAW > SM::NS ? SM::NS : NGRP_RAW);
  constexpr int GRP_WARPS = PHX_GEN_WARPS / NGRP;
  extern __shared__ unsigned char smem_raw[];
  unsigned char* smem = align1024(smem_raw);
  unsigned char* sR = smem;
  unsigned char* sL = sR + SM::NS * SM::R_BYTES;
  uint64_t* full = reinterpret_cast<uint64_t*>(sL + SM::NS * SM::L_BYTES);
  uint64_t* empty = full + SM::NS;

  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int n0 = blockIdx.x * NT, m0 = blockIdx.y * MT;
  const long long kb = static_cast<long long>(blockIdx.z) * a.k_chunk;
  const long long ke = min(a.K, kb + a.k_chunk);
  const int nk = kb < ke ? static_cast<int>((ke - kb + KT - 1) / KT) : 0;
  const uint32_t crank = CS > 1 ? cluster_ctarank() : 0;

  if (threadIdx.x == 0) {
#pragma unroll
    for (int s = 0; s < SM::NS; ++s) {
#ifdef RS_PHX_LOCAL_STS
      mbar_init(&full[s], 1 + GRP_WARPS);  // TMA producer + the stage's generator warps (+ peers' tx bytes)
#else
      mbar_init(&full[s], 1);  // the TMA producer's arrive; every Omega byte completes as tx (st.async)
#endif
      mbar_init(&empty[s], NCONS * CS);
    }
    fence_mbar_init();
  }
  if (CS > 1)
    cluster_sync_all();
  else
    __syncthreads();

  if (warp < PHX_GEN_WARPS) {
    // ------------------------- generator / TMA warpgroup -------------------------
    asm volatile("setmaxnreg.dec.sync.aligned.u32 %0;\n" ::"n"(PHX_GEN_REGS));
    // work item w = (row, q): Omega[row, 4q .. 4q+3] of the stage (one Philox block when the
    // row offset is a multiple of 4); items are spread over all 128 generator threads.
    const int grp = warp / GRP_WARPS;
    const int g = threadIdx.x - grp * GRP_WARPS * 32;  // thread index inside the group
    const int o = static_cast<int>(a.row_offset & 3);  // uniform
    constexpr int ITEMS = ROWS * 4;
    if (threadIdx.x == 0) tma_prefetch_desc(&tmR);
    for (int it = grp; it < nk; it += NGRP) {
      const int s = it % SM::NS;
      if (it >= SM::NS) {
        if (lane == 0) mbar_wait_sleep(&empty[s], ((it / SM::NS) - 1) & 1);
        __syncwarp();
      }
      if (g == 0) {
#ifdef RS_PHX_LOCAL_STS
        mbar_arrive_expect_tx(&full[s], SM::R_BYTES + (MT - ROWS) * KT * 8);  // A tile + peers' Omega rows
#else
        mbar_arrive_expect_tx(&full[s], SM::R_BYTES + MT * KT * 8);  // A tile + all Omega rows
#endif
        tma_load_2d(sR + s * SM::R_BYTES, &tmR, &full[s], static_cast<int>(kb + static_cast<long long>(it) * KT), n0);
      }
      const long long j0 = a.row_offset + kb + static_cast<long long>(it) * KT;  // global row of A
      const uint64_t t0 = static_cast<uint64_t>(j0 >> 2);
#pragma unroll 1
      for (int w = g; w < ITEMS; w += GRP_WARPS * 32) {
        const int lrow = static_cast<int>(crank) * ROWS + (w >> 2);
        const int q = w & 3;
        const int gi = m0 + lrow;
        double* dst = reinterpret_cast<double*>(sL + s * SM::L_BYTES) + lrow * PHX_LD + 4 * q;
        double v0 = 0.0, v1 = 0.0, v2 = 0.0, v3 = 0.0;
        if (gi < a.ell) {
          const float4 z = omega_block4f(static_cast<uint32_t>(a.omega_row0 + gi), t0 + q, a.tag, a.key);
          if (o == 0) {
            v0 = z.x, v1 = z.y, v2 = z.z, v3 = z.w;
          } else {
            const float4 z2 = omega_block4f(static_cast<uint32_t>(a.omega_row0 + gi), t0 + q + 1, a.tag, a.key);
            v0 = o + 0 < 4 ? f4_get(z, o + 0) : f4_get(z2, o - 4);
            v1 = o + 1 < 4 ? f4_get(z, o + 1) : f4_get(z2, o - 3);
            v2 = o + 2 < 4 ? f4_get(z, o + 2) : f4_get(z2, o - 2);
            v3 = f4_get(z2, o - 1);
          }
        }
#ifdef RS_PHX_LOCAL_STS
        reinterpret_cast<double2*>(dst)[0] = make_double2(v0, v1);
        reinterpret_cast<double2*>(dst)[1] = make_double2(v2, v3);
#else
        // own ring too by st.async completing tx bytes on full[s]: every Omega byte is counted by
        // the barrier the MMA warps wait on (no generator arrive to order the stores behind)
        st_async_v2(mapa_shared(smem_u32(dst), crank), v0, v1, mapa_shared(smem_u32(&full[s]), crank));
        st_async_v2(mapa_shared(smem_u32(dst), crank) + 16, v2, v3, mapa_shared(smem_u32(&full[s]), crank));
#endif
        if (CS > 1) {  // the same 32 bytes into every peer's ring; completes tx on its full[s]
          const uint32_t sa = smem_u32(dst);
          const uint32_t fb = smem_u32(&full[s]);
#pragma unroll
          for (int pc = 1; pc < CS; ++pc) {
            const uint32_t peer = (crank + pc) % CS;
            const uint32_t ra = mapa_shared(sa, peer);
            const uint32_t rb = mapa_shared(fb, peer);
            st_async_v2(ra, v0, v1, rb);
            st_async_v2(ra + 16, v2, v3, rb);
          }
        }
      }
#ifdef RS_PHX_LOCAL_STS
      __syncwarp();
      if (lane == 0) mbar_arrive(&full[s]);
#endif
    }
  } else {
    // ------------------------- MMA warpgroups -------------------------
    asm volatile("setmaxnreg.inc.sync.aligned.u32 %0;\n" ::"n"(PHX_MMA_REGS));
    const int w = warp - PHX_GEN_WARPS;
    const int wm = w >> 2, wn = w & 3;
    const int r = lane >> 2, kk = lane & 3;
    double acc[MFW][4][2];
#pragma unroll
    for (int mf = 0; mf < MFW; ++mf)
#pragma unroll
      for (int nf = 0; nf < 4; ++nf) acc[mf][nf][0] = acc[mf][nf][1] = 0.0;
    auto rowL = [&](int mf) { return 8 * (wm * MFW + mf) + r; };  // natural rows (padded layout)
    auto rowR = [&](int nf) {
      const int ng = wn * 4 + nf;
      return kc_row(ng >> 1, ng & 1, r);
    };
    for (int it = 0; it < nk; ++it) {
      const int s = it % SM::NS;
      // CTA-scope wait: the slot's data is in this CTA's shared memory (no L1 to invalidate);
      // the remote generators' stores are ordered before their release.cluster arrive
      mbar_wait(&full[s], (it / SM::NS) & 1);
      if (it > 0) {  // deferred release of stage it - 1 (ring_release_prev), here and in the peers
        const int sp = (it - 1) % SM::NS;
        __syncwarp();
        if (lane == 0) {
          mbar_arrive(&empty[sp]);
#pragma unroll
          for (int pc = 1; pc < CS; ++pc)
            mbar_arrive_remote_cta(mapa_shared(smem_u32(&empty[sp]), (crank + pc) % CS));
        }
      }
      const double* Ls = reinterpret_cast<const double*>(sL + s * SM::L_BYTES);
      const unsigned char* Rs = sR + s * SM::R_BYTES;
      kc_stage_mma<MFW>(
          acc,
          [&](int mf, int p) { return *reinterpret_cast<const double2*>(Ls + rowL(mf) * PHX_LD + 8 * p + 2 * kk); },
          [&](int nf, int p) { return *reinterpret_cast<const double2*>(Rs + kc_pair_off(rowR(nf), p, kk)); });
    }
    kc_store<MFW>(acc, a.out, m0, n0, wn, kk, rowL);
  }
  // no CTA may leave while cluster peers can still write its shared memory / barriers
  if (CS > 1) cluster_sync_all();
}

// ------------------------------------------------------------------------------------------
// MC family.  tmL: dims {M (contiguous), K}, box {16, 16};  tmR: dims {N (contiguous), K},
// box {16, 16}.  One 2 KB box per 16 rows of M (or N) per stage.
//  WM = 1: warp w owns N box w (16 columns, two fragments) and all MT rows (2*MFW fragments):
//          per k4 step (MFW + 1) LDS.128 feed 4*MFW DMMAs (small M).
//  WM = 2: warp (wm, wn) owns N boxes 2wn, 2wn+1 (32 columns) and M boxes [wm*BH, (wm+1)*BH),
//          BH = ceil(MFW/2): (BH + 2) LDS.128 feed 8*BH DMMAs -- fewer non-DMMA issue slots per
//          DMMA (profiles/r01_probe_dmma_interference.jsonl).  Warps w and w+4 share an SM
//          sub-partition and hold the two M halves, so the sub-partitions stay balanced for odd MFW.
// a.tri = 1: L is lower triangular (L[m][k] = 0 for k > m): an M box skips the K stages past its
//            last row (the C1 = L^{-1} C apply of CholQR);
// a.tri = 2: R is upper triangular (R[k][n] = 0 for k > n): an N box skips the K stages past its
//            last column (Q1 = X R^{-1}, step 3 of Fig. 2(b)).  Skipped terms are exact zeros.
// Epilogue: the accumulators go through shared memory (the drained ring) so every global store
// is a 16-byte run along the output's contiguous dimension.
// ------------------------------------------------------------------------------------------
#ifndef RS_MC_NS
#define RS_MC_NS 4
#endif
constexpr int MC_NS = RS_MC_NS;  // MC ring depth (-DRS_MC_NS only for ring-depth experiments)
template <int MFW, int WM>
struct MCSmem {
  static constexpr int MT = 16 * MFW;
  static constexpr int R_BYTES = NT * KT * 8;
  static constexpr int L_BYTES = MT * KT * 8;
  static constexpr int RING = MC_NS * (R_BYTES + L_BYTES);
  static constexpr int STAGE_LD = (MT > NT ? MT : NT) + 1;  // staged tile row (doubles; odd: fewer conflicts)
  static constexpr int STAGE = (MT > NT ? MT : NT) * STAGE_LD * 8;  // rows: MT (N-contiguous out) or NT
  static constexpr int BODY = RING > STAGE ? RING : STAGE;
  static constexpr int TOTAL = 1024 + BODY + 2 * MC_NS * 8;
};

// One stage of an MC operand (rows0 = first M or N index of the tile, nbx 16-wide boxes, K offset
// kc).  3-D form (when the contiguous dimension is a multiple of 16): the tensor map is
// {16, K, dim/16} with strides {ld, 16 elements} and box {16, 16, nbx}, so ONE TMA fills the
// nbx boxes in exactly the layout of nbx separate {16, 16} 2-D boxes (box b at b * 2048 bytes,
// 128B swizzle keyed by the K row) -- the issuing thread sits in an MMA warp, and 15 TMA issues
// per stage measurably delayed it.  2-D form otherwise.
RS_DEVINL void mc_load(unsigned char* dst, const CUtensorMap* tm, uint64_t* bar, bool is3d, int rows0, int nbx,
                       int kc) {
  if (is3d) {
    tma_load_3d(dst, tm, bar, 0, kc, rows0 >> 4);
  } else {
#pragma unroll 1
    for (int b = 0; b < nbx; ++b) tma_load_2d(dst + b * 2048, tm, bar, rows0 + 16 * b, kc);
  }
}

// One MC pipeline stage for a warp holding the NFR 8-row M fragments PHI0 .. PHI0+NFR-1 (fragment
// phi = rows 16*(phi/2) + 2r + phi%2 of the tile: box phi/2, parity phi%2) and NB N boxes from
// nbox0.  A box whose two parities both belong to the warp feeds both from one LDS.128; at an odd
// split the middle box serves one parity per warp half.  TRI != 0: warp-uniform skips of
// structurally zero K blocks (see a.tri).  acc[fl][nb][f2][e]: local fragment fl, N box nb,
// N parity f2, element e.
template <int NFR, int PHI0, int NB, int TRI>
RS_DEVINL void mc_stage(double (&acc)[NFR][NB][2][2], const unsigned char* Ls, const unsigned char* Rs, int nbox0,
                        int r, int kk, long long kc, int m0, int n0) {
  constexpr int B0 = PHI0 / 2, B1 = (PHI0 + NFR - 1) / 2;  // boxes touched
  bool nlive[NB];
#pragma unroll
  for (int nb = 0; nb < NB; ++nb) nlive[nb] = TRI != 2 || n0 + 16 * (nbox0 + nb) + 15 >= kc;
  if (TRI == 2) {
    bool any = false;
#pragma unroll
    for (int nb = 0; nb < NB; ++nb) any |= nlive[nb];
    if (!any) return;
  }
#pragma unroll
  for (int ks = 0; ks < KT / 4; ++ks) {
    const uint32_t krow = 8 * (ks >> 1) + 2 * kk + (ks & 1);
    const uint32_t off = krow * 128u + (((static_cast<uint32_t>(r) ^ krow) & 7u) << 4);
    double2 b2[NB];
#pragma unroll
    for (int nb = 0; nb < NB; ++nb) b2[nb] = *reinterpret_cast<const double2*>(Rs + (nbox0 + nb) * 2048 + off);
#pragma unroll
    for (int b = B0; b <= B1; ++b) {
      if (TRI == 1 && m0 + 16 * b + 15 < kc) continue;
      const double2 a2 = *reinterpret_cast<const double2*>(Ls + b * 2048 + off);
#pragma unroll
      for (int f = 0; f < 2; ++f) {
        const int fl = 2 * b + f - PHI0;
        if (fl < 0 || fl >= NFR) continue;
        const double av = f == 0 ? a2.x : a2.y;
#pragma unroll
        for (int nb = 0; nb < NB; ++nb) {
          if (TRI == 2 && !nlive[nb]) continue;
          dmma_8x8x4(acc[fl][nb][0][0], acc[fl][nb][0][1], av, b2[nb].x);
          dmma_8x8x4(acc[fl][nb][1][0], acc[fl][nb][1][1], av, b2[nb].y);
        }
      }
    }
  }
}

template <int MFW, int WM, int TRI>
__global__ void __launch_bounds__(GEMM_THREADS, 1)
    mc_gemm_kernel(const __grid_constant__ CUtensorMap tmL, const __grid_constant__ CUtensorMap tmR,
                   const GemmArgs a) {
  using SM = MCSmem<MFW, WM>;
  constexpr int MT = SM::MT;
  constexpr int NFR = WM == 1 ? 2 * MFW : MFW;  // 8-row M fragments per warp
  constexpr int NB = WM == 1 ? 1 : 2;            // N boxes per warp
  extern __shared__ unsigned char smem_raw[];
  unsigned char* smem = align1024(smem_raw);
  unsigned char* sR = smem;
  unsigned char* sL = sR + MC_NS * SM::R_BYTES;
  uint64_t* full = reinterpret_cast<uint64_t*>(smem + SM::BODY);
  uint64_t* empty = full + MC_NS;

  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int n0 = blockIdx.x * NT, m0 = blockIdx.y * MT;
  const long long kb = static_cast<long long>(blockIdx.z) * a.k_chunk;
  const long long ke = min(a.K, kb + a.k_chunk);
  const int nk = kb < ke ? static_cast<int>((ke - kb + KT - 1) / KT) : 0;

  if (threadIdx.x == 0) {
#pragma unroll
    for (int s = 0; s < MC_NS; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], NCONS);
    }
    fence_mbar_init();
  }
  __syncthreads();

  auto issue = [&](int it) {
    const int s = it % MC_NS;
    if (it >= MC_NS) mbar_wait_sleep(&empty[s], ((it / MC_NS) - 1) & 1);
    mbar_arrive_expect_tx(&full[s], SM::R_BYTES + SM::L_BYTES);
    const int kc = static_cast<int>(kb + static_cast<long long>(it) * KT);
    mc_load(sL + s * SM::L_BYTES, &tmL, &full[s], a.l3d, m0, MT / 16, kc);
    mc_load(sR + s * SM::R_BYTES, &tmR, &full[s], a.r3d, n0, NT / 16, kc);
  };
  if (threadIdx.x == 0) {
    tma_prefetch_desc(&tmL);
    tma_prefetch_desc(&tmR);
    for (int it = 0; it < MC_NS - 1 && it < nk; ++it) issue(it);
  }

  const int r = lane >> 2, kk = lane & 3;
  const int wm = WM == 1 ? 0 : warp >> 2;
  const int nbox0 = WM == 1 ? warp : 2 * (warp & 3);  // first N box of this warp
  const int phi0 = wm * NFR;                          // first M fragment of this warp
  double acc[NFR][NB][2][2];
#pragma unroll
  for (int fl = 0; fl < NFR; ++fl)
#pragma unroll
    for (int nb = 0; nb < NB; ++nb)
#pragma unroll
      for (int f2 = 0; f2 < 2; ++f2) acc[fl][nb][f2][0] = acc[fl][nb][f2][1] = 0.0;

  for (int it = 0; it < nk; ++it) {
    const int s = it % MC_NS;
    mbar_wait(&full[s], (it / MC_NS) & 1);
    ring_release_prev(empty, it, MC_NS, lane);
    if (threadIdx.x == 0 && it + MC_NS - 1 < nk) issue(it + MC_NS - 1);
    const long long kc = kb + static_cast<long long>(it) * KT;  // first K of the stage
    const unsigned char* Ls = sL + s * SM::L_BYTES;
    const unsigned char* Rs = sR + s * SM::R_BYTES;
    // compile-time fragment sets: the dense path has no per-box branches
    if (WM == 1 || wm == 0)
      mc_stage<NFR, 0, NB, TRI>(acc, Ls, Rs, nbox0, r, kk, kc, m0, n0);
    else
      mc_stage<NFR, NFR, NB, TRI>(acc, Ls, Rs, nbox0, r, kk, kc, m0, n0);
  }

  // ---- epilogue: stage the MT x NT tile in shared memory, then coalesced 16-byte stores ----
  const GemmOut& o = a.out;
  double* base = o.ptr + static_cast<long long>(blockIdx.z) * o.split_stride;
  const bool n_contig = o.ld_n == 1, m_contig = o.ld_m == 1;
  if (!n_contig && !m_contig) {  // generic strides: direct stores
#pragma unroll
    for (int fl = 0; fl < NFR; ++fl) {
      const int phi = phi0 + fl;
      const long long gm = m0 + 16 * (phi >> 1) + 2 * r + (phi & 1);
      if (gm >= o.m_store) continue;
#pragma unroll
      for (int nb = 0; nb < NB; ++nb)
#pragma unroll
        for (int f2 = 0; f2 < 2; ++f2)
#pragma unroll
          for (int e = 0; e < 2; ++e) {
            const long long gn = n0 + 16 * (nbox0 + nb) + 2 * (2 * kk + e) + f2;
            if (gn < o.n_store) gemm_put(base + gm * o.ld_m + gn * o.ld_n, acc[fl][nb][f2][e], o.mode);
          }
    }
    return;
  }
  __syncthreads();  // every warp is done with the ring
  double* st = reinterpret_cast<double*>(smem);
  // n_contig: st[m * LDS + n] (rows along N); else st[n * LDS + m] (rows along M)
  constexpr int LDS = SM::STAGE_LD;
#pragma unroll
  for (int fl = 0; fl < NFR; ++fl) {
    const int phi = phi0 + fl;
    const int lm = 16 * (phi >> 1) + 2 * r + (phi & 1);
#pragma unroll
    for (int nb = 0; nb < NB; ++nb)
#pragma unroll
      for (int f2 = 0; f2 < 2; ++f2)
#pragma unroll
        for (int e = 0; e < 2; ++e) {
          const int ln = 16 * (nbox0 + nb) + 2 * (2 * kk + e) + f2;
          st[n_contig ? lm * LDS + ln : ln * LDS + lm] = acc[fl][nb][f2][e];
        }
  }
  __syncthreads();
  // rows of the staged tile: n_contig -> MT rows of NT; else NT rows of MT
  const int nrows = n_contig ? MT : NT, rowlen = n_contig ? NT : MT;
  const long long row0 = n_contig ? m0 : n0, col0 = n_contig ? n0 : m0;
  const long long row_lim = n_contig ? o.m_store : o.n_store, col_lim = n_contig ? o.n_store : o.m_store;
  const long long ld_row = n_contig ? o.ld_m : o.ld_n;
  const int pairs = rowlen / 2;
  for (int idx = threadIdx.x; idx < nrows * pairs; idx += GEMM_THREADS) {
    const int lr = idx / pairs, lc = 2 * (idx - lr * pairs);
    const long long gr = row0 + lr, gc = col0 + lc;
    if (gr >= row_lim || gc >= col_lim) continue;
    double* p = base + gr * ld_row + gc;
    const double v0 = st[lr * LDS + lc], v1 = st[lr * LDS + lc + 1];
    if (gc + 1 < col_lim && (reinterpret_cast<uintptr_t>(p) & 15) == 0) {
      double2* p2 = reinterpret_cast<double2*>(p);
      if (o.mode) {
        double2 c = *p2;
        c.x -= v0;
        c.y -= v1;
        *p2 = c;
      } else {
        *p2 = make_double2(v0, v1);
      }
    } else {
      gemm_put(p, v0, o.mode);
      if (gc + 1 < col_lim) gemm_put(p + 1, v1, o.mode);
    }
  }
}

// MC with a dedicated producer warpgroup (warps 8-11, as kc_gemm_pwg_kernel): the MMA warps never
// carry the TMA issue; the epilogue synchronises the 8 MMA warps with a named barrier.
template <int MFW, int WM, int TRI>
__global__ void __launch_bounds__(KCP_THREADS, 1)
    mc_gemm_pwg_kernel(const __grid_constant__ CUtensorMap tmL, const __grid_constant__ CUtensorMap tmR,
                   const GemmArgs a) {
  using SM = MCSmem<MFW, WM>;
  constexpr int MT = SM::MT;
  constexpr int NFR = WM == 1 ? 2 * MFW : MFW;  // 8-row M fragments per warp
  constexpr int NB = WM == 1 ? 1 : 2;            // N boxes per warp
  extern __shared__ unsigned char smem_raw[];
  unsigned char* smem = align1024(smem_raw);
  unsigned char* sR = smem;
  unsigned char* sL = sR + MC_NS * SM::R_BYTES;
  uint64_t* full = reinterpret_cast<uint64_t*>(smem + SM::BODY);
  uint64_t* empty = full + MC_NS;

  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int n0 = blockIdx.x * NT, m0 = blockIdx.y * MT;
  const long long kb = static_cast<long long>(blockIdx.z) * a.k_chunk;
  const long long ke = min(a.K, kb + a.k_chunk);
  const int nk = kb < ke ? static_cast<int>((ke - kb + KT - 1) / KT) : 0;

  if (threadIdx.x == 0) {
#pragma unroll
    for (int s = 0; s < MC_NS; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], NCONS);
    }
    fence_mbar_init();
  }
  __syncthreads();

  auto issue = [&](int it) {
    const int s = it % MC_NS;
    if (it >= MC_NS) mbar_wait_sleep(&empty[s], ((it / MC_NS) - 1) & 1);
    mbar_arrive_expect_tx(&full[s], SM::R_BYTES + SM::L_BYTES);
    const int kc = static_cast<int>(kb + static_cast<long long>(it) * KT);
    mc_load(sL + s * SM::L_BYTES, &tmL, &full[s], a.l3d, m0, MT / 16, kc);
    mc_load(sR + s * SM::R_BYTES, &tmR, &full[s], a.r3d, n0, NT / 16, kc);
  };
  if (warp >= NCONS) {
    asm volatile("setmaxnreg.dec.sync.aligned.u32 %0;\n" ::"n"(MCP_PROD_REGS));
    if (warp == NCONS && lane == 0) {
      tma_prefetch_desc(&tmL);
      tma_prefetch_desc(&tmR);
      for (int it = 0; it < nk; ++it) issue(it);
    }
    return;
  }
  asm volatile("setmaxnreg.inc.sync.aligned.u32 %0;\n" ::"n"(MCP_MMA_REGS));

  const int r = lane >> 2, kk = lane & 3;
  const int wm = WM == 1 ? 0 : warp >> 2;
  const int nbox0 = WM == 1 ? warp : 2 * (warp & 3);  // first N box of this warp
  const int phi0 = wm * NFR;                          // first M fragment of this warp
  double acc[NFR][NB][2][2];
#pragma unroll
  for (int fl = 0; fl < NFR; ++fl)
#pragma unroll
    for (int nb = 0; nb < NB; ++nb)
#pragma unroll
      for (int f2 = 0; f2 < 2; ++f2) acc[fl][nb][f2][0] = acc[fl][nb][f2][1] = 0.0;

  for (int it = 0; it < nk; ++it) {
    const int s = it % MC_NS;
    mbar_wait(&full[s], (it / MC_NS) & 1);
#ifdef RS_MC_RELEASE_DEFERRED
    ring_release_prev(empty, it, MC_NS, lane);
#endif
    const long long kc = kb + static_cast<long long>(it) * KT;  // first K of the stage
    const unsigned char* Ls = sL + s * SM::L_BYTES;
    const unsigned char* Rs = sR + s * SM::R_BYTES;
    // compile-time fragment sets: the dense path has no per-box branches
    if (WM == 1 || wm == 0)
      mc_stage<NFR, 0, NB, TRI>(acc, Ls, Rs, nbox0, r, kk, kc, m0, n0);
    else
      mc_stage<NFR, NFR, NB, TRI>(acc, Ls, Rs, nbox0, r, kk, kc, m0, n0);
#ifndef RS_MC_RELEASE_DEFERRED
    // released at the end of its own stage behind a CTA fence (measured at cfg4: 30.83 ms against
    // 31.72 ms with the one-stage-deferred release on the same box; both pass the overlap stress)
    ring_release_fenced(empty, s, lane);
#endif
  }

  // ---- epilogue: stage the MT x NT tile in shared memory, then coalesced 16-byte stores ----
  const GemmOut& o = a.out;
  double* base = o.ptr + static_cast<long long>(blockIdx.z) * o.split_stride;
  const bool n_contig = o.ld_n == 1, m_contig = o.ld_m == 1;
  if (!n_contig && !m_contig) {  // generic strides: direct stores
#pragma unroll
    for (int fl = 0; fl < NFR; ++fl) {
      const int phi = phi0 + fl;
      const long long gm = m0 + 16 * (phi >> 1) + 2 * r + (phi & 1);
      if (gm >= o.m_store) continue;
#pragma unroll
      for (int nb = 0; nb < NB; ++nb)
#pragma unroll
        for (int f2 = 0; f2 < 2; ++f2)
#pragma unroll
          for (int e = 0; e < 2; ++e) {
            const long long gn = n0 + 16 * (nbox0 + nb) + 2 * (2 * kk + e) + f2;
            if (gn < o.n_store) gemm_put(base + gm * o.ld_m + gn * o.ld_n, acc[fl][nb][f2][e], o.mode);
          }
    }
    return;
  }
  named_bar_sync(1, GEMM_THREADS);  // every MMA warp is done with the ring
  double* st = reinterpret_cast<double*>(smem);
  // n_contig: st[m * LDS + n] (rows along N); else st[n * LDS + m] (rows along M)
  constexpr int LDS = SM::STAGE_LD;
#pragma unroll
  for (int fl = 0; fl < NFR; ++fl) {
    const int phi = phi0 + fl;
    const int lm = 16 * (phi >> 1) + 2 * r + (phi & 1);
#pragma unroll
    for (int nb = 0; nb < NB; ++nb)
#pragma unroll
      for (int f2 = 0; f2 < 2; ++f2)
#pragma unroll
        for (int e = 0; e < 2; ++e) {
          const int ln = 16 * (nbox0 + nb) + 2 * (2 * kk + e) + f2;
          st[n_contig ? lm * LDS + ln : ln * LDS + lm] = acc[fl][nb][f2][e];
        }
  }
  named_bar_sync(1, GEMM_THREADS);
  // rows of the staged tile: n_contig -> MT rows of NT; else NT rows of MT
  const int nrows = n_contig ? MT : NT, rowlen = n_contig ? NT : MT;
  const long long row0 = n_contig ? m0 : n0, col0 = n_contig ? n0 : m0;
  const long long row_lim = n_contig ? o.m_store : o.n_store, col_lim = n_contig ? o.n_store : o.m_store;
  const long long ld_row = n_contig ? o.ld_m : o.ld_n;
  const int pairs = rowlen / 2;
  for (int idx = threadIdx.x; idx < nrows * pairs; idx += GEMM_THREADS) {
    const int lr = idx / pairs, lc = 2 * (idx - lr * pairs);
    const long long gr = row0 + lr, gc = col0 + lc;
    if (gr >= row_lim || gc >= col_lim) continue;
    double* p = base + gr * ld_row + gc;
    const double v0 = st[lr * LDS + lc], v1 = st[lr * LDS + lc + 1];
    if (gc + 1 < col_lim && (reinterpret_cast<uintptr_t>(p) & 15) == 0) {
      double2* p2 = reinterpret_cast<double2*>(p);
      if (o.mode) {
        double2 c = *p2;
        c.x -= v0;
        c.y -= v1;
        *p2 = c;
      } else {
        *p2 = make_double2(v0, v1);
      }
    } else {
      gemm_put(p, v0, o.mode);
      if (gc + 1 < col_lim) gemm_put(p + 1, v1, o.mode);
    }
  }
}

// ------------------------------------------------------------------------------------------
// Persistent MC for the short-K products (K <= 128: C1 = L^{-1} C, Q1 = X R^{-1}): a CTA has
// only ceil(K/16) stages of work per tile, so one tile per CTA leaves the TMA round trip and the
// epilogue exposed.  Here each CTA walks tiles blockIdx.x, + gridDim.x, ...; the TMA thread keeps
// issuing the next tile's stages into the same ring while the warps finish and store the current
// one.  Epilogue: direct 16-byte stores of the fragment pairs adjacent along the contiguous output
// dimension (rows 2r, 2r+1 for M-contiguous, columns 2(2kk+e), +1 for N-contiguous).
// ------------------------------------------------------------------------------------------
// Short-K persistent layout: the operand shared by every tile (L when there is one M tile, R when
// there is one N tile) is loaded ONCE into a resident region (all K stages, <= 8 x 16 KB); only the
// other operand streams through a MCP_NS-deep ring, so twice the bytes are in flight per SM for
// the same shared memory and each stage needs 8 instead of 16 TMA boxes.
constexpr int MCP_NS = 6;
template <int MFW>
struct MCPSmem {
  static constexpr int MT = 16 * MFW;
  static constexpr int R_BYTES = NT * KT * 8;   // one K stage of R
  static constexpr int L_BYTES = MT * KT * 8;   // one K stage of L
  static constexpr int RES = 8 * (R_BYTES > L_BYTES ? R_BYTES : L_BYTES);  // resident operand, K <= 128
  static constexpr int SLOT = R_BYTES > L_BYTES ? R_BYTES : L_BYTES;
  static constexpr int RING = MCP_NS * SLOT;
  static constexpr int TOTAL = 1024 + RES + RING + (2 * MCP_NS + 1) * 8;
};

RS_DEVINL void put2(double* p, double v0, double v1, bool ok1, int mode) {
  if (ok1 && (reinterpret_cast<uintptr_t>(p) & 15) == 0) {
    double2* p2 = reinterpret_cast<double2*>(p);
    if (mode) {
      double2 c = *p2;
      c.x -= v0;
      c.y -= v1;
      *p2 = c;
    } else {
      *p2 = make_double2(v0, v1);
    }
  } else {
    gemm_put(p, v0, mode);
    if (ok1) gemm_put(p + 1, v1, mode);
  }
}

// Fragment sets of the two warp halves (wm = 0, 1) of the persistent 2 x 4 grid, as bit masks
// over the 8-row M fragments phi = 2 * box + parity.  Dense / N-triangular products: contiguous
// halves (the middle box split by parity at odd MFW).  M-triangular products (TRI == 1, box b is
// live in stages 0..b): whole boxes, greedily balanced so both halves carry the same number of
// live box-stages (MFW = 7: boxes {6, 3, 2} and {5, 4, 1, 0}, 14 each) -- with contiguous halves
// one half would carry 40 of 56 fragment-stages and the ring would advance at its pace.
template <int MFW, int TRI>
struct McpFrag {
  __host__ __device__ static constexpr unsigned mask(int wm) {
    if (TRI != 1) {
      unsigned m = 0;
      for (int phi = wm * MFW; phi < (wm + 1) * MFW; ++phi) m |= 1u << phi;
      return m;
    }
    unsigned m0 = 0, m1 = 0;
    int w0 = 0, w1 = 0;
    for (int bx = MFW - 1; bx >= 0; --bx) {
      if (w0 <= w1) {
        m0 |= 3u << (2 * bx);
        w0 += bx + 1;
      } else {
        m1 |= 3u << (2 * bx);
        w1 += bx + 1;
      }
    }
    return wm == 0 ? m0 : m1;
  }
  __host__ __device__ static constexpr int count(unsigned m) {
    int c = 0;
    for (int i = 0; i < 32; ++i) c += (m >> i) & 1u;
    return c;
  }
  __host__ __device__ static constexpr int nfr() {
    return count(mask(0)) > count(mask(1)) ? count(mask(0)) : count(mask(1));
  }
  // local accumulator slot of fragment phi in mask m
  __host__ __device__ static constexpr int slot(unsigned m, int phi) { return count(m & ((1u << phi) - 1u)); }
};

// One stage of the persistent MC kernel for a warp with compile-time fragment mask FM and the
// two N boxes nbx[0..1] (runtime; dead boxes -- past N or triangular-zero -- are skipped).
template <int MFW, int TRI, unsigned FM, int NFR>
RS_DEVINL void mcp_stage(double (&acc)[NFR][2][2][2], const unsigned char* Ls, const unsigned char* Rs,
                         const int (&nbx)[2], const bool (&nl)[2], int r, int kk, long long kc, int m0) {
  using F = McpFrag<MFW, TRI>;
#pragma unroll
  for (int ks = 0; ks < KT / 4; ++ks) {
    const uint32_t krow = 8 * (ks >> 1) + 2 * kk + (ks & 1);
    const uint32_t off = krow * 128u + (((static_cast<uint32_t>(r) ^ krow) & 7u) << 4);
    double2 b2[2];
#pragma unroll
    for (int nb = 0; nb < 2; ++nb)
      b2[nb] = nl[nb] ? *reinterpret_cast<const double2*>(Rs + nbx[nb] * 2048 + off) : make_double2(0.0, 0.0);
#pragma unroll
    for (int bx = 0; bx < MFW; ++bx) {
      if (((FM >> (2 * bx)) & 3u) == 0) continue;
      if (TRI == 1 && m0 + 16 * bx + 15 < kc) continue;
      const double2 a2 = *reinterpret_cast<const double2*>(Ls + bx * 2048 + off);
#pragma unroll
      for (int f = 0; f < 2; ++f) {
        if (((FM >> (2 * bx + f)) & 1u) == 0) continue;
        const int fl = F::slot(FM, 2 * bx + f);
        const double av = f == 0 ? a2.x : a2.y;
#pragma unroll
        for (int nb = 0; nb < 2; ++nb) {
          if (!nl[nb]) continue;
          dmma_8x8x4(acc[fl][nb][0][0], acc[fl][nb][0][1], av, b2[nb].x);
          dmma_8x8x4(acc[fl][nb][1][0], acc[fl][nb][1][1], av, b2[nb].y);
        }
      }
    }
  }
}

template <int MFW, int TRI, unsigned FM, int NFR>
RS_DEVINL void mcp_store(const double (&acc)[NFR][2][2][2], const GemmOut& o, const int (&nbx)[2], int r, int kk,
                         int m0, int n0) {
  using F = McpFrag<MFW, TRI>;
#pragma unroll
  for (int phi = 0; phi < 2 * MFW; ++phi) {
    if (((FM >> phi) & 1u) == 0) continue;
    const int fl = F::slot(FM, phi);
    const bool pair_m = (phi & 1) == 0 && ((FM >> (phi + 1)) & 1u);  // rows 2r, 2r+1 both here
    if ((phi & 1) == 1 && ((FM >> (phi - 1)) & 1u) && o.ld_m == 1) continue;  // stored with phi - 1
    const long long gm = m0 + 16 * (phi >> 1) + 2 * r + (phi & 1);
#pragma unroll
    for (int nb = 0; nb < 2; ++nb)
#pragma unroll
      for (int e = 0; e < 2; ++e) {
        const long long gn0 = n0 + 16 * nbx[nb] + 2 * (2 * kk + e);  // cols gn0 (f2 = 0), gn0 + 1
        if (o.ld_m == 1 && pair_m) {
#pragma unroll
          for (int f2 = 0; f2 < 2; ++f2) {
            const long long gn = gn0 + f2;
            if (gn >= o.n_store || gm >= o.m_store) continue;
            put2(o.ptr + gm + gn * o.ld_n, acc[fl][nb][f2][e], acc[fl + 1][nb][f2][e], gm + 1 < o.m_store, o.mode);
          }
        } else if (o.ld_n == 1) {
          if (gm < o.m_store && gn0 < o.n_store)
            put2(o.ptr + gm * o.ld_m + gn0, acc[fl][nb][0][e], acc[fl][nb][1][e], gn0 + 1 < o.n_store, o.mode);
        } else {
#pragma unroll
          for (int f2 = 0; f2 < 2; ++f2) {
            const long long gn = gn0 + f2;
            if (gm < o.m_store && gn < o.n_store)
              gemm_put(o.ptr + gm * o.ld_m + gn * o.ld_n, acc[fl][nb][f2][e], o.mode);
          }
        }
      }
  }
}

// byte 2 wn + nb of a.nmap: the N box of warp column wn (identity, or balanced pairs for TRI == 2).
// byte 2 wn + nb of a.nmap: the N box of warp column wn (identity, or balanced pairs for TRI == 2).
// res_l = 1: L (one M tile) is the resident operand and tiles walk N; res_l = 0: R (one N tile) is
// resident and tiles walk M.
template <int MFW, int TRI>
__global__ void __launch_bounds__(GEMM_THREADS, 1)
    mc_persist_kernel(const __grid_constant__ CUtensorMap tmL, const __grid_constant__ CUtensorMap tmR,
                      const GemmArgs a, int ntn, int ntiles, int res_l) {
  using SM = MCPSmem<MFW>;
  using F = McpFrag<MFW, TRI>;
  constexpr int MT = SM::MT;
  constexpr unsigned FM0 = F::mask(0), FM1 = F::mask(1);
  constexpr int NFR = F::nfr();
  extern __shared__ unsigned char smem_raw[];
  unsigned char* smem = align1024(smem_raw);
  unsigned char* sRes = smem;                 // resident operand, stage it at it * (its stage bytes)
  unsigned char* sRing = smem + SM::RES;      // streamed operand
  uint64_t* full = reinterpret_cast<uint64_t*>(sRing + SM::RING);
  uint64_t* empty = full + MCP_NS;
  uint64_t* resb = empty + MCP_NS;
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int nk = static_cast<int>((a.K + KT - 1) / KT);
  const int mytiles = blockIdx.x < ntiles ? (ntiles - blockIdx.x + gridDim.x - 1) / gridDim.x : 0;
  const int total = mytiles * nk;
  const int res_bytes = res_l ? SM::L_BYTES : SM::R_BYTES;   // per stage
  const int str_bytes = res_l ? SM::R_BYTES : SM::L_BYTES;
  const int str_boxes = res_l ? NT / 16 : MT / 16;

  if (threadIdx.x == 0) {
#pragma unroll
    for (int s = 0; s < MCP_NS; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], NCONS);
    }
    mbar_init(resb, 1);
    fence_mbar_init();
  }
  __syncthreads();
  auto tile_of = [&](int i, int& m0, int& n0) {
    const int T = blockIdx.x + i * gridDim.x;
    n0 = (T % ntn) * NT;
    m0 = (T / ntn) * MT;
  };
  auto issue = [&](int g) {
    const int s = g % MCP_NS;
    if (g >= MCP_NS) mbar_wait_sleep(&empty[s], ((g / MCP_NS) - 1) & 1);
    int m0, n0;
    tile_of(g / nk, m0, n0);
    const int kc = (g % nk) * KT;
    mbar_arrive_expect_tx(&full[s], str_bytes);
    unsigned char* dst = sRing + s * SM::SLOT;
    if (res_l)
      mc_load(dst, &tmR, &full[s], a.r3d, n0, str_boxes, kc);
    else
      mc_load(dst, &tmL, &full[s], a.l3d, m0, str_boxes, kc);
  };
  if (threadIdx.x == 0) {
    tma_prefetch_desc(&tmL);
    tma_prefetch_desc(&tmR);
    // the resident operand: all nk stages, one barrier
    mbar_arrive_expect_tx(resb, static_cast<uint32_t>(res_bytes * nk));
    const int rboxes = res_l ? MT / 16 : NT / 16;
#pragma unroll 1
    for (int it = 0; it < nk; ++it) {
      if (res_l)
        mc_load(sRes + it * res_bytes, &tmL, resb, a.l3d, 0, rboxes, it * KT);
      else
        mc_load(sRes + it * res_bytes, &tmR, resb, a.r3d, 0, rboxes, it * KT);
    }
    for (int g = 0; g < MCP_NS - 1 && g < total; ++g) issue(g);
  }
  mbar_wait(resb, 0);
  const int r = lane >> 2, kk = lane & 3;
  const int wm = warp >> 2, wn = warp & 3;  // (measured: wm = warp & 1, one code path per sub-partition, is slower)
  const int nbx[2] = {static_cast<int>((a.nmap >> (16 * wn)) & 0xffu), static_cast<int>((a.nmap >> (16 * wn + 8)) & 0xffu)};
  const GemmOut& o = a.out;
  for (int i = 0; i < mytiles; ++i) {
    int m0, n0;
    tile_of(i, m0, n0);
    double acc[NFR][2][2][2];
#pragma unroll
    for (int fl = 0; fl < NFR; ++fl)
#pragma unroll
      for (int nb = 0; nb < 2; ++nb)
#pragma unroll
        for (int f2 = 0; f2 < 2; ++f2) acc[fl][nb][f2][0] = acc[fl][nb][f2][1] = 0.0;
    for (int it = 0; it < nk; ++it) {
      const int g = i * nk + it;
      const int s = g % MCP_NS;
      mbar_wait(&full[s], (g / MCP_NS) & 1);
      ring_release_prev(empty, g, MCP_NS, lane);  // the ring runs on across tiles
      if (threadIdx.x == 0 && g + MCP_NS - 1 < total) issue(g + MCP_NS - 1);
      const long long kc = static_cast<long long>(it) * KT;
      bool nl[2];
#pragma unroll
      for (int nb = 0; nb < 2; ++nb)
        nl[nb] = n0 + 16 * nbx[nb] < a.N && (TRI != 2 || n0 + 16 * nbx[nb] + 15 >= kc);
      if (nl[0] || nl[1]) {
        const unsigned char* Ls = res_l ? sRes + it * SM::L_BYTES : sRing + s * SM::SLOT;
        const unsigned char* Rs = res_l ? sRing + s * SM::SLOT : sRes + it * SM::R_BYTES;
        if (wm == 0)
          mcp_stage<MFW, TRI, FM0, NFR>(acc, Ls, Rs, nbx, nl, r, kk, kc, m0);
        else
          mcp_stage<MFW, TRI, FM1, NFR>(acc, Ls, Rs, nbx, nl, r, kk, kc, m0);
      }
    }
    if (wm == 0)
      mcp_store<MFW, TRI, FM0, NFR>(acc, o, nbx, r, kk, m0, n0);
    else
      mcp_store<MFW, TRI, FM1, NFR>(acc, o, nbx, r, kk, m0, n0);
  }
}

// ------------------------------------------------------------------------------------------
// SYRK: the Gram matrix G = X X^T of the <= 128 rows of a K-contiguous X (CholQR step (i),
// G = C C^T of the distributed C, G = (A P1)^T (A P1) of step 3).  G is symmetric, so
// only the lower-triangle 16 x 16 blocks (I, J), J <= I, are computed -- R(R+1)/2 of R^2 blocks,
// and no N padding to 128 -- and each is stored to both triangles.  One operand tile per stage
// (TMA box {16 (K), 16R}, 128B swizzle; the KC fragment layout of kc_row / kc_pair_off): a
// thread's K pair of row kc_row(g, f, r) is both the A fragment (row r of the 8-row fragment)
// and the B fragment (column r) of a DMMA, so one LDS.128 per 8 rows feeds every block that row
// group takes part in.  Warp w takes a contiguous run of the row-major lower-triangle block list
// (runs differ by at most one block; warps w and w + 4 share an SM sub-partition and together
// hold about 2/8 of the blocks).  Each warp's block list and the row groups it must load are
// compile-time constants (one specialised main loop per warp), so every group is loaded once
// per K pair.  Split-K over blockIdx.z into partial Grams, reduced in a fixed order.
// ------------------------------------------------------------------------------------------
template <int R>
struct SyrkPlan {
  static constexpr int T = R * (R + 1) / 2;  // lower-triangle blocks
  static constexpr int MAXB = (T + 7) / 8;
  __host__ __device__ static constexpr int count(int w) { return T / 8 + (w < T % 8 ? 1 : 0); }
  __host__ __device__ static constexpr int start(int w) {
    int s = 0;
    for (int i = 0; i < w; ++i) s += count(i);
    return s;
  }
  __host__ __device__ static constexpr int blk_i(int idx) {
    int I = 0;
    while ((I + 1) * (I + 2) / 2 <= idx) ++I;
    return I;
  }
  __host__ __device__ static constexpr int blk_j(int idx) { return idx - blk_i(idx) * (blk_i(idx) + 1) / 2; }
  __host__ __device__ static constexpr bool need(int w, int g) {
    for (int s = 0; s < count(w); ++s) {
      const int idx = start(w) + s;
      if (blk_i(idx) == g || blk_j(idx) == g) return true;
    }
    return false;
  }
};

constexpr int SYRK_NS = 8;  // ring depth (stages are 16R x 16 doubles, <= 16 KB)

template <int R>
struct SyrkSmem {
  static constexpr int X_BYTES = 16 * R * KT * 8;
  static constexpr int TOTAL = 1024 + SYRK_NS * X_BYTES + 2 * SYRK_NS * 8;
};

template <int R, int W, typename Issue>
RS_DEVINL void syrk_warp(const unsigned char* sX, uint64_t* full, uint64_t* empty, int nk, int lane, Issue&& issue,
                         double* out, long long ld, int n_store) {
  using P = SyrkPlan<R>;
  constexpr int NB = P::count(W);
  if constexpr (NB == 0) {
    // no blocks: still release every slot so the producer can refill it
    for (int it = 0; it < nk; ++it) {
      const int s = it % SYRK_NS;
#ifndef RS_SYRK_RELEASE_DEFERRED
      if (threadIdx.x == 0 && it + SYRK_NS - 1 < nk) issue(it + SYRK_NS - 1);
#endif
      mbar_wait(&full[s], (it / SYRK_NS) & 1);
#ifdef RS_SYRK_RELEASE_DEFERRED
      ring_release_prev(empty, it, SYRK_NS, lane);
      if (threadIdx.x == 0 && it + SYRK_NS - 1 < nk) issue(it + SYRK_NS - 1);
#else
      ring_release_fenced(empty, s, lane);
#endif
    }
    return;
  } else {
    const int r = lane >> 2, kk = lane & 3;
    double acc[NB][2][2][2];
#pragma unroll
    for (int b = 0; b < NB; ++b)
#pragma unroll
      for (int f = 0; f < 2; ++f)
#pragma unroll
        for (int f2 = 0; f2 < 2; ++f2) acc[b][f][f2][0] = acc[b][f][f2][1] = 0.0;
    for (int it = 0; it < nk; ++it) {
      const int s = it % SYRK_NS;
#ifndef RS_SYRK_RELEASE_DEFERRED
      if (threadIdx.x == 0 && it + SYRK_NS - 1 < nk) issue(it + SYRK_NS - 1);  // slot of it - 1, released
#endif
      mbar_wait(&full[s], (it / SYRK_NS) & 1);
#ifdef RS_SYRK_RELEASE_DEFERRED
      ring_release_prev(empty, it, SYRK_NS, lane);
      if (threadIdx.x == 0 && it + SYRK_NS - 1 < nk) issue(it + SYRK_NS - 1);
#endif
      const unsigned char* Xs = sX + s * SyrkSmem<R>::X_BYTES;
#pragma unroll
      for (int p = 0; p < 2; ++p) {
        double2 fr[R][2];
#pragma unroll
        for (int g = 0; g < R; ++g) {
          if (P::need(W, g)) {
#pragma unroll
            for (int f = 0; f < 2; ++f)
              fr[g][f] = *reinterpret_cast<const double2*>(Xs + kc_pair_off(kc_row(g, f, r), p, kk));
          }
        }
#pragma unroll
        for (int b = 0; b < NB; ++b) {
          const int I = P::blk_i(P::start(W) + b), J = P::blk_j(P::start(W) + b);
#pragma unroll
          for (int f = 0; f < 2; ++f)
#pragma unroll
            for (int f2 = 0; f2 < 2; ++f2) {
              dmma_8x8x4(acc[b][f][f2][0], acc[b][f][f2][1], fr[I][f].x, fr[J][f2].x);
              dmma_8x8x4(acc[b][f][f2][0], acc[b][f][f2][1], fr[I][f].y, fr[J][f2].y);
            }
        }
      }
#ifndef RS_SYRK_RELEASE_DEFERRED
      ring_release_fenced(empty, s, lane);
#endif
    }
    // G[kc_row(I, f, r)][kc_row(J, f2, 2kk + e)] and its mirror
#pragma unroll
    for (int b = 0; b < NB; ++b) {
      const int I = P::blk_i(P::start(W) + b), J = P::blk_j(P::start(W) + b);
#pragma unroll
      for (int f = 0; f < 2; ++f)
#pragma unroll
        for (int f2 = 0; f2 < 2; ++f2)
#pragma unroll
          for (int e = 0; e < 2; ++e) {
            const int i = kc_row(I, f, r), j = kc_row(J, f2, 2 * kk + e);
            if (i < n_store && j < n_store) {
              out[i + j * ld] = acc[b][f][f2][e];
              out[j + i * ld] = acc[b][f][f2][e];
            }
          }
    }
  }
}

// tmX: dims {K (contiguous), rows}, box {16, 16R}.  out: partial Gram of split z at
// out + z * split_stride, element (i, j) at i + j * ld_n (i, j < n_store).
template <int R>
__global__ void __launch_bounds__(GEMM_THREADS, 1)
    syrk_kernel(const __grid_constant__ CUtensorMap tmX, const GemmArgs a) {
  using SM = SyrkSmem<R>;
  extern __shared__ unsigned char smem_raw[];
  unsigned char* smem = align1024(smem_raw);
  unsigned char* sX = smem;
  uint64_t* full = reinterpret_cast<uint64_t*>(sX + SYRK_NS * SM::X_BYTES);
  uint64_t* empty = full + SYRK_NS;
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const long long kb = static_cast<long long>(blockIdx.z) * a.k_chunk;
  const long long ke = min(a.K, kb + a.k_chunk);
  const int nk = kb < ke ? static_cast<int>((ke - kb + KT - 1) / KT) : 0;
  if (threadIdx.x == 0) {
#pragma unroll
    for (int s = 0; s < SYRK_NS; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], NCONS);
    }
    fence_mbar_init();
  }
  __syncthreads();
  auto issue = [&](int it) {
    const int s = it % SYRK_NS;
    if (it >= SYRK_NS) mbar_wait_sleep(&empty[s], ((it / SYRK_NS) - 1) & 1);
    mbar_arrive_expect_tx(&full[s], SM::X_BYTES);
    tma_load_2d(sX + s * SM::X_BYTES, &tmX, &full[s], static_cast<int>(kb + static_cast<long long>(it) * KT), 0);
  };
  if (threadIdx.x == 0) {
    tma_prefetch_desc(&tmX);
    for (int it = 0; it < SYRK_NS - 1 && it < nk; ++it) issue(it);
  }
  double* out = a.out.ptr + static_cast<long long>(blockIdx.z) * a.out.split_stride;
  const long long ld = a.out.ld_n;
  const int ns = a.out.n_store;
  switch (warp) {
    case 0: syrk_warp<R, 0>(sX, full, empty, nk, lane, issue, out, ld, ns); break;
    case 1: syrk_warp<R, 1>(sX, full, empty, nk, lane, issue, out, ld, ns); break;
    case 2: syrk_warp<R, 2>(sX, full, empty, nk, lane, issue, out, ld, ns); break;
    case 3: syrk_warp<R, 3>(sX, full, empty, nk, lane, issue, out, ld, ns); break;
    case 4: syrk_warp<R, 4>(sX, full, empty, nk, lane, issue, out, ld, ns); break;
    case 5: syrk_warp<R, 5>(sX, full, empty, nk, lane, issue, out, ld, ns); break;
    case 6: syrk_warp<R, 6>(sX, full, empty, nk, lane, issue, out, ld, ns); break;
    default: syrk_warp<R, 7>(sX, full, empty, nk, lane, issue, out, ld, ns); break;
  }
}

// ------------------------------------------------------------------------------------------
// TSA: Y = X U for a tall column-major X (m x k, k <= 128) and an upper-triangular U (k x k):
// the CholQR applies of Fig. 2 -- C1 = L^{-1} C of the power iteration, seen as
// C1^T = C^T L^{-T}, and Q1 = (A P1) R^{-1} of step 3.  Persistent CTAs
// walk 128-row tiles of X through a TMA ring (one dedicated producer warp) while U stays resident
// in shared memory.  MMA warp w owns rows 16w .. 16w + 15 of the tile and ALL NB column boxes,
// so every warp runs the same fully unrolled schedule with no runtime branches: column box nb is
// live in K stages 0..nb only (U[t][j] = 0 for t > j; the skipped terms are exact zeros).
// Operand layouts are the MC family's (X: M-contiguous boxes, U: N-contiguous boxes, 128B
// swizzle, fragment pairs by LDS.128).  The epilogue stores row pairs (2r, 2r+1) as 16-byte runs.
// ------------------------------------------------------------------------------------------
constexpr int TSA_NS = 6;
constexpr int TSA_THREADS = (NCONS + 1) * 32;  // 8 MMA warps + 1 producer warp

template <int NB>
struct TsaSmem {
  static constexpr int STAGE = 128 * KT * 8;  // one K stage of a 128-row X tile (8 boxes)
  static constexpr int UST = NB * 2048;       // one K stage of U (NB boxes)
  static constexpr int RES = NB * UST;
  static constexpr int TOTAL = 1024 + RES + TSA_NS * STAGE + (2 * TSA_NS + 1) * 8;
};

struct TsaArgs {
  double* y;
  long long ldy;
  int m, n_store, ntiles;
  int x3d, u3d;
};

// K-stage order of a tile: heavy and light stages interleaved -- stage s has NB - s live column
// boxes -- 0, NB-1, 1, NB-2, ... (measured at cfg4: factor 1.292 vs 1.31 / 1.317 ms, apply 0.601 vs
// 0.606 ms with 0, 1, 2, ...; -DRS_DEV_TSA_SEQ_ORDER restores the sequential order for A/B)
template <int NB>
__host__ __device__ constexpr int tsa_order(int i) {
#ifdef RS_DEV_TSA_SEQ_ORDER
  return i;
#else
  return (i & 1) ? NB - 1 - (i >> 1) : (i >> 1);
#endif
}

template <int NB>
__global__ void __launch_bounds__(TSA_THREADS, 1)
    tsa_kernel(const __grid_constant__ CUtensorMap tmX, const __grid_constant__ CUtensorMap tmU, const TsaArgs a) {
  using SM = TsaSmem<NB>;
  extern __shared__ unsigned char smem_raw[];
  unsigned char* smem = align1024(smem_raw);
  unsigned char* sU = smem;
  unsigned char* sX = smem + SM::RES;
  uint64_t* full = reinterpret_cast<uint64_t*>(sX + TSA_NS * SM::STAGE);
  uint64_t* empty = full + TSA_NS;
  uint64_t* resb = empty + TSA_NS;
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int mytiles = blockIdx.x < a.ntiles ? (a.ntiles - blockIdx.x + gridDim.x - 1) / gridDim.x : 0;
  const int total = mytiles * NB;
  if (threadIdx.x == 0) {
#pragma unroll
    for (int s = 0; s < TSA_NS; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], NCONS);
    }
    mbar_init(resb, 1);
    fence_mbar_init();
  }
  __syncthreads();
  if (warp == NCONS) {  // producer
    if (lane == 0) {
      tma_prefetch_desc(&tmX);
      tma_prefetch_desc(&tmU);
      mbar_arrive_expect_tx(resb, static_cast<uint32_t>(SM::RES));
#pragma unroll 1
      for (int s = 0; s < NB; ++s) mc_load(sU + s * SM::UST, &tmU, resb, a.u3d, 0, NB, s * KT);
#pragma unroll 1
      for (int g = 0; g < total; ++g) {
        const int s = g % TSA_NS;
        if (g >= TSA_NS) mbar_wait_sleep(&empty[s], ((g / TSA_NS) - 1) & 1);
        const int m0 = (blockIdx.x + (g / NB) * gridDim.x) * 128;
        mbar_arrive_expect_tx(&full[s], SM::STAGE);
        mc_load(sX + s * SM::STAGE, &tmX, &full[s], a.x3d, m0, 8, tsa_order<NB>(g % NB) * KT);
      }
    }
    return;
  }
  mbar_wait(resb, 0);
  const int r = lane >> 2, kk = lane & 3;
  int g = 0;
  int slot = 0;          // g % TSA_NS, kept incrementally (TSA_NS is not a power of two)
  uint32_t par = 0;      // (g / TSA_NS) & 1
  for (int i = 0; i < mytiles; ++i) {
    const int m0 = (blockIdx.x + i * gridDim.x) * 128;
    double acc[2][NB][2][2];
#pragma unroll
    for (int f = 0; f < 2; ++f)
#pragma unroll
      for (int nb = 0; nb < NB; ++nb)
#pragma unroll
        for (int f2 = 0; f2 < 2; ++f2) acc[f][nb][f2][0] = acc[f][nb][f2][1] = 0.0;
#pragma unroll
    for (int i2 = 0; i2 < NB; ++i2, ++g) {
      const int s = tsa_order<NB>(i2);
      mbar_wait(&full[slot], par);
#ifndef RS_RELEASE_FENCE_ALL
      if (g > 0) {  // ring_release_prev with the incrementally kept slot
        __syncwarp();
        if (lane == 0) mbar_arrive(&empty[slot == 0 ? TSA_NS - 1 : slot - 1]);
      }
#endif
      const unsigned char* Xs = sX + slot * SM::STAGE + warp * 2048;
      const unsigned char* Us = sU + s * SM::UST;
#pragma unroll
      for (int ks = 0; ks < KT / 4; ++ks) {
        const uint32_t krow = 8 * (ks >> 1) + 2 * kk + (ks & 1);
        const uint32_t off = krow * 128u + (((static_cast<uint32_t>(r) ^ krow) & 7u) << 4);
        // every load of the k-step first, then its DMMAs
        double2 b2[NB];
#pragma unroll
        for (int nb = s; nb < NB; ++nb) b2[nb] = *reinterpret_cast<const double2*>(Us + nb * 2048 + off);
        const double2 a2 = *reinterpret_cast<const double2*>(Xs + off);
#pragma unroll
        for (int nb = s; nb < NB; ++nb) {
          dmma_8x8x4(acc[0][nb][0][0], acc[0][nb][0][1], a2.x, b2[nb].x);
          dmma_8x8x4(acc[0][nb][1][0], acc[0][nb][1][1], a2.x, b2[nb].y);
          dmma_8x8x4(acc[1][nb][0][0], acc[1][nb][0][1], a2.y, b2[nb].x);
          dmma_8x8x4(acc[1][nb][1][0], acc[1][nb][1][1], a2.y, b2[nb].y);
        }
      }
#ifdef RS_RELEASE_FENCE_ALL
      ring_release_fenced(empty, slot, lane);
#endif
      if (++slot == TSA_NS) {
        slot = 0;
        par ^= 1u;
      }
    }
    // Y[row, col]: rows 2r (f = 0) and 2r + 1 (f = 1) of the warp's 16, col 16 nb + 2 (2 kk + e) + f2
    const long long row = static_cast<long long>(m0) + 16 * warp + 2 * r;
    if (row < a.m) {
      const bool ok1 = row + 1 < a.m;
#pragma unroll
      for (int nb = 0; nb < NB; ++nb)
#pragma unroll
        for (int e = 0; e < 2; ++e)
#pragma unroll
          for (int f2 = 0; f2 < 2; ++f2) {
            const int col = 16 * nb + 2 * (2 * kk + e) + f2;
            if (col < a.n_store) put2(a.y + row + col * a.ldy, acc[0][nb][f2][e], acc[1][nb][f2][e], ok1, 0);
          }
    }
  }
}

}  // namespace rs
