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
  int gen_mode;  // 0 = Philox + RS-BM32 (production); 1, 2 = generation-cost experiments only
};

template <int MFW, bool PHILOX>
struct KCSmem {
  static constexpr int MT = 16 * MFW;
  static constexpr int R_BYTES = NT * KT * 8;
  static constexpr int L_BYTES_TMA = MT * KT * 8;
  static constexpr int L_BYTES_RAW = PHILOX ? MT * PHX_LD * 8 : L_BYTES_TMA;
  static constexpr int L_BYTES = (L_BYTES_RAW + 1023) / 1024 * 1024;
  // small M (l <= 32): little MMA work per stage, so a deeper ring keeps more of A in flight and
  // lets several generator groups work on different stages at once
  static constexpr int NS = MFW <= 2 ? 8 : NSTAGE;
  static constexpr int TOTAL = 1024 + NS * (R_BYTES + L_BYTES) + 2 * NS * 8;
};

template <int MFW>
struct MCSmem {
  static constexpr int MT = 16 * MFW;
  static constexpr int R_BYTES = NT * KT * 8;
  static constexpr int L_BYTES = MT * KT * 8;
  static constexpr int TOTAL = 1024 + NSTAGE * (R_BYTES + L_BYTES) + 2 * NSTAGE * 8;
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
    if (it >= SM::NS) mbar_wait(&empty[s], ((it / SM::NS) - 1) & 1);
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
    if (threadIdx.x == 0 && it + SM::NS - 1 < nk) issue(it + SM::NS - 1);
    mbar_wait(&full[s], (it / SM::NS) & 1);
    const unsigned char* Ls = sL + s * SM::L_BYTES;
    const unsigned char* Rs = sR + s * SM::R_BYTES;
    kc_stage_mma<MFW>(
        acc, [&](int mf, int p) { return *reinterpret_cast<const double2*>(Ls + kc_pair_off(rowL(mf), p, kk)); },
        [&](int nf, int p) { return *reinterpret_cast<const double2*>(Rs + kc_pair_off(rowR(nf), p, kk)); });
    __syncwarp();
    if (lane == 0) mbar_arrive(&empty[s]);
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
      mbar_init(&full[s], 1 + GRP_WARPS);  // TMA producer + the stage's generator warps (+ peers' tx bytes)
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
        if (lane == 0) mbar_wait(&empty[s], ((it / SM::NS) - 1) & 1);
        __syncwarp();
      }
      if (g == 0) {
        mbar_arrive_expect_tx(&full[s], SM::R_BYTES + (MT - ROWS) * KT * 8);  // A tile + peers' Omega rows
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
        if (a.gen_mode != 0) {  // experiments: 1 = Philox words only, 2 = no generation
          if (a.gen_mode == 1 && gi < a.ell) {
            uint32_t c0 = static_cast<uint32_t>(t0 + q), c1 = static_cast<uint32_t>(gi), c2 = a.tag,
                     c3 = static_cast<uint32_t>((t0 + q) >> 32);
            philox4x32_10(c0, c1, c2, c3, a.key);
            v0 = static_cast<int>(c0) * 0x1p-31, v1 = static_cast<int>(c1) * 0x1p-31;
            v2 = static_cast<int>(c2) * 0x1p-31, v3 = static_cast<int>(c3) * 0x1p-31;
          } else if (gi < a.ell) {
            v0 = v1 = v2 = v3 = 1.0;
          }
        } else if (gi < a.ell) {
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
        reinterpret_cast<double2*>(dst)[0] = make_double2(v0, v1);
        reinterpret_cast<double2*>(dst)[1] = make_double2(v2, v3);
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
      __syncwarp();
      if (lane == 0) mbar_arrive(&full[s]);
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
      const double* Ls = reinterpret_cast<const double*>(sL + s * SM::L_BYTES);
      const unsigned char* Rs = sR + s * SM::R_BYTES;
      kc_stage_mma<MFW>(
          acc,
          [&](int mf, int p) { return *reinterpret_cast<const double2*>(Ls + rowL(mf) * PHX_LD + 8 * p + 2 * kk); },
          [&](int nf, int p) { return *reinterpret_cast<const double2*>(Rs + kc_pair_off(rowR(nf), p, kk)); });
      __syncwarp();
      if (lane == 0) {
        mbar_arrive(&empty[s]);
#pragma unroll
        for (int pc = 1; pc < CS; ++pc) mbar_arrive_remote_cta(mapa_shared(smem_u32(&empty[s]), (crank + pc) % CS));
      }
    }
    kc_store<MFW>(acc, a.out, m0, n0, wn, kk, rowL);
  }
  // no CTA may leave while cluster peers can still write its shared memory / barriers
  if (CS > 1) cluster_sync_all();
}

// ------------------------------------------------------------------------------------------
// MC family.  tmL: dims {M (contiguous), K}, box {16, 16};  tmR: dims {N (contiguous), K},
// box {16, 16}.  One 2 KB box per 16 rows of M (or N) per stage.  Warp w owns the N box w
// (16 columns, two fragments) and all MT rows (2*MFW fragments).
// ------------------------------------------------------------------------------------------
template <int MFW>
__global__ void __launch_bounds__(GEMM_THREADS, 1)
    mc_gemm_kernel(const __grid_constant__ CUtensorMap tmL, const __grid_constant__ CUtensorMap tmR,
                   const GemmArgs a) {
  using SM = MCSmem<MFW>;
  constexpr int MT = SM::MT;
  extern __shared__ unsigned char smem_raw[];
  unsigned char* smem = align1024(smem_raw);
  unsigned char* sR = smem;
  unsigned char* sL = sR + NSTAGE * SM::R_BYTES;
  uint64_t* full = reinterpret_cast<uint64_t*>(sL + NSTAGE * SM::L_BYTES);
  uint64_t* empty = full + NSTAGE;

  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int n0 = blockIdx.x * NT, m0 = blockIdx.y * MT;
  const long long kb = static_cast<long long>(blockIdx.z) * a.k_chunk;
  const long long ke = min(a.K, kb + a.k_chunk);
  const int nk = kb < ke ? static_cast<int>((ke - kb + KT - 1) / KT) : 0;

  if (threadIdx.x == 0) {
#pragma unroll
    for (int s = 0; s < NSTAGE; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], NCONS);
    }
    fence_mbar_init();
  }
  __syncthreads();

  auto issue = [&](int it) {
    const int s = it % NSTAGE;
    if (it >= NSTAGE) mbar_wait(&empty[s], ((it / NSTAGE) - 1) & 1);
    mbar_arrive_expect_tx(&full[s], SM::R_BYTES + SM::L_BYTES);
    const int kc = static_cast<int>(kb + static_cast<long long>(it) * KT);
#pragma unroll 1
    for (int b = 0; b < MT / 16; ++b) tma_load_2d(sL + s * SM::L_BYTES + b * 2048, &tmL, &full[s], m0 + 16 * b, kc);
#pragma unroll 1
    for (int b = 0; b < NT / 16; ++b) tma_load_2d(sR + s * SM::R_BYTES + b * 2048, &tmR, &full[s], n0 + 16 * b, kc);
  };
  if (threadIdx.x == 0) {
    tma_prefetch_desc(&tmL);
    tma_prefetch_desc(&tmR);
    for (int it = 0; it < NSTAGE - 1 && it < nk; ++it) issue(it);
  }

  const int r = lane >> 2, kk = lane & 3;
  // acc[b][f][f'][e]: M fragment (box b, parity f), N fragment (box warp, parity f'), element e
  double acc[MFW][2][2][2];
#pragma unroll
  for (int b = 0; b < MFW; ++b)
#pragma unroll
    for (int f = 0; f < 2; ++f)
#pragma unroll
      for (int f2 = 0; f2 < 2; ++f2) acc[b][f][f2][0] = acc[b][f][f2][1] = 0.0;

  for (int it = 0; it < nk; ++it) {
    const int s = it % NSTAGE;
    if (threadIdx.x == 0 && it + NSTAGE - 1 < nk) issue(it + NSTAGE - 1);
    mbar_wait(&full[s], (it / NSTAGE) & 1);
    const unsigned char* Ls = sL + s * SM::L_BYTES;
    const unsigned char* Rs = sR + s * SM::R_BYTES + warp * 2048;
#pragma unroll
    for (int ks = 0; ks < KT / 4; ++ks) {
      const uint32_t krow = 8 * (ks >> 1) + 2 * kk + (ks & 1);
      const uint32_t off = krow * 128u + (((static_cast<uint32_t>(r) ^ krow) & 7u) << 4);
      const double2 b2 = *reinterpret_cast<const double2*>(Rs + off);
#pragma unroll
      for (int b = 0; b < MFW; ++b) {
        const double2 a2 = *reinterpret_cast<const double2*>(Ls + b * 2048 + off);
        dmma_8x8x4(acc[b][0][0][0], acc[b][0][0][1], a2.x, b2.x);
        dmma_8x8x4(acc[b][0][1][0], acc[b][0][1][1], a2.x, b2.y);
        dmma_8x8x4(acc[b][1][0][0], acc[b][1][0][1], a2.y, b2.x);
        dmma_8x8x4(acc[b][1][1][0], acc[b][1][1][1], a2.y, b2.y);
      }
    }
    __syncwarp();
    if (lane == 0) mbar_arrive(&empty[s]);
  }

  const GemmOut& o = a.out;
  double* base = o.ptr + static_cast<long long>(blockIdx.z) * o.split_stride;
#pragma unroll
  for (int b = 0; b < MFW; ++b)
#pragma unroll
    for (int f = 0; f < 2; ++f) {
      const long long gm = m0 + 16 * b + 2 * r + f;
      if (gm >= o.m_store) continue;
#pragma unroll
      for (int f2 = 0; f2 < 2; ++f2)
#pragma unroll
        for (int e = 0; e < 2; ++e) {
          const long long gn = n0 + 16 * warp + 2 * (2 * kk + e) + f2;
          if (gn < o.n_store) gemm_put(base + gm * o.ld_m + gn * o.ld_n, acc[b][f][f2][e], o.mode);
        }
    }
}

}  // namespace rs
