// Sample GEMM B = Omega A (Fig. 2(b) lines 2-3) with Omega generated ONCE
// per split of K and shared by all N tiles through an L2-resident ring of chunks.
//
// The cluster kernel (kc_philox_kernel) regenerates every Omega value for each pair of N tiles --
// 20 times at n = 5 000 -- and the generator's INT/FP32 instructions cost the DMMA warps of the
// same SM ~9 % of their rate.  Here a persistent, cooperatively launched grid (one CTA per SM)
// walks units (split s of K, N tile nt).  The units of one split that run in the same round of
// the grid form a GROUP; the group's members generate the split's Omega in chunks of RG_CH rows
// of A (member i generates chunks i, i + |group|, ...) into the group's ring of RG_R chunk slots
// in global memory (L2-resident: a few MB in flight, never the whole Omega), publish each chunk
// with a release flag, and every member streams the chunks into its shared-memory ring by TMA
// next to its A tiles, exactly like the KC GEMM's C operand.  A slot is rewritten only after all
// members have counted it consumed.  Co-residency of all CTAs (cooperative launch) plus the
// rule that a member only waits for chunks of its own group, whose members are in the same round,
// make the waits deadlock-free: a round-j member waits at most for other members to finish
// round j - 1.
//
// Roles per CTA (384 threads): warps 0-7 run the DMMA tiles (kc_gemm_pwg_kernel's layout), lane 0
// of warp 8 issues the TMA loads (and waits for / signals the ring flags), warps 9-11 generate
// Omega (Philox4x32-10 + RS-BM32, bit-identical to kc_philox_kernel and the oracle).
#pragma once

namespace rs {

#ifndef RS_RG_CH
#define RS_RG_CH 256
#endif
#ifndef RS_RG_R
#define RS_RG_R 4
#endif
constexpr int RG_CH = RS_RG_CH;            // rows of A (K) per Omega chunk (-DRS_RG_CH: experiments)
constexpr int RG_R = RS_RG_R;              // chunk slots per group ring
constexpr int RG_GEN_WARPS = 3;            // warps 9..11
constexpr int RG_THREADS = (NCONS + 4) * 32;
constexpr int RG_AUX_REGS = 56;
constexpr int RG_MMA_REGS = 224;           // 4*32*56 + 8*32*224 = 64512 <= 65536

struct RingArgs {
  int ntn;               // N tiles
  int S;                 // K splits
  long long kspl;        // K rows per split (multiple of RG_CH)
  int nunits;            // ntn * S
  double* ring;          // [groups][RG_R][MT][RG_CH], rows >= ell stay zero
  unsigned int* ready;   // [groups][RG_R]: chunk index + 1 once published
  unsigned int* consumed;  // [groups][RG_R]: cumulative member count of consumed chunks
};

struct RgUnit {
  int s, nt, gid, mem, gsz;
  long long kb, ke;
  int nk, nch;
};

RS_DEVINL RgUnit rg_unit(const RingArgs& r, long long K, int u, int G) {
  RgUnit x;
  x.s = u / r.ntn;
  x.nt = u % r.ntn;
  const int j = u / G;
  x.gid = x.s + j;
  const int u0 = max(j * G, x.s * r.ntn), u1 = min((j + 1) * G, min((x.s + 1) * r.ntn, r.nunits));
  x.mem = u - u0;
  x.gsz = u1 - u0;
  x.kb = static_cast<long long>(x.s) * r.kspl;
  x.ke = min(K, x.kb + r.kspl);
  x.nk = x.kb < x.ke ? static_cast<int>((x.ke - x.kb + KT - 1) / KT) : 0;
  x.nch = x.kb < x.ke ? static_cast<int>((x.ke - x.kb + RG_CH - 1) / RG_CH) : 0;
  return x;
}

RS_DEVINL unsigned int rg_ld_acquire(const unsigned int* p) {
  unsigned int v;
  asm volatile("ld.acquire.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
RS_DEVINL void rg_st_release(unsigned int* p, unsigned int v) {
  asm volatile("st.release.gpu.global.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
RS_DEVINL void rg_red_release_add(unsigned int* p, unsigned int v) {
  asm volatile("red.release.gpu.global.add.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
RS_DEVINL void rg_wait_geq(const unsigned int* p, unsigned int target) {
  // (measured: relaxed polling with exponential back-off made cfg4 0.5 ms slower than this)
  while (rg_ld_acquire(p) < target) __nanosleep(64);
}

template <int MFW>
__global__ void __launch_bounds__(RG_THREADS, 1)
    kc_sample_ring_kernel(const __grid_constant__ CUtensorMap tmA, const __grid_constant__ CUtensorMap tmW,
                          const GemmArgs a, const RingArgs rg) {
  using SM = KCSmem<MFW, false>;
  constexpr int MT = SM::MT;
  extern __shared__ unsigned char smem_raw[];
  unsigned char* smem = align1024(smem_raw);
  unsigned char* sR = smem;                       // A tiles (16 K x 128 N)
  unsigned char* sL = sR + SM::NS * SM::R_BYTES;  // Omega tiles (16 K x MT rows)
  uint64_t* full = reinterpret_cast<uint64_t*>(sL + SM::NS * SM::L_BYTES);
  uint64_t* empty = full + SM::NS;
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int G = gridDim.x;
  if (threadIdx.x == 0) {
#pragma unroll
    for (int s = 0; s < SM::NS; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], NCONS);
    }
    fence_mbar_init();
  }
  __syncthreads();

  if (warp >= NCONS) {
    asm volatile("setmaxnreg.dec.sync.aligned.u32 %0;\n" ::"n"(RG_AUX_REGS));
    if (warp == NCONS) {
      // ------------------------- TMA producer (one thread) -------------------------
      if (lane != 0) return;
      tma_prefetch_desc(&tmA);
      tma_prefetch_desc(&tmW);
      // per smem slot: the ring chunk its stage came from, to count the chunk consumed once the
      // slot is handed back (the stage's TMA reads of the chunk completed long before)
      int hist_gid[8], hist_slot[8];
      bool hist_last[8];
#pragma unroll
      for (int i = 0; i < 8; ++i) hist_last[i] = false, hist_gid[i] = 0, hist_slot[i] = 0;
      int g = 0;
      for (int u = blockIdx.x; u < rg.nunits; u += G) {
        const RgUnit x = rg_unit(rg, a.K, u, G);
        for (int it = 0; it < x.nk; ++it, ++g) {
          const long long k = x.kb + static_cast<long long>(it) * KT;
          const int c = static_cast<int>((k - x.kb) / RG_CH);
          const int kin = static_cast<int>((k - x.kb) % RG_CH);
          const int slot = c % RG_R;
          if (kin == 0) {  // first stage of a chunk: wait until it is published
            rg_wait_geq(rg.ready + x.gid * RG_R + slot, static_cast<unsigned int>(c + 1));
            asm volatile("fence.proxy.async.global;" ::: "memory");  // generic writes -> TMA reads
          }
          const int s = g % SM::NS;
          if (g >= SM::NS) {
            mbar_wait_sleep(&empty[s], ((g / SM::NS) - 1) & 1);
            if (hist_last[s]) rg_red_release_add(rg.consumed + hist_gid[s] * RG_R + hist_slot[s], 1u);
          }
          hist_gid[s] = x.gid;
          hist_slot[s] = slot;
          hist_last[s] = kin + KT >= RG_CH || it + 1 == x.nk;
          mbar_arrive_expect_tx(&full[s], SM::R_BYTES + SM::L_BYTES_TMA);
          tma_load_2d(sR + s * SM::R_BYTES, &tmA, &full[s], static_cast<int>(k), x.nt * NT);
          tma_load_2d(sL + s * SM::L_BYTES, &tmW, &full[s], kin, (x.gid * RG_R + slot) * MT);
        }
      }
      // the last stages: their chunks are counted once their data has landed
      for (int d = 0; d < SM::NS && d < g; ++d) {
        const int gg = g - 1 - d, s = gg % SM::NS;
        mbar_wait(&full[s], (gg / SM::NS) & 1);
        if (hist_last[s]) rg_red_release_add(rg.consumed + hist_gid[s] * RG_R + hist_slot[s], 1u);
      }
      return;
    }
    // ------------------------- Omega generators (warps 9..11) -------------------------
    const int gt = threadIdx.x - (NCONS + 1) * 32;  // 0 .. 95
    constexpr int GT = RG_GEN_WARPS * 32;
    const int o = static_cast<int>(a.row_offset & 3);
    for (int u = blockIdx.x; u < rg.nunits; u += G) {
      const RgUnit x = rg_unit(rg, a.K, u, G);
      for (int c = x.mem; c < x.nch; c += x.gsz) {
        const int slot = c % RG_R;
        unsigned int* cons = rg.consumed + x.gid * RG_R + slot;
        if (gt == 0 && c >= RG_R) rg_wait_geq(cons, static_cast<unsigned int>(x.gsz * (c / RG_R)));
        named_bar_sync(1, GT);
        double* dst = rg.ring + static_cast<size_t>(x.gid * RG_R + slot) * MT * RG_CH;
        const long long kc0 = x.kb + static_cast<long long>(c) * RG_CH;  // first K row of the chunk
        const uint64_t t0 = static_cast<uint64_t>((a.row_offset + kc0) >> 2);
        constexpr int ITEMS_ROW = RG_CH / 4;
#pragma unroll 1
        for (int w = gt; w < a.ell * ITEMS_ROW; w += GT) {
          const int row = w / ITEMS_ROW, q = w % ITEMS_ROW;
          const long long kk = kc0 + 4 * q;
          double v0 = 0.0, v1 = 0.0, v2 = 0.0, v3 = 0.0;
          if (kk < x.ke) {  // rows past the split's (or A's) end multiply nothing: zeros
            const float4 z = omega_block4f(static_cast<uint32_t>(a.omega_row0 + row), t0 + q, a.tag, a.key);
            if (o == 0) {
              v0 = z.x, v1 = z.y, v2 = z.z, v3 = z.w;
            } else {
              const float4 z2 = omega_block4f(static_cast<uint32_t>(a.omega_row0 + row), t0 + q + 1, a.tag, a.key);
              v0 = o + 0 < 4 ? f4_get(z, o + 0) : f4_get(z2, o - 4);
              v1 = o + 1 < 4 ? f4_get(z, o + 1) : f4_get(z2, o - 3);
              v2 = o + 2 < 4 ? f4_get(z, o + 2) : f4_get(z2, o - 2);
              v3 = f4_get(z2, o - 1);
            }
            if (kk + 1 >= x.ke) v1 = 0.0;
            if (kk + 2 >= x.ke) v2 = 0.0;
            if (kk + 3 >= x.ke) v3 = 0.0;
          }
          double* p = dst + static_cast<size_t>(row) * RG_CH + 4 * q;
          reinterpret_cast<double2*>(p)[0] = make_double2(v0, v1);
          reinterpret_cast<double2*>(p)[1] = make_double2(v2, v3);
        }
        named_bar_sync(1, GT);  // every generator thread's stores precede the release below
        if (gt == 0) {
          __threadfence();
          rg_st_release(rg.ready + x.gid * RG_R + slot, static_cast<unsigned int>(c + 1));
        }
      }
    }
    return;
  }

  // ------------------------- MMA warps -------------------------
  asm volatile("setmaxnreg.inc.sync.aligned.u32 %0;\n" ::"n"(RG_MMA_REGS));
  const int wm = warp >> 2, wn = warp & 3;
  const int r = lane >> 2, kk = lane & 3;
  auto rowL = [&](int mf) {
    const int mg = wm * MFW + mf;
    return kc_row(mg >> 1, mg & 1, r);
  };
  auto rowR = [&](int nf) {
    const int ng = wn * 4 + nf;
    return kc_row(ng >> 1, ng & 1, r);
  };
  int g = 0;
  for (int u = blockIdx.x; u < rg.nunits; u += G) {
    const RgUnit x = rg_unit(rg, a.K, u, G);
    double acc[MFW][4][2];
#pragma unroll
    for (int mf = 0; mf < MFW; ++mf)
#pragma unroll
      for (int nf = 0; nf < 4; ++nf) acc[mf][nf][0] = acc[mf][nf][1] = 0.0;
    for (int it = 0; it < x.nk; ++it, ++g) {
      const int s = g % SM::NS;
      mbar_wait(&full[s], (g / SM::NS) & 1);
#ifdef RS_RING_RELEASE_DEFERRED
      ring_release_prev(empty, g, SM::NS, lane);
#endif
      const unsigned char* Ls = sL + s * SM::L_BYTES;
      const unsigned char* Rs = sR + s * SM::R_BYTES;
      kc_stage_mma<MFW>(
          acc, [&](int mf, int p) { return *reinterpret_cast<const double2*>(Ls + kc_pair_off(rowL(mf), p, kk)); },
          [&](int nf, int p) { return *reinterpret_cast<const double2*>(Rs + kc_pair_off(rowR(nf), p, kk)); });
#ifndef RS_RING_RELEASE_DEFERRED
      ring_release_fenced(empty, s, lane);  // measured 32.53 vs 32.68 ms (deferred) at cfg4
#endif
    }
    GemmOut o = a.out;
    o.ptr = a.out.ptr + static_cast<long long>(x.s) * a.out.split_stride;
    o.split_stride = 0;
    kc_store<MFW>(acc, o, 0, x.nt * NT, wn, kk, rowL);
  }
}

}  // namespace rs
