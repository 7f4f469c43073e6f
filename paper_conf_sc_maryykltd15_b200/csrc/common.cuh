// Device-side primitives for sm_100a: mbarrier, TMA (cp.async.bulk.tensor), FP64 DMMA,
// grid barrier.  Inline PTX only; no CUTLASS/CuTe.
#pragma once
#include <cstdint>
#include <cuda.h>
#include <cuda_runtime.h>

#define RS_DEVINL __device__ __forceinline__

namespace rs {

RS_DEVINL uint32_t smem_u32(const void* p) {
  return static_cast<uint32_t>(__cvta_generic_to_shared(p));
}

// ---- mbarrier ---------------------------------------------------------------------------
RS_DEVINL void mbar_init(uint64_t* bar, uint32_t count) {
  asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(count) : "memory");
}
RS_DEVINL void fence_mbar_init() {
  asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
}
RS_DEVINL void mbar_arrive_expect_tx(uint64_t* bar, uint32_t bytes) {
  asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes)
               : "memory");
}
RS_DEVINL void mbar_arrive(uint64_t* bar) {
  asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(smem_u32(bar)) : "memory");
}
RS_DEVINL void mbar_arrive_cnt(uint64_t* bar, uint32_t count) {
  asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(count) : "memory");
}
RS_DEVINL void mbar_wait(uint64_t* bar, uint32_t parity) {
  asm volatile(
      "{\n"
      ".reg .pred p;\n"
      "RS_WAIT_%=:\n"
      "mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n"
      "@!p bra RS_WAIT_%=;\n"
      "}\n" ::"r"(smem_u32(bar)),
      "r"(parity)
      : "memory");
}

// Producer-side wait (ring slot free): try_wait with a suspend-time hint, so a thread that is
// ahead of its consumers sleeps in the barrier until the phase completes instead of spinning --
// a spinning TRYWAIT / BRA / YIELD loop issues instructions on the SM sub-partition the DMMA warps
// share (measured in the Philox sample GEMM: 1.9e9 spin instructions per launch, ~0.8 per DMMA).
// -DRS_NO_WAIT_HINT restores the plain spin (A/B experiments only).
RS_DEVINL void mbar_wait_sleep(uint64_t* bar, uint32_t parity) {
#ifdef RS_NO_WAIT_HINT
  mbar_wait(bar, parity);
#else
  asm volatile(
      "{\n"
      ".reg .pred p;\n"
      "RS_WAITS_%=:\n"
      "mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1, %2;\n"
      "@!p bra RS_WAITS_%=;\n"
      "}\n" ::"r"(smem_u32(bar)),
      "r"(parity), "r"(0x989680u)
      : "memory");
#endif
}

// cluster-scope variants (thread-block clusters / distributed shared memory)
RS_DEVINL void mbar_wait_cluster(uint64_t* bar, uint32_t parity) {
  asm volatile(
      "{\n"
      ".reg .pred p;\n"
      "RS_WAITC_%=:\n"
      "mbarrier.try_wait.parity.acquire.cluster.shared::cta.b64 p, [%0], %1;\n"
      "@!p bra RS_WAITC_%=;\n"
      "}\n" ::"r"(smem_u32(bar)),
      "r"(parity)
      : "memory");
}
RS_DEVINL uint32_t cluster_ctarank() {
  uint32_t r;
  asm volatile("mov.u32 %0, %%cluster_ctarank;" : "=r"(r));
  return r;
}
RS_DEVINL uint32_t mapa_shared(uint32_t local_addr, uint32_t rank) {
  uint32_t r;
  asm volatile("mapa.shared::cluster.u32 %0, %1, %2;" : "=r"(r) : "r"(local_addr), "r"(rank));
  return r;
}
RS_DEVINL void st_cluster_v2(uint32_t addr, double a, double b) {
  asm volatile("st.shared::cluster.v2.f64 [%0], {%1, %2};" ::"r"(addr), "d"(a), "d"(b) : "memory");
}
RS_DEVINL void mbar_arrive_remote(uint32_t cluster_bar_addr) {
  asm volatile("mbarrier.arrive.release.cluster.shared::cluster.b64 _, [%0];" ::"r"(cluster_bar_addr) : "memory");
}
// asynchronous DSMEM store that completes 16 transaction bytes on the destination CTA's mbarrier
// (no fence, no arrive: the consumer's phase completes when all expected bytes have landed)
RS_DEVINL void st_async_v2(uint32_t remote_addr, double a, double b, uint32_t remote_mbar) {
  asm volatile("st.async.shared::cluster.mbarrier::complete_tx::bytes.v2.f64 [%0], {%1, %2}, [%3];" ::"r"(
                   remote_addr),
               "d"(a), "d"(b), "r"(remote_mbar)
               : "memory");
}
// remote arrive with the default (.release.cta) semantics: used by MMA warps to hand a ring slot
// back to a peer CTA -- the slot's smem reads have completed (their values were consumed by the
// DMMAs issued before the arrive), and no cluster-scope MEMBAR lands on the MMA warps
RS_DEVINL void mbar_arrive_remote_cta(uint32_t cluster_bar_addr) {
  asm volatile("mbarrier.arrive.shared::cluster.b64 _, [%0];" ::"r"(cluster_bar_addr) : "memory");
}
RS_DEVINL void cluster_sync_all() {
  asm volatile("barrier.cluster.arrive.release.aligned;\n\tbarrier.cluster.wait.acquire.aligned;" ::: "memory");
}

// ---- TMA -----------------------------------------------------------------------------------
RS_DEVINL void tma_prefetch_desc(const CUtensorMap* m) {
  asm volatile("prefetch.tensormap [%0];" ::"l"(reinterpret_cast<uint64_t>(m)) : "memory");
}
// 2-D tiled load: coordinates (c0 = innermost element index, c1 = row index), OOB -> zeros.
RS_DEVINL void tma_load_2d(void* smem_dst, const CUtensorMap* m, uint64_t* bar, int32_t c0, int32_t c1) {
  asm volatile(
      "cp.async.bulk.tensor.2d.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1, {%3, %4}], [%2];" ::"r"(
          smem_u32(smem_dst)),
      "l"(reinterpret_cast<uint64_t>(m)), "r"(smem_u32(bar)), "r"(c0), "r"(c1)
      : "memory");
}

// 3-D tiled load: coordinates (c0, c1, c2), OOB -> zeros.
RS_DEVINL void tma_load_3d(void* smem_dst, const CUtensorMap* m, uint64_t* bar, int32_t c0, int32_t c1, int32_t c2) {
  asm volatile(
      "cp.async.bulk.tensor.3d.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1, {%3, %4, %5}], [%2];" ::"r"(
          smem_u32(smem_dst)),
      "l"(reinterpret_cast<uint64_t>(m)), "r"(smem_u32(bar)), "r"(c0), "r"(c1), "r"(c2)
      : "memory");
}

// ---- FP64 tensor core: mma.sync m8n8k4 (lowers to DMMA.8x8x4 on sm_100a) ---------------
// A fragment: a = A[lane/4][lane%4]; B fragment: b = B[lane%4][lane/4];
// C/D: d0 = C[lane/4][2*(lane%4)], d1 = C[lane/4][2*(lane%4)+1].
// Consumer-side release of a TMA / generator ring slot, DEFERRED BY ONE STAGE: called right after
// the full-barrier wait of stage `it`, it releases the slot of stage it - 1.  A slot may only be
// refilled once every shared-memory load from it has completed.  Releasing at the end of the
// stage itself is not enough: ptxas schedules the (lane-0) arrive above the stage's DMMAs, right
// behind LDS.128s whose data is still in flight, and the producer's next TMA into the slot can
// then overwrite it before those loads read it -- rare wrong results that showed up with the
// ranks' kernels overlapping on one GPU.  Here the arrive sits in the basic block
// after the next stage's wait, so all of stage it - 1's DMMAs -- which consume every one of its
// loads -- have issued before it.
// The other safe form: release the slot at the end of its own stage, behind a CTA-scope fence
// (MEMBAR.CTA) that makes the warp wait for its outstanding shared-memory loads; ptxas keeps the
// stage's LDS before the fence.  Used by the dense MC GEMM (faster there), -DRS_RELEASE_FENCE for
// the KC kernels (measured equal).
RS_DEVINL void ring_release_fenced(uint64_t* empty, int s, int lane) {
  asm volatile("fence.acq_rel.cta;" ::: "memory");
  __syncwarp();
  if (lane == 0) mbar_arrive(&empty[s]);
}
RS_DEVINL void ring_release_prev(uint64_t* empty, int it, int ns, int lane) {
  if (it > 0) {
    __syncwarp();
    if (lane == 0) mbar_arrive(&empty[(it - 1) % ns]);
  }
}

RS_DEVINL void dmma_8x8x4(double& d0, double& d1, double a, double b) {
  asm volatile("mma.sync.aligned.m8n8k4.row.col.f64.f64.f64.f64 {%0,%1}, {%2}, {%3}, {%0,%1};"
               : "+d"(d0), "+d"(d1)
               : "d"(a), "d"(b));
}

RS_DEVINL void named_bar_sync(uint32_t id, uint32_t nthreads) {
  asm volatile("bar.sync %0, %1;" ::"r"(id), "r"(nthreads) : "memory");
}

// Byte offset of element (row, k) inside a 128B-swizzled TMA box whose rows are 128 B
// (16 doubles) long; the box base must be 1024-byte aligned.  (CU_TENSOR_MAP_SWIZZLE_128B:
// 16-byte chunk index XOR (row mod 8).)
RS_DEVINL uint32_t swz128_off(uint32_t row, uint32_t k) {
  return row * 128u + ((((k >> 1) ^ row) & 7u) << 4) + ((k & 1u) << 3);
}

// ---- grid-wide barrier for cooperative launches --------------------------------------------
struct GridBarrier {
  unsigned int count;
  unsigned int gen;
};
RS_DEVINL void grid_sync(GridBarrier* gb, unsigned int nblocks) {
  __syncthreads();
  if (threadIdx.x == 0) {
    volatile unsigned int* vgen = &gb->gen;
    unsigned int g = *vgen;
    __threadfence();
    if (atomicAdd(&gb->count, 1u) == nblocks - 1) {
      gb->count = 0;
      __threadfence();
      atomicAdd(&gb->gen, 1u);
    } else {
      while (*vgen == g) {
      }
    }
    __threadfence();
  }
  __syncthreads();
}

}  // namespace rs
