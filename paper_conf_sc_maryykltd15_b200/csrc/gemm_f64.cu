// Host launchers for the FP64 DMMA GEMM families (tensor-map encoding, tile/split choice).
#include <algorithm>
#include <cstdio>
#include <cstdlib>
#include <map>
#include <mutex>
#include <tuple>

#include "gemm_f64.cuh"
#include "internal.h"
#include "philox.cuh"
#include "sample_ring.cuh"

namespace rs {

cudaError_t ensure_func_attr(const void* fn, cudaFuncAttribute attr, int value) {
  static std::mutex mu;
  static std::map<std::tuple<int, const void*, int>, int> done;  // (device, kernel, attribute) -> value set
  int dev = 0;
  cudaError_t e = cudaGetDevice(&dev);
  if (e != cudaSuccess) return e;
  std::lock_guard<std::mutex> lk(mu);
  const auto key = std::make_tuple(dev, fn, static_cast<int>(attr));
  auto it = done.find(key);
  if (it != done.end() && it->second >= value) return cudaSuccess;
  e = cudaFuncSetAttribute(fn, attr, value);
  if (e == cudaSuccess) done[key] = value;
  return e;
}

namespace {

using EncodeTiledFn = CUresult (*)(CUtensorMap*, CUtensorMapDataType, cuuint32_t, void*, const cuuint64_t*,
                                   const cuuint64_t*, const cuuint32_t*, const cuuint32_t*, CUtensorMapInterleave,
                                   CUtensorMapSwizzle, CUtensorMapL2promotion, CUtensorMapFloatOOBfill);

EncodeTiledFn get_encode() {
  static EncodeTiledFn fn = nullptr;
  static std::once_flag once;
  std::call_once(once, [] {
    void* p = nullptr;
    cudaDriverEntryPointQueryResult q;
    if (cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &p, cudaEnableDefault, &q) == cudaSuccess &&
        q == cudaDriverEntryPointSuccess)
      fn = reinterpret_cast<EncodeTiledFn>(p);
  });
  return fn;
}

// 2-D FP64 tensor map, 128B swizzle, OOB -> zero.  box0 must be 16 (128 bytes).
bool make_tmap(CUtensorMap* m, const View2D& v, uint32_t box0, uint32_t box1) {
  EncodeTiledFn enc = get_encode();
  if (!enc) return false;
  cuuint64_t dims[2] = {static_cast<cuuint64_t>(v.dim0), static_cast<cuuint64_t>(v.dim1)};
  cuuint64_t strides[1] = {static_cast<cuuint64_t>(v.ld) * 8};
  cuuint32_t box[2] = {box0, box1};
  cuuint32_t estr[2] = {1, 1};
  CUresult r = enc(m, CU_TENSOR_MAP_DATA_TYPE_FLOAT64, 2, const_cast<double*>(v.base), dims, strides, box, estr,
                   CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_128B, CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
                   CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  return r == CUDA_SUCCESS;
}

// 3-D "stacked boxes" map of an MC operand (dim0 contiguous, a multiple of 16): dims {16, dim1,
// dim0/16}, strides {ld, 16} elements, box {16, 16, nbx}: one TMA = nbx {16, 16} boxes laid out
// back to back (see mc_load).
bool make_tmap3(CUtensorMap* m, const View2D& v, uint32_t nbx) {
  EncodeTiledFn enc = get_encode();
  if (!enc || v.dim0 % 16 != 0) return false;
  cuuint64_t dims[3] = {16, static_cast<cuuint64_t>(v.dim1), static_cast<cuuint64_t>(v.dim0 / 16)};
  cuuint64_t strides[2] = {static_cast<cuuint64_t>(v.ld) * 8, 128};
  cuuint32_t box[3] = {16, 16, nbx};
  cuuint32_t estr[3] = {1, 1, 1};
  CUresult r = enc(m, CU_TENSOR_MAP_DATA_TYPE_FLOAT64, 3, const_cast<double*>(v.base), dims, strides, box, estr,
                   CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_128B, CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
                   CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  return r == CUDA_SUCCESS;
}

template <int MFW>
cudaError_t launch_kc_tail_t(cudaStream_t st, dim3 grid, const CUtensorMap& tR, const CUtensorMap& tL,
                             const CUtensorMap& tT, const GemmArgs& a) {
  if constexpr (MFW >= 4) {
    constexpr int smem = KCSmem<MFW, false, true>::TOTAL;
    cudaError_t e = ensure_smem(kc_gemm_pwg_kernel<MFW, true>, smem);
    if (e != cudaSuccess) return e;
    kc_gemm_pwg_kernel<MFW, true><<<grid, KCP_THREADS, smem, st>>>(tR, tL, tT, a);
    count_launch();
    return cudaGetLastError();
  } else {
    return cudaErrorNotSupported;
  }
}

template <int MFW>
cudaError_t launch_kc_t(cudaStream_t st, dim3 grid, const CUtensorMap& tR, const CUtensorMap& tL, const GemmArgs& a) {
  constexpr int smem = KCSmem<MFW, false>::TOTAL;
  // producer warpgroup (default): with the producer sleeping in the slot wait (mbar_wait_sleep) the
  // MMA warps no longer carry the TMA issue; cfg4 B = C~ A 32.07 -> 31.36 ms.  -DRS_DEV_KC_NO_PWG:
  // TMA issued by thread 0 of MMA warp 0 (A/B switch)
#ifndef RS_DEV_KC_NO_PWG
  {
    cudaError_t e = ensure_smem(kc_gemm_pwg_kernel<MFW>, smem);
    if (e != cudaSuccess) return e;
    kc_gemm_pwg_kernel<MFW><<<grid, KCP_THREADS, smem, st>>>(tR, tL, tR, a);
    count_launch();
    return cudaGetLastError();
  }
#endif
  cudaError_t e = ensure_smem(kc_gemm_kernel<MFW>, smem);
  if (e != cudaSuccess) return e;
  kc_gemm_kernel<MFW><<<grid, GEMM_THREADS, smem, st>>>(tR, tL, a);
  count_launch();
  return cudaGetLastError();
}

template <int MFW, int CS>
cudaError_t launch_phx_cs(cudaStream_t st, dim3 grid, const CUtensorMap& tR, const GemmArgs& a) {
  constexpr int smem = KCSmem<MFW, true>::TOTAL;
  {
    cudaError_t e = ensure_smem(kc_philox_kernel<MFW, CS>, smem);
    if (e != cudaSuccess) return e;
  }
  grid.x = (grid.x + CS - 1) / CS * CS;  // whole clusters along N (extra CTAs store nothing)
  cudaLaunchConfig_t cfg = {};
  cfg.gridDim = grid;
  cfg.blockDim = dim3(PHX_THREADS);
  cfg.dynamicSmemBytes = smem;
  cfg.stream = st;
  cudaLaunchAttribute attr[1];
  attr[0].id = cudaLaunchAttributeClusterDimension;
  attr[0].val.clusterDim.x = CS;
  attr[0].val.clusterDim.y = 1;
  attr[0].val.clusterDim.z = 1;
  cfg.attrs = attr;
  cfg.numAttrs = 1;
  cudaError_t e = cudaLaunchKernelEx(&cfg, kc_philox_kernel<MFW, CS>, tR, a);
  count_launch();
  return e != cudaSuccess ? e : cudaGetLastError();
}

// Cluster size for Omega sharing (-DRS_DEV_PHILOX_CLUSTER=1, 2 or 4; default 2).
#ifndef RS_DEV_PHILOX_CLUSTER
#define RS_DEV_PHILOX_CLUSTER 2
#endif
constexpr int philox_cluster() { return RS_DEV_PHILOX_CLUSTER; }
static_assert(philox_cluster() == 1 || philox_cluster() == 2 || philox_cluster() == 4, "Philox cluster size");

template <int MFW>
cudaError_t launch_phx_t(cudaStream_t st, dim3 grid, const CUtensorMap& tR, const GemmArgs& a) {
  switch (philox_cluster()) {
    case 1:
      return launch_phx_cs<MFW, 1>(st, grid, tR, a);
    case 2:
      return launch_phx_cs<MFW, 2>(st, grid, tR, a);
    default:
      return launch_phx_cs<MFW, 4>(st, grid, tR, a);
  }
}

template <int MFW, int WM>
cudaError_t launch_mc_wm(cudaStream_t st, dim3 grid, const CUtensorMap& tL, const CUtensorMap& tR, const GemmArgs& a) {
  constexpr int smem = MCSmem<MFW, WM>::TOTAL;
  for (auto fn : {mc_gemm_kernel<MFW, WM, 0>, mc_gemm_kernel<MFW, WM, 1>, mc_gemm_kernel<MFW, WM, 2>}) {
    cudaError_t e = ensure_smem(fn, smem);
    if (e != cudaSuccess) return e;
  }
  // dense 1x8 products (C = B~ A^T): dedicated producer warpgroup; -DRS_DEV_MC_NO_PWG: A/B switch
#ifdef RS_DEV_MC_NO_PWG
  constexpr bool pwg = false;
#else
  constexpr bool pwg = true;
#endif
  if (WM == 1 && a.tri == 0 && pwg) {
    cudaError_t e = ensure_smem(mc_gemm_pwg_kernel<MFW, WM, 0>, smem);
    if (e != cudaSuccess) return e;
    mc_gemm_pwg_kernel<MFW, WM, 0><<<grid, KCP_THREADS, smem, st>>>(tL, tR, a);
    count_launch();
    return cudaGetLastError();
  }
  if (a.tri == 1)
    mc_gemm_kernel<MFW, WM, 1><<<grid, GEMM_THREADS, smem, st>>>(tL, tR, a);
  else if (a.tri == 2)
    mc_gemm_kernel<MFW, WM, 2><<<grid, GEMM_THREADS, smem, st>>>(tL, tR, a);
  else
    mc_gemm_kernel<MFW, WM, 0><<<grid, GEMM_THREADS, smem, st>>>(tL, tR, a);
  count_launch();
  return cudaGetLastError();
}

template <int MFW>
cudaError_t launch_mcp_t(cudaStream_t st, int grid, const CUtensorMap& tL, const CUtensorMap& tR, const GemmArgs& a,
                         int ntn, int ntiles, int res_l) {
  constexpr int smem = MCPSmem<MFW>::TOTAL;
  for (auto fn : {mc_persist_kernel<MFW, 0>, mc_persist_kernel<MFW, 1>, mc_persist_kernel<MFW, 2>}) {
    cudaError_t e = ensure_smem(fn, smem);
    if (e != cudaSuccess) return e;
  }
  if (a.tri == 1)
    mc_persist_kernel<MFW, 1><<<grid, GEMM_THREADS, smem, st>>>(tL, tR, a, ntn, ntiles, res_l);
  else if (a.tri == 2)
    mc_persist_kernel<MFW, 2><<<grid, GEMM_THREADS, smem, st>>>(tL, tR, a, ntn, ntiles, res_l);
  else
    mc_persist_kernel<MFW, 0><<<grid, GEMM_THREADS, smem, st>>>(tL, tR, a, ntn, ntiles, res_l);
  count_launch();
  return cudaGetLastError();
}

// N boxes of the four warp columns of the persistent kernel: identity, or -- for an upper-
// triangular R in a single N tile (box b is live in stages 0..b, boxes past N never) -- the
// pairing of the 8 boxes that minimises the largest pair's live stages (exhaustive over the 105
// pairings), so no warp column sets the ring's pace alone.
void mcp_nmap(GemmArgs& a, int N, long long K, int ntn) {
  auto pack = [&](const int* m) {
    a.nmap = 0;
    for (int b = 0; b < 8; ++b) a.nmap |= static_cast<unsigned long long>(m[b]) << (8 * b);
  };
  const int ident[8] = {0, 1, 2, 3, 4, 5, 6, 7};
  pack(ident);
  if (a.tri != 2 || ntn != 1) return;
  const int nk = static_cast<int>((K + KT - 1) / KT);
  int w[8];
  for (int b = 0; b < 8; ++b) w[b] = 16 * b < N ? std::min(b + 1, nk) : 0;
  int best = 1 << 30, bestp[8] = {0, 1, 2, 3, 4, 5, 6, 7};
  int p[8];
  bool used[8] = {false};
  // recursive pairing enumeration (first unused box with each later unused box)
  auto rec = [&](auto&& self, int depth, int cur) -> void {
    if (depth == 4) {
      if (cur < best) {
        best = cur;
        for (int i = 0; i < 8; ++i) bestp[i] = p[i];
      }
      return;
    }
    int f = 0;
    while (used[f]) ++f;
    used[f] = true;
    for (int s2 = f + 1; s2 < 8; ++s2) {
      if (used[s2]) continue;
      used[s2] = true;
      p[2 * depth] = f;
      p[2 * depth + 1] = s2;
      self(self, depth + 1, std::max(cur, w[f] + w[s2]));
      used[s2] = false;
    }
    used[f] = false;
  };
  rec(rec, 0, 0);
  pack(bestp);
}

// Warp grid.  Dense (long-K) products: 1 x 8 -- each warp 16 columns and all M fragments.  The
// 2 x 4 grid (each warp half of the M fragments, the middle box split by row parity at odd MFW,
// and 32 columns; (MFW/2 + 2) instead of (MFW + 1) LDS.128 per 4 MFW DMMAs) measured slower at
// cfg4 for C = B A^T (MFW = 7): 34.4 ms vs 33.5 ms with 1 x 8 (an earlier box-granular uneven
// split: 35.8 ms).  Short-K triangular products (and the persistent kernel): 2 x 4, measured
// faster for the L^-1 C apply (0.93 vs 1.18 ms at cfg4).  -DRS_DEV_MC_WM=1 / 2 forces a grid.
#ifndef RS_DEV_MC_WM
#define RS_DEV_MC_WM 0
#endif
constexpr int mc_wm_override() { return RS_DEV_MC_WM; }
template <int MFW>
cudaError_t launch_mc_t(cudaStream_t st, dim3 grid, const CUtensorMap& tL, const CUtensorMap& tR, const GemmArgs& a) {
  if constexpr (MFW < 3) {
    return launch_mc_wm<MFW, 1>(st, grid, tL, tR, a);
  } else {
    const int wm = mc_wm_override() ? mc_wm_override() : (a.tri != 0 ? 2 : 1);
    if (wm == 2) return launch_mc_wm<MFW, 2>(st, grid, tL, tR, a);
    return launch_mc_wm<MFW, 1>(st, grid, tL, tR, a);
  }
}

template <int R>
cudaError_t launch_syrk_t(cudaStream_t st, dim3 grid, const CUtensorMap& tX, const GemmArgs& a) {
  constexpr int smem = SyrkSmem<R>::TOTAL;
  {
    cudaError_t e = ensure_smem(syrk_kernel<R>, smem);
    if (e != cudaSuccess) return e;
  }
  syrk_kernel<R><<<grid, GEMM_THREADS, smem, st>>>(tX, a);
  count_launch();
  return cudaGetLastError();
}

}  // namespace

int num_sms_cached() {
  static int sms = [] {
    int dev = 0, n = 148;
    if (cudaGetDevice(&dev) == cudaSuccess) cudaDeviceGetAttribute(&n, cudaDevAttrMultiProcessorCount, dev);
    return n;
  }();
  return sms;
}

int gemm_mtile(int M) {
  if (M <= 128) return 16 * ((M + 15) / 16);
  const int mt = (M + 127) / 128;
  return 16 * ((M + 16 * mt - 1) / (16 * mt));
}

int gemm_choose_splits(int M, int N, long long K, int max_splits, int num_sms, bool tail) {
  const long long mtiles = (M + gemm_mtile(M) - 1) / gemm_mtile(M);
  const long long tiles = mtiles * (tail && kc_tail_applies(M, N) ? N / NT : (N + NT - 1) / NT);
#ifdef RS_DEV_KC_S
  if (tail && kc_tail_applies(M, N)) return std::min(max_splits, RS_DEV_KC_S);  // A/B experiments only
#endif
  if (tiles >= 2LL * num_sms || max_splits <= 1) return 1;
#ifndef RS_DEV_KC_SPLITS_OLD
  if (tail && kc_tail_applies(M, N)) {
    // B := C~ A with the tail fold: a time model in K rows per CTA, fitted to the measured split
    // sweeps (cfg4: S = 15 / 34 / 53 -> 31.37 / 31.15 / 31.10 ms; cfg2: 1.625 / 1.643 / 1.673 ms):
    // waves * (rows per split + ~48 rows of per-CTA start-up and epilogue) + the split-K reduce
    // (one l x N partial per split, ~N / 800 rows' worth of time each)
    int bs = 1;
    double bc = 1e300;
    for (int s = 1; s <= max_splits; ++s) {
      const long long chunk = ((K + s - 1) / s + KT - 1) / KT * KT;
      if (chunk < 8 * KT && s > 1) break;
      const long long real_s = (K + chunk - 1) / chunk;
      const long long waves = (tiles * real_s + num_sms - 1) / num_sms;
      const double cost = static_cast<double>(waves) * static_cast<double>(chunk + 48) +
                          static_cast<double>(real_s) * static_cast<double>(N) / 800.0;
      if (cost < bc - 1e-9) {
        bc = cost;
        bs = static_cast<int>(real_s);
      }
    }
    return bs;
  }
#endif
  int best = 1;
  double best_score = -1.0;
  for (int s = 1; s <= max_splits; ++s) {
    const long long chunk = ((K + s - 1) / s + KT - 1) / KT * KT;
    if (chunk < 8 * KT && s > 1) break;
    const long long real_s = (K + chunk - 1) / chunk;
    const long long ctas = tiles * real_s;
    const long long waves = (ctas + num_sms - 1) / num_sms;
    const double eff = static_cast<double>(ctas) / static_cast<double>(waves * num_sms);
    const double score = eff - 0.002 * static_cast<double>(waves);
    if (score > best_score + 1e-12) {
      best_score = score;
      best = static_cast<int>(real_s);
    }
  }
  return best;
}

bool kc_tail_applies(int M, int N) {
#if defined(RS_DEV_KC_NO_PWG) || defined(RS_DEV_NO_TAIL)
  return false;  // the fold lives in the producer-warpgroup kernels only (-DRS_DEV_NO_TAIL: A/B switch)
#else
  return M >= 1 && gemm_mtile(M) >= 64 && N > NT && N % NT != 0 && N % NT <= 16;
#endif
}

long long kc_tail_elems(int M, int N, int splits) {
  if (!kc_tail_applies(M, N)) return 0;
  const int MT = gemm_mtile(M);
  const long long mtiles = (M + MT - 1) / MT;
  return static_cast<long long>(splits) * mtiles * (N / NT) * MT * 16;
}

namespace {
// out(split s)[m, tail_n0 + c] (op)= sum over the N tiles nt = 0, 1, ... of the tail partials, in
// that fixed order (bitwise reproducible); one thread per (s, m, c)
__global__ void kc_tail_reduce_kernel(const GemmArgs a, int S, int mtiles, int MT, int w) {
  const int ntn = a.tail_ntn;
  const int mrows = min(a.out.m_store, mtiles * MT);
  const long long total = static_cast<long long>(S) * mrows * w;
  for (long long i = blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x; i < total;
       i += static_cast<long long>(gridDim.x) * blockDim.x) {
    const int c = static_cast<int>(i % w);
    const int m = static_cast<int>((i / w) % mrows);
    const int s = static_cast<int>(i / (static_cast<long long>(w) * mrows));
    const int n = a.tail_n0 + c;
    if (n >= a.out.n_store) continue;
    const int mt = m / MT, row = m % MT;
    const double* tp = a.tail_p + ((static_cast<long long>(s) * mtiles + mt) * ntn * MT + row) * 16 + c;
    double v = 0.0;
    for (int nt = 0; nt < ntn; ++nt) v += tp[static_cast<long long>(nt) * MT * 16];
    gemm_put(a.out.ptr + s * a.out.split_stride + m * a.out.ld_m + n * a.out.ld_n, v, a.out.mode);
  }
}

cudaError_t kc_tail_reduce(cudaStream_t st, const GemmArgs& a, int S, int mtiles, int MT, int N) {
  const int w = N - a.tail_n0;
  const long long total = static_cast<long long>(S) * std::min(a.out.m_store, mtiles * MT) * w;
  if (total <= 0) return cudaSuccess;
  const int blocks = static_cast<int>(std::min<long long>((total + 255) / 256, 148LL * 4));
  kc_tail_reduce_kernel<<<blocks, 256, 0, st>>>(a, S, mtiles, MT, w);
  count_launch();
  return cudaGetLastError();
}
}  // namespace

int gemm_nsplit(long long K, int splits) {
  const int s = splits < 1 ? 1 : splits;
  long long chunk = ((K + s - 1) / s + KT - 1) / KT * KT;
  if (chunk < KT) chunk = KT;
  const long long ns = (K + chunk - 1) / chunk;
  return ns < 1 ? 1 : static_cast<int>(ns);
}

static GemmArgs make_args(int M, int N, long long K, int splits, const GemmOutDesc& out) {
  GemmArgs a{};
  a.M = M;
  a.N = N;
  a.K = K;
  const int s = splits < 1 ? 1 : splits;
  a.k_chunk = ((K + s - 1) / s + KT - 1) / KT * KT;
  if (a.k_chunk < KT) a.k_chunk = KT;
  a.out.ptr = out.ptr;
  a.out.ld_m = out.ld_m;
  a.out.ld_n = out.ld_n;
  a.out.split_stride = out.split_stride;
  a.out.m_store = out.m_store;
  a.out.n_store = out.n_store;
  a.out.mode = out.mode;
  return a;
}

cudaError_t gemm_kc(cudaStream_t st, int M, int N, long long K, const View2D& Lv, const View2D& Rv,
                    const PhiloxDesc& phx, const GemmOutDesc& out, int splits) {
  const int MT = gemm_mtile(M);
  const int mfw = MT / 16;
  GemmArgs a = make_args(M, N, K, splits, out);
  const long long nsplit = (K + a.k_chunk - 1) / a.k_chunk;
  if (phx.enabled) {
    a.key.k0 = static_cast<uint32_t>(phx.seed);
    a.key.k1 = static_cast<uint32_t>(phx.seed >> 32);
    a.tag = phx.tag;
    a.row_offset = phx.row_offset;
    a.ell = phx.ell;
    a.omega_row0 = phx.omega_row0;
  }
  CUtensorMap tR, tL;
  if (!make_tmap(&tR, Rv, 16, NT)) return cudaErrorInvalidValue;
  if (phx.enabled) {
    tL = tR;
  } else if (!make_tmap(&tL, Lv, 16, MT)) {
    return cudaErrorInvalidValue;
  }
  dim3 grid((N + NT - 1) / NT, (M + MT - 1) / MT, static_cast<unsigned>(nsplit < 1 ? 1 : nsplit));
  // tail fold: N / 128 full tiles share the last N % 128 columns along K
  if (!phx.enabled && out.tail_ws && kc_tail_applies(M, N) &&
      kc_tail_elems(M, N, static_cast<int>(grid.z)) <= out.tail_cap) {
    CUtensorMap tT;
    if (!make_tmap(&tT, Rv, 16, 16)) return cudaErrorInvalidValue;
    grid.x = N / NT;
    a.tail_p = out.tail_ws;
    a.tail_n0 = static_cast<int>(grid.x) * NT;
    a.tail_ntn = static_cast<int>(grid.x);
    cudaError_t e;
    switch (mfw) {
      case 4: e = launch_kc_tail_t<4>(st, grid, tR, tL, tT, a); break;
      case 5: e = launch_kc_tail_t<5>(st, grid, tR, tL, tT, a); break;
      case 6: e = launch_kc_tail_t<6>(st, grid, tR, tL, tT, a); break;
      case 7: e = launch_kc_tail_t<7>(st, grid, tR, tL, tT, a); break;
      case 8: e = launch_kc_tail_t<8>(st, grid, tR, tL, tT, a); break;
      default: return cudaErrorInvalidConfiguration;
    }
    if (e != cudaSuccess) return e;
    return kc_tail_reduce(st, a, static_cast<int>(grid.z), static_cast<int>(grid.y), MT, N);
  }
#define RS_KC(W)                                                              \
  case W:                                                                     \
    return phx.enabled ? launch_phx_t<W>(st, grid, tR, a)                     \
                       : launch_kc_t<W>(st, grid, tR, tL, a);
  switch (mfw) {
    RS_KC(1) RS_KC(2) RS_KC(3) RS_KC(4) RS_KC(5) RS_KC(6) RS_KC(7) RS_KC(8)
    default:
      return cudaErrorInvalidConfiguration;
  }
#undef RS_KC
}

cudaError_t gemm_mc(cudaStream_t st, int M, int N, long long K, const View2D& Lv, const View2D& Rv,
                    const GemmOutDesc& out, int splits, int tri) {
  const int MT = gemm_mtile(M);
  const int mfw = MT / 16;
  GemmArgs a = make_args(M, N, K, splits, out);
  a.tri = tri;
  const long long nsplit = (K + a.k_chunk - 1) / a.k_chunk;
  CUtensorMap tL, tR;
#ifdef RS_DEV_MC_NO_TMA3D
  constexpr bool no3d = true;
#else
  constexpr bool no3d = false;
#endif
  a.l3d = !no3d && make_tmap3(&tL, Lv, static_cast<uint32_t>(MT / 16));
  a.r3d = !no3d && make_tmap3(&tR, Rv, static_cast<uint32_t>(NT / 16));
  if (!a.l3d && !make_tmap(&tL, Lv, 16, 16)) return cudaErrorInvalidValue;
  if (!a.r3d && !make_tmap(&tR, Rv, 16, 16)) return cudaErrorInvalidValue;
  dim3 grid((N + NT - 1) / NT, (M + MT - 1) / MT, static_cast<unsigned>(nsplit < 1 ? 1 : nsplit));
  // short K and many tiles: persistent CTAs (the ring runs on across tiles)
#ifdef RS_DEV_MC_NO_PERSIST
  constexpr bool no_persist = true;
#else
  constexpr bool no_persist = false;
#endif
  const long long ntiles = static_cast<long long>(grid.x) * grid.y;
  // (one of the two operands must be shared by every tile: a single M tile or a single N tile)
  // (measured: at 391 tiles (m = 50 000) the resident-operand start-up costs more than it saves;
  // at 7 813 tiles (m = 1e6) the factor's X R^-1 pair drops from 2.45 to 2.25 ms)
  if (!no_persist && nsplit <= 1 && K <= 8 * KT && ntiles >= 8LL * num_sms_cached() && (grid.y == 1 || grid.x == 1)) {
    const int pgrid = static_cast<int>(std::min<long long>(ntiles, num_sms_cached()));
    const int res_l = grid.y == 1 ? 1 : 0;
    mcp_nmap(a, N, K, static_cast<int>(grid.x));
#define RS_MCP(W) \
  case W:         \
    return launch_mcp_t<W>(st, pgrid, tL, tR, a, static_cast<int>(grid.x), static_cast<int>(ntiles), res_l);
    switch (mfw) {
      RS_MCP(1) RS_MCP(2) RS_MCP(3) RS_MCP(4) RS_MCP(5) RS_MCP(6) RS_MCP(7) RS_MCP(8)
      default:
        return cudaErrorInvalidConfiguration;
    }
#undef RS_MCP
  }
#define RS_MC(W) \
  case W:        \
    return launch_mc_t<W>(st, grid, tL, tR, a);
  switch (mfw) {
    RS_MC(1) RS_MC(2) RS_MC(3) RS_MC(4) RS_MC(5) RS_MC(6) RS_MC(7) RS_MC(8)
    default:
      return cudaErrorInvalidConfiguration;
  }
#undef RS_MC
}

template <int NB>
cudaError_t launch_tsa_t(cudaStream_t st, int grid, const CUtensorMap& tX, const CUtensorMap& tU, const TsaArgs& a) {
  constexpr int smem = TsaSmem<NB>::TOTAL;
  cudaError_t e = ensure_smem(tsa_kernel<NB>, smem);
  if (e != cudaSuccess) return e;
  tsa_kernel<NB><<<grid, TSA_THREADS, smem, st>>>(tX, tU, a);
  count_launch();
  return cudaGetLastError();
}

cudaError_t gemm_tsa(cudaStream_t st, long long m, int k, const View2D& Xv, const double* W, long long ldw, double* Y,
                     long long ldy, int n_store) {
  if (k < 1 || k > 128 || m < 0) return cudaErrorNotSupported;
  if (m == 0) return cudaSuccess;
  const int NB = (k + 15) / 16;
  TsaArgs a{};
  a.y = Y;
  a.ldy = ldy;
  a.m = static_cast<int>(m);
  a.n_store = std::min(n_store, 16 * NB);
  a.ntiles = static_cast<int>((m + 127) / 128);
  CUtensorMap tX, tU;
  const View2D Uv{W, k, k, ldw};
  a.x3d = make_tmap3(&tX, Xv, 8);
  a.u3d = make_tmap3(&tU, Uv, static_cast<uint32_t>(NB));
  if (!a.x3d && !make_tmap(&tX, Xv, 16, 16)) return cudaErrorInvalidValue;
  if (!a.u3d && !make_tmap(&tU, Uv, 16, 16)) return cudaErrorInvalidValue;
  const int grid = std::min(a.ntiles, num_sms_cached());
  switch (NB) {
    case 1: return launch_tsa_t<1>(st, grid, tX, tU, a);
    case 2: return launch_tsa_t<2>(st, grid, tX, tU, a);
    case 3: return launch_tsa_t<3>(st, grid, tX, tU, a);
    case 4: return launch_tsa_t<4>(st, grid, tX, tU, a);
    case 5: return launch_tsa_t<5>(st, grid, tX, tU, a);
    case 6: return launch_tsa_t<6>(st, grid, tX, tU, a);
    case 7: return launch_tsa_t<7>(st, grid, tX, tU, a);
    default: return launch_tsa_t<8>(st, grid, tX, tU, a);
  }
}

// ---- sample GEMM with an L2 ring of Omega chunks (sample_ring.cuh) ----
SampleRingPlan sample_ring_plan(int N, long long K, int max_splits, int G) {
  SampleRingPlan p{};
  p.ntn = (N + NT - 1) / NT;
  double best = -1.0;
  for (int s = 1; s <= max_splits; ++s) {
#ifdef RS_DEV_RING_S
    if (s != RS_DEV_RING_S) continue;  // A/B experiments only
#endif
    const long long kspl = ((K + s - 1) / s + RG_CH - 1) / RG_CH * RG_CH;
    if (kspl < 4 * RG_CH && s > 1) break;  // keep >= 4 chunks (128 stages) per unit
    const int sr = static_cast<int>((K + kspl - 1) / kspl);
    const long long units = static_cast<long long>(p.ntn) * sr;
    const long long rounds = (units + G - 1) / G;
    const double eff = static_cast<double>(units) / static_cast<double>(rounds * G) - 1e-4 * sr;
    if (eff > best + 1e-12) {
      best = eff;
      p.S = sr;
      p.kspl = kspl;
      p.rounds = static_cast<int>(rounds);
    }
  }
  p.ngroups = p.S + p.rounds;  // gid = split + round < S + rounds
  return p;
}

size_t sample_ring_bytes(int M, int N, long long K, int max_splits, int G) {
  if (M < 1 || M > 128 || K < 8 * RG_CH) return 0;
  const int MT = gemm_mtile(M);
  const SampleRingPlan p = sample_ring_plan(N, K, max_splits, G);
  return static_cast<size_t>(p.ngroups) * RG_R * MT * RG_CH * 8 + 2 * static_cast<size_t>(p.ngroups) * RG_R * 4 + 256;
}

template <int MFW>
cudaError_t launch_ring_t(cudaStream_t st, int grid, const CUtensorMap& tA, const CUtensorMap& tW, const GemmArgs& a,
                          const RingArgs& rg) {
  constexpr int smem = KCSmem<MFW, false>::TOTAL;
  cudaError_t e = ensure_smem(kc_sample_ring_kernel<MFW>, smem);
  if (e != cudaSuccess) return e;
  void* args[] = {const_cast<CUtensorMap*>(&tA), const_cast<CUtensorMap*>(&tW), const_cast<GemmArgs*>(&a),
                  const_cast<RingArgs*>(&rg)};
  e = cudaLaunchCooperativeKernel(reinterpret_cast<void*>(kc_sample_ring_kernel<MFW>), dim3(grid), dim3(RG_THREADS),
                                  args, smem, st);
  count_launch();
  return e != cudaSuccess ? e : cudaGetLastError();
}

cudaError_t gemm_sample_ring(cudaStream_t st, int M, int N, long long K, const View2D& Av, const PhiloxDesc& phx,
                             const GemmOutDesc& out, int max_splits, void* ring_ws, size_t ring_bytes,
                             int* nsplit_out) {
  const int G = num_sms_cached();
  if (M < 1 || M > 128 || K < 8 * RG_CH || !phx.enabled) return cudaErrorNotSupported;
  if (sample_ring_bytes(M, N, K, max_splits, G) > ring_bytes) return cudaErrorNotSupported;
  const int MT = gemm_mtile(M);
  // (no tail fold here: measured slower with it -- 34.29 vs 32.22 ms at cfg4, 33.84 with the tail
  // DMMAs skipped -- the ring couples the members of a group)
  const SampleRingPlan p = sample_ring_plan(N, K, max_splits, G);
  const int mfw = MT / 16;
  GemmArgs a = make_args(M, N, K, p.S, out);
  a.key.k0 = static_cast<uint32_t>(phx.seed);
  a.key.k1 = static_cast<uint32_t>(phx.seed >> 32);
  a.tag = phx.tag;
  a.row_offset = phx.row_offset;
  a.ell = phx.ell;
  a.omega_row0 = phx.omega_row0;
  RingArgs rg{};
  rg.ntn = p.ntn;
  rg.S = p.S;
  rg.kspl = p.kspl;
  rg.nunits = p.ntn * p.S;
  rg.ring = static_cast<double*>(ring_ws);
  const size_t ring_elems = static_cast<size_t>(p.ngroups) * RG_R * MT * RG_CH;
  rg.ready = reinterpret_cast<unsigned int*>(rg.ring + ring_elems);
  rg.consumed = rg.ready + p.ngroups * RG_R;
  cudaError_t e = cudaMemsetAsync(rg.ready, 0, 2 * static_cast<size_t>(p.ngroups) * RG_R * 4, st);
  if (e != cudaSuccess) return e;
  CUtensorMap tA, tW;
  if (!make_tmap(&tA, Av, 16, NT)) return cudaErrorInvalidValue;
  const View2D Wv{rg.ring, RG_CH, static_cast<long long>(p.ngroups) * RG_R * MT, RG_CH};
  if (!make_tmap(&tW, Wv, 16, static_cast<uint32_t>(MT))) return cudaErrorInvalidValue;
  if (nsplit_out) *nsplit_out = p.S;
  switch (mfw) {
    case 1: return launch_ring_t<1>(st, G, tA, tW, a, rg);
    case 2: return launch_ring_t<2>(st, G, tA, tW, a, rg);
    case 3: return launch_ring_t<3>(st, G, tA, tW, a, rg);
    case 4: return launch_ring_t<4>(st, G, tA, tW, a, rg);
    case 5: return launch_ring_t<5>(st, G, tA, tW, a, rg);
    case 6: return launch_ring_t<6>(st, G, tA, tW, a, rg);
    case 7: return launch_ring_t<7>(st, G, tA, tW, a, rg);
    default: return launch_ring_t<8>(st, G, tA, tW, a, rg);
  }
}

cudaError_t gemm_syrk(cudaStream_t st, int rows, long long K, const View2D& Xv, const GemmOutDesc& out, int splits) {
  if (rows < 1 || rows > 128) return cudaErrorInvalidValue;
  const int R = (rows + 15) / 16;
  GemmArgs a = make_args(rows, rows, K, splits, out);
  const long long nsplit = (K + a.k_chunk - 1) / a.k_chunk;
  CUtensorMap tX;
  if (!make_tmap(&tX, Xv, 16, static_cast<uint32_t>(16 * R))) return cudaErrorInvalidValue;
  dim3 grid(1, 1, static_cast<unsigned>(nsplit < 1 ? 1 : nsplit));
  switch (R) {
    case 1: return launch_syrk_t<1>(st, grid, tX, a);
    case 2: return launch_syrk_t<2>(st, grid, tX, a);
    case 3: return launch_syrk_t<3>(st, grid, tX, a);
    case 4: return launch_syrk_t<4>(st, grid, tX, a);
    case 5: return launch_syrk_t<5>(st, grid, tX, a);
    case 6: return launch_syrk_t<6>(st, grid, tX, a);
    case 7: return launch_syrk_t<7>(st, grid, tX, a);
    default: return launch_syrk_t<8>(st, grid, tX, a);
  }
}

}  // namespace rs
