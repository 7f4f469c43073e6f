// Probe: time the register-tile Cholesky + inverse kernel alone (n = 100, 110, 128).
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -I../paper_conf_sc_maryykltd15_b200/csrc chol_bench.cu
#include <cstdio>
#include <vector>

#include "../paper_conf_sc_maryykltd15_b200/csrc/chol.cu"

namespace rs {
void count_launch() {}
// chol.cu's 2 x 2 block path (n > 128) calls these; the probe only times n <= 128
cudaError_t small_gemm(cudaStream_t, int, int, int, const double*, long long, long long, const double*, long long,
                       long long, double*, long long, long long, bool, double) {
  return cudaErrorNotSupported;
}
cudaError_t copy_2d(cudaStream_t, const double*, long long, double*, long long, long long, long long) {
  return cudaErrorNotSupported;
}
cudaError_t ensure_func_attr(const void* fn, cudaFuncAttribute attr, int value) {
  return cudaFuncSetAttribute(fn, attr, value);
}
}  // namespace rs

int main() {
  for (int n : {54, 64, 100, 110}) {
    const int npad = (n + 15) / 16 * 16;
    std::vector<double> G(static_cast<size_t>(n) * n);
    unsigned s = 12345;
    std::vector<double> X(static_cast<size_t>(n) * 2 * n);
    for (auto& v : X) {
      s = s * 1664525u + 1013904223u;
      v = (s >> 8) * (1.0 / 16777216.0) - 0.5;
    }
    for (int i = 0; i < n; ++i)
      for (int j = 0; j < n; ++j) {
        double a = 0;
        for (int t = 0; t < 2 * n; ++t) a += X[i + t * n] * X[j + t * n];
        G[i + j * n] = a + (i == j ? 0.1 : 0.0);
      }
    double *dG, *dR, *dL;
    int* info;
    cudaMalloc(&dG, G.size() * 8);
    cudaMalloc(&dR, npad * npad * 8);
    cudaMalloc(&dL, npad * npad * 8);
    cudaMalloc(&info, 16);
    cudaMemset(info, 0, 16);
    cudaMemcpy(dG, G.data(), G.size() * 8, cudaMemcpyHostToDevice);
    const int np = (n + 3) / 4 * 4;
    const size_t smem = rs::ct_smem_doubles(np) * 8;
    for (auto fn : {rs::chol_tile_kernel<1, 256>, rs::chol_tile_kernel<1, 512>, rs::chol_tile_kernel<1, 832>,
                    rs::chol_tile_kernel<1, 1024>, rs::chol_tile_kernel<2, 416>, rs::chol_tile_kernel<2, 512>})
      cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, rs::ct_smem_doubles(128) * 8);
    const int tiles = (np / 4) * (np / 4 + 1);
    for (int nthr : {256, 512, 832, 1024, -416, -512}) {  // negative: two tiles per thread
      if (tiles > (nthr < 0 ? -2 * nthr : nthr)) continue;
      cudaEvent_t e0, e1;
      cudaEventCreate(&e0);
      cudaEventCreate(&e1);
      const int reps = 200;
      auto launch = [&] {
        if (nthr == 256) rs::chol_tile_kernel<1, 256><<<1, 256, smem>>>(dG, n, n, dR, npad, dL, npad, info, 5, npad, 0);
        else if (nthr == 512) rs::chol_tile_kernel<1, 512><<<1, 512, smem>>>(dG, n, n, dR, npad, dL, npad, info, 5, npad, 0);
        else if (nthr == 832) rs::chol_tile_kernel<1, 832><<<1, 832, smem>>>(dG, n, n, dR, npad, dL, npad, info, 5, npad, 0);
        else if (nthr == 1024) rs::chol_tile_kernel<1, 1024><<<1, 1024, smem>>>(dG, n, n, dR, npad, dL, npad, info, 5, npad, 0);
        else if (nthr == -416) rs::chol_tile_kernel<2, 416><<<1, 416, smem>>>(dG, n, n, dR, npad, dL, npad, info, 5, npad, 0);
        else rs::chol_tile_kernel<2, 512><<<1, 512, smem>>>(dG, n, n, dR, npad, dL, npad, info, 5, npad, 0);
      };
      for (int r = 0; r < 10; ++r) launch();
      cudaEventRecord(e0);
      for (int r = 0; r < reps; ++r) launch();
      cudaEventRecord(e1);
      cudaEventSynchronize(e1);
      float ms = 0;
      cudaEventElapsedTime(&ms, e0, e1);
      printf("{\"n\":%d,\"threads\":%d,\"us\":%.2f,\"err\":\"%s\"}\n", n, nthr, 1e3 * ms / reps,
             cudaGetErrorString(cudaGetLastError()));
    }
  }
  return 0;
}
