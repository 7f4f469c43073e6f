// Probe 0: FP64 DMMA vs DFMA throughput on sm_100a.
// Register-only loops; reports TFLOP/s per variant.  Build:
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o probes/fp64_peak probes/fp64_peak.cu
#include <cstdio>
#include <cuda_runtime.h>

template <int NACC>
__global__ void dmma_loop(double* out, int iters) {
  double a = 1.0 + threadIdx.x * 1e-9, b = 1.0 - threadIdx.x * 1e-9;
  double c[NACC][2];
#pragma unroll
  for (int i = 0; i < NACC; ++i) { c[i][0] = 0; c[i][1] = 0; }
  for (int it = 0; it < iters; ++it) {
#pragma unroll
    for (int i = 0; i < NACC; ++i) {
      asm volatile("mma.sync.aligned.m8n8k4.row.col.f64.f64.f64.f64 {%0,%1}, {%2}, {%3}, {%0,%1};"
                   : "+d"(c[i][0]), "+d"(c[i][1]) : "d"(a), "d"(b));
    }
  }
  double s = 0;
#pragma unroll
  for (int i = 0; i < NACC; ++i) s += c[i][0] + c[i][1];
  if (s == 12345.678) out[threadIdx.x] = s;
}

template <int NACC>
__global__ void dfma_loop(double* out, int iters) {
  double a = 1.0 + threadIdx.x * 1e-9, b = 1.0 - threadIdx.x * 1e-9;
  double c[NACC];
#pragma unroll
  for (int i = 0; i < NACC; ++i) c[i] = i;
  for (int it = 0; it < iters; ++it) {
#pragma unroll
    for (int i = 0; i < NACC; ++i) c[i] = fma(a, c[i], b);
  }
  double s = 0;
#pragma unroll
  for (int i = 0; i < NACC; ++i) s += c[i];
  if (s == 12345.678) out[threadIdx.x] = s;
}

// DMMA + concurrent FP32/INT work (Philox-like) in the same warp: does generation steal from DMMA?
template <int NACC>
__global__ void dmma_plus_int(double* out, int iters) {
  double a = 1.0 + threadIdx.x * 1e-9, b = 1.0 - threadIdx.x * 1e-9;
  double c[NACC][2];
  unsigned x = threadIdx.x, y = 12345u;
  float f = threadIdx.x * 0.5f;
#pragma unroll
  for (int i = 0; i < NACC; ++i) { c[i][0] = 0; c[i][1] = 0; }
  for (int it = 0; it < iters; ++it) {
#pragma unroll
    for (int i = 0; i < NACC; ++i) {
      asm volatile("mma.sync.aligned.m8n8k4.row.col.f64.f64.f64.f64 {%0,%1}, {%2}, {%3}, {%0,%1};"
                   : "+d"(c[i][0]), "+d"(c[i][1]) : "d"(a), "d"(b));
      x = __umulhi(x, 0xD2511F53u) ^ y; y = y * 0xCD9E8D57u + x;
      f = __fmaf_rn(f, 0.999f, 0.001f);
    }
  }
  double s = 0;
#pragma unroll
  for (int i = 0; i < NACC; ++i) s += c[i][0] + c[i][1];
  if (s == 12345.678 || x == 7u || f == 3.0f) out[threadIdx.x] = s + x + f;
}

int main() {
  int dev = 0; cudaDeviceProp p; cudaGetDeviceProperties(&p, dev);
  int clk = 0; cudaDeviceGetAttribute(&clk, cudaDevAttrClockRate, dev);
  int l2 = 0; cudaDeviceGetAttribute(&l2, cudaDevAttrL2CacheSize, dev);
  printf("{\"gpu\":\"%s\",\"sms\":%d,\"clock_khz\":%d,\"l2_bytes\":%d,\"smem_optin\":%zu}\n", p.name,
         p.multiProcessorCount, clk, l2, p.sharedMemPerBlockOptin);
  double* out; cudaMalloc(&out, 4096 * sizeof(double));
  cudaEvent_t e0, e1; cudaEventCreate(&e0); cudaEventCreate(&e1);
  int sms = p.multiProcessorCount;
  auto run = [&](const char* name, void (*k)(double*, int), int blocks, int threads, int iters, double flop_per_thread_iter) {
    k<<<blocks, threads>>>(out, 10); cudaDeviceSynchronize();
    float best = 1e30f;
    for (int r = 0; r < 5; ++r) {
      cudaEventRecord(e0); k<<<blocks, threads>>>(out, iters); cudaEventRecord(e1); cudaEventSynchronize(e1);
      float ms; cudaEventElapsedTime(&ms, e0, e1); if (ms < best) best = ms;
    }
    double flops = (double)blocks * threads * iters * flop_per_thread_iter;
    printf("{\"kernel\":\"%s\",\"blocks\":%d,\"threads\":%d,\"ms\":%.4f,\"tflops\":%.3f,\"err\":\"%s\"}\n", name, blocks,
           threads, best, flops / best / 1e9, cudaGetErrorString(cudaGetLastError()));
  };
  // m8n8k4: 8*8*4 = 256 FMA = 512 flop per warp instruction -> 16 flop per thread per mma
  for (int th : {128, 256, 512, 1024}) {
    run("dmma_acc8_sweep", dmma_loop<8>, sms * 4, th, 20000, 8 * 16.0);
  }
  run("dmma_acc4_b256", dmma_loop<4>, sms * 8, 256, 40000, 4 * 16.0);
  run("dmma_acc8_b256", dmma_loop<8>, sms * 8, 256, 20000, 8 * 16.0);
  run("dmma_acc16_b256", dmma_loop<16>, sms * 8, 256, 10000, 16 * 16.0);
  run("dmma_acc8_b128x1", dmma_loop<8>, sms, 128, 20000, 8 * 16.0);
  run("dmma_acc8_b256x1", dmma_loop<8>, sms, 256, 20000, 8 * 16.0);
  run("dfma_acc8_b256", dfma_loop<8>, sms * 8, 256, 20000, 8 * 2.0);
  run("dfma_acc16_b256", dfma_loop<16>, sms * 8, 256, 10000, 16 * 2.0);
  run("dfma_acc16_b512x2", dfma_loop<16>, sms * 2, 512, 10000, 16 * 2.0);
  run("dmma_plus_int_acc8_b256", dmma_plus_int<8>, sms * 8, 256, 20000, 8 * 16.0);
  return 0;
}
