// Probe: does INT/FP32 work in OTHER warps slow down FP64 DMMA warps on sm_100a?
// 8 DMMA warps + G "generator" warps per CTA (1 CTA/SM).  Generator warps run independent
// Philox-like chains (IMAD.WIDE + LOP3) or FP32 FMUL/FADD chains or MUFU.  Reports DMMA TFLOP/s.
#include <cstdio>
#include <cuda_runtime.h>

template <int MODE>
__global__ void __launch_bounds__(512, 1) probe(double* out, int iters, int gen_warps, int gen_work) {
  const int warp = threadIdx.x >> 5;
  if (warp >= 8) {
    if (warp >= 8 + gen_warps) return;
    unsigned x0 = threadIdx.x, x1 = 7, x2 = 11, x3 = 13;
    float f0 = threadIdx.x * 1e-3f, f1 = 1.f, f2 = 2.f, f3 = 3.f;
    for (int it = 0; it < iters * gen_work; ++it) {
      if (MODE == 0) {  // Philox round-like: 2 IMAD.WIDE + 2 LOP3 per round, 4 lanes of ILP
        unsigned long long p0 = 0xD2511F53ull * x0, p1 = 0xCD9E8D57ull * x2;
        x0 = (unsigned)(p1 >> 32) ^ x1 ^ 0x9E3779B9u;
        x1 = (unsigned)p1;
        x2 = (unsigned)(p0 >> 32) ^ x3 ^ 0xBB67AE85u;
        x3 = (unsigned)p0;
      } else if (MODE == 1) {  // FP32 mul/add chains
        f0 = __fadd_rn(__fmul_rn(f0, 0.999f), 1e-3f);
        f1 = __fadd_rn(__fmul_rn(f1, 0.998f), 2e-3f);
        f2 = __fadd_rn(__fmul_rn(f2, 0.997f), 3e-3f);
        f3 = __fadd_rn(__fmul_rn(f3, 0.996f), 4e-3f);
      } else {  // division + sqrt (MUFU + fixups)
        f0 = __fdiv_rn(f0 + 1.f, f1 + 2.f);
        f1 = __fsqrt_rn(f1 + f0);
      }
    }
    if (x0 == 12345u || f0 == 1.2345f || f1 == 3.3f || f2 == 3.3f || f3 == 3.3f || x1 + x2 + x3 == 9u) out[0] = 1;
    return;
  }
  double a = 1.0 + threadIdx.x * 1e-9, b = 1.0 - threadIdx.x * 1e-9;
  double c[8][2];
#pragma unroll
  for (int i = 0; i < 8; ++i) c[i][0] = c[i][1] = 0;
  for (int it = 0; it < iters; ++it) {
#pragma unroll
    for (int i = 0; i < 8; ++i)
      asm volatile("mma.sync.aligned.m8n8k4.row.col.f64.f64.f64.f64 {%0,%1}, {%2}, {%3}, {%0,%1};"
                   : "+d"(c[i][0]), "+d"(c[i][1]) : "d"(a), "d"(b));
  }
  double s = 0;
#pragma unroll
  for (int i = 0; i < 8; ++i) s += c[i][0] + c[i][1];
  if (s == 1.2345) out[1] = s;
}

int main() {
  int sms = 0;
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  double* out;
  cudaMalloc(&out, 64);
  cudaEvent_t e0, e1;
  cudaEventCreate(&e0);
  cudaEventCreate(&e1);
  const int iters = 20000;
  auto run = [&](int mode, int gw, int work) {
    auto k = mode == 0 ? probe<0> : (mode == 1 ? probe<1> : probe<2>);
    k<<<sms, 512>>>(out, 10, gw, work);
    cudaDeviceSynchronize();
    float best = 1e30f;
    for (int r = 0; r < 3; ++r) {
      cudaEventRecord(e0);
      k<<<sms, 512>>>(out, iters, gw, work);
      cudaEventRecord(e1);
      cudaEventSynchronize(e1);
      float ms;
      cudaEventElapsedTime(&ms, e0, e1);
      best = ms < best ? ms : best;
    }
    const double flops = (double)sms * 8 * 32 * iters * 8 * 16.0;
    // gen instructions per DMMA instruction (per SM): gw warps * iters*work * ~4 instr / (8 warps * iters * 8 dmma)
    printf("{\"mode\":%d,\"gen_warps\":%d,\"gen_work\":%d,\"gen_instr_per_dmma\":%.2f,\"ms\":%.3f,\"dmma_tflops\":%.2f,\"err\":\"%s\"}\n",
           mode, gw, work, gw * work * 4.0 / 64.0, best, flops / best / 1e9, cudaGetErrorString(cudaGetLastError()));
  };
  run(0, 0, 0);
  for (int mode = 0; mode < 3; ++mode)
    for (int gw : {4, 8})
      for (int work : {4, 8, 16, 32}) run(mode, gw, work);
  return 0;
}
