// Probe: single-warp latencies on sm_100a (cycles): dependent DFMA chain, DMUL, DP division,
// sqrt, LDS round trip, __syncthreads with 1024 threads, DMMA dependent chain.
#include <cstdio>
#include <cuda_runtime.h>

__global__ void lat(long long* out, double x, int n) {
  __shared__ double sm[1024];
  double a = x, b = 1.0000001, c = 1e-9;
  sm[threadIdx.x] = x;
  __syncthreads();
  long long t0, t1;
  // dependent DFMA
  t0 = clock64();
  for (int i = 0; i < n; ++i) a = fma(a, b, c);
  t1 = clock64();
  if (threadIdx.x == 0) out[0] = (t1 - t0) / n;
  // dependent DP division
  double d = a;
  t0 = clock64();
  for (int i = 0; i < n; ++i) d = 1.0 / (d + 1.0);
  t1 = clock64();
  if (threadIdx.x == 0) out[1] = (t1 - t0) / n;
  // dependent sqrt
  double s = d + 2.0;
  t0 = clock64();
  for (int i = 0; i < n; ++i) s = sqrt(s + 1.0);
  t1 = clock64();
  if (threadIdx.x == 0) out[2] = (t1 - t0) / n;
  // dependent LDS (pointer chase through smem)
  int* ism = reinterpret_cast<int*>(sm);
  __syncthreads();
  if (threadIdx.x < 32) ism[threadIdx.x] = (threadIdx.x + 1) % 32;
  __syncthreads();
  int p = threadIdx.x % 32;
  t0 = clock64();
  for (int i = 0; i < n; ++i) p = ism[p];
  t1 = clock64();
  if (threadIdx.x == 0) out[3] = (t1 - t0) / n;
  // __syncthreads
  t0 = clock64();
  for (int i = 0; i < n; ++i) __syncthreads();
  t1 = clock64();
  if (threadIdx.x == 0) out[4] = (t1 - t0) / n;
  // dependent DMUL
  double m = a;
  t0 = clock64();
  for (int i = 0; i < n; ++i) m = m * b;
  t1 = clock64();
  if (threadIdx.x == 0) out[5] = (t1 - t0) / n;
  // dependent DMMA (accumulator chain)
  double d0 = 0, d1 = 0;
  t0 = clock64();
  for (int i = 0; i < n; ++i)
    asm volatile("mma.sync.aligned.m8n8k4.row.col.f64.f64.f64.f64 {%0,%1}, {%2}, {%3}, {%0,%1};"
                 : "+d"(d0), "+d"(d1) : "d"(a), "d"(b));
  t1 = clock64();
  if (threadIdx.x == 0) out[6] = (t1 - t0) / n;
  // dependent FFMA
  float f = x;
  t0 = clock64();
  for (int i = 0; i < n; ++i) f = fmaf(f, 1.0001f, 1e-3f);
  t1 = clock64();
  if (threadIdx.x == 0) out[7] = (t1 - t0) / n;
  if (a + d + s + p + m + d0 + d1 + f == 12345.0) out[8] = 1;
}

int main() {
  long long* out;
  cudaMalloc(&out, 16 * sizeof(long long));
  long long h[16];
  const char* names[] = {"dfma", "ddiv", "dsqrt", "lds_chase", "syncthreads", "dmul", "dmma_chain", "ffma"};
  for (int threads : {32, 1024}) {
    lat<<<1, threads>>>(out, 1.5, 64);
    lat<<<1, threads>>>(out, 1.5, 4096);
    cudaMemcpy(h, out, 16 * sizeof(long long), cudaMemcpyDeviceToHost);
    printf("{\"threads\":%d", threads);
    for (int i = 0; i < 8; ++i) printf(",\"%s\":%lld", names[i], h[i]);
    printf(",\"err\":\"%s\"}\n", cudaGetErrorString(cudaGetLastError()));
  }
  return 0;
}
