// Microbenchmark: fp64 FMA throughput of one B200 (the "alu" roofline
// denominator of NAS EP).  Every thread runs 8 independent
// DFMA chains; grid = 8 CTAs of 256 per SM.  Prints DFMA/clk/SM (clock from
// clock64 inside the kernel) and TFLOP/s (2 flop per FMA, CUDA events).
#include <cstdio>

__global__ void __launch_bounds__(256) k_dfma(int iters, double a, double b, double* sink, long long* clk) {
  double x[8];
#pragma unroll
  for (int j = 0; j < 8; ++j) x[j] = threadIdx.x * 1e-9 + j;
  const long long t0 = clock64();
  for (int i = 0; i < iters; ++i) {
#pragma unroll
    for (int j = 0; j < 8; ++j) x[j] = fma(x[j], a, b);
  }
  const long long t1 = clock64();
  double s = 0;
#pragma unroll
  for (int j = 0; j < 8; ++j) s += x[j];
  if (s == 12345.678) sink[0] = s;
  if (threadIdx.x == 0 && blockIdx.x == 0) clk[0] = t1 - t0;
}

int main() {
  int sms = 0;
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  double* sink;
  long long* clk;
  cudaMalloc(&sink, 8);
  cudaMalloc(&clk, 8);
  const int grid = 8 * sms, iters = 20000;
  k_dfma<<<grid, 256>>>(100, 0.999999, 1e-7, sink, clk);
  cudaEvent_t e0, e1;
  cudaEventCreate(&e0);
  cudaEventCreate(&e1);
  float best = 1e30f;
  long long c = 0;
  for (int r = 0; r < 5; ++r) {
    cudaEventRecord(e0);
    k_dfma<<<grid, 256>>>(iters, 0.999999, 1e-7, sink, clk);
    cudaEventRecord(e1);
    cudaEventSynchronize(e1);
    float ms;
    cudaEventElapsedTime(&ms, e0, e1);
    if (ms < best) best = ms;
  }
  cudaMemcpy(&c, clk, 8, cudaMemcpyDeviceToHost);
  const double fmas = (double)grid * 256 * iters * 8;
  printf("{\"sms\": %d, \"dfma_per_clk_per_sm\": %.2f, \"tflops_fp64\": %.2f, \"ms\": %.3f, \"cta_clk\": %lld}\n",
         sms, fmas / sms / (double)c, 2 * fmas / (best * 1e-3) / 1e12, best, c);
  return 0;
}
