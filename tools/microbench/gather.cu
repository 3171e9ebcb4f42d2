// Microbenchmark: random 8-byte gather throughput on B200 (design input for
// the SpMV x-gather path).  Modes:
//   0: LDG from a 1.2 MB array (L2/L1)       -- the vector kernel's x path
//   1: LDS from own shared memory (150 KB)   -- x-stationary
//   2: DSMEM ld.shared::cluster from a random CTA of an 8-CTA cluster
//   3: DSMEM, own CTA only (mapa to self)
// Each thread performs ITERS dependent-free gathers with U in flight.
#include <cstdio>
#include <cstdint>
#include <cooperative_groups.h>
namespace cg = cooperative_groups;

constexpr int THREADS = 1024;
constexpr int ITERS = 2048;
constexpr int U = 8;
constexpr int SM_ELEMS = 18750;  // 150 KB of doubles

__device__ __forceinline__ uint32_t hash(uint32_t x) {
  x ^= x >> 16; x *= 0x7feb352dU; x ^= x >> 15; x *= 0x846ca68bU; x ^= x >> 16; return x;
}

template <int MODE>
__global__ void __launch_bounds__(THREADS, 1) k_gather(const double* __restrict__ g, int n, double* out) {
  extern __shared__ double xs[];
  cg::cluster_group cl = cg::this_cluster();
  for (int i = threadIdx.x; i < SM_ELEMS; i += blockDim.x) xs[i] = g[i % n] + blockIdx.x;
  cl.sync();
  uint32_t st = hash(blockIdx.x * THREADS + threadIdx.x);
  double acc = 0;
  for (int it = 0; it < ITERS; it += U) {
    double v[U];
#pragma unroll
    for (int u = 0; u < U; ++u) {
      st = hash(st + u);
      if (MODE == 0) v[u] = __ldg(g + (st % n));
      else if (MODE == 1) v[u] = xs[st % SM_ELEMS];
      else if (MODE == 2) v[u] = *cl.map_shared_rank(xs + ((st >> 3) % SM_ELEMS), st & 7);
      else v[u] = *cl.map_shared_rank(xs + (st % SM_ELEMS), cl.block_rank());
    }
#pragma unroll
    for (int u = 0; u < U; ++u) acc += v[u];
  }
  cl.sync();
  if (acc == 12345.0) out[0] = acc;
}

template <int MODE>
float run(const double* g, int n, double* out, int grid) {
  cudaLaunchConfig_t cfg = {};
  cfg.gridDim = grid; cfg.blockDim = THREADS; cfg.dynamicSmemBytes = SM_ELEMS * 8;
  cudaLaunchAttribute at[1];
  at[0].id = cudaLaunchAttributeClusterDimension;
  at[0].val.clusterDim.x = 8; at[0].val.clusterDim.y = 1; at[0].val.clusterDim.z = 1;
  cfg.attrs = at; cfg.numAttrs = 1;
  cudaFuncSetAttribute(k_gather<MODE>, cudaFuncAttributeMaxDynamicSharedMemorySize, SM_ELEMS * 8);
  cudaEvent_t a, b; cudaEventCreate(&a); cudaEventCreate(&b);
  cudaLaunchKernelEx(&cfg, k_gather<MODE>, g, n, out);
  cudaEventRecord(a);
  for (int r = 0; r < 5; ++r) cudaLaunchKernelEx(&cfg, k_gather<MODE>, g, n, out);
  cudaEventRecord(b); cudaEventSynchronize(b);
  float ms; cudaEventElapsedTime(&ms, a, b);
  cudaError_t e = cudaGetLastError();
  if (e != cudaSuccess) printf("error %s\n", cudaGetErrorString(e));
  return ms / 5;
}

int main() {
  int n = 150000;
  double *g, *out;
  cudaMalloc(&g, n * 8); cudaMemset(g, 0, n * 8); cudaMalloc(&out, 8);
  int clk; cudaDeviceGetAttribute(&clk, cudaDevAttrClockRate, 0);
  for (int grid : {8, 120}) {
    double gathers = double(grid) * THREADS * ITERS;
    float t0 = run<0>(g, n, out, grid), t1 = run<1>(g, n, out, grid), t2 = run<2>(g, n, out, grid),
          t3 = run<3>(g, n, out, grid);
    const char* nm[4] = {"LDG 1.2MB", "LDS local", "DSMEM random peer", "DSMEM self"};
    float ts[4] = {t0, t1, t2, t3};
    for (int m = 0; m < 4; ++m)
      printf("grid %3d %-18s %8.3f ms  %.3f gathers/clk/SM (clk %.0f MHz nominal)\n", grid, nm[m], ts[m],
             gathers / grid / (ts[m] * 1e-3 * clk * 1e3), clk / 1e3);
  }
  return 0;
}
