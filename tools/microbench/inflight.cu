// Microbenchmark: HBM read bandwidth of a TMA bulk-copy ring vs bytes in
// flight per SM (stages x stage bytes), with and without an L2 prefetch
// (cp.async.bulk.prefetch.L2) running D bytes ahead.  One producer lane, the
// consumer warps only release the slots.  Each CTA streams its own contiguous
// range of a 2 GB buffer.
#include <cstdint>
#include <cstdio>

__device__ __forceinline__ uint32_t smem_u32(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }
__device__ __forceinline__ void wait_par(uint64_t* b, uint32_t ph) {
  uint32_t ok = 0;
  while (!ok)
    asm volatile("{ .reg .pred p; mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2; selp.u32 %0,1,0,p; }"
                 : "=r"(ok) : "r"(smem_u32(b)), "r"(ph) : "memory");
}

__global__ void __launch_bounds__(128, 1) k_ring(const char* __restrict__ g, size_t per_cta, int stages, int sb,
                                                 size_t pf_dist, int hold, unsigned long long* sink) {
  extern __shared__ __align__(128) char sm[];
  __shared__ uint64_t full[16], empty[16];
  const int warp = threadIdx.x / 32, lane = threadIdx.x & 31;
  if (threadIdx.x == 0) {
    for (int s = 0; s < stages; ++s) {
      asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(&full[s])), "r"(1));
      asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(&empty[s])), "r"(3));
    }
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  __syncthreads();
  const char* base = g + blockIdx.x * per_cta;
  const int n = int(per_cta / sb);
  unsigned long long acc = 0;
  if (warp == 0) {
    if (lane == 0) {
      size_t pf = 0;
      for (int it = 0; it < n; ++it) {
        const int s = it % stages;
        if (it >= stages) wait_par(&empty[s], ((it / stages) - 1) & 1);
        if (pf_dist) {
          const size_t want = min(per_cta, size_t(it) * sb + pf_dist);
          while (pf < want) {
            asm volatile("cp.async.bulk.prefetch.L2.global [%0], %1;" ::"l"(base + pf), "r"(sb) : "memory");
            pf += sb;
          }
        }
        asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(&full[s])), "r"(sb) : "memory");
        asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];"
                     ::"r"(smem_u32(sm + size_t(s) * sb)), "l"(base + size_t(it) * sb), "r"(sb), "r"(smem_u32(&full[s]))
                     : "memory");
      }
    }
  } else {
    for (int it = 0; it < n; ++it) {
      const int s = it % stages;
      wait_par(&full[s], (it / stages) & 1);
      acc += ((volatile int*)(sm + size_t(s) * sb))[lane];
      if (hold) { long long t0 = clock64(); while (clock64() - t0 < hold) {} }
      __syncwarp();
      if (lane == 0) asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(smem_u32(&empty[s])) : "memory");
    }
  }
  if (acc == 0x1234567) sink[0] = acc;
}

int main() {
  size_t gbytes = size_t(2) << 30;
  char* g;
  cudaMalloc(&g, gbytes);
  cudaMemset(g, 1, gbytes);
  unsigned long long* sink;
  cudaMalloc(&sink, 8);
  cudaFuncSetAttribute(k_ring, cudaFuncAttributeMaxDynamicSharedMemorySize, 200 * 1024);
  const int grid = 120;
  size_t per_cta = (gbytes / grid) & ~size_t(65535);
  for (int hold : {0, 1000, 2000})
    for (size_t pf : {size_t(0), size_t(32) << 10, size_t(64) << 10, size_t(128) << 10})
      for (int cfg = 0; cfg < 3; ++cfg) {
        int sb = cfg == 2 ? 8192 : 16384, stages = cfg == 0 ? 4 : (cfg == 1 ? 8 : 8);
        cudaEvent_t a, b;
        cudaEventCreate(&a);
        cudaEventCreate(&b);
        k_ring<<<grid, 128, stages * sb>>>(g, per_cta, stages, sb, pf, hold, sink);
        cudaEventRecord(a);
        k_ring<<<grid, 128, stages * sb>>>(g, per_cta, stages, sb, pf, hold, sink);
        cudaEventRecord(b);
        cudaEventSynchronize(b);
        float ms;
        cudaEventElapsedTime(&ms, a, b);
        printf("hold %4d clk pf %4zu KB stage %5d x %d = %3d KB: %7.1f GB/s %s\n", hold, pf >> 10, sb, stages,
               stages * sb / 1024, double(grid) * per_cta / ms / 1e6, cudaGetErrorString(cudaGetLastError()));
      }
  return 0;
}
