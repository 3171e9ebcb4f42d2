// Microbenchmark: per-SM throughput of many small TMA 1-D bulk copies
// (cp.async.bulk global->shared, mbarrier complete_tx) of S bytes each, issued
// by the 32 lanes of one producer warp, from random 16-B aligned offsets of a
// 1 GB buffer (HBM-resident).  Reports GB/s and copies/clk/SM.
#include <cstdint>
#include <cstdio>

__device__ __forceinline__ uint32_t smem_u32(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }
__device__ __forceinline__ uint32_t hash(uint32_t x) {
  x ^= x >> 16; x *= 0x7feb352dU; x ^= x >> 15; x *= 0x846ca68bU; x ^= x >> 16; return x;
}

constexpr int STAGES = 4;
constexpr int STAGE_BYTES = 48 * 1024;

__global__ void __launch_bounds__(128, 1) k_bulk(const char* __restrict__ g, size_t gbytes, int S, int copies_per_cta,
                                                 int contiguous, unsigned long long* sink) {
  extern __shared__ __align__(128) char sm[];
  __shared__ uint64_t full[STAGES], empty[STAGES];
  const int warp = threadIdx.x / 32, lane = threadIdx.x & 31;
  const int per_stage = STAGE_BYTES / S;  // copies per stage
  if (threadIdx.x == 0) {
    for (int s = 0; s < STAGES; ++s) {
      asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(&full[s])), "r"(1));
      asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(&empty[s])), "r"(96));
    }
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  __syncthreads();
  const int nstage_iters = copies_per_cta / per_stage;
  unsigned long long acc = 0;
  if (warp == 0) {
    // producer
    for (int it = 0; it < nstage_iters; ++it) {
      const int s = it % STAGES;
      const uint32_t ph = (it / STAGES) & 1;
      if (it >= STAGES) {
        uint32_t ok = 0;
        while (!ok) asm volatile("{ .reg .pred p; mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2; selp.u32 %0,1,0,p; }"
                                 : "=r"(ok) : "r"(smem_u32(&empty[s])), "r"(ph ^ 1) : "memory");
      }
      if (lane == 0)
        asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(&full[s])),
                     "r"(per_stage * S) : "memory");
      __syncwarp();
      for (int c = lane; c < per_stage; c += 32) {
        size_t off;
        if (contiguous) off = ((size_t)blockIdx.x * copies_per_cta + (size_t)it * per_stage + c) * S % gbytes;
        else off = ((size_t)hash(blockIdx.x * 7919u + it * 131u + c) * 16) % (gbytes - S);
        off &= ~size_t(15);
        asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];"
                     ::"r"(smem_u32(sm + s * STAGE_BYTES + c * S)), "l"(g + off), "r"(S), "r"(smem_u32(&full[s]))
                     : "memory");
      }
    }
  } else {
    for (int it = 0; it < nstage_iters; ++it) {
      const int s = it % STAGES;
      const uint32_t ph = (it / STAGES) & 1;
      uint32_t ok = 0;
      while (!ok) asm volatile("{ .reg .pred p; mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2; selp.u32 %0,1,0,p; }"
                               : "=r"(ok) : "r"(smem_u32(&full[s])), "r"(ph) : "memory");
      acc += ((volatile int*)(sm + s * STAGE_BYTES))[threadIdx.x];
      asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(smem_u32(&empty[s])) : "memory");
    }
  }
  if (acc == 0x1234567) sink[0] = acc;
}

int main() {
  size_t gbytes = size_t(1) << 30;
  char* g;
  cudaMalloc(&g, gbytes);
  cudaMemset(g, 1, gbytes);
  unsigned long long* sink;
  cudaMalloc(&sink, 8);
  int sms;
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  cudaFuncSetAttribute(k_bulk, cudaFuncAttributeMaxDynamicSharedMemorySize, STAGES * STAGE_BYTES);
  for (int contiguous : {1, 0})
    for (int S : {128, 256, 512, 1024, 4096, 16384}) {
      int per_stage = STAGE_BYTES / S;
      int copies = per_stage * 200;
      cudaEvent_t a, b;
      cudaEventCreate(&a);
      cudaEventCreate(&b);
      k_bulk<<<sms, 128, STAGES * STAGE_BYTES>>>(g, gbytes, S, copies, contiguous, sink);
      cudaEventRecord(a);
      k_bulk<<<sms, 128, STAGES * STAGE_BYTES>>>(g, gbytes, S, copies, contiguous, sink);
      cudaEventRecord(b);
      cudaEventSynchronize(b);
      float ms;
      cudaEventElapsedTime(&ms, a, b);
      double bytes = double(sms) * copies * S;
      printf("%s S=%5d B: %.3f ms  %7.1f GB/s  %.4f copies/clk/SM  err=%s\n", contiguous ? "contig" : "random", S, ms,
             bytes / ms / 1e6, double(copies) / (ms * 1e-3 * 1.9e9), cudaGetErrorString(cudaGetLastError()));
    }
  return 0;
}
