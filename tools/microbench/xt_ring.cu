// Microbenchmark of the XT kernel's TMA ring in isolation:
// one 1024-thread CTA per SM, warp 0 lane 0 issues bulk copies of S bytes into
// an NS-slot ring (full/empty mbarriers + slot tags against parity ABA), the
// other 31 warps take "chunks" of C bytes in stream order (shared counter or
// round robin), wait for their stage, optionally read the chunk (LDS), and
// release it.  Reports HBM GB/s of the ring alone.
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o xt_ring xt_ring.cu
#include <cstdint>
#include <cstdio>

__device__ __forceinline__ uint32_t smem_u32(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }
__device__ __forceinline__ bool try_par(uint64_t* b, uint32_t ph) {
  uint32_t ok;
  asm volatile("{ .reg .pred p; mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2; selp.u32 %0,1,0,p; }"
               : "=r"(ok) : "r"(smem_u32(b)), "r"(ph) : "memory");
  return ok;
}
__device__ __forceinline__ void wait_par(uint64_t* b, uint32_t ph) {
  while (!try_par(b, ph)) {}
}

// mode: 0 = release at once, 1 = read every byte of the chunk (LDS.64 per lane), 2 = mode 1 + 8-B gathers
__global__ void __launch_bounds__(1024, 1) k_ring(const char* __restrict__ g, int nst, int NS, int S, int CPS,
                                                  int mode, int dyn, unsigned long long* sink, int ncons) {
  extern __shared__ __align__(128) char sm[];
  __shared__ uint64_t full[16], empty[16];
  __shared__ int tag[16];
  __shared__ int next;
  const int warp = threadIdx.x / 32, lane = threadIdx.x & 31;
  if (threadIdx.x == 0) {
    for (int s = 0; s < NS; ++s) {
      asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(&full[s])), "r"(1));
      asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(&empty[s])), "r"(CPS));
      tag[s] = -1;
    }
    next = ncons;
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  __syncthreads();
  const char* base = g + size_t(blockIdx.x) * size_t(nst) * S;
  const double* xs = reinterpret_cast<const double*>(sm + size_t(NS) * S);
  double acc = 0.0;
  if (warp == 0) {
    if (lane == 0)
      for (int s = 0; s < nst; ++s) {
        const int slot = s % NS;
        if (s >= NS) wait_par(&empty[slot], ((s / NS) - 1) & 1);
        *reinterpret_cast<volatile int*>(&tag[slot]) = s;
        asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(&full[slot])), "r"(S)
                     : "memory");
        asm volatile(
            "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
                smem_u32(sm + size_t(slot) * S)),
            "l"(base + size_t(s) * S), "r"(S), "r"(smem_u32(&full[slot]))
            : "memory");
      }
  } else if (warp <= ncons) {
    const int nch = nst * CPS, C = S / CPS;
    for (int c = warp - 1; c < nch;) {
      const int s = c / CPS, slot = s % NS;
      while (*reinterpret_cast<volatile int*>(&tag[slot]) != s) __nanosleep(64);
      wait_par(&full[slot], (s / NS) & 1);
      if (mode) {
        const char* cb = sm + size_t(slot) * S + size_t(c % CPS) * C;
        for (int o = lane * 8; o + 8 <= C; o += 256) {
          const double v = *reinterpret_cast<const double*>(cb + o);
          acc += mode == 2 ? v * xs[(__double_as_longlong(v) + o) & 4095] : v;
        }
      }
      __syncwarp();
      if (lane == 0) asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(smem_u32(&empty[slot])) : "memory");
      if (dyn) {
        int n = 0;
        if (lane == 0) n = atomicAdd(&next, 1);
        c = __shfl_sync(0xffffffffu, n, 0);
      } else {
        c += ncons;
      }
    }
  }
  if (acc == 1.2345) sink[0] = 1;
}

int main() {
  const size_t gbytes = size_t(480) << 20;
  char* g;
  cudaMalloc(&g, gbytes + (64 << 20));
  cudaMemset(g, 0, gbytes + (64 << 20));
  unsigned long long* sink;
  cudaMalloc(&sink, 8);
  char* flush;
  cudaMalloc(&flush, 256 << 20);
  cudaFuncSetAttribute(k_ring, cudaFuncAttributeMaxDynamicSharedMemorySize, 220 * 1024);
  struct Cfg { int grid, NS, S, CPS, mode, dyn, ncons, threads; };
  const Cfg cfgs[] = {{148, 7, 16384, 2, 0, 1, 31, 1024}, {148, 7, 16384, 2, 0, 1, 15, 1024},
                      {148, 7, 16384, 2, 0, 1, 7, 1024},  {148, 7, 16384, 2, 0, 1, 3, 1024},
                      {148, 7, 16384, 2, 0, 1, 1, 1024},  {148, 7, 16384, 2, 0, 1, 3, 128},
                      {148, 8, 16384, 1, 0, 1, 3, 128},   {148, 8, 16384, 1, 0, 1, 31, 1024},
                      {148, 7, 16384, 2, 1, 1, 7, 1024},  {148, 7, 16384, 2, 2, 1, 7, 1024},
                      {148, 7, 16384, 2, 2, 1, 31, 1024}};
  for (const Cfg& c : cfgs) {
    const int smem = c.NS * c.S + 32768;
    const int nst = int(gbytes / size_t(c.grid) / size_t(c.S));
    float best = 1e9;
    for (int rep = 0; rep < 5; ++rep) {
      // no write flush between launches (its dirty lines would be written back during the
      // timed kernel); the 480 MB stream is larger than L2 and read in the same order each time
      cudaEvent_t a, b;
      cudaEventCreate(&a);
      cudaEventCreate(&b);
      cudaEventRecord(a);
      k_ring<<<c.grid, c.threads, smem>>>(g, nst, c.NS, c.S, c.CPS, c.mode, c.dyn, sink, c.ncons);
      cudaEventRecord(b);
      cudaEventSynchronize(b);
      float ms;
      cudaEventElapsedTime(&ms, a, b);
      best = ms < best ? ms : best;
    }
    printf("grid %3d thr %4d consumers %2d NS %2d S %5d CPS %d mode %d dyn %d: %7.1f GB/s  %7.1f us  %s\n", c.grid,
           c.threads, c.ncons, c.NS, c.S, c.CPS, c.mode, c.dyn, double(c.grid) * nst * c.S / best / 1e6, best * 1e3, cudaGetErrorString(cudaGetLastError()));
  }
  return 0;
}
