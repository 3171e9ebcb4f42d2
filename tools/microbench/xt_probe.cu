// Probe for the TMA-streamed x-stationary SpMV design:
//  (1) how many clusters of B CTAs (1024 threads, ~210 KB smem) are co-resident;
//  (2) the HBM rate of a CTA-level TMA bulk ring of whole-chunk stages whose
//      chunks (32 lanes x L steps: f64 values [L][32], u16 columns [L][32]) are
//      consumed by 31 warps that gather x from a 75 KB shared block -- the
//      consumer side of the planned kernel, without the cluster exchange.
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o xt_probe xt_probe.cu
#include <cstdint>
#include <cstdio>
#include <vector>

__device__ __forceinline__ uint32_t smem_u32(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }
__device__ __forceinline__ void wait_par(uint64_t* b, uint32_t ph) {
  uint32_t ok = 0;
  while (!ok)
    asm volatile("{ .reg .pred p; mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2; selp.u32 %0,1,0,p; }"
                 : "=r"(ok) : "r"(smem_u32(b)), "r"(ph) : "memory");
}

constexpr int XW = 9376;  // x block (f64) = 75 KB

// stage = CPS chunks of L steps; chunk bytes = 32*L*10
template <int L, int CPS, bool GATHER>
__global__ void __launch_bounds__(1024, 1) k_xt(const char* __restrict__ g, int nstages_total, int NS,
                                               const double* __restrict__ xg, double* out) {
  extern __shared__ __align__(128) char sm[];
  __shared__ uint64_t full[16], empty[16];
  constexpr int CB = 32 * L * 10, SB = CB * CPS;
  double* xs = reinterpret_cast<double*>(sm);
  char* ring = sm + XW * 8;
  const int warp = threadIdx.x / 32, lane = threadIdx.x & 31;
  if (threadIdx.x == 0) {
    for (int s = 0; s < NS; ++s) {
      asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(&full[s])), "r"(1));
      asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(&empty[s])), "r"(CPS));
    }
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  for (int j = threadIdx.x; j < XW; j += blockDim.x) xs[j] = xg[j];
  __syncthreads();
  const char* base = g + size_t(blockIdx.x) * size_t(nstages_total) * SB;
  double acc = 0.0;
  if (warp == 31) {
    if (lane == 0) {
      for (int it = 0; it < nstages_total; ++it) {
        const int s = it % NS;
        if (it >= NS) wait_par(&empty[s], ((it / NS) - 1) & 1);
        asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(&full[s])), "r"(SB)
                     : "memory");
        asm volatile(
            "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
                smem_u32(ring + size_t(s) * SB)),
            "l"(base + size_t(it) * SB), "r"(SB), "r"(smem_u32(&full[s]))
            : "memory");
      }
    }
  } else {
    const int nchunks = nstages_total * CPS;
    for (int c = warp; c < nchunks; c += 31) {
      const int it = c / CPS, s = it % NS;
      wait_par(&full[s], (it / NS) & 1);
      const char* cb = ring + size_t(s) * SB + size_t(c % CPS) * CB;
      const double* V = reinterpret_cast<const double*>(cb);
      const uint16_t* C = reinterpret_cast<const uint16_t*>(cb + 32 * L * 8);
      double a = 0.0;
#pragma unroll
      for (int k = 0; k < L; ++k) {
        const double v = V[k * 32 + lane];
        const uint32_t col = C[k * 32 + lane];
        a = GATHER ? fma(v, xs[col % XW], a) : a + v * double(col);
      }
      acc += a;
      __syncwarp();
      if (lane == 0) asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(smem_u32(&empty[s])) : "memory");
    }
  }
  if (acc == 1.2345) out[0] = acc;
}

__global__ void k_dummy(int) {}

int main() {
  // (1) co-resident clusters
  for (int B : {1, 2, 4, 6, 8, 16})
    for (int smem : {150 * 1024, 200 * 1024, 215 * 1024}) {
      cudaFuncSetAttribute(k_xt<16, 3, true>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
      if (B > 8) cudaFuncSetAttribute(k_xt<16, 3, true>, cudaFuncAttributeNonPortableClusterSizeAllowed, 1);
      cudaLaunchConfig_t cfg = {};
      cfg.gridDim = dim3(B, 1, 1);
      cfg.blockDim = dim3(1024, 1, 1);
      cfg.dynamicSmemBytes = smem;
      cudaLaunchAttribute at[1];
      at[0].id = cudaLaunchAttributeClusterDimension;
      at[0].val.clusterDim.x = B;
      at[0].val.clusterDim.y = 1;
      at[0].val.clusterDim.z = 1;
      cfg.attrs = at;
      cfg.numAttrs = 1;
      int nc = -1;
      cudaError_t e = cudaOccupancyMaxActiveClusters(&nc, (void*)k_xt<16, 3, true>, &cfg);
      printf("cluster %2d smem %3d KB: max active clusters %3d (%3d SMs) %s\n", B, smem / 1024, nc, nc * B,
             cudaGetErrorString(e));
      cudaGetLastError();
    }
  // (2) ring rate
  const size_t gbytes = size_t(480) << 20;
  char* g;
  cudaMalloc(&g, gbytes + (64 << 20));
  cudaMemset(g, 0, gbytes + (64 << 20));
  double *xg, *out;
  cudaMalloc(&xg, XW * 8);
  cudaMemset(xg, 0, XW * 8);
  cudaMalloc(&out, 8);
  char* flush;
  cudaMalloc(&flush, 256 << 20);
  auto run = [&](auto kern, int grid, int NS, int SB, const char* name) {
    const int smem = XW * 8 + NS * SB;
    cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
    const int nst = int(gbytes / size_t(grid) / size_t(SB));
    float best = 1e9;
    for (int rep = 0; rep < 5; ++rep) {
      cudaMemset(flush, rep, 256 << 20);
      cudaEvent_t a, b;
      cudaEventCreate(&a);
      cudaEventCreate(&b);
      cudaEventRecord(a);
      kern<<<grid, 1024, smem>>>(g, nst, NS, xg, out);
      cudaEventRecord(b);
      cudaEventSynchronize(b);
      float ms;
      cudaEventElapsedTime(&ms, a, b);
      best = ms < best ? ms : best;
    }
    const double bytes = double(grid) * nst * SB;
    printf("%-22s grid %3d NS %d stage %6d B (%3d KB ring): %7.1f GB/s  %6.1f us  %s\n", name, grid, NS, SB,
           NS * SB / 1024, bytes / best / 1e6, best * 1e3, cudaGetErrorString(cudaGetLastError()));
  };
  for (int grid : {120, 144, 148}) {
    run(k_xt<16, 3, true>, grid, 7, 15360, "L16 x3 gather");
    run(k_xt<16, 3, true>, grid, 8, 15360, "L16 x3 gather");
    run(k_xt<16, 3, false>, grid, 7, 15360, "L16 x3 nogather");
    run(k_xt<12, 4, true>, grid, 7, 15360, "L12 x4 gather");
    run(k_xt<24, 2, true>, grid, 7, 15360, "L24 x2 gather");
    run(k_xt<8, 6, true>, grid, 7, 15360, "L8 x6 gather");
    run(k_xt<16, 2, true>, grid, 12, 10240, "L16 x2 gather");
  }
  return 0;
}
