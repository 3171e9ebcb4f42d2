// Minimal 3-D TMA tile load check: tma3d BX BY C0 C1 [grid_const=1|global=0]
#include <cuda.h>
#include <cuda_runtime.h>
#include <cstdio>
#include <cstdlib>
#include <cstdint>
__device__ __forceinline__ uint32_t sa(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }
__global__ void k(const __grid_constant__ CUtensorMap tm, const CUtensorMap* gtm, int use_g, int c0, int c1, int bytes, double* out) {
  __shared__ __align__(128) double buf[4096];
  __shared__ __align__(8) uint64_t bar;
  if (threadIdx.x == 0) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(sa(&bar)));
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  __syncthreads();
  const uint64_t t = use_g ? reinterpret_cast<uint64_t>(gtm) : reinterpret_cast<uint64_t>(&tm);
  if (threadIdx.x == 0) {
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(sa(&bar)), "r"(bytes) : "memory");
    asm volatile("cp.async.bulk.tensor.3d.shared::cluster.global.tile.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3, %4}], [%5];"
                 ::"r"(sa(buf)), "l"(t), "r"(c0), "r"(c1), "r"(0), "r"(sa(&bar)) : "memory");
  }
  uint32_t ok = 0;
  for (long i = 0; i < 100000000 && !ok; ++i)
    asm volatile("{.reg .pred p; mbarrier.try_wait.parity.shared::cta.b64 p, [%1], 0; selp.u32 %0,1,0,p;}" : "=r"(ok) : "r"(sa(&bar)) : "memory");
  if (!ok) { if (threadIdx.x == 0) printf("timeout\n"); return; }
  for (int i = threadIdx.x; i < bytes / 8; i += blockDim.x) out[i] = buf[i];
}
int main(int argc, char** argv) {
  int bx = atoi(argv[1]), by = atoi(argv[2]), c0 = atoi(argv[3]), c1 = atoi(argv[4]), use_g = argc > 5 ? atoi(argv[5]) : 0;
  const int nx = 256, ny = 256, nz = 4;
  double* x; cudaMalloc(&x, sizeof(double) * nx * ny * nz);
  double* h = (double*)malloc(sizeof(double) * nx * ny * nz);
  for (int i = 0; i < nx * ny * nz; ++i) h[i] = i + 1;
  cudaMemcpy(x, h, sizeof(double) * nx * ny * nz, cudaMemcpyHostToDevice);
  CUtensorMap tm;
  cuuint64_t dims[3] = {nx, ny, nz}, str[2] = {nx * 8, (cuuint64_t)nx * ny * 8};
  cuuint32_t box[3] = {(cuuint32_t)bx, (cuuint32_t)by, 1}, es[3] = {1, 1, 1};
  CUresult r = cuTensorMapEncodeTiled(&tm, CU_TENSOR_MAP_DATA_TYPE_FLOAT64, 3, x, dims, str, box, es, CU_TENSOR_MAP_INTERLEAVE_NONE,
                                      CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_L2_128B, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  printf("encode %d\n", (int)r);
  CUtensorMap* g; cudaMalloc(&g, sizeof(tm)); cudaMemcpy(g, &tm, sizeof(tm), cudaMemcpyHostToDevice);
  double* out; cudaMalloc(&out, 8 * 4096);
  int bytes = bx * by * 8;
  k<<<1, 128>>>(tm, g, use_g, c0, c1, bytes, out);
  cudaError_t e = cudaDeviceSynchronize();
  printf("bx %d by %d c0 %d c1 %d g %d: %s\n", bx, by, c0, c1, use_g, cudaGetErrorString(e));
  if (e == cudaSuccess) {
    double o[4096]; cudaMemcpy(o, out, bytes, cudaMemcpyDeviceToHost);
    printf("  o[0..2] %g %g %g  row1: %g %g %g %g  last %g\n", o[0], o[1], o[2], o[bx], o[bx + 1], o[bx + 2], o[bx + 3], o[bx * by - 1]);
  }
  return 0;
}
