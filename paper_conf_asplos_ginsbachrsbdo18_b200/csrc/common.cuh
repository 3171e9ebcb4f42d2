// common.cuh -- device helpers shared by the library's kernels (sm_100a).
// No code here is shared with oracle/ (the CPU oracle is a separate C file).
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

namespace spmv {

constexpr int kNumSMs = 148;  // B200: 2 dies x 74 SMs (queried at run time too)

__device__ __forceinline__ int64_t cmin64(int64_t a, int64_t b) { return a < b ? a : b; }
__device__ __forceinline__ int64_t cmax64(int64_t a, int64_t b) { return a > b ? a : b; }

// ---------------------------------------------------------------- loads
// Streamed operands (vals, colidx) are read exactly once per SpMV: bypass L1
// so the L1 capacity is left to the x gathers (ld.global.nc.L1::no_allocate).
__device__ __forceinline__ double ld_stream(const double* p) {
  double v;
  asm("ld.global.nc.L1::no_allocate.f64 %0, [%1];" : "=d"(v) : "l"(p));
  return v;
}
__device__ __forceinline__ float ld_stream(const float* p) {
  float v;
  asm("ld.global.nc.L1::no_allocate.f32 %0, [%1];" : "=f"(v) : "l"(p));
  return v;
}
__device__ __forceinline__ int ld_stream(const int* p) {
  int v;
  asm("ld.global.nc.L1::no_allocate.s32 %0, [%1];" : "=r"(v) : "l"(p));
  return v;
}
// x gathers: read-only path, L1-allocating (x is re-read across rows).
template <typename T>
__device__ __forceinline__ T ld_x(const T* p) { return __ldg(p); }

// ------------------------------------------------------------ reductions
template <int G>
__device__ __forceinline__ double group_sum(double v, unsigned mask) {
#pragma unroll
  for (int off = G / 2; off > 0; off >>= 1) v += __shfl_xor_sync(mask, v, off, G);
  return v;
}

__device__ __forceinline__ double warp_sum(double v) {
#pragma unroll
  for (int off = 16; off > 0; off >>= 1) v += __shfl_xor_sync(0xffffffffu, v, off);
  return v;
}

// Deterministic block sum (fixed tree); result valid in every thread.
// `red` must hold >= blockDim.x/32 doubles.
__device__ __forceinline__ double block_sum(double v, double* red) {
  const int lane = threadIdx.x & 31, wid = threadIdx.x >> 5, nw = blockDim.x >> 5;
  v = warp_sum(v);
  __syncthreads();
  if (lane == 0) red[wid] = v;
  __syncthreads();
  double t = (lane < nw) ? red[lane] : 0.0;
  t = warp_sum(t);
  return t;
}

// Deterministic sum over the first nw warps of the block only (named barrier
// 1), for warp-specialised kernels whose other warps do not participate.
__device__ __forceinline__ double block_sum_n(double v, double* red, int nw) {
  const int lane = threadIdx.x & 31, wid = threadIdx.x >> 5;
  v = warp_sum(v);
  asm volatile("bar.sync 1, %0;\n" ::"r"(nw * 32) : "memory");
  if (lane == 0) red[wid] = v;
  asm volatile("bar.sync 1, %0;\n" ::"r"(nw * 32) : "memory");
  double t = (lane < nw) ? red[lane] : 0.0;
  t = warp_sum(t);
  return t;
}

// A scalar source for the CG kernels: either `count` per-block partials to be
// summed (single GPU: every consuming block sums them in the same fixed order,
// so all blocks see bit-identical scalars), or count == 1 pointing at a
// finalized (and, in distributed mode, NCCL-all-reduced) value.
struct SumSrc {
  const double* p;
  int count;
};

// Sum of a SumSrc by warp 0 of the block; returns the value in every thread.
__device__ __forceinline__ double read_sum(SumSrc s, double* slot) {
  if (threadIdx.x < 32) {
    double a = 0.0;
    for (int i = threadIdx.x; i < s.count; i += 32) a += s.p[i];
    a = warp_sum(a);
    if (threadIdx.x == 0) *slot = a;
  }
  __syncthreads();
  double v = *slot;
  return v;
}

}  // namespace spmv
