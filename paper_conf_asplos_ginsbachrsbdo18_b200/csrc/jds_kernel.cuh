// jds_kernel.cuh -- SpMV on the jagged-diagonal JDS-32 layout (Parboil spmv's
// "unusual sparse matrix format"; reading R34; SURVEY 8(f)
// NEXT-4).  No code here is shared with oracle/.
//
// Layout: rows sorted by decreasing length (perm), slices of 32 sorted rows,
// diagonal k stored contiguously for all positions of the slices that reach
// it.  A warp owns a slice, lane = row: every diagonal step is one coalesced
// load of 32 consecutive values and 32 consecutive column indices, and the
// warp never diverges (all rows of a slice run zcnt steps; the shorter ones
// on zero padding).  Long slices (the power-law head: rows up to 10,000) are
// cut into units of <= JDS_SEG diagonal steps so no warp serialises a whole
// 10,000-step row; the units of one slice write per-lane partials that a
// fix-up pass adds in unit order (deterministic, no atomics).
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

#include "common.cuh"

namespace spmv {

#ifndef JDS_SEG_DEF
#define JDS_SEG_DEF 64
#endif
constexpr int JDS_SEG = JDS_SEG_DEF;  // diagonal steps per warp unit
constexpr int JDS_THREADS = 256;
#ifndef JDS_PRED
#define JDS_PRED 1
#endif
#ifndef JDS_B
#define JDS_B 4   // diagonal steps per predicated batch
#endif

// unit: {slice, k0, k1, part}; part < 0: the slice's only unit (writes y)
template <typename T>
__global__ void __launch_bounds__(JDS_THREADS)
k_spmv_jds(const int4* __restrict__ units, int nunits, int64_t m, const long long* __restrict__ jds_ptr,
           const int32_t* __restrict__ idx, const T* __restrict__ data, const T* __restrict__ x,
           const int32_t* __restrict__ perm, T* __restrict__ y, double alpha, double beta,
           double* __restrict__ parts) {
  const int warp = (int)(((int64_t)blockIdx.x * JDS_THREADS + threadIdx.x) >> 5);
  const int lane = threadIdx.x & 31;
  if (warp >= nunits) return;
  const int4 u = units[warp];
  const int64_t i = (int64_t)u.x * 32 + lane;
  double acc = 0.0;
#if JDS_PRED
  // batches of JDS_B steps, the tail batch predicated (no step-by-step tail)
  for (int k = u.y; k < u.z; k += JDS_B) {
    long long jp[JDS_B];
#pragma unroll
    for (int q = 0; q < JDS_B; ++q) jp[q] = k + q < u.z ? __ldg(jds_ptr + k + q) : 0;
    T d[JDS_B];
    int c[JDS_B];
#pragma unroll
    for (int q = 0; q < JDS_B; ++q) {
      d[q] = T(0);
      c[q] = 0;
      if (k + q < u.z) {
        d[q] = ld_stream(data + jp[q] + i);
        c[q] = ld_stream(idx + jp[q] + i);
      }
    }
    T xv[JDS_B];
#pragma unroll
    for (int q = 0; q < JDS_B; ++q) xv[q] = ld_x(x + c[q]);   // c = 0 on masked steps (x[0] valid)
#pragma unroll
    for (int q = 0; q < JDS_B; ++q)
      if (k + q < u.z) acc = fma((double)d[q], (double)xv[q], acc);
  }
#else
  int k = u.y;
  for (; k + 4 <= u.z; k += 4) {
    T d[4];
    int c[4];
#pragma unroll
    for (int q = 0; q < 4; ++q) {
      const int64_t j = __ldg(jds_ptr + k + q) + i;
      d[q] = ld_stream(data + j);
      c[q] = ld_stream(idx + j);
    }
    T xv[4];
#pragma unroll
    for (int q = 0; q < 4; ++q) xv[q] = ld_x(x + c[q]);
#pragma unroll
    for (int q = 0; q < 4; ++q) acc = fma((double)d[q], (double)xv[q], acc);
  }
  for (; k < u.z; ++k) {
    const int64_t j = __ldg(jds_ptr + k) + i;
    acc = fma((double)ld_stream(data + j), (double)ld_x(x + ld_stream(idx + j)), acc);
  }
#endif
  if (u.w < 0) {
    if (i < m) {
      const int row = perm[i];
      const double yo = beta != 0.0 ? beta * (double)y[row] : 0.0;
      y[row] = (T)(alpha * acc + yo);
    }
  } else {
    parts[(int64_t)u.w * 32 + lane] = acc;
  }
}

// fix-up of the split slices: {slice, first part, #parts}
template <typename T>
__global__ void __launch_bounds__(JDS_THREADS)
k_jds_fixup(const int4* __restrict__ fix, int nfix, int64_t m, const double* __restrict__ parts,
            const int32_t* __restrict__ perm, T* __restrict__ y, double alpha, double beta) {
  const int warp = (int)(((int64_t)blockIdx.x * JDS_THREADS + threadIdx.x) >> 5);
  const int lane = threadIdx.x & 31;
  if (warp >= nfix) return;
  const int4 f = fix[warp];
  const int64_t i = (int64_t)f.x * 32 + lane;
  double acc = 0.0;
  for (int p = 0; p < f.z; ++p) acc += parts[(int64_t)(f.y + p) * 32 + lane];
  if (i < m) {
    const int row = perm[i];
    const double yo = beta != 0.0 ? beta * (double)y[row] : 0.0;
    y[row] = (T)(alpha * acc + yo);
  }
}

}  // namespace spmv
