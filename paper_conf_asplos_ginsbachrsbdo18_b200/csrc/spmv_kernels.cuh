// spmv_kernels.cuh -- CSR SpMV kernels for sm_100a (no tensor cores: SpMV is
// not a dense contraction; it is HBM-bound at 2 flop / 12 B for fp64).
//
// All kernels compute, for each row i they own (Fig. 4; alpha/beta
// of DotProductLoop):
//     y[i] = alpha * sum_{k=rowptr[i]}^{rowptr[i+1]-1} vals[k]*x[colidx[k]] + beta*y[i]
// with k absolute (rowptr[0] may be != 0), rows accumulated in double (also
// for fp32 data, rounded once), beta == 0 meaning y is write-only.
//
// Optional fused epilogue (CG): DOT=true also accumulates
// sum_i w[i]*y[i] (w = p, giving p.q) into one double partial per CTA,
// part[blockIdx.x]; rows are assigned to CTAs by a fixed grid-stride so the
// partials (and the CG scalars) are deterministic.
#pragma once
#include "common.cuh"

namespace spmv {

struct SpmvArgs {
  int64_t m;              // rows to process (local rows in distributed mode)
  const int* rowptr;      // rowptr[0..m], absolute k
  const int* colidx;      // indexed by absolute k
  const void* vals;       // indexed by absolute k
  const void* x;
  void* y;
  double alpha, beta;
  const void* w;          // DOT: w[i] for local row i
  double* part;           // DOT: one partial per CTA
  P2PHook hk;             // p2p transport: wait for x / push the dot (common.cuh)
};

// ----------------------------------------------------------------------------
// VECTOR<G, U>: G lanes (a power of two, 1..32) cooperate on one row; each
// lane streams U strided elements per step with all loads issued before any
// use (U independent colidx->x gather chains per lane), guarded, so a row of
// L elements takes ceil(L/(G*U)) steps.  The G-lane partial sums are combined
// with __shfl_xor_sync.  G = 1 is the scalar-row kernel.
template <typename T, int G, int U, bool DOT>
__global__ void __launch_bounds__(256)
k_spmv_vector(SpmvArgs a) {
  __shared__ double red[8];
  p2p_prologue_wait(a.hk);
  const T* __restrict__ vals = static_cast<const T*>(a.vals);
  const T* __restrict__ x = static_cast<const T*>(a.x);
  T* __restrict__ y = static_cast<T*>(a.y);
  const int* __restrict__ rowptr = a.rowptr;
  const int* __restrict__ colidx = a.colidx;

  const int lane = threadIdx.x & (G - 1);
  const unsigned wl = threadIdx.x & 31;
  const unsigned gmask = (G == 32) ? 0xffffffffu : (((1u << G) - 1u) << (wl & ~(unsigned)(G - 1)));
  const int64_t group = (int64_t(blockIdx.x) * blockDim.x + threadIdx.x) / G;
  const int64_t ngroups = int64_t(gridDim.x) * blockDim.x / G;
  const double alpha = a.alpha, beta = a.beta;
  double dacc = 0.0;

  for (int64_t i = group; i < a.m; i += ngroups) {
    const int k0 = __ldg(rowptr + i);
    const int k1 = __ldg(rowptr + i + 1);
    double s = 0.0;
    for (int kb = k0 + lane; kb < k1; kb += G * U) {
      int c[U];
      T v[U];
#pragma unroll
      for (int u = 0; u < U; ++u) {
        const int k = kb + u * G;
        c[u] = (k < k1) ? ld_stream(colidx + k) : -1;
        v[u] = (k < k1) ? ld_stream(vals + k) : T(0);
      }
      T xv[U];
#pragma unroll
      for (int u = 0; u < U; ++u) xv[u] = (c[u] >= 0) ? ld_x(x + c[u]) : T(0);
#pragma unroll
      for (int u = 0; u < U; ++u) s += double(v[u]) * double(xv[u]);
    }
    if (G > 1) s = group_sum<G>(s, gmask);
    if (lane == 0) {
      double r = alpha * s;
      if (beta != 0.0) r += beta * double(y[i]);
      const T out = T(r);
      y[i] = out;
      if (DOT) dacc += double(static_cast<const T*>(a.w)[i]) * double(out);
    }
  }
  if (DOT) {
    const double t = block_sum(dacc, red);
    if (threadIdx.x == 0) a.part[blockIdx.x] = t;
    p2p_push_partials_last(a.hk, a.part, gridDim.x);
  }
}

// y <- beta*y (alpha == 0: A and x are not read; beta == 0: y <- 0).
template <typename T>
__global__ void __launch_bounds__(256) k_scale(int64_t m, T* y, double beta) {
  for (int64_t i = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; i < m;
       i += int64_t(gridDim.x) * blockDim.x)
    y[i] = (beta == 0.0) ? T(0) : T(beta * double(y[i]));
}

}  // namespace spmv
