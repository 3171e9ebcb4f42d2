// sell_kernel.cuh -- SELL-32 (sigma = 1) device plan of A with x gathered
// from global memory, for regular matrices whose x is too large for the
// x-stationary cluster plan (the 27-point stencil of BJ.cfg[4]: x = 134 MB).
//
// Plan (built once at create, the paper's device-resident "lazy copy" of A,
// P:1175-1184, reading R26): rows are cut into chunks of 32 consecutive rows
// (no sorting, so lane j of a chunk is row 32c + j and the x gathers of a
// step stay as local as the matrix makes them); chunk c stores len_c (even)
// steps column-major in step pairs:
//     vals  [len/2][32 lanes][2]   (16 B per lane per pair for fp64)
//     cols  [len/2][32 lanes][2]   int32, -1 = padding (not read)
// Step s of lane j is entry s of row 32c + j in CSR order, so every row is
// still summed left to right as Fig. 4 writes it.
//
// Kernel: warp per chunk, chunks dealt round-robin over all warps of the grid
// (so all SMs sweep the matrix together and the x window stays in L2),
// lane = row (no intra-row reduction), U pairs = 2U independent 16-B value
// loads + 8-B column loads issued before any gather, x gathered with
// ld.global.nc (L1-allocating: neighbouring steps of a stencil row share
// lines), coalesced y stores, fused CG dot partial per CTA.
#pragma once
#include "common.cuh"
#include "xplan_kernel.cuh"  // Pair<T>, streaming loads

namespace spmv {

constexpr int SELL_NT = 256;  // threads per CTA
#ifndef SELL_U_DEF
#define SELL_U_DEF 4
#endif
constexpr int SELL_U = SELL_U_DEF;  // step pairs in flight per lane

struct SellArgs {
  int64_t m;                   // local rows
  int64_t nchunks;             // ceil(m / 32)
  const unsigned char* vals;   // pair slots, sizeof(T)*2 bytes each
  const int2* cols;            // pair slots
  const long long* pair_off;   // [nchunks + 1]: first pair of chunk c (x32 lanes = slot)
  const void* x;
  void* y;
  double alpha, beta;
  const void* w;               // DOT: w[i]
  double* part;                // DOT: one partial per CTA
  P2PHook hk;
};

template <typename T, bool DOT>
__global__ void __launch_bounds__(SELL_NT)
k_spmv_sell(SellArgs a) {
  __shared__ double red[SELL_NT / 32];
  p2p_prologue_wait(a.hk);
  const T* __restrict__ x = static_cast<const T*>(a.x);
  const int lane = threadIdx.x & 31;
  const int64_t gw = (int64_t(blockIdx.x) * SELL_NT + threadIdx.x) >> 5;
  const int64_t nw = (int64_t(gridDim.x) * SELL_NT) >> 5;
  const double alpha = a.alpha, beta = a.beta;
  double dacc = 0.0;
  for (int64_t c = gw; c < a.nchunks; c += nw) {
    const long long p0 = a.pair_off[c], p1 = a.pair_off[c + 1];
    const int np = int(p1 - p0);
    const unsigned char* V = a.vals + (size_t(p0) * 32 + lane) * 2 * sizeof(T);
    const int2* C = a.cols + size_t(p0) * 32 + lane;
    double acc = 0.0;
    for (int p = 0; p < np; p += SELL_U) {
      Pair<T> v[SELL_U];
      int2 cc[SELL_U];
#pragma unroll
      for (int u = 0; u < SELL_U; ++u) {
        if (p + u < np) {
          v[u] = Pair<T>::load(V + size_t(p + u) * 32 * 2 * sizeof(T));
          const uint2 r = ldg_stream8(C + size_t(p + u) * 32);
          cc[u] = make_int2(int(r.x), int(r.y));
        } else {
          v[u] = Pair<T>{T(0), T(0)};
          cc[u] = make_int2(-1, -1);
        }
      }
      T xa[SELL_U], xb[SELL_U];
#pragma unroll
      for (int u = 0; u < SELL_U; ++u) {
        xa[u] = cc[u].x >= 0 ? ld_x(x + cc[u].x) : T(0);
        xb[u] = cc[u].y >= 0 ? ld_x(x + cc[u].y) : T(0);
      }
#pragma unroll
      for (int u = 0; u < SELL_U; ++u) {
        if (cc[u].x >= 0) acc += double(v[u].a) * double(xa[u]);
        if (cc[u].y >= 0) acc += double(v[u].b) * double(xb[u]);
      }
    }
    const int64_t i = c * 32 + lane;
    if (i < a.m) {
      T* y = static_cast<T*>(a.y);
      double r = alpha * acc;
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

// ---------------------------------------------------------------- builders
// pairs[c] = ceil(max row length of chunk c / 2)
__global__ void k_sell_pairs(int64_t m, const int* __restrict__ rowptr, int64_t nchunks, long long* __restrict__ pairs) {
  for (int64_t c = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; c < nchunks; c += int64_t(gridDim.x) * blockDim.x) {
    int L = 0;
    const int64_t r1 = cmin64(m, c * 32 + 32);
    for (int64_t i = c * 32; i < r1; ++i) L = max(L, rowptr[i + 1] - rowptr[i]);
    pairs[c] = (L + 1) >> 1;
  }
}

// Thread per row: entry s of row i -> slot (pair_off[c] + s/2)*32 + lane, half s&1.
template <typename T>
__global__ void k_sell_pack(int64_t m, const int* __restrict__ rowptr, const int* __restrict__ colidx,
                            const T* __restrict__ vals, const long long* __restrict__ pair_off,
                            T* __restrict__ pv, int* __restrict__ pc, int values_only) {
  for (int64_t i = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; i < m; i += int64_t(gridDim.x) * blockDim.x) {
    const int64_t c = i >> 5;
    const int lane = int(i & 31);
    const int k0 = rowptr[i], k1 = rowptr[i + 1];
    const size_t base = size_t(pair_off[c]) * 32 + lane;
    for (int k = k0; k < k1; ++k) {
      const int s = k - k0;
      const size_t e = (base + size_t(s >> 1) * 32) * 2 + (s & 1);
      pv[e] = vals[k];
      if (!values_only) pc[e] = colidx[k];
    }
  }
}

}  // namespace spmv
