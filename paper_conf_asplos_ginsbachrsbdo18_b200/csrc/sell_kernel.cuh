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
// Sorted variant (skewed rows: the Parboil-shaped power law, BJ.cfg[2]; the
// "CSR-adaptive for skewed rows" of BJ.ns): rows are ordered by length,
// descending, over the whole matrix (sigma = m, a stable device radix sort), so
// the 32 rows of a chunk have nearly equal lengths and padding vanishes; the
// nlong rows longer than SELL_LONG come first and are processed straight from
// the CSR arrays, cut into segments of at most SELL_SEG entries, one warp per
// segment (32 lanes x 2*SELL_U coalesced loads, shuffle reduction), longest
// rows first; a row's segment partials go to a buffer and the warp that
// completes the row (ticket counter) sums them in segment order, so the
// result does not depend on which warp finishes last; y is written through
// the permutation.  (One warp per whole 10,000-entry row was the critical
// path: 157 us on the Parboil-shaped matrix.)  x gathers cannot be avoided for random columns
// (4 MB of x, more than a cluster's shared memory): the bound is one L1
// wavefront per gather.
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
#define SELL_U_DEF 2
#endif
constexpr int SELL_U = SELL_U_DEF;  // step pairs in flight per lane

#ifndef SELL_LONG_DEF
#define SELL_LONG_DEF 64
#endif
#ifndef SELL_SEG_DEF
#define SELL_SEG_DEF 1024
#endif
constexpr int SELL_LONG = SELL_LONG_DEF;  // sorted variant: rows longer than this are processed from the CSR by warps
constexpr int SELL_SEG = SELL_SEG_DEF;    // ... in segments of at most this many entries

// one long-row segment (sorted variant)
struct SellSeg {
  int row, k0, k1;  // row and its entries [k0, k1) of this segment
  int pbase;        // -1: the row has one segment; else first slot of the row's partials
  int sidx, nseg;   // segment index, segments of the row
  int cslot;        // ticket counter of the row (multi-segment rows)
  int pad;
};

struct SellArgs {
  int64_t m;                   // local rows
  int64_t nchunks;             // chunks of 32 (sorted) rows
  const int* perm;             // sorted variant: row of sorted position s (NULL: identity, no long rows)
  int64_t nlong;               // sorted variant: rows perm[0..nlong) are long
  int64_t nseg;                // sorted variant: long-row segments (work items before the chunks)
  const SellSeg* seg;
  double* seg_part;            // partials of multi-segment rows
  int* seg_cnt;                // ticket counters (0 between launches)
  const int* colidx;           // long rows: CSR (absolute k)
  const void* csr_vals;
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
  T* __restrict__ y = static_cast<T*>(a.y);
  auto finish = [&](int64_t i, double acc) {
    double r = alpha * acc;
    if (beta != 0.0) r += beta * double(y[i]);
    const T out = T(r);
    y[i] = out;
    if (DOT) dacc += double(static_cast<const T*>(a.w)[i]) * double(out);
  };
  // work items: the long-row segments (warp per segment), then the chunks (warp per chunk)
  const int64_t nitems = a.nseg + a.nchunks;
  for (int64_t it = gw; it < nitems; it += nw) {
    if (it < a.nseg) {
      const SellSeg sg = a.seg[it];
      const T* __restrict__ cv = static_cast<const T*>(a.csr_vals);
      double acc = 0.0;
      for (int kb = sg.k0 + lane; kb < sg.k1; kb += 32 * 2 * SELL_U) {
        int c[2 * SELL_U];
        T v[2 * SELL_U];
#pragma unroll
        for (int u = 0; u < 2 * SELL_U; ++u) {
          const int k = kb + 32 * u;
          c[u] = k < sg.k1 ? ld_stream(a.colidx + k) : -1;
          v[u] = k < sg.k1 ? ld_stream(cv + k) : T(0);
        }
        T xv[2 * SELL_U];
#pragma unroll
        for (int u = 0; u < 2 * SELL_U; ++u) xv[u] = c[u] >= 0 ? ld_x(x + c[u]) : T(0);
#pragma unroll
        for (int u = 0; u < 2 * SELL_U; ++u)
          if (c[u] >= 0) acc += double(v[u]) * double(xv[u]);
      }
      acc = warp_sum(acc);
      if (lane == 0) {
        if (sg.pbase < 0) {
          finish(sg.row, acc);
        } else {
          a.seg_part[sg.pbase + sg.sidx] = acc;
          __threadfence();
          if (atomicAdd(a.seg_cnt + sg.cslot, 1) == sg.nseg - 1) {
            __threadfence();
            double tot = 0.0;
            for (int q = 0; q < sg.nseg; ++q) tot += __ldcg(a.seg_part + sg.pbase + q);  // segment order
            a.seg_cnt[sg.cslot] = 0;
            finish(sg.row, tot);
          }
        }
      }
      continue;
    }
    const int64_t c = it - a.nseg;
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
    const int64_t s_ = c * 32 + lane;  // position among the short rows
    if (a.perm) {
      if (a.nlong + s_ < a.m) finish(a.perm[a.nlong + s_], acc);
    } else if (s_ < a.m) {
      finish(s_, acc);
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
static __global__ void k_sell_pairs(int64_t m, const int* __restrict__ rowptr, int64_t nchunks, long long* __restrict__ pairs) {
  for (int64_t c = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; c < nchunks; c += int64_t(gridDim.x) * blockDim.x) {
    int L = 0;
    const int64_t r1 = cmin64(m, c * 32 + 32);
    for (int64_t i = c * 32; i < r1; ++i) L = max(L, rowptr[i + 1] - rowptr[i]);
    pairs[c] = (L + 1) >> 1;
  }
}

// pairs[c] = ceil(longest row of sorted chunk c / 2); rows are perm[nlong + 32c ..]
static __global__ void k_sell_pairs_sorted(int64_t m, const int* __restrict__ rowptr, const int* __restrict__ perm,
                                    int64_t nlong, int64_t nchunks, long long* __restrict__ pairs) {
  for (int64_t c = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; c < nchunks; c += int64_t(gridDim.x) * blockDim.x) {
    int L = 0;
    const int64_t s1 = cmin64(m, nlong + c * 32 + 32);
    for (int64_t s = nlong + c * 32; s < s1; ++s) {
      const int i = perm[s];
      L = max(L, rowptr[i + 1] - rowptr[i]);
    }
    pairs[c] = (L + 1) >> 1;
  }
}

// Thread per (sorted) short row: entry s of the row -> slot (pair_off[c] + s/2)*32 + lane, half s&1.
// perm == NULL: identity order, no long rows.
template <typename T>
__global__ void k_sell_pack(int64_t m, const int* __restrict__ rowptr, const int* __restrict__ colidx,
                            const T* __restrict__ vals, const long long* __restrict__ pair_off,
                            const int* __restrict__ perm, int64_t nlong,
                            T* __restrict__ pv, int* __restrict__ pc, int values_only) {
  for (int64_t q = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; q < m - nlong; q += int64_t(gridDim.x) * blockDim.x) {
    const int64_t c = q >> 5;
    const int lane = int(q & 31);
    const int64_t i = perm ? perm[nlong + q] : q;
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

// Row lengths (sort keys) and identity row ids for the sorted variant.
static __global__ void k_row_len_ids(int64_t m, const int* __restrict__ rowptr, int* __restrict__ len, int* __restrict__ ids) {
  for (int64_t i = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; i < m; i += int64_t(gridDim.x) * blockDim.x) {
    len[i] = rowptr[i + 1] - rowptr[i];
    ids[i] = int(i);
  }
}

}  // namespace spmv
