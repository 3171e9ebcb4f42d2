// merge_kernel.cuh -- merge-path CSR SpMV for skewed row lengths (Parboil-
// shaped power law, BJ.cfg[2], reading R21).
//
// The merge path of the row-end list A = rowptr[1..m]-base and the nonzero
// indices B = 0..nnz-1 is cut into tiles of exactly D = NT*IPT items (rows +
// nonzeros), so a 10,000-entry row costs the same per item as a 5-entry row
// and every CTA does the same work.  Per tile (one CTA):
//   1. stage the tile's row ends and the products vals[k]*x[colidx[k]] (in
//      double; coalesced loads of vals/colidx, x gathered through L1) in
//      shared memory;
//   2. each thread finds its diagonal (binary search in shared memory) and
//      walks IPT items: a row end closes a row, a nonzero adds its product;
//   3. a block-wide segmented scan of the threads' carry-outs (head flag =
//      "the thread closed a row") gives each thread the partial of the row it
//      starts in, deterministically (fixed shuffle tree);
//   4. closed rows are written (y = alpha*sum + beta*y); the first row of a
//      tile that began in an earlier tile is deferred: its in-tile partial goes
//      to head[t], and the tile's open row at the end goes to carry[t].
// A fix-up kernel then finishes the deferred rows: one thread per tile sums
// carry[] of the preceding tiles that the row spans, in tile order, plus
// head[t] -- deterministic, no atomics.
#pragma once
#include "common.cuh"

namespace spmv {

constexpr int MG_NT = 256;
constexpr int MG_IPT = 8;
constexpr int MG_D = MG_NT * MG_IPT;

struct MergeArgs {
  int64_t m;
  int ntiles;
  const int* rowptr;         // absolute k
  const int* colidx;
  const void* vals;
  const long long* split_row;  // [ntiles+1] rows consumed before tile t
  const long long* split_nz;   // [ntiles+1] nonzeros consumed before tile t (relative to rowptr[0])
  const void* x;
  void* y;
  double alpha, beta;
  double* head;              // [ntiles] in-tile partial of a deferred first row
  double* carry;             // [ntiles] partial of the row open at the tile end
  int* head_flag;            // [ntiles] 1 if the tile's first closed row is deferred
  P2PHook hk;                // p2p transport: wait for x
};

struct SegPair {
  int f;
  double v;
};
__device__ __forceinline__ SegPair seg_op(SegPair a, SegPair b) {
  return SegPair{a.f | b.f, b.f ? b.v : a.v + b.v};
}

template <typename T>
__global__ void __launch_bounds__(MG_NT)
k_spmv_merge(MergeArgs a) {
  __shared__ int s_end[MG_D + 1];
  __shared__ double s_prod[MG_D];
  __shared__ SegPair s_warp[MG_NT / 32];
  const int t = blockIdx.x;
  const int tid = threadIdx.x, lane = tid & 31, wid = tid >> 5;
  const int* __restrict__ rowptr = a.rowptr;
  const T* __restrict__ vals = static_cast<const T*>(a.vals);
  const T* __restrict__ x = static_cast<const T*>(a.x);
  const int base = __ldg(rowptr);
  const int64_t r0 = a.split_row[t], r1 = a.split_row[t + 1];
  const int64_t k0 = a.split_nz[t], k1 = a.split_nz[t + 1];
  const int nr = int(r1 - r0), nn = int(k1 - k0);
  p2p_prologue_wait(a.hk);

  // 1. stage row ends (relative nz index) and products
  // all IPT colidx/vals loads of a thread are issued before the x gathers,
  // and all gathers before any use (IPT independent chains in flight)
  for (int i = tid; i < nr; i += MG_NT) s_end[i] = __ldg(rowptr + r0 + 1 + i) - base;
  {
    int c[MG_IPT];
    T v[MG_IPT];
#pragma unroll
    for (int u = 0; u < MG_IPT; ++u) {
      const int j = tid + u * MG_NT;
      const int64_t k = base + k0 + j;
      c[u] = (j < nn) ? ld_stream(a.colidx + k) : -1;
      v[u] = (j < nn) ? ld_stream(vals + k) : T(0);
    }
    T xv[MG_IPT];
#pragma unroll
    for (int u = 0; u < MG_IPT; ++u) xv[u] = (c[u] >= 0) ? __ldg(x + c[u]) : T(0);
#pragma unroll
    for (int u = 0; u < MG_IPT; ++u) {
      const int j = tid + u * MG_NT;
      if (j < nn) s_prod[j] = double(v[u]) * double(xv[u]);
    }
  }
  __syncthreads();

  // 2. merge-path search for this thread's diagonal inside the tile:
  //    largest i in [max(0, d-nn), min(d, nr)] with end(i-1) <= k0 + (d - i)
  const int d = min(tid * MG_IPT, nr + nn);
  int lo = max(0, d - nn), hi = min(d, nr);
  while (lo < hi) {
    const int i = (lo + hi + 1) >> 1;
    if (int64_t(s_end[i - 1]) <= k0 + (d - i)) lo = i; else hi = i - 1;
  }
  const int i_start = lo, j_start = d - lo;
  const int dend = min(d + MG_IPT, nr + nn);

  // walk (fully unrolled, so the emitted partials stay in registers):
  // item `it` closes row i_start+ (number of earlier closes) when it is a row end
  int i = i_start, j = j_start;
  double run = 0.0;
  int closed = 0;
  double emit[MG_IPT];
  uint32_t cmask = 0;  // bit it: item it closed a row
#pragma unroll
  for (int it = 0; it < MG_IPT; ++it) {
    emit[it] = 0.0;
    if (d + it < dend) {
      if (i < nr && int64_t(s_end[i]) <= k0 + j) {
        emit[it] = run;
        cmask |= 1u << it;
        ++i;
        run = 0.0;
        closed = 1;
      } else {
        run += s_prod[j];
        ++j;
      }
    }
  }

  // 3. block-wide exclusive segmented scan of (closed, run) -> carry-in
  SegPair v{closed, run};
  SegPair inc = v;
#pragma unroll
  for (int off = 1; off < 32; off <<= 1) {
    SegPair o;
    o.f = __shfl_up_sync(0xffffffffu, inc.f, off);
    o.v = __shfl_up_sync(0xffffffffu, inc.v, off);
    if (lane >= off) inc = seg_op(o, inc);
  }
  if (lane == 31) s_warp[wid] = inc;
  __syncthreads();
  SegPair wpre{0, 0.0};  // exclusive prefix of the previous warps
  for (int w = 0; w < wid; ++w) wpre = seg_op(wpre, s_warp[w]);
  SegPair exc;
  exc.f = __shfl_up_sync(0xffffffffu, inc.f, 1);
  exc.v = __shfl_up_sync(0xffffffffu, inc.v, 1);
  if (lane == 0) exc = SegPair{0, 0.0};
  exc = seg_op(wpre, exc);  // carry-in of this thread (partial of row i_start)

  // 4. emit closed rows (the first one receives the carry-in)
  T* __restrict__ y = static_cast<T*>(a.y);
  const bool head_deferred = (int64_t(__ldg(rowptr + r0)) - base) < k0;  // row r0 began earlier
  {
    int row_i = i_start;
    bool first = true;
#pragma unroll
    for (int it = 0; it < MG_IPT; ++it) {
      if (cmask & (1u << it)) {
        const double val = first ? emit[it] + exc.v : emit[it];
        first = false;
        const int64_t row = r0 + row_i;
        if (row_i == 0 && head_deferred) {
          a.head[t] = val;
        } else {
          double r = a.alpha * val;
          if (a.beta != 0.0) r += a.beta * double(y[row]);
          y[row] = T(r);
        }
        ++row_i;
      }
    }
  }
  if (tid == MG_NT - 1) {
    // inclusive total of the last thread = partial of the row open at the end
    const SegPair tot = seg_op(wpre, inc);
    a.carry[t] = (r1 < a.m) ? tot.v : 0.0;
    a.head_flag[t] = (nr > 0 && head_deferred) ? 1 : 0;
  }
}

// Finish the deferred first rows: y[r0] = alpha*(carries of the preceding
// tiles the row spans, in tile order, + head[t]) + beta*y.
template <typename T>
__global__ void __launch_bounds__(256)
k_merge_fixup(MergeArgs a) {
  const int t = blockIdx.x * blockDim.x + threadIdx.x;
  if (t >= a.ntiles || !a.head_flag[t]) return;
  const int64_t row = a.split_row[t];
  double sum = 0.0;
  int u = t - 1;
  // tiles u < t that end with `row` open; stop after the tile where it began
  while (u >= 0) {
    sum += a.carry[u];
    if (a.split_row[u] < row) break;
    --u;
  }
  sum += a.head[t];
  T* y = static_cast<T*>(a.y);
  double r = a.alpha * sum;
  if (a.beta != 0.0) r += a.beta * double(y[row]);
  y[row] = T(r);
}

// Merge-path splits (reading R21) on the device, bit-exact with the host
// spmv_csr_merge_splits: thread c finds the split of diagonal floor(c*(m+nnz)/C).
// With C = ceil((m+nnz)/D) every tile holds at most D items.
static __global__ void k_merge_splits(int64_t m, const int* __restrict__ rowptr, int64_t C,
                               long long* __restrict__ split_row, long long* __restrict__ split_nz) {
  const int64_t c = int64_t(blockIdx.x) * blockDim.x + threadIdx.x;
  if (c > C) return;
  const int64_t base = rowptr[0];
  const int64_t nnz = int64_t(rowptr[m]) - base;
  const int64_t d = (c * (m + nnz)) / C;
  int64_t lo = cmax64(0, d - nnz), hi = cmin64(d, m);
  while (lo < hi) {
    const int64_t i = lo + ((hi - lo + 1) >> 1);
    if (int64_t(rowptr[i]) - base <= d - i) lo = i; else hi = i - 1;
  }
  split_row[c] = lo;
  split_nz[c] = d - lo;
}

}  // namespace spmv
