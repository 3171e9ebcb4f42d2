// analysis_kernels.cuh -- ingest + analyse: row statistics,
// optional structure validation, device nnz-balanced partition (reading R20)
// and the column renumbering of a rank's row block (distributed mode).
#pragma once
#include "common.cuh"

namespace spmv {

// Per-CTA partial row statistics: [min, max, sum, sumsq, unsorted_rows].
// Reduced on the host in CTA order (deterministic on every rank).
static __global__ void __launch_bounds__(256)
k_row_stats(int64_t m, const int* __restrict__ rowptr, const int* __restrict__ colidx,
            int check_sorted, double* __restrict__ part /* 5 * gridDim.x */) {
  __shared__ double red[8];
  __shared__ double s_min[8], s_max[8];
  double mn = 1e300, mx = -1e300, sum = 0.0, sq = 0.0, uns = 0.0;
  for (int64_t i = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; i < m;
       i += int64_t(gridDim.x) * blockDim.x) {
    const int k0 = rowptr[i], k1 = rowptr[i + 1];
    const double L = double(int64_t(k1) - int64_t(k0));
    mn = fmin(mn, L);
    mx = fmax(mx, L);
    sum += L;
    sq += L * L;
    if (check_sorted) {
      for (int k = k0 + 1; k < k1; ++k)
        if (colidx[k] <= colidx[k - 1]) { uns += 1.0; break; }
    }
  }
  // min / max via shuffles
  for (int off = 16; off > 0; off >>= 1) {
    mn = fmin(mn, __shfl_xor_sync(0xffffffffu, mn, off));
    mx = fmax(mx, __shfl_xor_sync(0xffffffffu, mx, off));
  }
  const int lane = threadIdx.x & 31, wid = threadIdx.x >> 5;
  if (lane == 0) { s_min[wid] = mn; s_max[wid] = mx; }
  sum = block_sum(sum, red);
  sq = block_sum(sq, red);
  uns = block_sum(uns, red);
  if (threadIdx.x == 0) {
    double a = 1e300, b = -1e300;
    for (int w = 0; w < int(blockDim.x >> 5); ++w) { a = fmin(a, s_min[w]); b = fmax(b, s_max[w]); }
    part[5 * blockIdx.x + 0] = a;
    part[5 * blockIdx.x + 1] = b;
    part[5 * blockIdx.x + 2] = sum;
    part[5 * blockIdx.x + 3] = sq;
    part[5 * blockIdx.x + 4] = uns;
  }
}

// validate=1: flags[0] |= 1 if rowptr decreases, flags[0] |= 2 if a column
// index is outside [0, n).
static __global__ void __launch_bounds__(256)
k_validate(int64_t m, int64_t n, const int* __restrict__ rowptr, const int* __restrict__ colidx,
           int* __restrict__ flags) {
  const int64_t stride = int64_t(gridDim.x) * blockDim.x;
  const int64_t t0 = int64_t(blockIdx.x) * blockDim.x + threadIdx.x;
  int bad = 0;
  for (int64_t i = t0; i < m; i += stride)
    if (rowptr[i + 1] < rowptr[i]) bad |= 1;
  if (!(bad & 1)) {
    const int64_t kb = rowptr[0], ke = rowptr[m];
    for (int64_t k = kb + t0; k < ke; k += stride) {
      const int c = colidx[k];
      if (c < 0 || int64_t(c) >= n) { bad |= 2; break; }
    }
  }
  if (bad) atomicOr(flags, bad);
}

// Device nnz-balanced partition (R20): thread r finds
//   b_r = min{ i in [0,m] : rowptr[i] - rowptr[0] >= floor(r*nnz/P) }
// by binary search; b_0 = 0, b_P = m.
static __global__ void k_partition(int64_t m, const int* __restrict__ rowptr, int P,
                            long long* __restrict__ bounds) {
  const int r = blockIdx.x * blockDim.x + threadIdx.x;
  if (r > P) return;
  if (r == 0) { bounds[0] = 0; return; }
  if (r == P) { bounds[P] = m; return; }
  const long long base = rowptr[0];
  const long long nnz = (long long)rowptr[m] - base;
  const long long t = ((long long)r * nnz) / P;
  long long lo = 0, hi = m;  // answer in [lo, hi]; prefix(m) = nnz >= t
  while (lo < hi) {
    const long long mid = lo + ((hi - lo) >> 1);
    if ((long long)rowptr[mid] - base >= t) hi = mid; else lo = mid + 1;
  }
  bounds[r] = lo;
}

// Renumber the columns of a rank's row block into the padded gather layout:
// column c owned by rank s (bounds[s] <= c < bounds[s+1]) -> s*maxlen + (c - bounds[s]).
static __global__ void __launch_bounds__(256)
k_renumber(int64_t k0, int64_t k1, const int* __restrict__ colidx, const long long* __restrict__ bounds,
           int P, long long maxlen, int* __restrict__ out) {
  extern __shared__ long long sb[];
  for (int i = threadIdx.x; i <= P; i += blockDim.x) sb[i] = bounds[i];
  __syncthreads();
  for (int64_t k = k0 + int64_t(blockIdx.x) * blockDim.x + threadIdx.x; k < k1;
       k += int64_t(gridDim.x) * blockDim.x) {
    const long long c = colidx[k];
    int lo = 0, hi = P - 1;  // largest s with sb[s] <= c
    while (lo < hi) {
      const int mid = (lo + hi + 1) >> 1;
      if (sb[mid] <= c) lo = mid; else hi = mid - 1;
    }
    out[k - k0] = int(lo * maxlen + (c - sb[lo]));
  }
}

// Halo intervals (NEXT-2, reading R27): for destination rank r and source rank
// s != r, tab[(r*P+s)*2 .. +1] = min / max local index (c - bounds[s]) over the
// columns c of rank r's rows owned by s (INT_MAX / -1 when there are none).
// Warp per row over the GLOBAL matrix (every rank computes the whole table,
// identically: min/max do not depend on the order).  Smem table per CTA,
// updates only when they change it, then global atomics.
static __global__ void __launch_bounds__(256)
k_halo_bounds(int64_t m, const int* __restrict__ rowptr, const int* __restrict__ colidx,
              const long long* __restrict__ bounds, int P, int* __restrict__ tab) {
  extern __shared__ long long sb[];  // [P+1] bounds, then int [P*P*2]
  int* st = reinterpret_cast<int*>(sb + P + 1);
  for (int i = threadIdx.x; i <= P; i += blockDim.x) sb[i] = bounds[i];
  for (int i = threadIdx.x; i < P * P; i += blockDim.x) {
    st[2 * i] = 0x7fffffff;
    st[2 * i + 1] = -1;
  }
  __syncthreads();
  auto owner = [&](long long c) {
    int lo = 0, hi = P - 1;  // largest s with sb[s] <= c
    while (lo < hi) {
      const int mid = (lo + hi + 1) >> 1;
      if (sb[mid] <= c) lo = mid; else hi = mid - 1;
    }
    return lo;
  };
  const int lane = threadIdx.x & 31;
  const int64_t w0 = (int64_t(blockIdx.x) * blockDim.x + threadIdx.x) >> 5;
  const int64_t nw = (int64_t(gridDim.x) * blockDim.x) >> 5;
  for (int64_t i = w0; i < m; i += nw) {
    const int r = owner(i);
    const int k0 = rowptr[i], k1 = rowptr[i + 1];
    for (int k = k0 + lane; k < k1; k += 32) {
      const long long c = colidx[k];
      const int sidx = owner(c);
      if (sidx == r) continue;
      const int li = int(c - sb[sidx]);
      int* e = st + 2 * (r * P + sidx);
      if (li < e[0]) atomicMin(e, li);
      if (li > e[1]) atomicMax(e + 1, li);
    }
  }
  __syncthreads();
  for (int i = threadIdx.x; i < P * P; i += blockDim.x)
    if (st[2 * i + 1] >= 0) {
      atomicMin(tab + 2 * i, st[2 * i]);
      atomicMax(tab + 2 * i + 1, st[2 * i + 1]);
    }
}

}  // namespace spmv
