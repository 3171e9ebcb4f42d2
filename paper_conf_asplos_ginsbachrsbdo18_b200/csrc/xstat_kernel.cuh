// xstat_kernel.cuh -- x-stationary CSR SpMV with thread-block clusters (sm_100a).
//
// Why: the vector kernel's x gathers cost one L1TEX wavefront per nonzero
// (random columns never share a 128-B line), capping a B200 SM at ~1 gather
// per cycle -- 36.1M gathers of NAS class C take ~128 us, twice the HBM time
// of the 436 MB the SpMV must stream (ncu: L1TEX 80% busy, DRAM 31%).
// Here a cluster of B CTAs (one per SM) keeps x resident in shared memory,
// column block b (width W) in CTA rank b, loaded once per launch with one TMA
// bulk copy (cp.async.bulk + mbarrier).  Each CTA streams, for the rows of its
// cluster, only the part of every row whose columns fall in its block (split
// points precomputed at create from the sorted colidx), gathers x from its
// own shared memory (bank-conflict-limited, ~4x the L1 rate), and writes one
// partial per row into a triple-buffered shared array.  After a split cluster
// barrier (arrive ... wait, hidden behind the next tile), CTA b reduces rows
// [b*R/B, (b+1)*R/B) of the tile by reading the B partials of every peer
// through DSMEM in rank order -- deterministic, no atomics, no extra HBM
// traffic.  Semantics are those of Fig. 4 with alpha/beta.
#pragma once
#include <cooperative_groups.h>

#include "common.cuh"

namespace spmv {

namespace cgx = cooperative_groups;

struct XstatArgs {
  int64_t m;              // local rows
  int64_t nx;             // length of x
  int W;                  // column block width (multiple of 4)
  int R;                  // rows per tile
  const int* rowptr;      // absolute k
  const int* colidx;
  const void* vals;
  const int* seg;         // (B-1) x m interior split points (absolute k), block-major
  const long long* crow;  // cluster row ranges [nclusters+1]
  const void* x;
  void* y;
  double alpha, beta;
  const void* w;          // DOT
  double* part;           // DOT: one partial per CTA
  P2PHook hk;
};

__device__ __forceinline__ uint32_t smem_u32(const void* p) {
  return static_cast<uint32_t>(__cvta_generic_to_shared(p));
}
// Cluster barrier halves.  The non-.aligned forms plus __syncwarp(): the
// callers reach them from divergent code, and inline asm gives the compiler
// no reason to reconverge the warp before an .aligned barrier.
__device__ __forceinline__ void cluster_arrive() {
  __syncwarp();
  asm volatile("barrier.cluster.arrive.release;\n" ::: "memory");
}
__device__ __forceinline__ void cluster_wait() {
  __syncwarp();
  asm volatile("barrier.cluster.wait.acquire;\n" ::: "memory");
}
__device__ __forceinline__ uint32_t cluster_rank() {
  uint32_t r;
  asm volatile("mov.u32 %0, %%cluster_ctarank;\n" : "=r"(r));
  return r;
}
__device__ __forceinline__ uint32_t cluster_id() {
  uint32_t r;
  asm volatile("mov.u32 %0, %%clusterid.x;\n" : "=r"(r));
  return r;
}

// TMA 1-D bulk copy global -> own shared memory, completing on an mbarrier.
__device__ __forceinline__ void bulk_g2s(void* dst, const void* src, uint32_t bytes, uint64_t* bar) {
  asm volatile(
      "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];\n" ::"r"(
          smem_u32(dst)),
      "l"(src), "r"(bytes), "r"(smem_u32(bar))
      : "memory");
}
__device__ __forceinline__ void mbar_init(uint64_t* bar, uint32_t count) {
  asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;\n" ::"r"(smem_u32(bar)), "r"(count) : "memory");
}
__device__ __forceinline__ void mbar_expect_tx(uint64_t* bar, uint32_t bytes) {
  asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;\n" ::"r"(smem_u32(bar)), "r"(bytes)
               : "memory");
}
// Wait for the phase of `parity` to complete.  Watchdog: a wait that spins for
// more than ~4e9 cycles (~2 s) reports the barrier and traps, turning a
// deadlock into a launch error instead of a hung GPU.
__device__ __forceinline__ void mbar_wait(uint64_t* bar, uint32_t parity, int tag = -1) {
  uint32_t ok = 0;
  long long t0 = 0;
  for (uint32_t spin = 0; !ok; ++spin) {
    asm volatile(
        "{\n .reg .pred p;\n mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2;\n selp.u32 %0, 1, 0, p;\n}\n"
        : "=r"(ok)
        : "r"(smem_u32(bar)), "r"(parity)
        : "memory");
    if (!ok && (spin & 1023) == 1023) {
      const long long now = clock64();
      if (t0 == 0) t0 = now;
      else if (now - t0 > 4000000000LL) {
        printf("spmv: mbarrier wait timeout block %d thread %d bar smem 0x%x parity %u tag %d\n", blockIdx.x,
               threadIdx.x, smem_u32(bar), parity, tag);
        __trap();
      }
    }
  }
}

// Dynamic shared memory: [xs: W*sizeof(T), 16-B aligned][pbuf: 3*R doubles]
//                        [bnd: 2 x 2 x R ints (double-buffered segment bounds)]
template <typename T, int G, int U, bool DOT>
__global__ void __launch_bounds__(1024, 1)
k_spmv_xstat(XstatArgs a) {
  extern __shared__ __align__(128) unsigned char smem[];
  __shared__ uint64_t bar;
  __shared__ double red[32];
  cgx::cluster_group cluster = cgx::this_cluster();
  const int B = (int)cluster.num_blocks();
  const int b = (int)cluster_rank();
  const int c = (int)cluster_id();
  const int R = a.R;
  p2p_prologue_wait(a.hk);

  T* xs = reinterpret_cast<T*>(smem);
  double* pbuf = reinterpret_cast<double*>(smem + ((size_t(a.W) * sizeof(T) + 15) & ~size_t(15)));
  int* bnd = reinterpret_cast<int*>(pbuf + 3 * R);  // [2][2][R]
  const T* __restrict__ vals = static_cast<const T*>(a.vals);
  const T* __restrict__ xg = static_cast<const T*>(a.x);
  const int* __restrict__ colidx = a.colidx;
  const int* __restrict__ rowptr = a.rowptr;
  const int* __restrict__ seg = a.seg;
  const int64_t m = a.m;

  // ---- x column block b -> shared memory (one TMA bulk copy + scalar tail)
  const int64_t col0 = int64_t(b) * a.W;
  const int64_t ncols = cmax64(0, cmin64(a.W, a.nx - col0));
  const int64_t bulk_elems = ((reinterpret_cast<uintptr_t>(xg + col0) & 15) == 0)
                                 ? ((ncols * int64_t(sizeof(T))) & ~int64_t(15)) / int64_t(sizeof(T))
                                 : 0;
  if (threadIdx.x == 0) {
    mbar_init(&bar, 1);
    asm volatile("fence.mbarrier_init.release.cluster;\n" ::: "memory");
  }
  __syncthreads();
  if (threadIdx.x == 0) {
    const uint32_t bytes = uint32_t(bulk_elems * sizeof(T));
    mbar_expect_tx(&bar, bytes);
    if (bytes) bulk_g2s(xs, xg + col0, bytes, &bar);
  }
  for (int64_t j = bulk_elems + threadIdx.x; j < ncols; j += blockDim.x) xs[j] = xg[col0 + j];

  const int lane = threadIdx.x & (G - 1);
  const unsigned wl = threadIdx.x & 31;
  const unsigned gmask = (G == 32) ? 0xffffffffu : (((1u << G) - 1u) << (wl & ~(unsigned)(G - 1)));
  const int group = threadIdx.x / G;
  const int ngroups = blockDim.x / G;
  const int64_t r0c = a.crow[c], r1c = a.crow[c + 1];
  const int ntiles = int((r1c - r0c + R - 1) / R);
  const double alpha = a.alpha, beta = a.beta;
  const int fin_lo = (b * R) / B, fin_hi = ((b + 1) * R) / B;
  double dacc = 0.0;

  // segment bounds of tile t: every thread loads rows j = tid, tid+blockDim ...
  auto load_bounds = [&](int t, int* dst) {
    const int64_t rt = r0c + int64_t(t) * R;
    const int nrows = int(cmin64(R, r1c - rt));
    for (int j = threadIdx.x; j < nrows; j += blockDim.x) {
      const int64_t i = rt + j;
      dst[j] = (b == 0) ? __ldg(rowptr + i) : __ldg(seg + int64_t(b - 1) * m + i);
      dst[R + j] = (b == B - 1) ? __ldg(rowptr + i + 1) : __ldg(seg + int64_t(b) * m + i);
    }
  };
  if (ntiles > 0) load_bounds(0, bnd);

  mbar_wait(&bar, 0);
  __syncthreads();

  auto process = [&](int t) {
    double* pb = pbuf + (t % 3) * R;
    const int* bb = bnd + (t & 1) * 2 * R;
    const int64_t rt = r0c + int64_t(t) * R;
    const int nrows = int(cmin64(R, r1c - rt));
    // prefetch the bounds of tile t+1 into registers; stored after the tile
    int pf0 = 0, pf1 = 0;
    const bool has_next = (t + 1 < ntiles);
    const int64_t rn = rt + R;
    const int nnext = has_next ? int(cmin64(R, r1c - rn)) : 0;
    const int jn = threadIdx.x;  // R <= blockDim.x is not assumed: loop below covers the rest
    if (jn < nnext) {
      pf0 = (b == 0) ? __ldg(rowptr + rn + jn) : __ldg(seg + int64_t(b - 1) * m + rn + jn);
      pf1 = (b == B - 1) ? __ldg(rowptr + rn + jn + 1) : __ldg(seg + int64_t(b) * m + rn + jn);
    }
    for (int j = group; j < nrows; j += ngroups) {
      const int k0 = bb[j], k1 = bb[R + j];
      double s = 0.0;
      for (int kb = k0 + lane; kb < k1; kb += G * U) {
        int cc[U];
        T v[U];
#pragma unroll
        for (int u = 0; u < U; ++u) {
          const int k = kb + u * G;
          cc[u] = (k < k1) ? ld_stream(colidx + k) - int(col0) : -1;
          v[u] = (k < k1) ? ld_stream(vals + k) : T(0);
        }
#pragma unroll
        for (int u = 0; u < U; ++u) s += double(v[u]) * double(cc[u] >= 0 ? xs[cc[u]] : T(0));
      }
      if (G > 1) s = group_sum<G>(s, gmask);
      if (lane == 0) pb[j] = s;
    }
    if (has_next) {
      int* nb = bnd + ((t + 1) & 1) * 2 * R;
      if (jn < nnext) { nb[jn] = pf0; nb[R + jn] = pf1; }
      for (int j = jn + blockDim.x; j < nnext; j += blockDim.x) {
        nb[j] = (b == 0) ? __ldg(rowptr + rn + j) : __ldg(seg + int64_t(b - 1) * m + rn + j);
        nb[R + j] = (b == B - 1) ? __ldg(rowptr + rn + j + 1) : __ldg(seg + int64_t(b) * m + rn + j);
      }
    }
  };

  auto finalize = [&](int t) {
    const double* pb = pbuf + (t % 3) * R;
    const int64_t rt = r0c + int64_t(t) * R;
    const int nrows = int(cmin64(R, r1c - rt));
    for (int j = fin_lo + threadIdx.x; j < min(fin_hi, nrows); j += blockDim.x) {
      double s = 0.0;
      for (int q = 0; q < B; ++q) s += *cluster.map_shared_rank(pb + j, q);
      const int64_t i = rt + j;
      T* y = static_cast<T*>(a.y);
      double r = alpha * s;
      if (beta != 0.0) r += beta * double(y[i]);
      const T out = T(r);
      y[i] = out;
      if (DOT) dacc += double(static_cast<const T*>(a.w)[i]) * double(out);
    }
  };

  // The bounds of tile t+1 are written during process(t) by every thread, so
  // all threads of the CTA must finish process(t) before any starts
  // process(t+1) (__syncthreads); the split cluster barrier alone only orders
  // tiles t-1 and t+1.
  if (ntiles > 0) {
    process(0);
    __syncthreads();
    cluster_arrive();
    for (int t = 1; t < ntiles; ++t) {
      process(t);
      __syncthreads();
      cluster_wait();
      finalize(t - 1);
      cluster_arrive();
    }
    cluster_wait();
    finalize(ntiles - 1);
  }
  // peers may still read this CTA's pbuf: leave together
  cluster_arrive();
  cluster_wait();
  if (DOT) {
    const double tsum = block_sum(dacc, red);
    if (threadIdx.x == 0) a.part[blockIdx.x] = tsum;
    p2p_push_partials_last(a.hk, a.part, gridDim.x);
  }
}

// Split points of every row at the column-block boundaries b*W (b = 1..B-1):
// seg[(b-1)*m + i] = first k in [rowptr[i], rowptr[i+1]) with colidx[k] >= b*W
// (binary search; needs ascending columns in each row).
static __global__ void __launch_bounds__(256)
k_xstat_splits(int64_t m, const int* __restrict__ rowptr, const int* __restrict__ colidx, int B, int W,
               int* __restrict__ seg) {
  for (int64_t i = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; i < m;
       i += int64_t(gridDim.x) * blockDim.x) {
    const int k0 = rowptr[i], k1 = rowptr[i + 1];
    for (int b = 1; b < B; ++b) {
      const long long bound = (long long)b * W;
      int lo = k0, hi = k1;
      while (lo < hi) {
        const int mid = lo + ((hi - lo) >> 1);
        if ((long long)colidx[mid] >= bound) hi = mid; else lo = mid + 1;
      }
      seg[int64_t(b - 1) * m + i] = lo;
    }
  }
}

}  // namespace spmv
