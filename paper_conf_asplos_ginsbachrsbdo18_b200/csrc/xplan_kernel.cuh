// xplan_kernel.cuh -- x-stationary SpMV over a column-blocked device plan of A.
//
// Measured on B200 (tools/microbench): random 8-B gathers run at ~1/clk/SM
// through L1 (one wavefront per line), ~5/clk/SM from local shared memory and
// ~0.35/clk/SM through DSMEM; TMA bulk copies sustain only ~1 request per 65
// clk per SM, so they stream HBM at 6.6-7.2 TB/s only in chunks of >= 4 KB.
// NAS-CG rows (random columns) therefore need x in LOCAL shared memory and
// the nonzeros in large CONTIGUOUS chunks.  The plan (built once at create --
// the paper's device-resident "lazy copy" of A) re-lays the
// nonzeros out so that both hold:
//
//   clusters of B CTAs; CTA rank b holds x[b*W, (b+1)*W) in shared memory;
//   cluster c owns rows [crow[c], crow[c+1]) (nnz-balanced), cut into tiles of
//   R rows; for every (tile, b) the entries of those rows whose column lies in
//   block b are stored contiguously (row-major inside the tile), values in
//   the matrix precision and columns as uint16 offsets inside the block; the
//   streams of one CTA (all its tiles) are contiguous in HBM.
//
// Kernel: one producer warp streams the CTA's tiles through an S-stage ring
// with cp.async.bulk (chunks of CH entries, mbarrier full/empty pipeline) plus
// the per-tile row offsets; 16 consumer warps form groups of G lanes, each
// group owns R/NG fixed rows of every tile and accumulates their partial sums
// in registers over the chunks (deterministic order); at the end of a tile
// the partials go to a triple-buffered shared array and, after a split
// cluster barrier, CTA b reduces rows [b*R/B, (b+1)*R/B) of the tile over the
// B CTAs by DSMEM reads in rank order and writes y (+ the fused CG dot).
#pragma once
#include <cooperative_groups.h>

#include "common.cuh"
#include "xstat_kernel.cuh"  // cluster/mbarrier/bulk helpers

namespace spmv {

constexpr int XP_R = 256;          // rows per tile
constexpr int XP_CONSUMERS = 512;  // consumer threads (16 warps)
constexpr int XP_THREADS = XP_CONSUMERS + 32;
constexpr int XP_S = 4;            // pipeline stages

struct XplanArgs {
  int64_t nx;               // length of x
  int W;                    // column block width
  int CH;                   // entries per chunk (multiple of 8)
  const void* pvals;        // plan values (T)
  const uint16_t* pcols;    // plan column offsets inside the block
  const int* rofs;          // [tile][b][R+1] row offsets inside the tile stream
  const long long* toff;    // [tile][b] entry offset of the tile stream (multiple of 8)
  const int* tlen;          // [tile][b] padded entry count (multiple of 8)
  const long long* crow;    // [ncl+1] cluster row ranges
  const int* tile0;         // [ncl+1] first global tile of each cluster
  const void* x;
  void* y;
  double alpha, beta;
  const void* w;            // DOT: w[i]
  double* part;             // DOT: one partial per CTA
};

__device__ __forceinline__ void mbar_arrive(uint64_t* bar) {
  asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];\n" ::"r"(smem_u32(bar)) : "memory");
}

// smem layout (dynamic): xs [W*sizeof(T) rounded to 128] | stage vals [S][CH] T |
// stage cols [S][CH] u16 | rofs [3][R+1] int | pbuf [3][R] double
template <typename T, int G, bool DOT>
__global__ void __launch_bounds__(XP_THREADS, 1)
k_spmv_xplan(XplanArgs a) {
  extern __shared__ __align__(128) unsigned char smem[];
  __shared__ uint64_t full[XP_S], empty[XP_S], rbar[3], xbar;
  __shared__ double red[32];
  cgx::cluster_group cluster = cgx::this_cluster();
  const int B = (int)cluster.num_blocks();
  const int b = (int)cluster_rank();
  const int c = (int)cluster_id();
  constexpr int R = XP_R;
  constexpr int NG = XP_CONSUMERS / G;
  constexpr int RPG = R / NG;  // rows per group per tile
  const int CH = a.CH;

  const size_t xbytes = (size_t(a.W) * sizeof(T) + 127) & ~size_t(127);
  T* xs = reinterpret_cast<T*>(smem);
  T* sv = reinterpret_cast<T*>(smem + xbytes);
  uint16_t* sc = reinterpret_cast<uint16_t*>(smem + xbytes + size_t(XP_S) * CH * sizeof(T));
  int* srofs = reinterpret_cast<int*>(smem + xbytes + size_t(XP_S) * CH * (sizeof(T) + 2));
  double* pbuf = reinterpret_cast<double*>(smem + xbytes + size_t(XP_S) * CH * (sizeof(T) + 2) + 3 * (R + 4) * 4);

  const int warp = threadIdx.x >> 5;
  const bool producer = warp == XP_CONSUMERS / 32;
  const int64_t r0c = a.crow[c], r1c = a.crow[c + 1];
  const int ntiles = int((r1c - r0c + R - 1) / R);
  const int tbase = a.tile0[c];

  const int64_t col0 = int64_t(b) * a.W;
  const int64_t ncols = cmax64(0, cmin64(a.W, a.nx - col0));
  const T* __restrict__ xg = static_cast<const T*>(a.x);
  const bool x_aligned = (reinterpret_cast<uintptr_t>(xg + col0) & 15) == 0;
  const int64_t bulk_elems = x_aligned ? ((ncols * int64_t(sizeof(T))) & ~int64_t(15)) / int64_t(sizeof(T)) : 0;

  if (threadIdx.x == 0) {
    for (int s = 0; s < XP_S; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], XP_CONSUMERS / 32);
    }
    for (int s = 0; s < 3; ++s) mbar_init(&rbar[s], 1);
    mbar_init(&xbar, 1);
    asm volatile("fence.mbarrier_init.release.cluster;\n" ::: "memory");
  }
  __syncthreads();

  if (producer) {
    // ------------------------------------------------------------ producer
    const int lane = threadIdx.x & 31;
    if (lane == 0) {
      const uint32_t xb = uint32_t(bulk_elems * sizeof(T));
      mbar_expect_tx(&xbar, xb);
      if (xb) bulk_g2s(xs, xg + col0, xb, &xbar);
    }
    const T* __restrict__ pv = static_cast<const T*>(a.pvals);
    int gc = 0;  // global chunk counter of this CTA
    for (int t = 0; t < ntiles; ++t) {
      const int tg = tbase + t;
      const int64_t off = a.toff[int64_t(tg) * B + b];
      const int len = a.tlen[int64_t(tg) * B + b];
      if (lane == 0) {
        const int rs = t % 3;
        // R+1 offsets, stored padded to R+4 ints (1040 B, a 16-B multiple)
        mbar_expect_tx(&rbar[rs], uint32_t((R + 4) * 4));
        bulk_g2s(srofs + rs * (R + 4), a.rofs + (int64_t(tg) * B + b) * (R + 4), uint32_t((R + 4) * 4), &rbar[rs]);
      }
      for (int e0 = 0; e0 < len; e0 += CH, ++gc) {
        const int n = min(CH, len - e0);
        const int s = gc % XP_S;
        if (gc >= XP_S) mbar_wait(&empty[s], ((gc / XP_S) - 1) & 1);
        if (lane == 0) {
          const uint32_t vb = uint32_t(n * sizeof(T)), cb = uint32_t(n * 2);
          mbar_expect_tx(&full[s], vb + cb);
          bulk_g2s(sv + size_t(s) * CH, pv + off + e0, vb, &full[s]);
          bulk_g2s(sc + size_t(s) * CH, a.pcols + off + e0, cb, &full[s]);
        }
        __syncwarp();
      }
      // tile t issued
      if (t == 0) {
        cluster_arrive();
      } else {
        cluster_wait();
        cluster_arrive();
      }
    }
    if (ntiles > 0) cluster_wait();
  } else {
    // ----------------------------------------------------------- consumers
    const int lane = threadIdx.x & (G - 1);
    const unsigned wl = threadIdx.x & 31;
    const unsigned gmask = (G == 32) ? 0xffffffffu : (((1u << G) - 1u) << (wl & ~(unsigned)(G - 1)));
    const int group = threadIdx.x / G;
    const double alpha = a.alpha, beta = a.beta;
    const int fin_lo = (b * R) / B, fin_hi = ((b + 1) * R) / B;
    double dacc = 0.0;
    // tail of the x block not covered by the bulk copy
    for (int64_t j = bulk_elems + threadIdx.x; j < ncols; j += XP_CONSUMERS) xs[j] = xg[col0 + j];
    asm volatile("bar.sync 1, %0;\n" ::"r"(XP_CONSUMERS) : "memory");
    mbar_wait(&xbar, 0);

    int gc = 0;
    auto process = [&](int t) {
      const int tg = tbase + t;
      const int len = a.tlen[int64_t(tg) * B + b];
      const int64_t rt = r0c + int64_t(t) * R;
      const int nrows = int(cmin64(R, r1c - rt));
      const int rs = t % 3;
      mbar_wait(&rbar[rs], (t / 3) & 1);
      const int* ro = srofs + rs * (R + 4);
      int lo[RPG], hi[RPG];
      double acc[RPG];
#pragma unroll
      for (int i = 0; i < RPG; ++i) {
        const int j = group + i * NG;
        lo[i] = (j < nrows) ? ro[j] : 0;
        hi[i] = (j < nrows) ? ro[j + 1] : 0;
        acc[i] = 0.0;
      }
      for (int e0 = 0; e0 < len; e0 += CH, ++gc) {
        const int s = gc % XP_S;
        mbar_wait(&full[s], (gc / XP_S) & 1);
        const T* v = sv + size_t(s) * CH - e0;
        const uint16_t* cc = sc + size_t(s) * CH - e0;
        const int e1 = e0 + CH;
#pragma unroll
        for (int i = 0; i < RPG; ++i) {
          const int l0 = max(lo[i], e0), l1 = min(hi[i], e1);
          int e = l0 + lane;
          for (; e + G < l1; e += 2 * G) {
            const uint16_t c0 = cc[e], c1 = cc[e + G];
            const T v0 = v[e], v1 = v[e + G];
            acc[i] += double(v0) * double(xs[c0]);
            acc[i] += double(v1) * double(xs[c1]);
          }
          if (e < l1) acc[i] += double(v[e]) * double(xs[cc[e]]);
        }
        __syncwarp();
        if ((threadIdx.x & 31) == 0) mbar_arrive(&empty[s]);
      }
      double* pb = pbuf + (t % 3) * R;
#pragma unroll
      for (int i = 0; i < RPG; ++i) {
        double sum = (G > 1) ? group_sum<G>(acc[i], gmask) : acc[i];
        const int j = group + i * NG;
        if (lane == 0 && j < nrows) pb[j] = sum;
      }
    };
    auto finalize = [&](int t) {
      const double* pb = pbuf + (t % 3) * R;
      const int64_t rt = r0c + int64_t(t) * R;
      const int nrows = int(cmin64(R, r1c - rt));
      for (int j = fin_lo + threadIdx.x; j < min(fin_hi, nrows); j += XP_CONSUMERS) {
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
    if (ntiles > 0) {
      process(0);
      cluster_arrive();
      for (int t = 1; t < ntiles; ++t) {
        process(t);
        cluster_wait();
        finalize(t - 1);
        cluster_arrive();
      }
      cluster_wait();
      finalize(ntiles - 1);
    }
    if (DOT) {
      const double tsum = block_sum_n(dacc, red, XP_CONSUMERS / 32);
      if (threadIdx.x == 0) a.part[blockIdx.x] = tsum;
    }
  }
  // peers may still read this CTA's pbuf: leave together
  cluster_arrive();
  cluster_wait();
}

// ---------------------------------------------------------------- builders
// Per (tile, b): row lengths inside block b -> row offsets (exclusive scan)
// and the tile's entry count.  One CTA (R threads) per (global tile, b).
__global__ void __launch_bounds__(XP_R)
k_xplan_rofs(const int* __restrict__ rowptr, const int* __restrict__ seg, int64_t m, int B,
             const long long* __restrict__ crow, const int* __restrict__ tile0, int ncl,
             int* __restrict__ rofs, int* __restrict__ tlen_raw) {
  __shared__ int sc[XP_R];
  const int tg = blockIdx.x / B, b = blockIdx.x % B;
  int c = 0;
  while (c + 1 < ncl && tile0[c + 1] <= tg) ++c;
  const int t = tg - tile0[c];
  const int64_t rt = crow[c] + int64_t(t) * XP_R;
  const int nrows = int(cmin64(XP_R, crow[c + 1] - rt));
  const int j = threadIdx.x;
  int L = 0;
  if (j < nrows) {
    const int64_t i = rt + j;
    const int k0 = (b == 0) ? rowptr[i] : seg[int64_t(b - 1) * m + i];
    const int k1 = (b == B - 1) ? rowptr[i + 1] : seg[int64_t(b) * m + i];
    L = k1 - k0;
  }
  sc[j] = L;
  __syncthreads();
  for (int d = 1; d < XP_R; d <<= 1) {  // inclusive Hillis-Steele scan
    const int v = (j >= d) ? sc[j - d] : 0;
    __syncthreads();
    sc[j] += v;
    __syncthreads();
  }
  int* ro = rofs + (int64_t(tg) * B + b) * (XP_R + 4);
  ro[j + 1] = sc[j];
  if (j == 0) ro[0] = 0;
  if (j < 3) ro[XP_R + 1 + j] = sc[XP_R - 1];  // padding of the 16-B copy
  if (j == XP_R - 1) tlen_raw[int64_t(tg) * B + b] = sc[j];
}

// Scatter every nonzero into its (tile, block) stream: warp per row.
template <typename T>
__global__ void __launch_bounds__(256)
k_xplan_pack(const int* __restrict__ rowptr, const int* __restrict__ colidx, const T* __restrict__ vals,
             const int* __restrict__ seg, int64_t m, int B, int W, const long long* __restrict__ crow,
             const int* __restrict__ tile0, int ncl, const int* __restrict__ rofs,
             const long long* __restrict__ toff, T* __restrict__ pv, uint16_t* __restrict__ pc, int values_only) {
  const int lane = threadIdx.x & 31;
  for (int64_t i = (int64_t(blockIdx.x) * blockDim.x + threadIdx.x) / 32; i < m;
       i += int64_t(gridDim.x) * blockDim.x / 32) {
    // cluster of row i (binary search in crow) and its tile
    int lo = 0, hi = ncl - 1;
    while (lo < hi) {
      const int mid = (lo + hi + 1) >> 1;
      if (crow[mid] <= i) lo = mid; else hi = mid - 1;
    }
    const int c = lo;
    const int t = int((i - crow[c]) / XP_R);
    const int j = int((i - crow[c]) % XP_R);
    const int tg = tile0[c] + t;
    const int k0 = rowptr[i], k1 = rowptr[i + 1];
    for (int k = k0 + lane; k < k1; k += 32) {
      const int col = colidx[k];
      const int bb = col / W;
      const int s0 = (bb == 0) ? k0 : seg[int64_t(bb - 1) * m + i];
      const int64_t dst = toff[int64_t(tg) * B + bb] + rofs[(int64_t(tg) * B + bb) * (XP_R + 4) + j] + (k - s0);
      pv[dst] = vals[k];
      if (!values_only) pc[dst] = uint16_t(col - bb * W);
    }
  }
}

}  // namespace spmv
