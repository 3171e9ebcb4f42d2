// xplan_kernel.cuh -- x-stationary SpMV over a column-blocked device plan of A.
//
// Measured on B200 (tools/microbench):
//   * random 8-B gathers: ~1/clk/SM through L1 (one wavefront per line),
//     ~5/clk/SM from local shared memory, ~0.35/clk/SM through DSMEM;
//   * TMA bulk copies: ~1 request per 65 clk per SM; a ring of 4 x 16 KB
//     copies per SM streams HBM at 6.7 TB/s on 120 SMs, 8 KB copies cap at
//     ~4.5 TB/s.
// NAS-CG rows (random columns) therefore need x in LOCAL shared memory and
// the nonzeros in large contiguous records.  The plan (built once at create:
// the paper's device-resident "lazy copy" of A) re-lays A out:
//
//   clusters of B CTAs; CTA rank b keeps x[b*W, (b+1)*W) in shared memory;
//   cluster c owns rows [crow[c], crow[c+1]) (nnz-balanced), cut into tiles of
//   R rows; for every (cluster, b) the entries of its rows whose column lies
//   in block b form one contiguous stream of RECORDS, each <= SB bytes and
//   holding whole rows of one tile:
//       int32 header {tile, j0 (first row in tile), nr (rows), n (entries,
//       multiple of 8)}, uint16 ofs[nr+1] (row starts, padded to 16 B),
//       T vals[n], uint16 cols[n] (column offsets inside block b).
//
// Kernel (one CTA per SM, clusters of B): one producer warp streams the CTA's
// records through S slots with one cp.async.bulk each (mbarrier full/empty);
// slot s is consumed by its own WPS warps, which split the record's rows,
// gather x from shared memory and write each row's block partial into a
// triple-buffered receive array of the CTA that owns the row (rows
// [q*R/B, (q+1)*R/B) of a tile belong to CTA q) with st.async, which completes
// transaction bytes on the owner's mbarrier of that tile.  The owner waits for
// all B partials of its rows, sums them in rank order and writes y (+ the
// fused CG dot).  A relaxed split cluster barrier (arrive after tile t, wait
// after tile t+1) bounds how far a CTA may run ahead, so a receive buffer is
// never overwritten before its tile was reduced.  No fences on the steady
// path, deterministic (fixed row->lane mapping and summation order).
#pragma once
#include <cooperative_groups.h>

#include "common.cuh"
#include "xstat_kernel.cuh"  // cluster / mbarrier / bulk-copy helpers

namespace spmv {

constexpr int XP_R = 256;   // rows per tile
constexpr int XP_S = 4;     // record slots (pipeline stages)
constexpr int XP_WPS = 4;   // consumer warps per slot
constexpr int XP_CONSUMERS = XP_S * XP_WPS * 32;
constexpr int XP_THREADS = XP_CONSUMERS + 32;
constexpr int XP_HDR = 16;  // record header bytes

__host__ __device__ constexpr int xp_ofs_bytes(int nr) { return ((nr + 1) * 2 + 15) & ~15; }

struct XplanArgs {
  int64_t nx;                  // length of x
  int W;                       // column block width
  int SB;                      // slot bytes (max record size)
  const unsigned char* plan;   // record streams
  const long long* rec_off;    // [nrec+1] byte offset of every record
  const int* rec_tile;         // [nrec] tile (within the cluster) of every record
  const int* cta_rec;          // [ncl*B+1] first record of CTA (c, b)
  const long long* crow;       // [ncl+1] cluster row ranges
  const void* x;
  void* y;
  double alpha, beta;
  const void* w;               // DOT: w[i]
  double* part;                // DOT: one partial per CTA
};

__device__ __forceinline__ void mbar_arrive(uint64_t* bar) {
  asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];\n" ::"r"(smem_u32(bar)) : "memory");
}

// Relaxed cluster-barrier arrive: no memory ordering (the .release form and
// fence.acq_rel.cluster both lower to MEMBAR.ALL.GPU, which waits for every
// outstanding global store).  Used only for buffer back-pressure; the row
// partials travel by st.async with mbarrier transaction counts.
__device__ __forceinline__ void cluster_arrive_relaxed() {
  asm volatile("barrier.cluster.arrive.relaxed.aligned;\n" ::: "memory");
}
__device__ __forceinline__ uint32_t mapa_u32(uint32_t laddr, uint32_t rank) {
  uint32_t r;
  asm volatile("mapa.shared::cluster.u32 %0, %1, %2;\n" : "=r"(r) : "r"(laddr), "r"(rank));
  return r;
}
// 8-byte store into a peer CTA's shared memory that completes `bytes` on the
// peer's mbarrier (no fence needed, the mbarrier phase orders it).
__device__ __forceinline__ void st_async_f64(uint32_t raddr, double v, uint32_t rbar) {
  asm volatile("st.async.shared::cluster.mbarrier::complete_tx::bytes.b64 [%0], %1, [%2];\n" ::"r"(raddr),
               "l"(__double_as_longlong(v)), "r"(rbar)
               : "memory");
}

// smem (dynamic): xs [W*sizeof(T) rounded to 128] | slots [S][SB] | recv [3][R] double
//                 (recv[t%3][b*(R/B) + jl]: partial of CTA b for owned row jl)
template <typename T, int G, bool DOT>
__global__ void __launch_bounds__(XP_THREADS, 1)
k_spmv_xplan(XplanArgs a) {
  extern __shared__ __align__(128) unsigned char smem[];
  __shared__ uint64_t full[XP_S], empty[XP_S], xbar, tbar[3];
  __shared__ double red[32];
  cgx::cluster_group cluster = cgx::this_cluster();
  const int B = (int)cluster.num_blocks();
  const int b = (int)cluster_rank();
  const int c = (int)cluster_id();
  constexpr int R = XP_R;
  const int SB = a.SB;

  const size_t xbytes = (size_t(a.W) * sizeof(T) + 127) & ~size_t(127);
  T* xs = reinterpret_cast<T*>(smem);
  unsigned char* slots = smem + xbytes;
  double* recv = reinterpret_cast<double*>(slots + size_t(XP_S) * SB);
  const int RB = R / B;  // rows of a tile owned by each CTA

  const int warp = threadIdx.x >> 5;
  const bool producer = warp == XP_CONSUMERS / 32;
  const int64_t r0c = a.crow[c], r1c = a.crow[c + 1];
  const int ntiles = int((r1c - r0c + R - 1) / R);
  const int rb = a.cta_rec[c * B + b], re = a.cta_rec[c * B + b + 1];

  const int64_t col0 = int64_t(b) * a.W;
  const int64_t ncols = cmax64(0, cmin64(a.W, a.nx - col0));
  const T* __restrict__ xg = static_cast<const T*>(a.x);
  const bool x_aligned = (reinterpret_cast<uintptr_t>(xg + col0) & 15) == 0;
  const int64_t bulk_elems = x_aligned ? ((ncols * int64_t(sizeof(T))) & ~int64_t(15)) / int64_t(sizeof(T)) : 0;

  if (threadIdx.x == 0) {
    for (int s = 0; s < XP_S; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], XP_WPS);
    }
    mbar_init(&xbar, 1);
    for (int q = 0; q < 3; ++q) mbar_init(&tbar[q], 1);
    asm volatile("fence.mbarrier_init.release.cluster;\n" ::: "memory");
  }
  __syncthreads();
  // bytes of partials this CTA receives for tile t: B per owned existing row
  auto recv_bytes = [&](int t) -> uint32_t {
    const int nrows = int(cmin64(R, r1c - (r0c + int64_t(t) * R)));
    const int own = max(0, min((b + 1) * RB, nrows) - b * RB);
    return uint32_t(own * B * 8);
  };
  if (threadIdx.x == 0)
    for (int t = 0; t < 3 && t < ntiles; ++t) mbar_expect_tx(&tbar[t], recv_bytes(t));
  // every CTA of the cluster must have initialised its barriers before peers
  // send partials to it
  cluster_arrive();
  cluster_wait();

  if (producer) {
    // ------------------------------------------------------------ producer
    const int lane = threadIdx.x & 31;
    if (lane == 0) {
      const uint32_t xb = uint32_t(bulk_elems * sizeof(T));
      mbar_expect_tx(&xbar, xb);
      if (xb) bulk_g2s(xs, xg + col0, xb, &xbar);
    }
    int t = 0;
    for (int k = rb; k <= re; ++k) {
      const int tk = (k < re) ? a.rec_tile[k] : ntiles;
      for (; t < tk; ++t) {  // all records of tile t issued
        if (t > 0) cluster_wait();
        cluster_arrive_relaxed();
      }
      if (k == re) break;
      const int j = k - rb, s = j % XP_S;
      if (j >= XP_S) mbar_wait(&empty[s], ((j / XP_S) - 1) & 1);
      if (lane == 0) {
        const uint32_t bytes = uint32_t(a.rec_off[k + 1] - a.rec_off[k]);
        mbar_expect_tx(&full[s], bytes);
        bulk_g2s(slots + size_t(s) * SB, a.plan + a.rec_off[k], bytes, &full[s]);
      }
      __syncwarp();
    }
    if (ntiles > 0) cluster_wait();
  } else {
    // ----------------------------------------------------------- consumers
    const int s = warp / XP_WPS, sub = warp % XP_WPS;
    const int lane = threadIdx.x & (G - 1);
    const unsigned wl = threadIdx.x & 31;
    const unsigned gmask = (G == 32) ? 0xffffffffu : (((1u << G) - 1u) << (wl & ~(unsigned)(G - 1)));
    const int gw = (threadIdx.x & 31) / G;  // group inside the warp
    constexpr int GPW = 32 / G;             // groups per warp
    const double alpha = a.alpha, beta = a.beta;
    const int fin_lo = (b * R) / B, fin_hi = ((b + 1) * R) / B;
    double dacc = 0.0;
    for (int64_t j = bulk_elems + threadIdx.x; j < ncols; j += XP_CONSUMERS) xs[j] = xg[col0 + j];
    asm volatile("bar.sync 1, %0;\n" ::"r"(XP_CONSUMERS) : "memory");
    mbar_wait(&xbar, 0);

    auto finalize = [&](int t) {
      const double* rv = recv + (t % 3) * R;
      const int64_t rt = r0c + int64_t(t) * R;
      const int nrows = int(cmin64(R, r1c - rt));
      mbar_wait(&tbar[t % 3], (t / 3) & 1);
      for (int jl = threadIdx.x; jl < RB && b * RB + jl < nrows; jl += XP_CONSUMERS) {
        double sum = 0.0;
        for (int q = 0; q < B; ++q) sum += rv[q * RB + jl];
        const int64_t i = rt + b * RB + jl;
        T* y = static_cast<T*>(a.y);
        double r = alpha * sum;
        if (beta != 0.0) r += beta * double(y[i]);
        const T out = T(r);
        y[i] = out;
        if (DOT) dacc += double(static_cast<const T*>(a.w)[i]) * double(out);
      }
      // re-arm the buffer for tile t+3 (its partials can only arrive after
      // this CTA's next arrive, see the barrier argument above)
      asm volatile("bar.sync 1, %0;\n" ::"r"(XP_CONSUMERS) : "memory");
      if (threadIdx.x == 0 && t + 3 < ntiles) mbar_expect_tx(&tbar[t % 3], recv_bytes(t + 3));
    };
    // every row of a tile lies in exactly one record of this CTA (empty
    // segments included), so each pbuf entry is written before it is read.
    int t = 0;
    int tk = (rb + s < re) ? a.rec_tile[rb + s] : ntiles;
    for (int k = rb + s; ; k += XP_S) {
      for (; t < tk; ++t) {  // tile boundary after tile t
        if (t > 0) {
          cluster_wait();
          finalize(t - 1);
        }
        cluster_arrive_relaxed();
      }
      if (k >= re) break;
      const int tk_next = (k + XP_S < re) ? a.rec_tile[k + XP_S] : ntiles;  // prefetch
      const int j = k - rb;
      mbar_wait(&full[s], (j / XP_S) & 1);
      const unsigned char* rec = slots + size_t(s) * SB;
      const int* hdr = reinterpret_cast<const int*>(rec);
      const int j0 = hdr[1], nr = hdr[2], n = hdr[3];
      const uint16_t* ofs = reinterpret_cast<const uint16_t*>(rec + XP_HDR);
      const T* v = reinterpret_cast<const T*>(rec + XP_HDR + xp_ofs_bytes(nr));
      const uint16_t* cc = reinterpret_cast<const uint16_t*>(rec + XP_HDR + xp_ofs_bytes(nr) + size_t(n) * sizeof(T));
      const uint32_t rbase = smem_u32(recv + (hdr[0] % 3) * R + b * RB);
      const uint32_t rbar_l = smem_u32(&tbar[hdr[0] % 3]);
      // rows r = sub*GPW + gw + m*(WPS*GPW)
      for (int r = sub * GPW + gw; r < nr; r += XP_WPS * GPW) {
        const int e0 = ofs[r], e1 = ofs[r + 1];
        double acc = 0.0;
        int e = e0 + lane;
        for (; e + G < e1; e += 2 * G) {
          const uint16_t c0 = cc[e], c1 = cc[e + G];
          const T v0 = v[e], v1 = v[e + G];
          acc += double(v0) * double(xs[c0]);
          acc += double(v1) * double(xs[c1]);
        }
        if (e < e1) acc += double(v[e]) * double(xs[cc[e]]);
        if (G > 1) acc = group_sum<G>(acc, gmask);
        if (lane == 0) {
          const int j = j0 + r, q = j / RB, jl = j - q * RB;
          // same layout in every CTA: slot [t%3][b*RB + jl] of the owner q
          st_async_f64(mapa_u32(rbase + uint32_t(jl * 8), q), acc, mapa_u32(rbar_l, q));
        }
      }
      __syncwarp();
      if ((threadIdx.x & 31) == 0) mbar_arrive(&empty[s]);
      tk = tk_next;
    }
    if (ntiles > 0) {
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
// Row segment [k0, k1) of row i in column block b.
__device__ __forceinline__ void xp_seg(const int* rowptr, const int* seg, int64_t m, int B, int b, int64_t i,
                                       int* k0, int* k1) {
  *k0 = (b == 0) ? rowptr[i] : seg[int64_t(b - 1) * m + i];
  *k1 = (b == B - 1) ? rowptr[i + 1] : seg[int64_t(b) * m + i];
}

__device__ __forceinline__ int xp_rec_bytes(int nr, int n, int ts) {
  return XP_HDR + xp_ofs_bytes(nr) + n * ts + n * 2;
}

// Greedy cut of the rows of (tile, b) into records of <= SB bytes, whole rows
// only.  pass 0: counts records and bytes (too-long row -> *bad = 1);
// pass 1: writes headers/offsets, the record table and every row's
// (record, position) for the pack kernel.  One thread per (tile, b).
__global__ void k_xplan_records(const int* __restrict__ rowptr, const int* __restrict__ seg, int64_t m, int B,
                                const long long* __restrict__ crow, const int* __restrict__ tile0, int ncl,
                                int ntiles, int ts, int SB, int pass, int* __restrict__ nrec,
                                long long* __restrict__ bytes, const int* __restrict__ rec_first,
                                const long long* __restrict__ byte_first, long long* __restrict__ rec_off,
                                int* __restrict__ rec_tile, unsigned char* __restrict__ plan,
                                int* __restrict__ row_rec, int* __restrict__ row_pos, int* __restrict__ bad) {
  const int64_t id = int64_t(blockIdx.x) * blockDim.x + threadIdx.x;
  if (id >= int64_t(ntiles) * B) return;
  const int tg = int(id / B), b = int(id % B);
  int c = 0;
  while (c + 1 < ncl && tile0[c + 1] <= tg) ++c;
  const int t = tg - tile0[c];
  const int64_t rt = crow[c] + int64_t(t) * XP_R;
  const int nrows = int(cmin64(XP_R, crow[c + 1] - rt));
  int cnt = 0;
  long long tot = 0;
  int r = 0;
  int rec = pass ? rec_first[id] : 0;
  long long off = pass ? byte_first[id] : 0;
  while (r < nrows) {
    // grow a record from row r
    int nr = 0, n = 0;
    while (r + nr < nrows) {
      int k0, k1;
      xp_seg(rowptr, seg, m, B, b, rt + r + nr, &k0, &k1);
      const int L = k1 - k0;
      const int n2 = (n + L + 7) & ~7;
      if (xp_rec_bytes(nr + 1, n2, ts) > SB) {
        if (nr == 0) { atomicExch(bad, 1); return; }
        break;
      }
      n += L;
      ++nr;
    }
    const int np = (n + 7) & ~7;
    const int nb = xp_rec_bytes(nr, np, ts);
    if (pass) {
      unsigned char* p = plan + off;
      int* hdr = reinterpret_cast<int*>(p);
      hdr[0] = t;
      hdr[1] = r;
      hdr[2] = nr;
      hdr[3] = np;
      uint16_t* ofs = reinterpret_cast<uint16_t*>(p + XP_HDR);
      int e = 0;
      for (int q = 0; q < nr; ++q) {
        int k0, k1;
        xp_seg(rowptr, seg, m, B, b, rt + r + q, &k0, &k1);
        ofs[q] = uint16_t(e);
        row_rec[int64_t(b) * m + rt + r + q] = rec;
        row_pos[int64_t(b) * m + rt + r + q] = e;
        e += k1 - k0;
      }
      ofs[nr] = uint16_t(e);
      rec_off[rec] = off;
      rec_tile[rec] = t;
      ++rec;
      off += nb;
    }
    ++cnt;
    tot += nb;
    r += nr;
  }
  if (!pass) {
    nrec[id] = cnt;
    bytes[id] = tot;
  }
}

// Scatter every nonzero into its record: warp per row.
template <typename T>
__global__ void __launch_bounds__(256)
k_xplan_pack(const int* __restrict__ rowptr, const int* __restrict__ colidx, const T* __restrict__ vals,
             const int* __restrict__ seg, int64_t m, int B, int W, const long long* __restrict__ rec_off,
             const int* __restrict__ row_rec, const int* __restrict__ row_pos, unsigned char* __restrict__ plan,
             int values_only) {
  const int lane = threadIdx.x & 31;
  for (int64_t i = (int64_t(blockIdx.x) * blockDim.x + threadIdx.x) / 32; i < m;
       i += int64_t(gridDim.x) * blockDim.x / 32) {
    const int k0 = rowptr[i], k1 = rowptr[i + 1];
    for (int k = k0 + lane; k < k1; k += 32) {
      const int col = colidx[k];
      const int bb = col / W;
      const int s0 = (bb == 0) ? k0 : seg[int64_t(bb - 1) * m + i];
      const int rec = row_rec[int64_t(bb) * m + i];
      unsigned char* p = plan + rec_off[rec];
      const int* hdr = reinterpret_cast<const int*>(p);
      const int nr = hdr[2], n = hdr[3];
      const int pos = row_pos[int64_t(bb) * m + i] + (k - s0);
      T* v = reinterpret_cast<T*>(p + XP_HDR + xp_ofs_bytes(nr));
      v[pos] = vals[k];
      if (!values_only) {
        uint16_t* cc = reinterpret_cast<uint16_t*>(p + XP_HDR + xp_ofs_bytes(nr) + size_t(n) * sizeof(T));
        cc[pos] = uint16_t(col - bb * W);
      }
    }
  }
}

}  // namespace spmv
