// xplan_kernel.cuh -- x-stationary SpMV over a column-blocked SELL-32 plan of A.
//
// Measured on B200 (tools/microbench):
//   * random 8-B gathers: ~1/clk/SM through L1 (one wavefront per line),
//     ~5/clk/SM from local shared memory, ~0.35/clk/SM through DSMEM;
//   * a TMA bulk-copy ring needs >= 64 KB of 16-KB copies in flight per SM to
//     approach HBM bandwidth -- which does not fit next to a resident x block.
// NAS-CG rows (random columns) therefore need x in LOCAL shared memory, and
// the nonzeros must stream with deep memory-level parallelism without shared
// memory staging.  The plan (built once at create: the paper's
// device-resident "lazy copy" of A) re-lays A out as
//
//   clusters of B CTAs; CTA rank b keeps x[b*W, (b+1)*W) (+ a zero pad at W)
//   in shared memory; cluster c owns rows [crow[c], crow[c+1]) (nnz-balanced),
//   cut into tiles of R = 32*NW rows; inside a tile the rows are sorted by the
//   length of their segment in block b (SELL-C-sigma with C = 32, sigma = R)
//   and cut into NW chunks of 32 rows.  Chunk (tile, b, w) stores len
//   steps column-major: vals as [len/2][32 lanes][2] (2 values per lane per
//   step pair; an odd last step as one [32] row) then columns as
//   [len/2][32][2] uint16 offsets inside the block (odd last step [32]);
//   padding entries have value 0 and column W (x pad 0.0).
//
// Kernel (one CTA of NW warps per SM, clusters of B): per tile, warp w streams
// chunk w with coalesced 16-B loads, 4 step pairs in flight, lane = row, so no
// reduction is needed inside a row; the lane's block partial is pushed to the
// CTA that owns the row (rows [q*R/B, (q+1)*R/B) of a tile belong to CTA q)
// with st.async, completing transaction bytes on the owner's mbarrier of that
// tile.  The owner sums the B partials of its rows in rank order and writes y
// (+ the fused CG dot).  A relaxed split cluster barrier (arrive after tile t,
// wait after tile t+1) bounds how far a CTA runs ahead, so receive buffers are
// reused safely.  No fences on the steady path, deterministic.
#pragma once
#include <cooperative_groups.h>

#include "common.cuh"
#include "xstat_kernel.cuh"  // cluster / mbarrier / bulk-copy helpers

namespace spmv {

#ifndef XP_NW_DEF
#define XP_NW_DEF 32
#endif
constexpr int XP_NW = XP_NW_DEF;     // warps per CTA
#ifndef XP_CPW_DEF
#define XP_CPW_DEF 2
#endif
constexpr int XP_CPW = XP_CPW_DEF;   // chunks per warp per tile (paired longest + shortest)
constexpr int XP_CPT = XP_NW * XP_CPW;  // chunks per tile
constexpr int XP_R = 32 * XP_CPT;    // rows per tile
constexpr int XP_THREADS = 32 * XP_NW;
constexpr int XP_K = 3;              // receive buffers
#ifndef XP_U_DEF
#define XP_U_DEF 9
#endif
constexpr int XP_U = XP_U_DEF;       // step pairs (16-B loads) in flight per lane
#ifndef XP_ODD
#define XP_ODD 0  // 1: odd chunk lengths (no even-rounding padding: measured 87.0 vs 78.9 us on C); 0: even
#endif

struct XplanArgs {
  int64_t nx;                  // length of x
  int W;                       // column block width (pad column = W)
  const unsigned char* plan;   // chunk data
  const long long* chunk_off;  // [tile][b][chunk] byte offset of chunk data
  const int* chunk_len;        // [tile][b][chunk] steps (the chunk's longest segment)
  const uint16_t* chunk_row;   // [tile][b][chunk][32] tile-local row of each lane (0xffff = none)
  const long long* crow;       // [ncl+1] cluster row ranges
  const int* tile0;            // [ncl+1] first global tile of each cluster
  const void* x;
  void* y;
  double alpha, beta;
  const void* w;               // DOT: w[i]
  double* part;                // DOT: one partial per CTA
  P2PHook hk;                  // p2p transport: wait for x / push the dot
  int dbg;
  int prefetch;                // 1: L2-prefetch the warp's chunk of the next tile
  const long long* cta_range;  // small plans (nullable): [grid][2] byte range of each CTA's chunks, prefetched
                               // into L2 whole at kernel start
  unsigned long long* tstamp;  // diagnostics (nullable): per CTA {start, x ready, streaming done, end} globaltimer
  // DYN (dynamic tile scheduling): the plan is one row range of ntiles_total
  // tiles; clusters pop tiles from *tq (rank 0, K tiles ahead) and the last
  // CTA resets tq/tq_done for the next launch; the fused dot is one partial
  // per (tile, owner CTA): part[tile * B + b]
  int* tq;
  int* tq_done;
  int ntiles_total;
};

// Arguments of the persistent CG kernel (persist_kernel.cuh, NEXT-1).
struct PersistArgs {
  XplanArgs sp;                 // the plan; sp.x = the SpMV input (r, or the padded buffer holding r)
  int64_t n;                    // local vector length (rows)
  int iters;
  double* r;                    // the SpMV input slice (cg_p): r
  double* p;                    // p
  double* s;                    // s = A p (recurrence)
  double* w;                    // w = A r (the SpMV output)
  double* z;                    // solution
  double* part_d;               // [grid] delta partials
  double* part_g;               // [3][pstride] gamma partials (rotating)
  int64_t pstride;
  const double* gam0;           // k_cg_init's r.r partials
  int gam0_count;
  double* alpha2;               // [2] alpha of the last two iterations (for the host-side status)
  int* flags;                   // [0] breakdown, [2] iterations done
  unsigned int* gbar;           // grid barrier counter (zeroed before the launch)
};

__device__ __forceinline__ unsigned long long gtimer() {
  unsigned long long t;
  asm volatile("mov.u64 %0, %globaltimer;" : "=l"(t));
  return t;
}

__device__ __forceinline__ void cluster_arrive_relaxed() {
  __syncwarp();
#ifdef XP_RELEASE_ARRIVE
  asm volatile("barrier.cluster.arrive.release;\n" ::: "memory");
#else
  asm volatile("barrier.cluster.arrive.relaxed;\n" ::: "memory");
#endif
}
__device__ __forceinline__ uint32_t mapa_u32(uint32_t laddr, uint32_t rank) {
  uint32_t r;
  asm volatile("mapa.shared::cluster.u32 %0, %1, %2;\n" : "=r"(r) : "r"(laddr), "r"(rank));
  return r;
}
// 8-byte store into a peer CTA's shared memory that completes 8 transaction
// bytes on the peer's mbarrier (ordered by the mbarrier phase, no fence).
__device__ __forceinline__ void st_async_f64(uint32_t raddr, double v, uint32_t rbar) {
  asm volatile("st.async.shared::cluster.mbarrier::complete_tx::bytes.b64 [%0], %1, [%2];\n" ::"r"(raddr),
               "l"(__double_as_longlong(v)), "r"(rbar)
               : "memory");
}
__device__ __forceinline__ int4 ldg_stream16(const void* p) {
  int4 r;
  asm("ld.global.nc.L1::no_allocate.v4.s32 {%0, %1, %2, %3}, [%4];"
      : "=r"(r.x), "=r"(r.y), "=r"(r.z), "=r"(r.w)
      : "l"(p));
  return r;
}
__device__ __forceinline__ uint32_t ldg_stream4(const void* p) {
  uint32_t r;
  asm("ld.global.nc.L1::no_allocate.u32 %0, [%1];" : "=r"(r) : "l"(p));
  return r;
}
__device__ __forceinline__ uint2 ldg_stream8(const void* p) {
  uint2 r;
  asm("ld.global.nc.L1::no_allocate.v2.u32 {%0, %1}, [%2];" : "=r"(r.x), "=r"(r.y) : "l"(p));
  return r;
}

// two consecutive values of a lane (one step pair)
template <typename T>
struct Pair;
template <>
struct Pair<double> {
  double a, b;
  __device__ __forceinline__ static Pair load(const unsigned char* p) {
    const int4 r = ldg_stream16(p);
    return {__hiloint2double(r.y, r.x), __hiloint2double(r.w, r.z)};
  }
};
template <>
struct Pair<float> {
  float a, b;
  __device__ __forceinline__ static Pair load(const unsigned char* p) {
    const uint2 r = ldg_stream8(p);
    return {__uint_as_float(r.x), __uint_as_float(r.y)};
  }
};

// The block partial of one chunk for the calling lane: len steps in the
// chunk's layout -- vals [len/2][32 lanes][2] then, for odd len, the last step
// [32]; cols likewise ([len/2][32][2] u16, then [32] u16), starting at
// base + len*32*sizeof(T).  XP_U step pairs of 16-B loads in flight per lane
// (the tail batch predicated: masked pairs add 0 * x[W] = 0); the odd last
// step is loaded with the first batch and added last (the chunk's step order).
template <typename T>
__device__ __forceinline__ double xplan_chunk_dot(const unsigned char* base, int len, int lane, const T* xs, int W) {
  const unsigned char* V = base + size_t(lane) * 2 * sizeof(T);
  const unsigned char* C = base + size_t(len) * 32 * sizeof(T) + size_t(lane) * 4;
  constexpr size_t VS = 32 * 2 * sizeof(T);  // bytes per step pair (vals)
  const int np = len >> 1;                   // step pairs
  T vt = T(0);
  uint32_t ct = uint32_t(W);
  if (XP_ODD && (len & 1)) {  // the odd last step, issued ahead of the pairs
    vt = *reinterpret_cast<const T*>(base + size_t(np) * VS + size_t(lane) * sizeof(T));
    ct = *reinterpret_cast<const uint16_t*>(base + size_t(len) * 32 * sizeof(T) + size_t(np) * 128 + size_t(lane) * 2);
  }
  double acc = 0.0;
  const uint32_t padcc = uint32_t(W) | (uint32_t(W) << 16);  // both steps -> x pad 0.0
  for (int p = 0; p < np; p += XP_U) {
    Pair<T> v[XP_U];
    uint32_t cc[XP_U];
#pragma unroll
    for (int u = 0; u < XP_U; ++u) {
      if (p + u < np) {
        v[u] = Pair<T>::load(V + size_t(p + u) * VS);
        cc[u] = ldg_stream4(C + size_t(p + u) * 128);
      } else {
        v[u] = Pair<T>{T(0), T(0)};
        cc[u] = padcc;
      }
    }
#pragma unroll
    for (int u = 0; u < XP_U; ++u) {
      acc += double(v[u].a) * double(xs[cc[u] & 0xffffu]);
      acc += double(v[u].b) * double(xs[cc[u] >> 16]);
    }
  }
  if (XP_ODD && (len & 1)) acc += double(vt) * double(xs[ct]);
  return acc;
}

// smem (dynamic): xs [(W+1)*sizeof(T) rounded to 16] | recv [K][R] double
//   recv[t%K][b*(R/B) + jl]: partial of CTA b for owned row jl
constexpr int XP_TQ = 8;  // DYN: tile-id ring (local tile k in slot k % 8)

template <typename T, bool DOT, bool DYN>
__global__ void __launch_bounds__(XP_THREADS, 1)
k_spmv_xplan(XplanArgs a) {
  extern __shared__ __align__(128) unsigned char smem[];
  __shared__ uint64_t xbar, tbar[XP_K];
  __shared__ uint64_t qbar[XP_TQ];
  __shared__ int tileid[XP_TQ];
  __shared__ double red[32];
  const int B = (int)cgx::this_cluster().num_blocks();
  const int b = (int)cluster_rank();
  const int c = (int)cluster_id();
  constexpr int R = XP_R;
  const int RB = R / B;
  const int W = a.W;

  T* xs = reinterpret_cast<T*>(smem);
  double* recv = reinterpret_cast<double*>(smem + ((size_t(W + 1) * sizeof(T) + 15) & ~size_t(15)));
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  // static: cluster c owns tiles [tile0[c], tile0[c+1]) of rows [crow[c], crow[c+1]);
  // DYN: one range [crow[0], crow[1]), tiles handed out at run time
  const int64_t r0c = DYN ? a.crow[0] : a.crow[c], r1c = DYN ? a.crow[1] : a.crow[c + 1];
  const int ntiles = DYN ? a.ntiles_total : int((r1c - r0c + R - 1) / R);
  const int tbase = DYN ? 0 : a.tile0[c];

  const int64_t col0 = int64_t(b) * W;
  const int64_t ncols = cmax64(0, cmin64(W, a.nx - col0));
  const T* __restrict__ xg = static_cast<const T*>(a.x);
  const bool x_aligned = (reinterpret_cast<uintptr_t>(xg + col0) & 15) == 0;
  const int64_t bulk_elems = x_aligned ? ((ncols * int64_t(sizeof(T))) & ~int64_t(15)) / int64_t(sizeof(T)) : 0;

  if (a.tstamp && threadIdx.x == 0) {
    uint32_t smid;
    asm volatile("mov.u32 %0, %%smid;" : "=r"(smid));
    a.tstamp[4 * blockIdx.x] = (gtimer() & ~0xffull) | smid;  // low byte: the SM (diagnostics)
  }
  if (a.cta_range && warp == 1) {
    // small plan (a few tiles per cluster, latency-bound): ask the TMA unit to
    // stream the CTA's whole chunk range into L2 now, so the warps' dependent
    // load batches hit L2 instead of waiting on HBM one round trip at a time
    const long long r0 = a.cta_range[2 * blockIdx.x], r1 = a.cta_range[2 * blockIdx.x + 1];
    for (long long o = r0 + int64_t(lane) * 65536; o < r1; o += 32 * 65536) {
      const uint32_t nb = uint32_t(cmin64(65536, r1 - o));
      asm volatile("cp.async.bulk.prefetch.L2.global [%0], %1;" ::"l"(a.plan + o), "r"(nb) : "memory");
    }
  }
  auto recv_bytes = [&](int t) -> uint32_t {
    const int nrows = int(cmin64(R, r1c - (r0c + int64_t(t) * R)));
    const int own = max(0, min((b + 1) * RB, nrows) - b * RB);
    return uint32_t(own * B * 8);
  };
  // barrier set-up reads nothing a predecessor writes: it runs before pdl_wait
  // (overlapping the previous kernel's tail under PDL)
  if (threadIdx.x == 0) {
    mbar_init(&xbar, 1);
    for (int q = 0; q < XP_K; ++q) mbar_init(&tbar[q], 1);
    if (DYN)
      for (int q = 0; q < XP_TQ; ++q) mbar_init(&qbar[q], 1);
    asm volatile("fence.mbarrier_init.release.cluster;\n" ::: "memory");
    if (DYN) {
      for (int q = 0; q < XP_TQ; ++q) mbar_expect_tx(&qbar[q], 4);  // tile ids of local tiles 0..7
    } else {
      for (int t = 0; t < XP_K && t < ntiles; ++t) mbar_expect_tx(&tbar[t], recv_bytes(t));
    }
  }
  pdl_wait();               // x (and w, y) of the predecessor kernel
  pdl_trigger();
  p2p_prologue_wait(a.hk);  // x slices of the peers (p2p transport)
  if (threadIdx.x == 0) {
    const uint32_t xb = uint32_t(bulk_elems * sizeof(T));
    mbar_expect_tx(&xbar, xb);
    if (xb) bulk_g2s(xs, xg + col0, xb, &xbar);
  }
  for (int64_t j = bulk_elems + threadIdx.x; j <= W; j += blockDim.x) xs[j] = (j < ncols) ? xg[col0 + j] : T(0);
  // peers must have initialised their barriers before partials are sent
  cluster_arrive();
  cluster_wait();
  // DYN: rank 0 pops the cluster's tiles K ahead and stores each id into every
  // CTA of the cluster (st.async, 4 transaction bytes on the slot's qbar)
  bool popped_end = false;
  auto pop_send = [&](int k) {  // rank 0, thread 0: the tile of local index k (-1: none left)
    int tid = -1;
    if (!popped_end) {
      tid = atomicAdd(a.tq, 1);
      if (tid >= ntiles) {
        tid = -1;
        popped_end = true;
      }
    }
    const uint32_t la = smem_u32(&tileid[k % XP_TQ]), lb = smem_u32(&qbar[k % XP_TQ]);
    for (int p = 0; p < B; ++p)
      asm volatile("st.async.shared::cluster.mbarrier::complete_tx::bytes.b32 [%0], %1, [%2];\n" ::"r"(
                       mapa_u32(la, uint32_t(p))),
                   "r"(tid), "r"(mapa_u32(lb, uint32_t(p)))
                   : "memory");
  };
  auto tile_of = [&](int k) -> int {  // every thread: wait for the id of local tile k
    mbar_wait(&qbar[k % XP_TQ], uint32_t(k / XP_TQ) & 1u, 5000000 + k);
    return *reinterpret_cast<volatile int*>(&tileid[k % XP_TQ]);
  };
  if (DYN) {
    if (b == 0 && threadIdx.x == 0)
      for (int k = 0; k < XP_K; ++k) pop_send(k);
    if (threadIdx.x == 0)
      for (int k = 0; k < XP_K; ++k) {
        const int tk = tile_of(k);
        if (tk >= 0) mbar_expect_tx(&tbar[k], recv_bytes(tk));
      }
    // every CTA armed its receive barriers before any partial is sent
    cluster_arrive();
    cluster_wait();
  }
  mbar_wait(&xbar, 0, 1);
  if (a.tstamp && threadIdx.x == 0) a.tstamp[4 * blockIdx.x + 1] = gtimer();

  const double alpha = a.alpha, beta = a.beta;
  double dacc = 0.0;

  // t: tile index (relative to tbase), k: local sequence number (receive slot k % K)
  auto process_chunk = [&](int t, int k, int ch) {
    const int64_t cid = (int64_t(tbase + t) * B + b) * XP_CPT + ch;
    const int len = a.chunk_len[cid];
    const int row = a.chunk_row[cid * 32 + lane];
    const unsigned char* base = a.plan + a.chunk_off[cid];
    if (!DYN && a.prefetch && lane == 0 && t + 1 < ntiles) {
      const int64_t nid = cid + int64_t(B) * XP_CPT;
      const uint32_t nb = uint32_t(a.chunk_len[nid]) * 32u * uint32_t(sizeof(T) + 2);
      if (nb) asm volatile("cp.async.bulk.prefetch.L2.global [%0], %1;" ::"l"(a.plan + a.chunk_off[nid]), "r"(nb)
                           : "memory");
    }
    const double acc = xplan_chunk_dot<T>(base, len, lane, xs, W);
    if (row != 0xffff) {
      const int q = row / RB, jl = row - q * RB;
      const uint32_t laddr = smem_u32(recv + (k % XP_K) * R + b * RB + jl);
      st_async_f64(mapa_u32(laddr, q), acc, mapa_u32(smem_u32(&tbar[k % XP_K]), q));
    }
  };
  // chunks are sorted longest first: warp w takes chunk w and chunk CPT-1-w
  auto process = [&](int t, int k) {
#pragma unroll 1
    for (int h = 0; h < XP_CPW; h += 2) {
      process_chunk(t, k, h * XP_NW / 2 + warp);
      if (h + 1 < XP_CPW) process_chunk(t, k, XP_CPT - 1 - (h * XP_NW / 2 + warp));
    }
  };

  // Only the RB finalizer threads (rounded up to whole warps) wait on the
  // tile's mbarrier; all of them pass the wait before thread 0 re-arms it for
  // tile t+K.  (If every thread waited, a late warp could miss the phase: a
  // re-arm that expects 0 bytes completes the next phase at once and flips
  // the parity back -- an ABA deadlock seen on CTAs owning no rows of a
  // cluster's last tile.)
  const int nfin = min((RB + 31) & ~31, XP_THREADS);
  // t: tile index, k: local sequence number, t_next: tile of local k + K (< 0: none)
  auto finalize = [&](int t, int k, int t_next) {
    if (int(threadIdx.x) >= nfin) return;
    const double* rv = recv + (k % XP_K) * R;
    const int64_t rt = r0c + int64_t(t) * R;
    const int nrows = int(cmin64(R, r1c - rt));
    // the fused dot's w[i] (and beta*y[i]) do not depend on the partials: for
    // the first row of each finalizer thread (all of them when RB <= nfin) the
    // loads are issued before the wait so their latency hides behind it
    const int jl0 = threadIdx.x;
    const bool has0 = jl0 < RB && b * RB + jl0 < nrows;
    double w0 = 0.0, y0 = 0.0;
    if (has0) {
      const int64_t i0 = rt + b * RB + jl0;
      if (DOT) w0 = double(static_cast<const T*>(a.w)[i0]);
      if (beta != 0.0) y0 = double(static_cast<const T*>(a.y)[i0]);
    }
    mbar_wait(&tbar[k % XP_K], (k / XP_K) & 1, 1000000 * ntiles + 1000 * t + int(recv_bytes(t) / 8));
    double tacc = 0.0;  // DYN: this tile's share of the fused dot
    for (int jl = threadIdx.x; jl < RB && b * RB + jl < nrows; jl += nfin) {
      double sum = 0.0;
      for (int q = 0; q < B; ++q) sum += rv[q * RB + jl];
      const int64_t i = rt + b * RB + jl;
      T* y = static_cast<T*>(a.y);
      const bool first = jl == jl0;
      double r = alpha * sum;
      if (beta != 0.0) r += beta * (first ? y0 : double(y[i]));
      const T out = T(r);
      y[i] = out;
      if (DOT) (DYN ? tacc : dacc) += (first ? w0 : double(static_cast<const T*>(a.w)[i])) * double(out);
    }
    if (DOT && DYN) {
      // one partial per (tile, owner): the dot does not depend on which cluster ran the tile
      const double ts = block_sum_n(tacc, red, nfin / 32);
      if (threadIdx.x == 0) a.part[int64_t(t) * B + b] = ts;
    }
    asm volatile("bar.sync 2, %0;\n" ::"r"(nfin) : "memory");
    if (threadIdx.x == 0 && t_next >= 0) mbar_expect_tx(&tbar[k % XP_K], recv_bytes(t_next));
  };

  // Buffer reuse: partials of local tile k+K (K = 3) are sent only after the
  // sender passed wait(k+1), i.e. after every CTA arrived(k+1), which each
  // does after finalize(k) (reads of recv[k%K] + re-arm of tbar[k%K]).
  if (DYN) {
    // tiles handed out at run time; local k's tile id arrives in slot k % 8
    int t_cur = tile_of(0);
    if (t_cur >= 0) {
      if (b == 0 && threadIdx.x == 0) pop_send(XP_K);
      process(t_cur, 0);
      cluster_arrive_relaxed();
      int k = 1;
      for (;; ++k) {
        const int t_k = tile_of(k);
        if (t_k < 0) break;
        if (b == 0 && threadIdx.x == 0) pop_send(k + XP_K);
        process(t_k, k);
        cluster_wait();
        // tile of local k-1+K, popped at local k-1 (arrived by now or shortly)
        const int t_next = (threadIdx.x == 0) ? tile_of(k - 1 + XP_K) : -1;
        finalize(t_cur, k - 1, t_next);
        // slot (k-1) % 8 is free: every thread read it before the cluster barrier above
        if (threadIdx.x == 0) mbar_expect_tx(&qbar[(k - 1) % XP_TQ], 4);
        cluster_arrive_relaxed();
        t_cur = t_k;
      }
      if (a.tstamp && lane == 0) atomicMax(a.tstamp + 4 * blockIdx.x + 2, gtimer());
      cluster_wait();
      const int t_next = (threadIdx.x == 0) ? tile_of(k - 1 + XP_K) : -1;
      finalize(t_cur, k - 1, t_next);
    }
  } else if (ntiles > 0) {
    process(0, 0);
    cluster_arrive_relaxed();
    for (int t = 1; t < ntiles; ++t) {
      process(t, t);
      cluster_wait();
      finalize(t - 1, t - 1, t - 1 + XP_K < ntiles ? t - 1 + XP_K : -1);
      cluster_arrive_relaxed();
    }
    if (a.tstamp && lane == 0) atomicMax(a.tstamp + 4 * blockIdx.x + 2, gtimer());  // last warp done streaming
    cluster_wait();
    finalize(ntiles - 1, ntiles - 1, -1);
  }
  if (DOT && !DYN) {
    const double tsum = block_sum(dacc, red);
    if (threadIdx.x == 0) a.part[blockIdx.x] = tsum;
  }
  // leave together (peers may still be sending to / reading this CTA)
  cluster_arrive();
  cluster_wait();
  if (a.tstamp && threadIdx.x == 0) a.tstamp[4 * blockIdx.x + 3] = gtimer();
  if (DYN && threadIdx.x == 0) {
    // the last CTA of the launch (every pop done) re-arms the tile queue
    __threadfence();
    if (atomicAdd(a.tq_done, 1) == int(gridDim.x) - 1) {
      *a.tq = 0;
      *a.tq_done = 0;
      __threadfence();
    }
  }
  if (DOT) p2p_push_partials_last(a.hk, a.part, DYN ? ntiles * B : int(gridDim.x));
}

// ---------------------------------------------------------------- builders
__device__ __forceinline__ void xp_seg(const int* rowptr, const int* seg, int64_t m, int B, int b, int64_t i,
                                       int* k0, int* k1) {
  *k0 = (b == 0) ? rowptr[i] : seg[int64_t(b - 1) * m + i];
  *k1 = (b == B - 1) ? rowptr[i + 1] : seg[int64_t(b) * m + i];
}

// One CTA (XP_THREADS threads, R/XP_THREADS rows each) per (global tile, b):
// sort the tile's rows by segment length (descending, ties by row: bitonic
// sort of (len, row) keys), cut into CPT chunks of 32 lanes, record each
// chunk's step count and each row's slot (chunk = slot/32, lane = slot%32).
static __global__ void __launch_bounds__(XP_THREADS)
k_xplan_sell(const int* __restrict__ rowptr, const int* __restrict__ seg, int64_t m, int B,
             const long long* __restrict__ crow, const int* __restrict__ tile0, int ncl, int* __restrict__ chunk_len,
             uint16_t* __restrict__ chunk_row, int* __restrict__ row_slot) {
  // bitonic sort over the next power of two >= R (XP_R need not be one: the
  // tile height must be a multiple of the cluster size B); padding sorts last
  constexpr int PR = XP_R <= 1024 ? 1024 : XP_R <= 2048 ? 2048 : 4096;
  static_assert(XP_R <= PR, "tile too tall");
  __shared__ unsigned long long key[PR];
  constexpr int PER = (PR + XP_THREADS - 1) / XP_THREADS;
  const int tg = blockIdx.x / B, b = blockIdx.x % B;
  int c = 0;
  while (c + 1 < ncl && tile0[c + 1] <= tg) ++c;
  const int t = tg - tile0[c];
  const int64_t rt = crow[c] + int64_t(t) * XP_R;
  const int nrows = int(cmin64(XP_R, crow[c + 1] - rt));
  for (int e = 0; e < PER; ++e) {
    const int j = threadIdx.x + e * XP_THREADS;
    if (j >= PR) continue;
    if (j >= XP_R) {
      key[j] = ~0ull;  // power-of-two padding
      continue;
    }
    int L = -1;  // absent rows sort last
    if (j < nrows) {
      int k0, k1;
      xp_seg(rowptr, seg, m, B, b, rt + j, &k0, &k1);
      L = k1 - k0;
    }
    // descending by L, then ascending by row: key = (~(L+1)) << 32 | j, ascending
    key[j] = (static_cast<unsigned long long>(~static_cast<uint32_t>(L + 1)) << 32) | uint32_t(j);
  }
  __syncthreads();
  for (int k = 2; k <= PR; k <<= 1)
    for (int s = k >> 1; s > 0; s >>= 1) {
      for (int e = 0; e < PER; ++e) {
        const int j = threadIdx.x + e * XP_THREADS;
        if (j >= PR) continue;
        const int p = j ^ s;
        if (p > j) {
          const bool up = (j & k) == 0;
          const unsigned long long a0 = key[j], a1 = key[p];
          if ((a0 > a1) == up) { key[j] = a1; key[p] = a0; }
        }
      }
      __syncthreads();
    }
  for (int e = 0; e < PER; ++e) {
    const int j = threadIdx.x + e * XP_THREADS;
    if (j >= XP_R) continue;
    const unsigned long long kk = key[j];
    const int row = int(kk & 0xffffffffu);
    const int Ls = int(~uint32_t(kk >> 32)) - 1;
    const int w = j / 32, ln = j % 32;
    const int64_t cid = (int64_t(tg) * B + b) * XP_CPT + w;
    chunk_row[cid * 32 + ln] = (Ls >= 0) ? uint16_t(row) : uint16_t(0xffff);
    if (Ls >= 0) row_slot[int64_t(b) * m + rt + row] = j;
    // chunk length = the first (longest) lane's length
    if (ln == 0) chunk_len[cid] = XP_ODD ? max(Ls, 0) : (max(Ls, 0) + 1) & ~1;  // the longest segment
  }
}

// Scatter every nonzero into its chunk slot: warp per row.
template <typename T>
__global__ void __launch_bounds__(256)
k_xplan_pack(const int* __restrict__ rowptr, const int* __restrict__ colidx, const T* __restrict__ vals,
             const int* __restrict__ seg, int64_t m, int B, int W, const long long* __restrict__ crow,
             const int* __restrict__ tile0, int ncl, const long long* __restrict__ chunk_off,
             const int* __restrict__ chunk_len, const int* __restrict__ row_slot, unsigned char* __restrict__ plan,
             int values_only, int64_t mplan /* rows [0, mplan) are in the plan */) {
  const int lane = threadIdx.x & 31;
  for (int64_t i = (int64_t(blockIdx.x) * blockDim.x + threadIdx.x) / 32; i < mplan;
       i += int64_t(gridDim.x) * blockDim.x / 32) {
    int lo = 0, hi = ncl - 1;
    while (lo < hi) {
      const int mid = (lo + hi + 1) >> 1;
      if (crow[mid] <= i) lo = mid; else hi = mid - 1;
    }
    const int tg = tile0[lo] + int((i - crow[lo]) / XP_R);
    const int k0 = rowptr[i], k1 = rowptr[i + 1];
    for (int k = k0 + lane; k < k1; k += 32) {
      const int col = colidx[k];
      const int bb = col / W;
      const int s0 = (bb == 0) ? k0 : seg[int64_t(bb - 1) * m + i];
      const int slot = row_slot[int64_t(bb) * m + i];
      const int64_t cid = (int64_t(tg) * B + bb) * XP_CPT + slot / 32;
      const int ln = slot % 32, len = chunk_len[cid];
      const int s = k - s0;  // step
      unsigned char* base = plan + chunk_off[cid];
      unsigned char* cbase = base + size_t(len) * 32 * sizeof(T);
      const bool tail = (len & 1) && s == len - 1;  // odd last step: its own [32] row of vals and cols
      T* v = tail ? reinterpret_cast<T*>(base + size_t(s >> 1) * 64 * sizeof(T) + size_t(ln) * sizeof(T))
                  : reinterpret_cast<T*>(base + (size_t(s >> 1) * 32 + ln) * 2 * sizeof(T)) + (s & 1);
      *v = vals[k];
      if (!values_only) {
        uint16_t* cc = tail ? reinterpret_cast<uint16_t*>(cbase + size_t(s >> 1) * 128 + size_t(ln) * 2)
                            : reinterpret_cast<uint16_t*>(cbase + (size_t(s >> 1) * 32 + ln) * 4) + (s & 1);
        *cc = uint16_t(col - bb * W);
      }
    }
  }
}

// Bank spreading (create time, after k_xplan_pack): inside each lane (row) of
// a chunk, the order of the row's nonzeros over the chunk's steps is free --
// the SPMV idiom's DotProductLoop is a sum (Fig. 12), and the
// per-row tolerance of BJ.ns bounds any summation order.  The kernel reorders
// them so that the x gathers of one step (xs[col] in shared memory, 8-B words
// for fp64 = bank pair col % 16 per half-warp, 4-B words for fp32 = bank
// col % 32 per warp) hit distinct banks.  Step by step, in up to BP_ROUNDS
// rounds, every unplaced lane proposes its first remaining nonzero whose bank
// is still free in this step; lanes proposing the same bank are resolved in
// favour of the lowest lane (the others retry against the grown set of taken
// banks); lanes left over keep their next entry.  Pads (column W, value 0)
// share one word.  One warp per chunk; deterministic (it depends only on the
// columns and their CSR order), so a values-only re-pack followed by this pass
// reproduces it.
constexpr int BP_ROUNDS = 4;
constexpr int BP_MAXLEN = 512;  // longer chunks keep CSR order (the pass is quadratic in the chunk length)
template <typename T>
__global__ void __launch_bounds__(256)
k_xplan_bankperm(unsigned char* __restrict__ plan, const long long* __restrict__ chunk_off,
                 const int* __restrict__ chunk_len, int64_t nchunks, int W) {
  constexpr int NG = sizeof(T) == 8 ? 16 : 32;  // conflict-free slots per lane group (half-warp for fp64)
  const int lane = threadIdx.x & 31;
  const int grp = lane / NG;
  const uint32_t gshift = uint32_t(grp * NG);   // this group's bits in a warp-wide 32-bit mask
  const int64_t warps = int64_t(gridDim.x) * (blockDim.x >> 5);
  for (int64_t c = int64_t(blockIdx.x) * (blockDim.x >> 5) + (threadIdx.x >> 5); c < nchunks; c += warps) {
    const int len = chunk_len[c];
    if (len < 2 || len > BP_MAXLEN) continue;
    unsigned char* base = plan + chunk_off[c];
    T* V = reinterpret_cast<T*>(base);
    uint16_t* C = reinterpret_cast<uint16_t*>(base + size_t(len) * 32 * sizeof(T));
    auto at = [&](int st) { return (size_t(st >> 1) * 32 + lane) * 2 + (st & 1); };
    for (int st = 0; st < len - 1; ++st) {
      uint32_t taken = 0;  // warp-wide: bit (grp*NG + slot)
      uint32_t padded = 0;  // warp-wide: bit grp*NG set once a pad holds the group's pad slot
      bool placed = false;
#pragma unroll 1
      for (int r = 0; r < BP_ROUNDS; ++r) {
        int cand = -1, slot = 0;
        bool pad = false;
        if (!placed) {
          for (int e = st; e < len; ++e) {
            const int col = C[at(e)];
            const int sl = col % NG;
            const bool isp = col == W;
            const bool free_ = !(taken & (1u << (gshift + sl))) || (isp && (padded & (1u << gshift)));
            if (free_) {
              cand = e;
              slot = sl;
              pad = isp;
              break;
            }
          }
        }
        // lowest lane per (group, slot) wins; pads of a group all win together
        const bool want = cand >= 0;
        const uint32_t key = want ? (pad ? 0x10000u + uint32_t(grp) : uint32_t(grp * 64 + slot)) : 0xffffffffu;
        const uint32_t peers = __match_any_sync(0xffffffffu, key);
        const bool win = want && (pad || (__ffs(peers) - 1) == lane);
        if (win) {
          if (cand != st) {
            const size_t i0 = at(st), i1 = at(cand);
            const T tv = V[i0];
            V[i0] = V[i1];
            V[i1] = tv;
            const uint16_t tc = C[i0];
            C[i0] = C[i1];
            C[i1] = tc;
          }
          placed = true;
        }
        taken |= __reduce_or_sync(0xffffffffu, win ? (1u << (gshift + slot)) : 0u);
        padded |= __reduce_or_sync(0xffffffffu, (win && pad) ? (1u << gshift) : 0u);
        if (__all_sync(0xffffffffu, placed)) break;
      }
    }
  }
}

// Padding: value regions 0, column regions the pad column W (x pad 0.0).
// Chunk c of the plan spans [chunk_off[c], chunk_off[c] + len*32*(ts+2)).
static __global__ void k_xplan_fill(unsigned char* __restrict__ plan, const long long* __restrict__ chunk_off,
                             const int* __restrict__ chunk_len, int64_t nchunks, int ts, uint16_t pad) {
  for (int64_t c = blockIdx.x; c < nchunks; c += gridDim.x) {
    const int len = chunk_len[c];
    unsigned char* base = plan + chunk_off[c];
    const int64_t vbytes = int64_t(len) * 32 * ts, cn = int64_t(len) * 32;
    for (int64_t i = threadIdx.x; i < vbytes / 4; i += blockDim.x) reinterpret_cast<uint32_t*>(base)[i] = 0u;
    uint16_t* cc = reinterpret_cast<uint16_t*>(base + vbytes);
    for (int64_t i = threadIdx.x; i < cn; i += blockDim.x) cc[i] = pad;
  }
}

}  // namespace spmv
