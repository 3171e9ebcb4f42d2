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
//   in shared memory; the rows are cut into tiles of R = 32*CPT rows, claimed
//   dynamically by the clusters (see below); inside a tile the rows are sorted by the
//   length of their segment in block b (SELL-C-sigma with C = 32, sigma = R)
//   and cut into NW chunks of 32 rows.  Chunk (tile, b, w) stores len (even)
//   steps column-major: vals as [len/2][32 lanes][2] (2 values per lane per
//   step pair) then columns as [len/2][32][2] uint16 offsets inside the
//   block; padding entries have value 0 and column W (x pad 0.0).
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
#define XP_U_DEF 8
#endif
constexpr int XP_U = XP_U_DEF;       // step pairs (16-B loads) in flight per lane

struct XplanArgs {
  int64_t nx;                  // length of x
  int W;                       // column block width (pad column = W)
  const unsigned char* plan;   // chunk data
  const long long* chunk_off;  // [tile][b][chunk] byte offset of chunk data
  const int* chunk_len;        // [tile][b][chunk] steps (even)
  const uint16_t* chunk_row;   // [tile][b][chunk][32] tile-local row of each lane (0xffff = none)
  int64_t m;                   // rows
  int ntiles;                  // ceil(m / R)
  int* counter;                // tile counter (zeroed before every launch)
  const void* x;
  void* y;
  double alpha, beta;
  const void* w;               // DOT: w[i]
  double* part;                // DOT: one partial per (tile, b): part[tile*B + b]
  int dbg;
};

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

// st.async of a 4-byte value into a peer CTA, completing 4 transaction bytes.
__device__ __forceinline__ void st_async_u32(uint32_t raddr, uint32_t v, uint32_t rbar) {
  asm volatile("st.async.shared::cluster.mbarrier::complete_tx::bytes.b32 [%0], %1, [%2];\n" ::"r"(raddr), "r"(v),
               "r"(rbar)
               : "memory");
}

// smem (dynamic): xs [(W+1)*sizeof(T) rounded to 16] | recv [K][R] double
//   recv[s%K][b*(R/B) + jl]: partial of CTA b for owned row jl of the tile of step s
//
// Scheduling: tiles (R consecutive rows) are claimed dynamically: the leader
// thread of every cluster (rank 0, thread 0) takes the next tile with an
// atomicAdd one step ahead and sends its id to the B CTAs with st.async into
// a ring of 4 slots (mbarrier transaction bytes), so fast clusters take more
// tiles and the kernel ends together.  Protocol (s = step):
//   init: every CTA arms slots 0..3; after the first cluster barrier the
//         leader sends the tiles of steps 0 and 1;
//   step s: all threads wait slot s%4 (tile of step s; >= ntiles ends the
//         loop), process it, and in the finalize section (after the cluster
//         barrier wait of step s-1) thread 0 re-arms slot (s+2)%4 for step s+2
//         (its last reader, step s-2, is over for every thread) and the leader
//         sends the tile of step s+1 into slot (s+1)%4 (armed at step s-1 or at
//         init, i.e. before every CTA's arrive that the leader waited for).
// Every tile row is sent exactly B partials (absent rows of the last tile send
// 0.0), so the receive byte count of a step is constant.
template <typename T, bool DOT>
__global__ void __launch_bounds__(XP_THREADS, 1)
k_spmv_xplan(XplanArgs a) {
  extern __shared__ __align__(128) unsigned char smem[];
  __shared__ uint64_t xbar, tbar[XP_K], sbar[4];
  __shared__ int stile[4];
  __shared__ double red[32];
  const int B = (int)cgx::this_cluster().num_blocks();
  const int b = (int)cluster_rank();
  constexpr int R = XP_R;
  const int RB = R / B;
  const int W = a.W;
  const int ntiles = a.ntiles;
  const int64_t m = a.m;

  T* xs = reinterpret_cast<T*>(smem);
  double* recv = reinterpret_cast<double*>(smem + ((size_t(W + 1) * sizeof(T) + 15) & ~size_t(15)));
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const bool leader = (b == 0 && threadIdx.x == 0);

  const int64_t col0 = int64_t(b) * W;
  const int64_t ncols = cmax64(0, cmin64(W, a.nx - col0));
  const T* __restrict__ xg = static_cast<const T*>(a.x);
  const bool x_aligned = (reinterpret_cast<uintptr_t>(xg + col0) & 15) == 0;
  const int64_t bulk_elems = x_aligned ? ((ncols * int64_t(sizeof(T))) & ~int64_t(15)) / int64_t(sizeof(T)) : 0;
  const uint32_t recv_bytes = uint32_t(RB * B * 8);

  if (threadIdx.x == 0) {
    mbar_init(&xbar, 1);
    for (int q = 0; q < XP_K; ++q) mbar_init(&tbar[q], 1);
    for (int q = 0; q < 4; ++q) mbar_init(&sbar[q], 1);
    asm volatile("fence.mbarrier_init.release.cluster;\n" ::: "memory");
    const uint32_t xb = uint32_t(bulk_elems * sizeof(T));
    mbar_expect_tx(&xbar, xb);
    if (xb) bulk_g2s(xs, xg + col0, xb, &xbar);
    for (int q = 0; q < XP_K; ++q) mbar_expect_tx(&tbar[q], recv_bytes);
    for (int q = 0; q < 4; ++q) mbar_expect_tx(&sbar[q], 4);
  }
  for (int64_t j = bulk_elems + threadIdx.x; j <= W; j += blockDim.x) xs[j] = (j < ncols) ? xg[col0 + j] : T(0);
  int next_tile = 0;
  if (leader) next_tile = atomicAdd(a.counter, 1);
  // peers must have initialised their barriers before anything is sent
  cluster_arrive();
  cluster_wait();
  auto send_tile = [&](int step, int tile) {
    const uint32_t slot = smem_u32(&stile[step & 3]), bar = smem_u32(&sbar[step & 3]);
    for (int q = 0; q < B; ++q) st_async_u32(mapa_u32(slot, q), uint32_t(tile), mapa_u32(bar, q));
  };
  if (leader) {
    send_tile(0, next_tile);
    send_tile(1, atomicAdd(a.counter, 1));
    next_tile = atomicAdd(a.counter, 1);  // tile of step 2
  }
  mbar_wait(&xbar, 0, 1);

  const double alpha = a.alpha, beta = a.beta;
  double dacc = 0.0;

  auto process_chunk = [&](int s, int tile, int ch) {
    const int64_t cid = (int64_t(tile) * B + b) * XP_CPT + ch;
    const int len = a.chunk_len[cid];
    const int row = a.chunk_row[cid * 32 + lane];
    const unsigned char* base = a.plan + a.chunk_off[cid];
    const unsigned char* V = base + size_t(lane) * 2 * sizeof(T);
    const unsigned char* C = base + size_t(len) * 32 * sizeof(T) + size_t(lane) * 4;
    constexpr size_t VS = 32 * 2 * sizeof(T);  // bytes per step pair (vals)
    double acc = 0.0;
    const int np = len >> 1;  // step pairs
    const uint32_t padcc = uint32_t(W) | (uint32_t(W) << 16);  // both steps -> x pad 0.0
    // every batch issues up to XP_U independent 16-B loads (the tail batch is
    // predicated: masked pairs contribute 0 * x[W] = 0), so a chunk costs
    // ceil(np / XP_U) memory round trips
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
    // every row slot of the tile gets B partials (absent rows: 0.0)
    const int j = row & 0x7fff, q = j / RB, jl = j - q * RB;
    const uint32_t laddr = smem_u32(recv + (s % XP_K) * R + b * RB + jl);
    st_async_f64(mapa_u32(laddr, q), (row & 0x8000) ? 0.0 : acc, mapa_u32(smem_u32(&tbar[s % XP_K]), q));
  };
  // chunks are sorted longest first: warp w takes chunk w and chunk CPT-1-w
  auto process = [&](int s, int tile) {
#pragma unroll 1
    for (int h = 0; h < XP_CPW; h += 2) {
      process_chunk(s, tile, h * XP_NW / 2 + warp);
      if (h + 1 < XP_CPW) process_chunk(s, tile, XP_CPT - 1 - (h * XP_NW / 2 + warp));
    }
  };

  // Only the RB finalizer threads (whole warps) wait on the step's receive
  // mbarrier, and all of them pass it before thread 0 re-arms it (a late
  // waiter could otherwise miss the phase: parity ABA).  The dot partial of
  // (tile, b) goes to part[tile*B + b]: deterministic whichever cluster ran it.
  const int nfin = min((RB + 31) & ~31, XP_THREADS);
  auto finalize = [&](int s, int tile) {
    if (int(threadIdx.x) < nfin) {
      const double* rv = recv + (s % XP_K) * R;
      const int64_t rt = int64_t(tile) * R;
      const int nrows = int(cmin64(R, m - rt));
      mbar_wait(&tbar[s % XP_K], (s / XP_K) & 1, 1000000 + 1000 * tile + s);
      double dt = 0.0;
      for (int jl = threadIdx.x; jl < RB && b * RB + jl < nrows; jl += nfin) {
        double sum = 0.0;
        for (int q = 0; q < B; ++q) sum += rv[q * RB + jl];
        const int64_t i = rt + b * RB + jl;
        T* y = static_cast<T*>(a.y);
        double r = alpha * sum;
        if (beta != 0.0) r += beta * double(y[i]);
        const T out = T(r);
        y[i] = out;
        if (DOT) dt += double(static_cast<const T*>(a.w)[i]) * double(out);
      }
      if (DOT) {
        dt = warp_sum(dt);
        if (lane == 0) red[warp] = dt;
      }
      asm volatile("bar.sync 2, %0;\n" ::"r"(nfin) : "memory");
      if (threadIdx.x == 0) {
        mbar_expect_tx(&tbar[s % XP_K], recv_bytes);  // re-arm for step s+K
        if (DOT) {
          double tot = 0.0;
          for (int w = 0; w < nfin / 32; ++w) tot += red[w];
          a.part[int64_t(tile) * B + b] = tot;
        }
      }
    }
  };
  auto next_step_tile = [&](int s) -> int {  // tile of step s (waits for the leader's id)
    mbar_wait(&sbar[s & 3], (s >> 2) & 1, 2000000 + s);
    return stile[s & 3];
  };
  auto boundary = [&](int s) {  // after the cluster-barrier wait of step s-1
    if (threadIdx.x == 0 && s >= 2) mbar_expect_tx(&sbar[(s + 2) & 3], 4);  // slot for step s+2
    if (leader) {
      send_tile(s + 1, next_tile);
      next_tile = atomicAdd(a.counter, 1);
    }
  };

  int s = 0;
  int tile = next_step_tile(0);
  int prev = -1;
  if (tile < ntiles) {
    process(0, tile);
    cluster_arrive_relaxed();
    prev = tile;
    for (s = 1;; ++s) {
      // the tile of step s was sent during step s-1 (or at init for s = 1)
      tile = next_step_tile(s);
      if (tile >= ntiles) break;
      process(s, tile);
      cluster_wait();
      finalize(s - 1, prev);
      boundary(s);
      cluster_arrive_relaxed();
      prev = tile;
    }
    cluster_wait();
    finalize(s - 1, prev);
  }
  // leave together (peers may still be sending to / reading this CTA)
  cluster_arrive();
  cluster_wait();
}

// ---------------------------------------------------------------- builders
__device__ __forceinline__ void xp_seg(const int* rowptr, const int* seg, int64_t m, int B, int b, int64_t i,
                                       int* k0, int* k1) {
  *k0 = (b == 0) ? rowptr[i] : seg[int64_t(b - 1) * m + i];
  *k1 = (b == B - 1) ? rowptr[i + 1] : seg[int64_t(b) * m + i];
}

// One CTA (XP_THREADS threads, R/XP_THREADS rows each) per (tile, b), tile g =
// rows [g*R, (g+1)*R): sort the tile's rows by segment length (descending, ties
// by row: bitonic sort of (len, row) keys), cut into CPT chunks of 32 lanes,
// record each chunk's even step count, each lane's tile row (bit 15 set for
// rows beyond m, which send 0.0) and each row's slot (chunk slot/32, lane slot%32).
__global__ void __launch_bounds__(XP_THREADS)
k_xplan_sell(const int* __restrict__ rowptr, const int* __restrict__ seg, int64_t m, int B,
             int* __restrict__ chunk_len, uint16_t* __restrict__ chunk_row, int* __restrict__ row_slot) {
  __shared__ unsigned long long key[XP_R];
  constexpr int PER = XP_R / XP_THREADS;
  const int tg = blockIdx.x / B, b = blockIdx.x % B;
  const int64_t rt = int64_t(tg) * XP_R;
  const int nrows = int(cmin64(XP_R, m - rt));
  for (int e = 0; e < PER; ++e) {
    const int j = threadIdx.x + e * XP_THREADS;
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
  for (int k = 2; k <= XP_R; k <<= 1)
    for (int s = k >> 1; s > 0; s >>= 1) {
      for (int e = 0; e < PER; ++e) {
        const int j = threadIdx.x + e * XP_THREADS;
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
    const unsigned long long kk = key[j];
    const int row = int(kk & 0xffffffffu);
    const int Ls = int(~uint32_t(kk >> 32)) - 1;
    const int w = j / 32, ln = j % 32;
    const int64_t cid = (int64_t(tg) * B + b) * XP_CPT + w;
    chunk_row[cid * 32 + ln] = uint16_t(row) | ((Ls >= 0) ? uint16_t(0) : uint16_t(0x8000));
    if (Ls >= 0) row_slot[int64_t(b) * m + rt + row] = j;
    // chunk length = the first (longest) lane's length, rounded up to even
    if (ln == 0) chunk_len[cid] = (max(Ls, 0) + 1) & ~1;
  }
}

// Scatter every nonzero into its chunk slot: warp per row.
template <typename T>
__global__ void __launch_bounds__(256)
k_xplan_pack(const int* __restrict__ rowptr, const int* __restrict__ colidx, const T* __restrict__ vals,
             const int* __restrict__ seg, int64_t m, int B, int W, const long long* __restrict__ chunk_off,
             const int* __restrict__ chunk_len, const int* __restrict__ row_slot, unsigned char* __restrict__ plan,
             int values_only) {
  const int lane = threadIdx.x & 31;
  for (int64_t i = (int64_t(blockIdx.x) * blockDim.x + threadIdx.x) / 32; i < m;
       i += int64_t(gridDim.x) * blockDim.x / 32) {
    const int tg = int(i / XP_R);
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
      T* v = reinterpret_cast<T*>(base + (size_t(s >> 1) * 32 + ln) * 2 * sizeof(T));
      v[s & 1] = vals[k];
      if (!values_only) {
        uint16_t* cc = reinterpret_cast<uint16_t*>(base + size_t(len) * 32 * sizeof(T) + (size_t(s >> 1) * 32 + ln) * 4);
        cc[s & 1] = uint16_t(col - bb * W);
      }
    }
  }
}

// Padding: value regions 0, column regions the pad column W (x pad 0.0).
// Chunk c of the plan spans [chunk_off[c], chunk_off[c] + len*32*(ts+2)).
__global__ void k_xplan_fill(unsigned char* __restrict__ plan, const long long* __restrict__ chunk_off,
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
