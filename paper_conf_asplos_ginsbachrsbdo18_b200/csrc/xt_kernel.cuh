// xt_kernel.cuh -- x-stationary SpMV over a TMA-streamed, column-parted plan of A
// (SPMV_KERNEL_XT).  Semantics: Fig. 4 with the
// alpha/beta of DotProductLoop; the loop is "the performance
// bottleneck of the NAS CG benchmark".
//
// Why a second x-stationary kernel (measured on this GPU, DESIGN.md 5.1/5.2):
//   * the SpMV is HBM-bound; LDG streaming measured ~5.9 TB/s and TMA bulk
//     copies of >= 16 KB with >= 64 KB in flight per SM 6.7-7.2 TB/s (both
//     re-measured in round 2 without a write flush: LDG 6.4-6.8, the XT ring
//     alone 6.6-6.8 TB/s -- DESIGN.md 5.2b/5.2c);
//   * random 8-B gathers of x run at ~5/clk/SM from local shared memory, ~1
//     through L1 and ~0.35 through DSMEM, so x must sit in each CTA's own
//     shared memory;
//   * clusters of 2 CTAs tile all 148 SMs (74 clusters), clusters of 8 only
//     120.  A TMA ring next to x needs x blocks of <= ~80 KB.
// Hence: the columns are cut into NB = Q*B blocks (Q "parts" of B blocks, a
// part per cluster), x block g lives in the shared memory of its CTA, and the
// CTA's slice of the matrix streams through a ring of <= 16 KB TMA stages.
//
// Plan (built once at create -- the paper's device-resident "lazy copy",
// P:1175-1184): cluster c owns part q(c) and rows [r0, r1) (nnz-balanced within
// the part, multiples of 32); its rows are cut into tiles of XT_R = 1024 rows;
// CTA b of the cluster holds column block g = q*B + b.  For tile t, block g the
// tile's rows are sorted by the length of their segment in g (descending) and
// cut into 32 chunks of 32 rows (SELL-32-sigma, sigma = 1024).  A chunk is
//   [row map: 32 x u16 tile-local rows, 0xffff = none]
//   [piece 0: vals [L0][32] T, cols [L0][32] u16 (offset in the block)] [piece 1] ...
// with len = the longest segment of the chunk, pieces of <= XT_LMAX steps, and
// padding entries value 0 / column W_g (the zero pad of x).  The chunks of a
// CTA (tile-major, longest first) are cut into stages of whole chunks of <=
// XT_SMAX bytes (a multi-piece chunk: one stage per piece) -- the units of the
// CTA's TMA ring.
//
// Kernel (one 1024-thread CTA per SM, clusters of B): warp 0 lane 0 streams
// the stages into an NS-slot ring (mbarrier full/empty, a stage's piece count
// pre-arrived on its empty barrier); warps 1..31 take the CTA's chunks round
// robin (lane = row, the step loop in the chunk's column order, x from shared
// memory) and push the row's block partial into the receive array of the
// owning CTA with st.async (transaction bytes on the owner's per-tile-slot
// mbarrier).  The owner sums the B partials of each row in rank order.  With
// Q = 1 that is y; with Q > 1 it is written to ypart[q][i] and the last of the
// Q owners of a 32-row group (a global atomic ticket) sums the Q partials in
// part order and writes y.  Every summation order is fixed: results are
// deterministic.  Receive slots are recycled by mbarrier signals (free[slot],
// one remote arrive per owner CTA), not cluster barriers, so the producer warp
// never joins a barrier in the steady state.  Every wait has a watchdog.
#pragma once
#include <cooperative_groups.h>

#include "common.cuh"
#include "xstat_kernel.cuh"  // cluster / mbarrier / bulk-copy helpers

namespace spmv {

constexpr int XT_THREADS = 1024;
constexpr int XT_NFW = 4;            // finalizer warps (the last ones)
constexpr int XT_NWC = XT_THREADS / 32 - 1 - XT_NFW;  // consumer warps (warp 0 = producer)
constexpr int XT_NC = 32;            // chunks per tile per CTA
constexpr int XT_R = 32 * XT_NC;     // rows per tile
constexpr int XT_K = 3;              // receive slots
constexpr int XT_NS_MAX = 12;        // ring slots (runtime NS <= this)
constexpr int XT_SMAX = 16384;       // bytes per ring slot / stage
constexpr int XT_HDR = 64;           // row map at the start of every chunk
constexpr int XT_EMPTY = 128;        // empty-barrier arrival count (>= pieces per stage)
#ifndef XT_U_DEF
#define XT_U_DEF 4
#endif
constexpr int XT_U = XT_U_DEF;       // steps of loads issued together per lane

// steps per piece: the row map and one piece fit one stage
template <typename T>
__host__ __device__ constexpr int xt_lmax() {
  return (XT_SMAX - XT_HDR) / (32 * int(sizeof(T) + 2));
}

struct XtArgs {
  int64_t m;                    // rows of the handle (ypart stride)
  int Q;                        // column parts
  int NS;                       // ring slots
  int dyn;                      // 1: consumer warps take chunks in stream order from a shared counter
  int xcap;                     // elements of the x smem block (max block width + 1, rounded)
  int64_t nx;                   // length of x
  const unsigned char* plan;    // stage data
  const int* cl_part;           // [ncl] part of cluster c
  const long long* cl_rows;     // [ncl][2] row range of cluster c
  const int* cl_tile0;          // [ncl] first global tile of cluster c
  const long long* cta_col0;    // [grid] first column of the CTA's block
  const int* cta_w;             // [grid] block width W_g (pad column index)
  const int* cta_st0;           // [grid + 1] first stage of each CTA
  const long long* st_off;      // [stages] byte offset in plan
  const uint32_t* st_info;      // [stages] bytes | pieces << 16
  const uint2* ck_meta;         // [chunks] {stage (CTA-relative), off16 | len << 16}
  const void* x;
  void* y;
  double alpha, beta;
  double* ypart;                // Q > 1: [Q][m] part partials
  int* gcnt;                    // Q > 1: [ceil(m/32)] group tickets (zero between launches)
  const void* w;                // DOT: w[i]
  double* part;                 // DOT: one partial per CTA
  P2PHook hk;
  unsigned long long* prof;     // -DXT_PROF builds: per warp {tag, full, proc, fbar, fin, rbar, total, chunks} clocks
};

// diagnostics of -DXT_PROF variant builds (tools/build_variants.sh): per-warp clock accounting
#ifdef XT_PROF
#define XT_T0(v) const long long v = clock64()
#define XT_ACC(i, t0) pr[i] += (unsigned long long)(clock64() - (t0))
#else
#define XT_T0(v)
#define XT_ACC(i, t0)
#endif

__device__ __forceinline__ void mbar_arrive_cnt(uint64_t* bar, uint32_t cnt) {
  asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0], %1;\n" ::"r"(smem_u32(bar)), "r"(cnt) : "memory");
}
// Arrive on the mbarrier at the same offset in cluster CTA `rank` (release at cluster scope).
__device__ __forceinline__ void mbar_arrive_remote(uint64_t* bar, uint32_t rank) {
  uint32_t r;
  asm volatile("mapa.shared::cluster.u32 %0, %1, %2;\n" : "=r"(r) : "r"(smem_u32(bar)), "r"(rank));
  asm volatile("mbarrier.arrive.release.cluster.shared::cluster.b64 _, [%0];\n" ::"r"(r) : "memory");
}
__device__ __forceinline__ uint32_t xt_mapa(uint32_t laddr, uint32_t rank) {
  uint32_t r;
  asm volatile("mapa.shared::cluster.u32 %0, %1, %2;\n" : "=r"(r) : "r"(laddr), "r"(rank));
  return r;
}
__device__ __forceinline__ void xt_st_async(uint32_t raddr, double v, uint32_t rbar) {
  asm volatile("st.async.shared::cluster.mbarrier::complete_tx::bytes.b64 [%0], %1, [%2];\n" ::"r"(raddr),
               "l"(__double_as_longlong(v)), "r"(rbar)
               : "memory");
}
template <typename T>
__device__ __forceinline__ T xt_lds(const unsigned char* p) {
  return *reinterpret_cast<const T*>(p);
}

// dynamic smem: xs [xcap T, 16-B rounded] | ring [NS][XT_SMAX] | recv [K][R] double
template <typename T, bool DOT>
__global__ void __launch_bounds__(XT_THREADS, 1)
k_spmv_xt(XtArgs a) {
  extern __shared__ __align__(128) unsigned char smem[];
  __shared__ uint64_t xbar, full[XT_NS_MAX], empty[XT_NS_MAX], rbar[XT_K], fbar[XT_K];
  __shared__ int fincnt[XT_K];
  __shared__ int stag[XT_NS_MAX];  // stage currently issued into each ring slot
  __shared__ int next_chunk;       // dyn: next chunk (stream order) to hand out
  __shared__ double red[32];
  constexpr int R = XT_R;
  constexpr int LMAX = xt_lmax<T>();
  const int B = (int)cgx::this_cluster().num_blocks();
  const int b = (int)cluster_rank();
  const int c = (int)cluster_id();
  const int RB = R / B;
  const int NS = a.NS;
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int q = a.cl_part[c];
  const int64_t r0 = a.cl_rows[2 * c], r1 = a.cl_rows[2 * c + 1];
  const int ntiles = int((r1 - r0 + R - 1) / R);
  const int tile0 = a.cl_tile0[c];
  const int cta = blockIdx.x;
  const int64_t col0 = a.cta_col0[cta];
  const int Wg = a.cta_w[cta];
  const int st0 = a.cta_st0[cta], nst = a.cta_st0[cta + 1] - st0;

  T* xs = reinterpret_cast<T*>(smem);
  unsigned char* ring = smem + ((size_t(a.xcap) * sizeof(T) + 127) & ~size_t(127));
  double* recv = reinterpret_cast<double*>(ring + size_t(NS) * XT_SMAX);

  // rows of tile t owned by this CTA: [b*RB, (b+1)*RB) of the tile
  auto tile_rows = [&](int t) -> int { return int(cmin64(R, r1 - (r0 + int64_t(t) * R))); };
  auto own_rows = [&](int t) -> int { return max(0, min((b + 1) * RB, tile_rows(t)) - b * RB); };

  p2p_prologue_wait(a.hk);  // x slices of the peers (p2p transport)
  const int64_t ncols = cmax64(0, cmin64(Wg, a.nx - col0));
  const T* __restrict__ xg = static_cast<const T*>(a.x);
  const bool x_aligned = (reinterpret_cast<uintptr_t>(xg + col0) & 15) == 0;
  const int64_t bulk_elems = x_aligned ? ((ncols * int64_t(sizeof(T))) & ~int64_t(15)) / int64_t(sizeof(T)) : 0;
  if (threadIdx.x == 0) {
    mbar_init(&xbar, 1);
    for (int s = 0; s < NS; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], XT_EMPTY);
      stag[s] = -1;
    }
    for (int k = 0; k < XT_K; ++k) {
      mbar_init(&rbar[k], 1);
      mbar_init(&fbar[k], B);
      fincnt[k] = 0;
    }
    next_chunk = XT_NWC;  // chunks 0..NWC-1 go to consumer warps 0..NWC-1
    asm volatile("fence.mbarrier_init.release.cluster;\n" ::: "memory");
    const uint32_t xb = uint32_t(bulk_elems * sizeof(T));
    mbar_expect_tx(&xbar, xb);
    if (xb) bulk_g2s(xs, xg + col0, xb, &xbar);
    for (int t = 0; t < XT_K && t < ntiles; ++t) mbar_expect_tx(&rbar[t], uint32_t(own_rows(t) * B * 8));
  }
  for (int64_t j = bulk_elems + threadIdx.x; j <= Wg; j += blockDim.x) xs[j] = (j < ncols) ? xg[col0 + j] : T(0);
  // peers must have initialised their barriers before partials or signals arrive
  cluster_arrive();
  cluster_wait();

  double dacc = 0.0;
#ifdef XT_PROF
  unsigned long long pr[8] = {0, 0, 0, 0, 0, 0, 0, 0};
  XT_T0(tk0);
#endif
  if (warp == 0) {
    // ---------------------------------------------------------- producer
    // Lane 0 issues the stages in order; the whole warp fetches the stage
    // metadata 32 stages at a time (one LDG per lane, a batch ahead), so no
    // global-load latency sits between two bulk copies.
    uint32_t inf_n = 0;
    long long off_n = 0;
    if (lane < nst) {
      inf_n = a.st_info[st0 + lane];
      off_n = a.st_off[st0 + lane];
    }
    for (int s0 = 0; s0 < nst; s0 += 32) {
      const uint32_t inf_c = inf_n;
      const long long off_c = off_n;
      if (s0 + 32 + lane < nst) {  // next batch, in flight while this one is issued
        inf_n = a.st_info[st0 + s0 + 32 + lane];
        off_n = a.st_off[st0 + s0 + 32 + lane];
      }
      const int nb = min(32, nst - s0);
      for (int k = 0; k < nb; ++k) {
        const uint32_t info = __shfl_sync(0xffffffffu, inf_c, k);
        const long long off = __shfl_sync(0xffffffffu, off_c, k);
        if (lane == 0) {
          const int s = s0 + k, slot = s % NS;
          if (s >= NS) mbar_wait(&empty[slot], uint32_t((s / NS) - 1) & 1u, 100000 + s);
          const uint32_t bytes = info & 0xffffu, np = info >> 16;
          if (np < uint32_t(XT_EMPTY)) mbar_arrive_cnt(&empty[slot], uint32_t(XT_EMPTY) - np);
          // the slot's tag is published before the arrive (release): a consumer that is
          // more than NS stages ahead of the oldest unreleased stage sees a stale tag and
          // keeps waiting instead of mistaking an older phase of the same parity (ABA)
          atomicExch(&stag[slot], s);  // atomic: the tag is a flag read concurrently by consumers
          mbar_expect_tx(&full[slot], bytes);
          bulk_g2s(ring + size_t(slot) * XT_SMAX, a.plan + off, bytes, &full[slot]);
        }
        __syncwarp();
      }
    }
  } else {
    const double alpha = a.alpha, beta = a.beta;
    const int NG = RB / 32;  // 32-row groups owned per tile
    T* __restrict__ y = static_cast<T*>(a.y);
    if (warp >= XT_THREADS / 32 - XT_NFW) {
      // -------------------------------------------------------- finalizers
      // Tile t: wait for the B partials of every owned row, sum them in rank
      // order, write y (Q = 1) or this part's partial (Q > 1, then one ticket
      // per 32-row group: the last of the Q owners combines the parts in part
      // order), then free the receive slot in every peer.  Off the ring's
      // critical path: the consumer warps never wait for this work.
      const int fw = warp - (XT_THREADS / 32 - XT_NFW);
      for (int t = 0; t < ntiles; ++t) {
        const int slot = t % XT_K;
        XT_T0(tf0);
        mbar_wait(&rbar[slot], uint32_t(t / XT_K) & 1u, 200000 + t);
        XT_ACC(5, tf0);
        const double* rv = recv + size_t(slot) * R;
        const int nrows = tile_rows(t);
        const int64_t tr0 = r0 + int64_t(t) * R + b * RB;  // first global row owned in this tile
        for (int g = fw; g < NG; g += XT_NFW) {
          const int jl = g * 32 + lane;
          const bool valid = b * RB + jl < nrows;
          const int64_t i = tr0 + jl;
          if (!valid) continue;
          double sum = 0.0;
          for (int p = 0; p < B; ++p) sum += rv[p * RB + jl];
          if (a.Q == 1) {
            double r = alpha * sum;
            if (beta != 0.0) r += beta * double(y[i]);
            const T out = T(r);
            y[i] = out;
            if (DOT) dacc += double(static_cast<const T*>(a.w)[i]) * double(out);
          } else {
            a.ypart[int64_t(q) * a.m + i] = sum;
            // DOT with Q > 1 (beta == 0, enforced by the host): this part's share of w.y
            if (DOT) dacc += double(static_cast<const T*>(a.w)[i]) * (alpha * sum);
          }
        }
        if (a.Q > 1) {
          // group tickets, one lane per group of this warp (groups past the
          // cluster's last row belong to the next cluster of the part: none)
          __syncwarp();
          __threadfence();
          const int g = fw + lane * XT_NFW;
          const int64_t grow = tr0 + int64_t(g) * 32;
          bool last = false;
          if (g < NG && grow < r1) last = atomicAdd(a.gcnt + (grow >> 5), 1) == a.Q - 1;
          unsigned mask = __ballot_sync(0xffffffffu, last);
          if (mask) __threadfence();
          while (mask) {
            const int k = __ffs(mask) - 1;
            mask &= mask - 1;
            const int gk = fw + k * XT_NFW;
            const int64_t i = tr0 + int64_t(gk) * 32 + lane;
            if (i < r1) {
              double s2 = 0.0;
              for (int p = 0; p < a.Q; ++p) s2 += __ldcg(a.ypart + int64_t(p) * a.m + i);
              double r = alpha * s2;
              if (beta != 0.0) r += beta * double(y[i]);
              y[i] = T(r);
            }
            if (lane == k) a.gcnt[grow >> 5] = 0;  // re-armed for the next launch (stream order)
          }
        }
        // the last finalizer re-arms the slot for tile t+K and frees it in every peer
        __syncwarp();
        int lastw = 0;
        if (lane == 0) {
          __threadfence_block();
          lastw = atomicAdd(&fincnt[slot], 1) == XT_NFW - 1;
        }
        lastw = __shfl_sync(0xffffffffu, lastw, 0);
        if (lastw && lane == 0) {
          fincnt[slot] = 0;
          if (t + XT_K < ntiles) mbar_expect_tx(&rbar[slot], uint32_t(own_rows(t + XT_K) * B * 8));
          for (int p = 0; p < B; ++p) mbar_arrive_remote(&fbar[slot], uint32_t(p));
        }
        XT_ACC(4, tf0);
      }
    } else {
      // -------------------------------------------------------- consumers
      const int cw = warp - 1;
      const uint32_t recv_l = smem_u32(recv);
      const uint32_t rbar_l = smem_u32(&rbar[0]);
      mbar_wait(&xbar, 0, 1);
      const int nchunks = ntiles * XT_NC;
      for (int j = cw; j < nchunks;) {
        const int t = j / XT_NC;
        const int64_t cid = (int64_t(tile0 + t) * B + b) * XT_NC + (j % XT_NC);
        const uint2 meta = a.ck_meta[cid];
        const int stage = int(meta.x);
        const int len = int(meta.y >> 16);
        const int npc = max(1, (len + LMAX - 1) / LMAX);
        double acc0 = 0.0, acc1 = 0.0;  // two chains: even / odd steps (fixed order, deterministic)
        int row = 0xffff;
        for (int pc = 0; pc < npc; ++pc) {
          const int s = stage + pc, slot = s % NS;
          XT_T0(tt0);
          {  // wait until stage s is the slot's current occupant (see the producer), then its data
            long long t0 = 0;
            for (uint32_t spin = 0; atomicOr(&stag[slot], 0) != s; ++spin) {
              __nanosleep(64);  // back off: spinning warps would steal issue and LDS slots
              if ((spin & 255) == 255) {
                const long long now = clock64();
                if (t0 == 0) t0 = now;
                else if (now - t0 > 4000000000LL) {
                  printf("spmv: xt stage tag timeout block %d warp %d stage %d slot %d tag %d\n", blockIdx.x, warp,
                         s, slot, atomicOr(&stag[slot], 0));
                  __trap();
                }
              }
            }
          }
          XT_ACC(0, tt0);
          XT_T0(tw0);
          mbar_wait(&full[slot], uint32_t(s / NS) & 1u, 300000 + s);
          XT_ACC(1, tw0);
          XT_T0(tp0);
          const unsigned char* base = ring + size_t(slot) * XT_SMAX;
          if (pc == 0) {
            base += size_t(meta.y & 0xffffu) * 16;
            row = reinterpret_cast<const uint16_t*>(base)[lane];
            base += XT_HDR;
          }
          int L = min(LMAX, len - pc * LMAX);
#ifdef XT_NOPROC  // diagnostic variant builds only: ring throughput without the step loop
          L = 0;
#endif
          const unsigned char* V = base + size_t(lane) * sizeof(T);
          const unsigned char* C = base + size_t(L) * 32 * sizeof(T) + size_t(lane) * 2;
          for (int k = 0; k < L; k += XT_U) {
            T v[XT_U];
            uint32_t cc[XT_U];
#pragma unroll
            for (int u = 0; u < XT_U; ++u) {
              if (k + u < L) {
                v[u] = xt_lds<T>(V + size_t(k + u) * 32 * sizeof(T));
                cc[u] = xt_lds<uint16_t>(C + size_t(k + u) * 64);
              } else {
                v[u] = T(0);
                cc[u] = uint32_t(Wg);
              }
            }
            T xv[XT_U];
#pragma unroll
            for (int u = 0; u < XT_U; ++u) {
#ifdef XT_NOGATHER  // diagnostic variant builds only: no x gathers
              xv[u] = T(cc[u]);
#else
              xv[u] = xs[cc[u]];
#endif
            }
#pragma unroll
            for (int u = 0; u < XT_U; u += 2) {
              acc0 = fma(double(v[u]), double(xv[u]), acc0);
              if (u + 1 < XT_U) acc1 = fma(double(v[u + 1]), double(xv[u + 1]), acc1);
            }
          }
          __syncwarp();
          if (lane == 0) mbar_arrive_cnt(&empty[slot], 1u);
          XT_ACC(2, tp0);
        }
#ifdef XT_PROF
        pr[7] += 1;
#endif
        // push the block partial of the lane's row to its owner (once the slot of tile t is free)
        const double acc = acc0 + acc1;
        const int slot = t % XT_K;
        XT_T0(tb0);
        if (t >= XT_K && __any_sync(0xffffffffu, row != 0xffff))
          mbar_wait(&fbar[slot], uint32_t(t / XT_K - 1) & 1u, 400000 + t);
        XT_ACC(3, tb0);
        if (row != 0xffff) {
          const int own = row / RB, jl = row - own * RB;
          const uint32_t laddr = recv_l + uint32_t((slot * R + b * RB + jl) * 8);
          xt_st_async(xt_mapa(laddr, own), acc, xt_mapa(rbar_l + uint32_t(slot * 8), own));
        }
        if (a.dyn) {  // the next chunk in stream order: the oldest ring stages are served first
          int nj = 0;
          if (lane == 0) nj = atomicAdd(&next_chunk, 1);
          j = __shfl_sync(0xffffffffu, nj, 0);
        } else {
          j += XT_NWC;
        }
      }
    }
  }
#ifdef XT_PROF
  XT_ACC(6, tk0);
  if (lane == 0 && a.prof)
    for (int i = 0; i < 8; ++i) a.prof[(size_t(blockIdx.x) * 32 + warp) * 8 + i] = pr[i];
#endif
  if (DOT) {
    const double tsum = block_sum(dacc, red);
    if (threadIdx.x == 0) a.part[blockIdx.x] = tsum;
  }
  // leave together: peers may still signal this CTA's barriers
  cluster_arrive();
  cluster_wait();
  if (DOT) p2p_push_partials_last(a.hk, a.part, gridDim.x);
}

// ---------------------------------------------------------------- builders
// Segment of row i in block g: [k0, k1) (absolute k).  bseg: (NB-1) x m
// interior split points, block-major.
__device__ __forceinline__ void xt_seg(const int* rowptr, const int* bseg, int64_t m, int NB, int g, int64_t i,
                                       int* k0, int* k1) {
  *k0 = (g == 0) ? rowptr[i] : bseg[int64_t(g - 1) * m + i];
  *k1 = (g == NB - 1) ? rowptr[i + 1] : bseg[int64_t(g) * m + i];
}

// Interior split points: bseg[g-1][i] = first k of row i with colidx[k] >= bcol[g]
// (columns ascending), g = 1..NB-1.  Thread per row, binary search per boundary.
static __global__ void __launch_bounds__(256)
k_xt_splits(int64_t m, const int* __restrict__ rowptr, const int* __restrict__ colidx, int NB,
            const long long* __restrict__ bcol, int* __restrict__ bseg) {
  for (int64_t i = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; i < m; i += int64_t(gridDim.x) * blockDim.x) {
    const int k0 = rowptr[i], k1 = rowptr[i + 1];
    int lo = k0;
    for (int g = 1; g < NB; ++g) {
      const long long cb = bcol[g];
      int hi = k1;
      while (lo < hi) {
        const int mid = lo + ((hi - lo) >> 1);
        if (colidx[mid] < cb) lo = mid + 1; else hi = mid;
      }
      bseg[int64_t(g - 1) * m + i] = lo;
    }
  }
}

// One CTA (1024 threads) per (cluster, tile, b): sort the tile's rows by the
// length of their segment in block g = part*B + b (descending, ties by row),
// cut into XT_NC chunks of 32; chunk length = its longest segment; each row's
// slot (chunk*32 + lane) for the pack.  tiles: [ntiles_total] cluster of each
// global tile.
static __global__ void __launch_bounds__(1024)
k_xt_sell(const int* __restrict__ rowptr, const int* __restrict__ bseg, int64_t m, int NB, int B,
          const int* __restrict__ tile_cl, const int* __restrict__ cl_tile0, const int* __restrict__ cl_part,
          const long long* __restrict__ cl_rows, int* __restrict__ ck_len, uint16_t* __restrict__ ck_row,
          int* __restrict__ row_slot) {
  __shared__ unsigned long long key[XT_R];
  const int tg = blockIdx.x / B, b = blockIdx.x % B;
  const int c = tile_cl[tg];
  const int t = tg - cl_tile0[c];
  const int g = cl_part[c] * B + b;
  const int64_t rt = cl_rows[2 * c] + int64_t(t) * XT_R;
  const int nrows = int(cmin64(XT_R, cl_rows[2 * c + 1] - rt));
  const int j = threadIdx.x;
  int L = -1;  // absent rows sort last
  if (j < nrows) {
    int k0, k1;
    xt_seg(rowptr, bseg, m, NB, g, rt + j, &k0, &k1);
    L = k1 - k0;
  }
  key[j] = (static_cast<unsigned long long>(~static_cast<uint32_t>(L + 1)) << 32) | uint32_t(j);
  __syncthreads();
  for (int k = 2; k <= XT_R; k <<= 1)
    for (int s = k >> 1; s > 0; s >>= 1) {
      const int p = j ^ s;
      if (p > j) {
        const bool up = (j & k) == 0;
        const unsigned long long a0 = key[j], a1 = key[p];
        if ((a0 > a1) == up) { key[j] = a1; key[p] = a0; }
      }
      __syncthreads();
    }
  const unsigned long long kk = key[j];
  const int row = int(kk & 0xffffffffu);
  const int Ls = int(~uint32_t(kk >> 32)) - 1;
  const int w = j / 32, ln = j % 32;
  const int64_t cid = (int64_t(tg) * B + b) * XT_NC + w;
  ck_row[cid * 32 + ln] = (Ls >= 0) ? uint16_t(row) : uint16_t(0xffff);
  if (Ls >= 0) row_slot[int64_t(g) * m + rt + row] = j;
  if (ln == 0) ck_len[cid] = max(Ls, 0);
}

// Byte offset of step s (lane ln) of a chunk starting at `off` with `len`
// steps: pieces of LMAX steps after the row map; vals then cols per piece.
template <typename T>
__device__ __forceinline__ void xt_addr(long long off, int len, int s, int ln, long long* voff, long long* coff) {
  constexpr int LMAX = xt_lmax<T>();
  const int pc = s / LMAX, sl = s - pc * LMAX;
  const int L = min(LMAX, len - pc * LMAX);
  const long long pbase = off + XT_HDR + (long long)pc * LMAX * 32 * (long long)(sizeof(T) + 2);
  *voff = pbase + ((long long)sl * 32 + ln) * (long long)sizeof(T);
  *coff = pbase + (long long)L * 32 * (long long)sizeof(T) + ((long long)sl * 32 + ln) * 2;
}

// Row maps and padding of every chunk (value 0, column = the block's pad column).
template <typename T>
__global__ void k_xt_fill(unsigned char* __restrict__ plan, const long long* __restrict__ ck_off,
                          const int* __restrict__ ck_len, const uint16_t* __restrict__ ck_row,
                          const int* __restrict__ ck_pad, int64_t nchunks) {
  for (int64_t c = blockIdx.x; c < nchunks; c += gridDim.x) {
    const long long off = ck_off[c];
    const int len = ck_len[c];
    const uint16_t pad = uint16_t(ck_pad[c]);
    if (threadIdx.x < 32) reinterpret_cast<uint16_t*>(plan + off)[threadIdx.x] = ck_row[c * 32 + threadIdx.x];
    for (int e = threadIdx.x; e < len * 32; e += blockDim.x) {
      long long vo, co;
      xt_addr<T>(off, len, e / 32, e % 32, &vo, &co);
      *reinterpret_cast<T*>(plan + vo) = T(0);
      *reinterpret_cast<uint16_t*>(plan + co) = pad;
    }
  }
}

// Scatter every nonzero into its chunk slot: warp per row.  For each part,
// the row's cluster is found by binary search in that part's cluster ranges.
template <typename T>
__global__ void __launch_bounds__(256)
k_xt_pack(const int* __restrict__ rowptr, const int* __restrict__ colidx, const T* __restrict__ vals,
          const int* __restrict__ bseg, int64_t m, int NB, int B, const long long* __restrict__ bcol,
          const int* __restrict__ part_cl0, const long long* __restrict__ cl_rows, const int* __restrict__ cl_tile0,
          const long long* __restrict__ ck_off, const int* __restrict__ ck_len, const int* __restrict__ row_slot,
          unsigned char* __restrict__ plan, int values_only) {
  const int lane = threadIdx.x & 31;
  for (int64_t i = (int64_t(blockIdx.x) * blockDim.x + threadIdx.x) / 32; i < m;
       i += int64_t(gridDim.x) * blockDim.x / 32) {
    for (int g = 0; g < NB; ++g) {
      int k0, k1;
      xt_seg(rowptr, bseg, m, NB, g, i, &k0, &k1);
      if (k1 <= k0) continue;
      const int qq = g / B, b = g % B;
      int lo = part_cl0[qq], hi = part_cl0[qq + 1] - 1;
      while (lo < hi) {
        const int mid = (lo + hi + 1) >> 1;
        if (cl_rows[2 * mid] <= i) lo = mid; else hi = mid - 1;
      }
      const int c = lo;
      const int t = int((i - cl_rows[2 * c]) / XT_R);
      const int slot = row_slot[int64_t(g) * m + i];
      const int64_t cid = (int64_t(cl_tile0[c] + t) * B + b) * XT_NC + slot / 32;
      const int ln = slot % 32, len = ck_len[cid];
      const long long off = ck_off[cid];
      for (int k = k0 + lane; k < k1; k += 32) {
        long long vo, co;
        xt_addr<T>(off, len, k - k0, ln, &vo, &co);
        *reinterpret_cast<T*>(plan + vo) = vals[k];
        if (!values_only) *reinterpret_cast<uint16_t*>(plan + co) = uint16_t(colidx[k] - bcol[g]);
      }
    }
  }
}

// Column histogram (nnz per column) for the part split points.
static __global__ void k_col_count(int64_t k0, int64_t k1, const int* __restrict__ colidx, int* __restrict__ cnt) {
  for (int64_t k = k0 + int64_t(blockIdx.x) * blockDim.x + threadIdx.x; k < k1; k += int64_t(gridDim.x) * blockDim.x)
    atomicAdd(cnt + colidx[k], 1);
}

}  // namespace spmv
