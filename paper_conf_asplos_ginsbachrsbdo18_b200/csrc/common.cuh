// common.cuh -- device helpers shared by the library's kernels (sm_100a).
// No code here is shared with oracle/ (the CPU oracle is a separate C file).
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

namespace spmv {

constexpr int kNumSMs = 148;  // B200: 2 dies x 74 SMs (queried at run time too)

__device__ __forceinline__ int64_t cmin64(int64_t a, int64_t b) { return a < b ? a : b; }
__device__ __forceinline__ int64_t cmax64(int64_t a, int64_t b) { return a > b ? a : b; }

// ---------------------------------------------------------------- loads
// Streamed operands (vals, colidx) are read exactly once per SpMV: bypass L1
// so the L1 capacity is left to the x gathers (ld.global.nc.L1::no_allocate).
__device__ __forceinline__ double ld_stream(const double* p) {
  double v;
  asm("ld.global.nc.L1::no_allocate.f64 %0, [%1];" : "=d"(v) : "l"(p));
  return v;
}
__device__ __forceinline__ float ld_stream(const float* p) {
  float v;
  asm("ld.global.nc.L1::no_allocate.f32 %0, [%1];" : "=f"(v) : "l"(p));
  return v;
}
__device__ __forceinline__ int ld_stream(const int* p) {
  int v;
  asm("ld.global.nc.L1::no_allocate.s32 %0, [%1];" : "=r"(v) : "l"(p));
  return v;
}
// x gathers: read-only path, L1-allocating (x is re-read across rows).
template <typename T>
__device__ __forceinline__ T ld_x(const T* p) { return __ldg(p); }

// ------------------------------------------------------------ reductions
template <int G>
__device__ __forceinline__ double group_sum(double v, unsigned mask) {
#pragma unroll
  for (int off = G / 2; off > 0; off >>= 1) v += __shfl_xor_sync(mask, v, off, G);
  return v;
}

__device__ __forceinline__ double warp_sum(double v) {
#pragma unroll
  for (int off = 16; off > 0; off >>= 1) v += __shfl_xor_sync(0xffffffffu, v, off);
  return v;
}

// Deterministic block sum (fixed tree); result valid in every thread.
// `red` must hold >= blockDim.x/32 doubles.
__device__ __forceinline__ double block_sum(double v, double* red) {
  const int lane = threadIdx.x & 31, wid = threadIdx.x >> 5, nw = blockDim.x >> 5;
  v = warp_sum(v);
  __syncthreads();
  if (lane == 0) red[wid] = v;
  __syncthreads();
  double t = (lane < nw) ? red[lane] : 0.0;
  t = warp_sum(t);
  return t;
}

// Deterministic sum over the first nw warps of the block only (named barrier
// 1), for warp-specialised kernels whose other warps do not participate.
__device__ __forceinline__ double block_sum_n(double v, double* red, int nw) {
  const int lane = threadIdx.x & 31, wid = threadIdx.x >> 5;
  v = warp_sum(v);
  asm volatile("bar.sync 1, %0;\n" ::"r"(nw * 32) : "memory");
  if (lane == 0) red[wid] = v;
  asm volatile("bar.sync 1, %0;\n" ::"r"(nw * 32) : "memory");
  double t = (lane < nw) ? red[lane] : 0.0;
  t = warp_sum(t);
  return t;
}

__device__ __forceinline__ void st_release_sys_u64(unsigned long long* p, unsigned long long v) {
  asm volatile("st.release.sys.global.u64 [%0], %1;\n" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ unsigned long long ld_acquire_sys_u64(const unsigned long long* p) {
  unsigned long long v;
  asm volatile("ld.acquire.sys.global.u64 %0, [%1];\n" : "=l"(v) : "l"(p) : "memory");
  return v;
}

// Wait until every peer completed exchange epoch `e` (watchdog: trap after ~2 s).
__device__ __forceinline__ void p2p_wait_flags(const unsigned long long* flags, int me, int P,
                                               unsigned long long e) {
  for (int q = 0; q < P; ++q) {
    if (q == me) continue;
    long long t0 = 0;
    for (uint32_t spin = 0; ld_acquire_sys_u64(flags + q) < e; ++spin) {
      if ((spin & 1023) == 1023) {
        const long long now = clock64();
        if (t0 == 0) t0 = now;
        else if (now - t0 > 4000000000LL) {
          printf("spmv: p2p wait timeout rank %d waits rank %d for epoch %llu (has %llu)\n", me, q, e,
                 ld_acquire_sys_u64(flags + q));
          __trap();
        }
      }
    }
  }
}

// Last-CTA ticket with acquire-release semantics at GPU scope: the CTA's
// writes (ordered before thread 0 by the preceding bar.sync) happen-before the
// increment, and the CTA drawing the last ticket has acquired every other
// CTA's writes.  Only that CTA then fences at system scope and publishes with
// st.release.sys (p2p_signal): causality is transitive across the two scopes
// (PTX memory model), so one system-scope fence per kernel replaces one per CTA.
__device__ __forceinline__ int ticket_acq_rel_gpu(int* t) {
  int old;
  asm volatile("atom.add.acq_rel.gpu.global.s32 %0, [%1], 1;\n" : "=r"(old) : "l"(t) : "memory");
  return old;
}

constexpr int P2P_NSLOT = 8;       // scalar slots (same ids as reduce_src slots)
constexpr int P2P_XSLOT = P2P_NSLOT;  // slot_epoch index of the x exchange
constexpr int P2P_PMAX = 1024;     // partials per rank per slot: exch is [NSLOT][P][PMAX] doubles

struct P2PCtx {
  unsigned char* const* peer;      // device array [P]: fabric base of every rank (own included)
  size_t off_exch, off_flags;      // byte offsets inside a fabric
  unsigned long long* epoch;       // local exchange counter
  unsigned long long* slot_epoch;  // local [P2P_NSLOT + 1]
  int* ticket;                     // local last-CTA ticket
  const int2* send_iv;             // [P] halo: elements [x, y) of this rank's slice go to rank q (NULL = all)
  int me, P;
};

// Does element j of this rank's x slice go to rank q (halo interval, NEXT-2)?
__device__ __forceinline__ bool p2p_sends(const P2PCtx& c, int q, int64_t j) {
  if (!c.send_iv) return true;
  const int2 iv = c.send_iv[q];
  return j >= iv.x && j < iv.y;
}

// Publish: bump the local epoch, record it for `slot`, flag every peer.  The
// flag stores are releases at system scope: they order every write this
// thread made or acquired (the other CTAs' stores, through their acq_rel GPU
// tickets) before the flag -- no separate fence; with one rank nothing is
// stored and nothing is fenced.
__device__ __forceinline__ void p2p_signal(const P2PCtx& c, int slot, int slot2 = -1) {
  unsigned long long e = *c.epoch + 1;
  c.slot_epoch[slot] = e;
  if (slot2 >= 0) c.slot_epoch[slot2] = ++e;  // a second slot in the same publication
  *c.epoch = e;
  for (int q = 0; q < c.P; ++q) {
    if (q == c.me) continue;
    unsigned long long* f = reinterpret_cast<unsigned long long*>(c.peer[q] + c.off_flags);
    st_release_sys_u64(f + c.me, e);
  }
}

// Exchange hook carried by the compute kernels in the p2p transport (all
// zero / disabled otherwise):
//   wait_x    -- the kernel reads x from xpad: thread 0 of every CTA first
//                waits until every peer published the latest x exchange;
//   push_slot -- the kernel writes one dot partial per CTA into part[]:
//                push_per == gridDim.x (round 2): every CTA stores its partial
//                into entry blockIdx.x of this rank's row of `push_slot` in
//                every rank, the last CTA only publishes (consumers sum the
//                P x push_per values); push_per == 0: the last CTA to finish
//                sums them (read_sum order) and pushes the one value.
struct P2PHook {
  P2PCtx c;
  int enabled = 0;
  int wait_x = 0;
  int push_slot = -1;
  int push_per = 0;
};

// Programmatic dependent launch (PDL): a kernel launched with
// cudaLaunchAttributeProgrammaticStreamSerialization may start while its
// predecessor in the stream is still running; pdl_wait() blocks until the
// predecessor grid has completed and its memory is visible (a no-op when the
// kernel was launched without the attribute).  pdl_trigger() lets the NEXT
// kernel start launching; called only after pdl_wait(), so a kernel's
// successor can never overlap its predecessor.
__device__ __forceinline__ void pdl_wait() { asm volatile("griddepcontrol.wait;\n" ::: "memory"); }
__device__ __forceinline__ void pdl_trigger() { asm volatile("griddepcontrol.launch_dependents;\n" ::: "memory"); }

__device__ __forceinline__ void p2p_prologue_wait(const P2PHook& h) {
  if (h.enabled && h.wait_x) {
    if (threadIdx.x == 0) {
      const unsigned long long* flags =
          reinterpret_cast<const unsigned long long*>(h.c.peer[h.c.me] + h.c.off_flags);
      p2p_wait_flags(flags, h.c.me, h.c.P, h.c.slot_epoch[P2P_XSLOT]);
    }
    __syncthreads();
  }
}

// Call from every thread of every CTA after part[blockIdx.x] was written.
// also_slot >= 0: the last CTA publishes that slot too (its data written before
// every CTA's ticket), with one flag store per peer.
__device__ __forceinline__ void p2p_push_partials_last(const P2PHook& h, const double* part, int count,
                                                       int also_slot = -1) {
  if (!h.enabled || h.push_slot < 0) return;
  __shared__ int s_last;
  const bool per_cta = h.push_per == int(gridDim.x) && count == int(gridDim.x);
  if (per_cta && threadIdx.x == 0) {
    // this CTA's partial straight into every rank (plain stores, ordered before
    // the ticket below and, through the last CTA's release, before the flag)
    const double v = part[blockIdx.x];
    for (int q = 0; q < h.c.P; ++q) {
      double* ex = reinterpret_cast<double*>(h.c.peer[q] + h.c.off_exch);
      ex[(size_t(h.push_slot) * h.c.P + h.c.me) * P2P_PMAX + blockIdx.x] = v;
    }
  }
  // part[blockIdx.x] was stored by thread 0; the acq_rel ticket orders it
  // before the increment and gives the last CTA every other CTA's partial
  __syncthreads();
  if (threadIdx.x == 0) {
    const int tk = ticket_acq_rel_gpu(h.c.ticket);
    s_last = (tk == int(gridDim.x) - 1);
  }
  __syncthreads();
  if (!s_last) return;
  if (per_cta) {
    if (threadIdx.x == 0) {
      *h.c.ticket = 0;
      p2p_signal(h.c, h.push_slot, also_slot);
    }
    return;
  }
  if (threadIdx.x < 32) {
    double a = 0.0;
#pragma unroll 4
    for (int i = threadIdx.x; i < count; i += 32) a += __ldcg(part + i);  // L2: other CTAs' stores
    a = warp_sum(a);
    if (threadIdx.x == 0) {
      *h.c.ticket = 0;
      for (int q = 0; q < h.c.P; ++q) {
        double* ex = reinterpret_cast<double*>(h.c.peer[q] + h.c.off_exch);
        ex[(size_t(h.push_slot) * h.c.P + h.c.me) * P2P_PMAX] = a;
      }
      p2p_signal(h.c, h.push_slot, also_slot);
    }
  }
}

// A scalar source for the CG kernels: either `count` > 0 per-block partials to
// be summed (single GPU: every consuming block sums them in the same fixed
// order, so all blocks see bit-identical scalars), count == 1 pointing at a
// finalized (NCCL-all-reduced) value, or count == -P: the values pushed by
// the ranks over peer memory (p2p_kernels.cuh), `per` per rank at stride
// P2P_PMAX, read once flags[q] >= *epoch for every other rank q and summed
// rank by rank (per == 1: one value each, in rank order; per > 1: lane-strided
// within each rank, then the warp tree) -- identical on all ranks.
struct SumSrc {
  const double* p;
  int count;
  const unsigned long long* flags = nullptr;
  const unsigned long long* epoch = nullptr;
  int me = 0;
  int per = 1;
};

// Warp-wide sum of the pushed values of a p2p source (after its flags).
__device__ __forceinline__ double pushed_sum(const SumSrc& s, int P) {
  const int lane = threadIdx.x & 31;
  double a = 0.0;
  if (s.per <= 1) {
    if (lane == 0)
      for (int q = 0; q < P; ++q) a += s.p[size_t(q) * P2P_PMAX];  // rank order
    return __shfl_sync(0xffffffffu, a, 0);
  }
  for (int q = 0; q < P; ++q)
    for (int i = lane; i < s.per; i += 32) a += s.p[size_t(q) * P2P_PMAX + i];
  return warp_sum(a);
}

// Sum of a SumSrc by warp 0 of the block; returns the value in every thread.
__device__ __forceinline__ double read_sum(SumSrc s, double* slot) {
  if (threadIdx.x < 32) {
    int n = s.count;
    double a = 0.0;
    if (n < 0) {
      if (threadIdx.x == 0) p2p_wait_flags(s.flags, s.me, -n, *s.epoch);
      __syncwarp();
      a = pushed_sum(s, -n);
    } else {
#pragma unroll 4
      for (int i = threadIdx.x; i < n; i += 32) a += s.p[i];
      a = warp_sum(a);
    }
    if (threadIdx.x == 0) *slot = a;
  }
  __syncthreads();
  double v = *slot;
  return v;
}

// The same sum as read_sum (same order, bit-identical), computed by ONE warp
// without a block barrier, so several warps can read different sources at
// once; the value is returned in every lane of the calling warp.
__device__ __forceinline__ double warp_read_sum(SumSrc s) {
  const int lane = threadIdx.x & 31;
  int n = s.count;
  double a = 0.0;
  if (n < 0) {
    if (lane == 0) p2p_wait_flags(s.flags, s.me, -n, *s.epoch);
    __syncwarp();
    return pushed_sum(s, -n);
  }
#pragma unroll 4
  for (int i = lane; i < n; i += 32) a += s.p[i];
  return warp_sum(a);
}

}  // namespace spmv
