// idiom_kernels.cuh -- sm_100a kernels of the histogram (Fig. 11),
// scalar-reduction (Fig. 14) idioms and NAS EP [ext:NPB-EP]
// (include/idioms.h states the semantics).
// No code here is shared with oracle/ (the CPU oracle is oracle_idioms.c).
//
// All three are reductions of a long stream into a few (or many) bins, so the
// design is: read the stream once, coalesced and with enough bytes in flight
// for HBM (16-B vector loads, several per thread before use); privatise the
// bins where they fit (shared memory) and combine privately held partials in
// a FIXED order (per-thread sequential -> fixed warp/block trees -> per-CTA
// partials summed by the last CTA in CTA order) so every float result is
// bit-identical run to run.  EP is fp64-ALU bound (log, div, sqrt per
// accepted pair), not memory bound: its random numbers are generated in
// registers by jumping the LCG to each thread's first pair.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

#include "common.cuh"

namespace spmv {

constexpr int kRedThreads = 512;
constexpr int kRedMaxGrid = 1024;   // partial slots in the workspace
constexpr int kWsHeader = 16;       // bytes: ticket (u32) + pad

// Last-CTA-done ticket: returns true in every thread of the CTA that arrives
// last (after its partials are visible); that CTA re-arms the ticket.
__device__ __forceinline__ bool last_cta(unsigned* ticket, unsigned nblocks) {
  __shared__ bool last;
  __syncthreads();
  if (threadIdx.x == 0) {
    __threadfence();
    const unsigned t = atomicAdd(ticket, 1u);
    last = (t == nblocks - 1);
  }
  __syncthreads();
  if (last) __threadfence();
  return last;
}

// ---------------------------------------------------------- scalar reduction
template <typename T> struct Vec16;
template <> struct Vec16<double> { using V = double2; static constexpr int W = 2; };
template <> struct Vec16<float> { using V = float4; static constexpr int W = 4; };

template <typename T>
__device__ __forceinline__ double vterm(const typename Vec16<T>::V& a, const typename Vec16<T>::V& b, bool dot,
                                        double acc);
template <>
__device__ __forceinline__ double vterm<double>(const double2& a, const double2& b, bool dot, double acc) {
  if (dot) {
    acc = fma(a.x, b.x, acc);
    return fma(a.y, b.y, acc);
  }
  return (acc + a.x) + a.y;
}
template <>
__device__ __forceinline__ double vterm<float>(const float4& a, const float4& b, bool dot, double acc) {
  if (dot) {
    acc = fma((double)a.x, (double)b.x, acc);
    acc = fma((double)a.y, (double)b.y, acc);
    acc = fma((double)a.z, (double)b.z, acc);
    return fma((double)a.w, (double)b.w, acc);
  }
  return (((acc + (double)a.x) + (double)a.y) + (double)a.z) + (double)a.w;
}

// CTA c reduces the contiguous range [c*chunk, min(n, (c+1)*chunk)) (chunk a
// multiple of the vector width); VEC: a (and b) 16-B aligned.
template <typename T, bool DOT, bool VEC>
__global__ void __launch_bounds__(kRedThreads)
k_reduce(int64_t n, int64_t chunk, const T* __restrict__ a, const T* __restrict__ b, double* __restrict__ out,
         unsigned* __restrict__ ticket, double* __restrict__ part) {
  __shared__ double red[kRedThreads / 32];
  const int64_t lo = (int64_t)blockIdx.x * chunk;
  const int64_t hi = cmin64(n, lo + chunk);
  double acc = 0.0;
  if (VEC) {
    using V = typename Vec16<T>::V;
    constexpr int W = Vec16<T>::W;
    constexpr int U = 4;
    const V* av = reinterpret_cast<const V*>(a + lo);
    const V* bv = DOT ? reinterpret_cast<const V*>(b + lo) : nullptr;
    const int64_t nv = hi > lo ? (hi - lo) / W : 0;
    int64_t i = threadIdx.x;
    for (; i + (U - 1) * kRedThreads < nv; i += U * kRedThreads) {
      V x[U], y[U];
#pragma unroll
      for (int u = 0; u < U; ++u) {
        x[u] = __ldcs(av + i + u * kRedThreads);
        if (DOT) y[u] = __ldcs(bv + i + u * kRedThreads);
      }
#pragma unroll
      for (int u = 0; u < U; ++u) acc = vterm<T>(x[u], DOT ? y[u] : x[u], DOT, acc);
    }
    for (; i < nv; i += kRedThreads) {
      V x = __ldcs(av + i);
      V y = DOT ? __ldcs(bv + i) : x;
      acc = vterm<T>(x, y, DOT, acc);
    }
    for (int64_t k = lo + nv * W + threadIdx.x; k < hi; k += kRedThreads)
      acc = DOT ? fma((double)a[k], (double)b[k], acc) : acc + (double)a[k];
  } else {
    for (int64_t k = lo + threadIdx.x; k < hi; k += kRedThreads)
      acc = DOT ? fma((double)a[k], (double)b[k], acc) : acc + (double)a[k];
  }
  const double s = block_sum(acc, red);
  if (threadIdx.x == 0) part[blockIdx.x] = s;
  if (last_cta(ticket, gridDim.x)) {
    double t = 0.0;
    for (int c = threadIdx.x; c < (int)gridDim.x; c += kRedThreads) t += __ldcg(part + c);
    t = block_sum(t, red);
    if (threadIdx.x == 0) {
      *out = t;
      *ticket = 0u;
    }
  }
}

// ---------------------------------------------------------------- histogram
// Kinds (include/idioms.h): 0 count u32, 1 saturating u8 (counted in a u32
// workspace, then min(255, old + count)), 2 weighted f64.
constexpr int kHistThreads = 1024;

template <int KIND>
struct HistBin { using T = unsigned; };
template <>
struct HistBin<2> { using T = double; };

// Per-key update of a privatised (shared) or global bin.
template <int KIND>
__device__ __forceinline__ void hist_add(typename HistBin<KIND>::T* bin, const double* w, int64_t i) {
  if (KIND == 2) atomicAdd(reinterpret_cast<double*>(bin), __ldcs(w + i));
  else atomicAdd(reinterpret_cast<unsigned*>(bin), 1u);
}

// Visit the keys of [lo, hi) with 16-B loads when `vec` (keys 16-B aligned).
template <typename F>
__device__ __forceinline__ void for_keys(const int32_t* __restrict__ keys, int64_t lo, int64_t hi, int64_t stride0,
                                         int64_t stride, bool vec, F&& f) {
  if (vec) {
    const int64_t vlo = (lo + 3) & ~int64_t(3), vhi = hi & ~int64_t(3);
    if (vlo < vhi) {
      for (int64_t k = lo + stride0; k < vlo; k += stride) f(k, __ldcs(keys + k));
      const int4* kv = reinterpret_cast<const int4*>(keys);
      int64_t j = vlo / 4 + stride0;
      for (; j + stride < vhi / 4; j += 2 * stride) {
        const int4 a = __ldcs(kv + j), b = __ldcs(kv + j + stride);
        f(4 * j, a.x); f(4 * j + 1, a.y); f(4 * j + 2, a.z); f(4 * j + 3, a.w);
        const int64_t jb = j + stride;
        f(4 * jb, b.x); f(4 * jb + 1, b.y); f(4 * jb + 2, b.z); f(4 * jb + 3, b.w);
      }
      for (; j < vhi / 4; j += stride) {
        const int4 a = __ldcs(kv + j);
        f(4 * j, a.x); f(4 * j + 1, a.y); f(4 * j + 2, a.z); f(4 * j + 3, a.w);
      }
      for (int64_t k = vhi + stride0; k < hi; k += stride) f(k, __ldcs(keys + k));
      return;
    }
  }
  for (int64_t k = lo + stride0; k < hi; k += stride) f(k, __ldcs(keys + k));
}

// Shared-memory privatised histogram (nbins fits the CTA's shared memory):
// CTA c counts the contiguous key range [c*chunk, ...) into its own bins and
// then adds its nonzero bins to the global (or workspace) bins.
template <int KIND>
__global__ void __launch_bounds__(kHistThreads)
k_hist_smem(int64_t n, int64_t chunk, int nbins, const int32_t* __restrict__ keys, const double* __restrict__ w,
            typename HistBin<KIND>::T* __restrict__ dst, int vec) {
  using B = typename HistBin<KIND>::T;
  extern __shared__ __align__(16) unsigned char sm_raw[];
  B* sh = reinterpret_cast<B*>(sm_raw);
  for (int b = threadIdx.x; b < nbins; b += kHistThreads) sh[b] = B(0);
  __syncthreads();
  const int64_t lo = (int64_t)blockIdx.x * chunk, hi = cmin64(n, lo + chunk);
  for_keys(keys, lo, hi, threadIdx.x, kHistThreads, vec != 0, [&](int64_t i, int k) {
    if ((unsigned)k < (unsigned)nbins) hist_add<KIND>(sh + k, w, i);
  });
  __syncthreads();
  for (int b = threadIdx.x; b < nbins; b += kHistThreads) {
    const B v = sh[b];
    if (v != B(0)) atomicAdd(dst + b, v);
  }
}

// Global-memory histogram (bins beyond shared memory; they stay L2-resident
// while hot).  AGG: warp-aggregate equal keys (__match_any_sync) so hot bins
// (Parboil-histo hot spots) take one atomic per warp instead of one per key.
template <int KIND, bool AGG>
__global__ void __launch_bounds__(256)
k_hist_global(int64_t n, int nbins, const int32_t* __restrict__ keys, const double* __restrict__ w,
              typename HistBin<KIND>::T* __restrict__ dst, int vec) {
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  const int64_t t0 = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
  if (!AGG) {
    for_keys(keys, 0, n, t0, stride, vec != 0, [&](int64_t i, int k) {
      if ((unsigned)k < (unsigned)nbins) hist_add<KIND>(dst + k, w, i);
    });
    return;
  }
  // AGG (counting kinds): the warp walks the keys in lockstep, 32 consecutive keys per step
  const int lane = threadIdx.x & 31;
  const int64_t wid = t0 >> 5, nwarps = stride >> 5;
  for (int64_t base = wid * 32; base < n; base += nwarps * 32) {
    const int64_t i = base + lane;
    const int k = i < n ? __ldcs(keys + i) : -1;
    const bool ok = (unsigned)k < (unsigned)nbins;
    const unsigned same = __match_any_sync(0xffffffffu, ok ? k : -1);
    if (ok && lane == __ffs(same) - 1) atomicAdd(reinterpret_cast<unsigned*>(dst + k), (unsigned)__popc(same));
  }
}

// Saturating finalize: bins8[b] = min(255, bins8[b] + cnt[b]); cnt re-zeroed.
static __global__ void __launch_bounds__(256)
k_hist_sat_fin(int64_t nbins, unsigned* __restrict__ cnt, uint8_t* __restrict__ bins8) {
  for (int64_t b = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; b < nbins; b += (int64_t)gridDim.x * blockDim.x) {
    const unsigned c = cnt[b];
    if (c) {
      const unsigned v = (unsigned)bins8[b] + c;
      bins8[b] = (uint8_t)(v < c || v > 255u ? 255u : v);
      cnt[b] = 0u;
    }
  }
}

// ----------------------------------------------- bucketed counting histogram
// For bin arrays far beyond shared memory with many keys per bin (NAS IS:
// 2^27 keys into 2^23 bins), one global atomic per key is bound by the L2
// atomic units (measured 182 G/s, lts 79 %).  Instead the keys are
// partitioned by bucket = key >> HB_SHIFT (2^HB_SHIFT bins per bucket, one
// CTA's shared memory), then every bucket is counted in shared memory by one
// CTA that owns its bins (plain read-add-write, no global atomics):
//   K1 hb_count  : per-CTA bucket counts (contiguous key chunks), bucket-major
//   K2 hb_scan   : per bucket, exclusive scan over the CTAs + bucket total
//   K3 hb_scatter: keys staged per 4096-key tile in shared memory, sorted by
//                  bucket, written as 16-bit in-bucket offsets in runs
//                  (coalesced) at the bucket's cursor
//   K4 hb_bins   : one CTA per bucket: shared-memory counts, then
//                  bins[b*BW + j] += count (KIND 0) or min(255, old + count)
//                  (KIND 1, Parboil's saturating uint8 bins)
// Integer counts, so the result is exact whatever the order.
constexpr int HB_SHIFT = 15;               // 32768 bins per bucket (128 KB of uint32 in K4)
constexpr int HB_BW = 1 << HB_SHIFT;
constexpr int HB_MAXB = 1024;              // buckets (nbins <= 2^25)
constexpr int HB_THREADS = 1024;
constexpr int HB_TILE = 4096;              // keys staged per tile in K3 (16 KB of shared memory)

static __global__ void __launch_bounds__(HB_THREADS)
k_hb_count(int64_t n, int64_t chunk, int nbins, int nb, const int32_t* __restrict__ keys,
           unsigned* __restrict__ cnt /* [nb][G] */, int vec) {
  __shared__ unsigned sc[HB_MAXB];
  for (int b = threadIdx.x; b < nb; b += HB_THREADS) sc[b] = 0;
  __syncthreads();
  const int64_t lo = (int64_t)blockIdx.x * chunk, hi = cmin64(n, lo + chunk);
  for_keys(keys, lo, hi, threadIdx.x, HB_THREADS, vec != 0, [&](int64_t, int k) {
    if ((unsigned)k < (unsigned)nbins) atomicAdd(&sc[k >> HB_SHIFT], 1u);
  });
  __syncthreads();
  for (int b = threadIdx.x; b < nb; b += HB_THREADS) cnt[(size_t)b * gridDim.x + blockIdx.x] = sc[b];
}

// grid = nb; block scans the G counts of bucket b (G <= HB_THREADS)
static __global__ void __launch_bounds__(HB_THREADS)
k_hb_scan(int G, unsigned* __restrict__ cnt, unsigned* __restrict__ total) {
  __shared__ unsigned ws[32];
  const int b = blockIdx.x, t = threadIdx.x, lane = t & 31, w = t >> 5;
  const unsigned v = t < G ? cnt[(size_t)b * G + t] : 0u;
  unsigned x = v;
#pragma unroll
  for (int o = 1; o < 32; o <<= 1) {
    const unsigned y = __shfl_up_sync(0xffffffffu, x, o);
    if (lane >= o) x += y;
  }
  if (lane == 31) ws[w] = x;
  __syncthreads();
  if (w == 0) {
    unsigned z = ws[lane];
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      const unsigned y = __shfl_up_sync(0xffffffffu, z, o);
      if (lane >= o) z += y;
    }
    ws[lane] = z;
  }
  __syncthreads();
  const unsigned incl = x + (w ? ws[w - 1] : 0u);
  if (t < G) cnt[(size_t)b * G + t] = incl - v;  // exclusive offset inside the bucket
  if (t == HB_THREADS - 1) total[b] = incl;
}

// exclusive scan of up to HB_MAXB values in shared memory by the whole block
__device__ __forceinline__ void block_excl_scan(unsigned* a, int nb, unsigned* ws) {
  const int t = threadIdx.x, lane = t & 31, w = t >> 5;
  const unsigned v = t < nb ? a[t] : 0u;
  unsigned x = v;
#pragma unroll
  for (int o = 1; o < 32; o <<= 1) {
    const unsigned y = __shfl_up_sync(0xffffffffu, x, o);
    if (lane >= o) x += y;
  }
  if (lane == 31) ws[w] = x;
  __syncthreads();
  if (w == 0) {
    unsigned z = ws[lane];
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      const unsigned y = __shfl_up_sync(0xffffffffu, z, o);
      if (lane >= o) z += y;
    }
    ws[lane] = z;
  }
  __syncthreads();
  if (t < nb) a[t] = x - v + (w ? ws[w - 1] : 0u);
  __syncthreads();
}

static __global__ void __launch_bounds__(HB_THREADS)
k_hb_scatter(int64_t n, int64_t chunk, int nbins, int nb, const int32_t* __restrict__ keys,
             const unsigned* __restrict__ off /* [nb][G] exclusive */, const unsigned* __restrict__ total,
             uint16_t* __restrict__ out) {
  __shared__ unsigned cursor[HB_MAXB], tcnt[HB_MAXB], tbase[HB_MAXB], ws[32];
  extern __shared__ __align__(16) unsigned stage[];  // HB_TILE entries (dynamic)
  const int t = threadIdx.x;
  // global start of bucket b = sum of the totals before it; cursor = start + this CTA's offset
  for (int b = t; b < HB_MAXB; b += HB_THREADS) cursor[b] = b < nb ? total[b] : 0u;
  __syncthreads();
  block_excl_scan(cursor, nb, ws);
  for (int b = t; b < nb; b += HB_THREADS) {
    cursor[b] += off[(size_t)b * gridDim.x + blockIdx.x];
    tcnt[b] = 0u;
  }
  __syncthreads();
  const int64_t lo = (int64_t)blockIdx.x * chunk, hi = cmin64(n, lo + chunk);
  constexpr int KPT = HB_TILE / HB_THREADS;  // keys per thread per tile
  for (int64_t base = lo; base < hi; base += HB_TILE) {
    int kk[KPT];
    unsigned rk[KPT];
#pragma unroll
    for (int q = 0; q < KPT; ++q) {
      const int64_t i = base + (int64_t)q * HB_THREADS + t;
      kk[q] = i < hi ? __ldcs(keys + i) : -1;
      if ((unsigned)kk[q] < (unsigned)nbins) rk[q] = atomicAdd(&tcnt[kk[q] >> HB_SHIFT], 1u);
    }
    __syncthreads();
    for (int b = t; b < nb; b += HB_THREADS) tbase[b] = tcnt[b];
    __syncthreads();
    block_excl_scan(tbase, nb, ws);
#pragma unroll
    for (int q = 0; q < KPT; ++q)
      if ((unsigned)kk[q] < (unsigned)nbins) {
        const unsigned b = (unsigned)kk[q] >> HB_SHIFT;
        stage[tbase[b] + rk[q]] = (b << 16) | ((unsigned)kk[q] & (HB_BW - 1));
      }
    __syncthreads();
    const unsigned staged = nb ? tbase[nb - 1] + tcnt[nb - 1] : 0u;
    for (unsigned p = t; p < staged; p += HB_THREADS) {
      const unsigned e = stage[p], b = e >> 16;
      out[cursor[b] + (p - tbase[b])] = (uint16_t)(e & 0xffffu);
    }
    __syncthreads();
    for (int b = t; b < nb; b += HB_THREADS) {
      cursor[b] += tcnt[b];
      tcnt[b] = 0u;
    }
    __syncthreads();
  }
}

template <int KIND>
__global__ void __launch_bounds__(HB_THREADS)
k_hb_bins(int nbins, int nb, const unsigned* __restrict__ total, const uint16_t* __restrict__ sorted,
          void* __restrict__ bins) {
  extern __shared__ __align__(16) unsigned char hb_raw[];
  unsigned* sh = reinterpret_cast<unsigned*>(hb_raw);
  __shared__ unsigned start_s[HB_MAXB], ws[32];
  const int t = threadIdx.x, b = blockIdx.x;
  for (int q = t; q < HB_MAXB; q += HB_THREADS) start_s[q] = q < nb ? total[q] : 0u;
  for (int j = t; j < HB_BW; j += HB_THREADS) sh[j] = 0u;
  __syncthreads();
  block_excl_scan(start_s, nb, ws);
  const int64_t lo = start_s[b], hi = lo + total[b];
  for (int64_t p = lo + t; p < hi; p += HB_THREADS) atomicAdd(&sh[sorted[p]], 1u);
  __syncthreads();
  const int64_t b0 = (int64_t)b * HB_BW;
  const int w = (int)cmin64(HB_BW, nbins - b0);
  for (int j = t; j < w; j += HB_THREADS) {
    const unsigned c = sh[j];
    if (KIND == 0) {
      unsigned* B = reinterpret_cast<unsigned*>(bins);
      if (c) B[b0 + j] += c;
    } else {
      uint8_t* B = reinterpret_cast<uint8_t*>(bins);
      if (c) {
        const unsigned v = (unsigned)B[b0 + j] + c;
        B[b0 + j] = (uint8_t)(v < c || v > 255u ? 255u : v);
      }
    }
  }
}

// ----------------------------------------------------------------------- EP
constexpr int kEpThreads = 256;
constexpr uint64_t kEpMask46 = (1ULL << 46) - 1;
constexpr uint64_t kEpA = 1220703125ULL;   // 5^13
constexpr uint64_t kEpS = 271828183ULL;

// (a*b) mod 2^46: the low 64 bits of the product already hold it (2^46 | 2^64)
__device__ __forceinline__ uint64_t mul46(uint64_t a, uint64_t b) { return (a * b) & kEpMask46; }

__device__ __forceinline__ uint64_t pow46(uint64_t base, uint64_t e) {
  uint64_t r = 1;
  while (e) {
    if (e & 1) r = mul46(r, base);
    base = mul46(base, base);
    e >>= 1;
  }
  return r;
}

// Thread t of the grid owns pairs [p0 + t*chunk, ...); out of the CTA: 12
// partial sums (q[0..9] as exact integer-valued doubles, sx, sy) in part[c*12].
template <bool EP_COMPACT>
__global__ void __launch_bounds__(kEpThreads)
k_ep(int64_t p0, int64_t count, int64_t chunk, double* __restrict__ out, unsigned* __restrict__ ticket,
     double* __restrict__ part) {
  __shared__ double red[kEpThreads / 32];
  __shared__ unsigned long long qrare[10];
  if (threadIdx.x < 10) qrare[threadIdx.x] = 0ull;
  __syncthreads();
  const int64_t t = (int64_t)blockIdx.x * kEpThreads + threadIdx.x;
  const int64_t lo = cmin64(count, t * chunk), hi = cmin64(count, lo + chunk);
  // seed before pair p: S * A^(2p) (the pair uses the next two draws)
  uint64_t s = mul46(kEpS, pow46(kEpA, 2ull * (uint64_t)(p0 + lo)));
  double sx = 0.0, sy = 0.0;
  unsigned q0 = 0, q1 = 0, q2 = 0, q3 = 0;
  // x = 2u - 1 with u = s * 2^-46, exactly, without an int->double convert:
  // the bits 0x3FF.. | s << 6 are the double 1 + s * 2^-46, and 2v - 3 = 2u - 1
  auto draw = [&](double& x1, double& x2) {
    s = mul46(s, kEpA);
    const double v1 = __longlong_as_double((long long)(0x3FF0000000000000ULL | (s << 6)));
    s = mul46(s, kEpA);
    const double v2 = __longlong_as_double((long long)(0x3FF0000000000000ULL | (s << 6)));
    x1 = fma(2.0, v1, -3.0);   // exact
    x2 = fma(2.0, v2, -3.0);
  };
  auto tally = [&](double x1, double x2) {
    const double tt = __dadd_rn(__dmul_rn(x1, x1), __dmul_rn(x2, x2));  // NPB's rounding, no FMA
    const double f = sqrt(-2.0 * log(tt) / tt);
    const double X = x1 * f, Y = x2 * f;
    const int l = (int)fmax(fabs(X), fabs(Y));
    q0 += (l == 0);
    q1 += (l == 1);
    q2 += (l == 2);
    q3 += (l == 3);
    if (l >= 4 && l < 10) atomicAdd(&qrare[l], 1ull);
    sx += X;
    sy += Y;
  };
  if (EP_COMPACT) {
    // warp-level compaction: accepted pairs (t <= 1, ~pi/4 of them) are queued
    // in shared memory and tallied 32 at a time by the whole warp, so the
    // log/div/sqrt body never runs with idle lanes
    __shared__ double2 queue[kEpThreads / 32][64];
    double2* qw = queue[threadIdx.x >> 5];
    const int lane = threadIdx.x & 31;
    const unsigned lt = (1u << lane) - 1u;
    int cnt = 0;  // warp-uniform
    for (int64_t it = 0; it < chunk; ++it) {
      double x1 = 0.0, x2 = 0.0;
      bool acc = false;
      if (lo + it < hi) {
        draw(x1, x2);
        acc = __dadd_rn(__dmul_rn(x1, x1), __dmul_rn(x2, x2)) <= 1.0;
      }
      const unsigned m = __ballot_sync(0xffffffffu, acc);
      if (acc) qw[cnt + __popc(m & lt)] = make_double2(x1, x2);
      cnt += __popc(m);
      if (cnt >= 32) {
        __syncwarp();
        const double2 e = qw[lane];
        tally(e.x, e.y);
        __syncwarp();
        if (lane < cnt - 32) qw[lane] = qw[32 + lane];
        __syncwarp();
        cnt -= 32;
      }
    }
    __syncwarp();
    if (lane < cnt) {
      const double2 e = qw[lane];
      tally(e.x, e.y);
    }
  } else {
    for (int64_t p = lo; p < hi; ++p) {
      double x1, x2;
      draw(x1, x2);
      if (__dadd_rn(__dmul_rn(x1, x1), __dmul_rn(x2, x2)) <= 1.0) tally(x1, x2);
    }
  }
  double v[12];
  v[0] = block_sum((double)q0, red);
  v[1] = block_sum((double)q1, red);
  v[2] = block_sum((double)q2, red);
  v[3] = block_sum((double)q3, red);
  v[10] = block_sum(sx, red);
  v[11] = block_sum(sy, red);
  __syncthreads();
  if (threadIdx.x == 0) {
    for (int j = 4; j < 10; ++j) v[j] = (double)qrare[j];
    for (int j = 0; j < 12; ++j) part[(size_t)blockIdx.x * 12 + j] = v[j];
  }
  if (last_cta(ticket, gridDim.x)) {
    // sum the CTA partials in CTA order: warp j < 12 owns value j
    const int lane = threadIdx.x & 31, j = threadIdx.x >> 5;
    for (int jj = j; jj < 12; jj += kEpThreads / 32) {
      double a = 0.0;
      for (int c = lane; c < (int)gridDim.x; c += 32) a += __ldcg(part + (size_t)c * 12 + jj);
      a = warp_sum(a);
      if (lane == 0) out[jj] = a;
    }
    if (threadIdx.x == 0) *ticket = 0u;
  }
}

}  // namespace spmv
