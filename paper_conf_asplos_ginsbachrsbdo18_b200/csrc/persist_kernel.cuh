// persist_kernel.cuh -- persistent, device-driven single-reduction CG over the
// XPLAN plan.  ONE launch runs all
// `iters` CG iterations of cg_solve / the NAS outer iteration (the loop the
// paper's lazy copying keeps on the device; its SpMV is "the
// performance bottleneck of the NAS CG benchmark"):
//
//   for k in 0..iters-1:
//     (A) w = A r: every CTA reloads its x block of r into shared memory and
//         streams its tiles of the XPLAN plan (the k_spmv_xplan tile loop,
//         receive slots and mbarrier phases continuing across iterations);
//         delta partial = w.r per CTA
//     -- grid barrier --
//     (B) the k_cgcg update on a grid-stride slice: gamma = r.r (the previous
//         (B)'s partials; k = 0: k_cg_init's), delta, beta = gamma/gamma_old,
//         alpha = gamma/(delta - beta*gamma/alpha_old); p = r + beta p,
//         s = w + beta s, z += alpha p, r -= alpha s; partial r.r
//     -- grid barrier --
//
// Every CTA sums the same partials in the same order, so all CTAs (and all
// runs) get bit-identical alpha, beta -- the iterates equal those of the
// k_spmv_xplan + k_cgcg graph path up to the per-CTA dot partition of (A),
// which is the same (one partial per CTA of the same grid).  The grid is the
// plan's co-resident clusters (one CTA per SM), so the software grid barrier
// (a monotonic counter, zeroed before the launch) cannot deadlock.
#pragma once
#include "xplan_kernel.cuh"

namespace spmv {


// Grid-wide barrier over a grid whose CTAs are all co-resident: the counter
// only grows; barrier number `e` (1, 2, ...) completes at e * gridDim.x arrivals.
__device__ __forceinline__ void grid_barrier(unsigned int* ctr, unsigned int e) {
  __syncthreads();
  if (threadIdx.x == 0) {
    __threadfence();
    atomicAdd(ctr, 1u);
    const unsigned int target = e * gridDim.x;
    long long t0 = 0;
    for (uint32_t spin = 0;; ++spin) {
      unsigned int v;
      asm volatile("ld.acquire.gpu.global.u32 %0, [%1];\n" : "=r"(v) : "l"(ctr) : "memory");
      if (v >= target) break;
      if ((spin & 1023) == 1023) {
        const long long now = clock64();
        if (t0 == 0) t0 = now;
        else if (now - t0 > 4000000000LL) {
          printf("spmv: grid barrier timeout block %d epoch %u (%u of %u)\n", blockIdx.x, e, v, target);
          __trap();
        }
      }
    }
  }
  __syncthreads();
}

// Sum of `count` partials in a fixed order (the order of warp_read_sum), by warp
// 0, broadcast through shared memory.
__device__ __forceinline__ double persist_sum(const double* src, int count, double* slot) {
  if (threadIdx.x < 32) {
    double a = 0.0;
#pragma unroll 4
    for (int i = threadIdx.x; i < count; i += 32) a += __ldcg(src + i);
    a = warp_sum(a);
    if (threadIdx.x == 0) *slot = a;
  }
  __syncthreads();
  return *slot;
}

static __global__ void __launch_bounds__(XP_THREADS, 1)
k_cg_persist(PersistArgs pa) {
  extern __shared__ __align__(128) unsigned char smem[];
  __shared__ uint64_t xbar, tbar[XP_K];
  __shared__ double red[32];
  __shared__ double sc[4];
  using T = double;
  const XplanArgs& a = pa.sp;
  const int B = (int)cgx::this_cluster().num_blocks();
  const int b = (int)cluster_rank();
  const int c = (int)cluster_id();
  constexpr int R = XP_R;
  const int RB = R / B;
  const int W = a.W;
  T* xs = reinterpret_cast<T*>(smem);
  double* recv = reinterpret_cast<double*>(smem + ((size_t(W + 1) * sizeof(T) + 15) & ~size_t(15)));
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int64_t r0c = a.crow[c], r1c = a.crow[c + 1];
  const int ntiles = int((r1c - r0c + R - 1) / R);
  const int tbase = a.tile0[c];
  const int64_t col0 = int64_t(b) * W;
  const int64_t ncols = cmax64(0, cmin64(W, a.nx - col0));
  const T* __restrict__ xg = static_cast<const T*>(a.x);
  const bool x_aligned = (reinterpret_cast<uintptr_t>(xg + col0) & 15) == 0;
  const int64_t bulk_elems = x_aligned ? ((ncols * int64_t(sizeof(T))) & ~int64_t(15)) / int64_t(sizeof(T)) : 0;
  const int64_t total_tiles = int64_t(ntiles) * pa.iters;  // tiles over all iterations (receive slot sequence)
  auto recv_bytes = [&](int t) -> uint32_t {
    const int nrows = int(cmin64(R, r1c - (r0c + int64_t(t) * R)));
    const int own = max(0, min((b + 1) * RB, nrows) - b * RB);
    return uint32_t(own * B * 8);
  };
  if (threadIdx.x == 0) {
    mbar_init(&xbar, 1);
    for (int q = 0; q < XP_K; ++q) mbar_init(&tbar[q], 1);
    asm volatile("fence.mbarrier_init.release.cluster;\n" ::: "memory");
    for (int q = 0; q < XP_K && q < total_tiles; ++q) mbar_expect_tx(&tbar[q], recv_bytes(q % ntiles));
  }
  cluster_arrive();
  cluster_wait();

  const int nfin = min((RB + 31) & ~31, XP_THREADS);
  unsigned int gepoch = 0;
  double alpha_old = 1.0;
  const int64_t G = gridDim.x;
  const int64_t gstride = G * blockDim.x;

  // diagnostics (tuning builds, cg_solve only): per-CTA phase stamps of iteration iters/2
  const int tk = pa.iters / 2;
  auto stamp = [&](int k, int i) {
    if (a.tstamp && k == tk && threadIdx.x == 0) a.tstamp[8 * blockIdx.x + i] = gtimer();
  };
  for (int k = 0; k < pa.iters; ++k) {
    // ---------------------------------------------------------- (A) w = A r
    stamp(k, 0);
    if (a.cta_range && warp == 1) {  // small plan: the CTA's chunk range into L2 (see k_spmv_xplan)
      const long long q0 = a.cta_range[2 * blockIdx.x], q1 = a.cta_range[2 * blockIdx.x + 1];
      for (long long o = q0 + int64_t(lane) * 65536; o < q1; o += 32 * 65536)
        asm volatile("cp.async.bulk.prefetch.L2.global [%0], %1;" ::"l"(a.plan + o), "r"(uint32_t(cmin64(65536, q1 - o)))
                     : "memory");
    }
    if (threadIdx.x == 0) {
      const uint32_t xb = uint32_t(bulk_elems * sizeof(T));
      mbar_expect_tx(&xbar, xb);
      if (xb) bulk_g2s(xs, xg + col0, xb, &xbar);
    }
    for (int64_t j = bulk_elems + threadIdx.x; j <= W; j += blockDim.x) xs[j] = (j < ncols) ? xg[col0 + j] : T(0);
    __syncthreads();
    mbar_wait(&xbar, uint32_t(k) & 1u, 7000000 + k);
    stamp(k, 1);
    double dacc = 0.0;
    const int64_t tg0 = int64_t(k) * ntiles;  // global sequence number of this iteration's tile 0

    auto process_chunk = [&](int t, int ch) {
      const int64_t seq = tg0 + t;
      const int64_t cid = (int64_t(tbase + t) * B + b) * XP_CPT + ch;
      const int len = a.chunk_len[cid];
      const int row = a.chunk_row[cid * 32 + lane];
      const unsigned char* base = a.plan + a.chunk_off[cid];
      const double acc = xplan_chunk_dot<T>(base, len, lane, xs, W);
      if (row != 0xffff) {
        const int q = row / RB, jl = row - q * RB;
        const uint32_t laddr = smem_u32(recv + int(seq % XP_K) * R + b * RB + jl);
        st_async_f64(mapa_u32(laddr, q), acc, mapa_u32(smem_u32(&tbar[seq % XP_K]), q));
      }
    };
    auto process = [&](int t) {
#pragma unroll 1
      for (int h = 0; h < XP_CPW; h += 2) {
        process_chunk(t, h * XP_NW / 2 + warp);
        if (h + 1 < XP_CPW) process_chunk(t, XP_CPT - 1 - (h * XP_NW / 2 + warp));
      }
    };
    auto finalize = [&](int t) {
      if (int(threadIdx.x) >= nfin) return;
      const int64_t seq = tg0 + t;
      const double* rv = recv + int(seq % XP_K) * R;
      const int64_t rt = r0c + int64_t(t) * R;
      const int nrows = int(cmin64(R, r1c - rt));
      mbar_wait(&tbar[seq % XP_K], uint32_t(seq / XP_K) & 1u, 8000000 + t);
      for (int jl = threadIdx.x; jl < RB && b * RB + jl < nrows; jl += nfin) {
        double sum = 0.0;
        for (int q = 0; q < B; ++q) sum += rv[q * RB + jl];
        const int64_t i = rt + b * RB + jl;
        pa.w[i] = sum;
        dacc += pa.r[i] * sum;  // delta = w.r (alpha = 1, beta = 0)
      }
      asm volatile("bar.sync 2, %0;\n" ::"r"(nfin) : "memory");
      // re-arm the slot for the tile K later in the sequence (next iteration's first tiles included)
      if (threadIdx.x == 0 && seq + XP_K < total_tiles)
        mbar_expect_tx(&tbar[seq % XP_K], recv_bytes(int((seq + XP_K) % ntiles)));
    };
    if (ntiles > 0) {
      process(0);
      cluster_arrive_relaxed();
      for (int t = 1; t < ntiles; ++t) {
        process(t);
        cluster_wait();
        finalize(t - 1);
        cluster_arrive_relaxed();
      }
      if (a.tstamp && k == tk && lane == 0) atomicMax(a.tstamp + 8 * blockIdx.x + 2, gtimer());
      cluster_wait();
      finalize(ntiles - 1);
    }
    {
      const double ts = block_sum(dacc, red);
      if (threadIdx.x == 0) pa.part_d[blockIdx.x] = ts;
    }
    stamp(k, 3);
    grid_barrier(pa.gbar, ++gepoch);
    stamp(k, 4);

    // ---------------------------------------------------------- (B) update
    {
      const int wid = threadIdx.x >> 5;
      double v = 0.0;
      const double* gk = k == 0 ? pa.gam0 : pa.part_g + (k % 3) * pa.pstride;
      const int gkc = k == 0 ? pa.gam0_count : int(G);
      const double* go = k <= 1 ? pa.gam0 : pa.part_g + ((k - 1) % 3) * pa.pstride;
      const int goc = k <= 1 ? pa.gam0_count : int(G);
      if (wid < 3) {
        const double* src = wid == 0 ? gk : wid == 1 ? pa.part_d : go;
        const int cnt = wid == 0 ? gkc : wid == 1 ? int(G) : goc;
        double a2 = 0.0;
#pragma unroll 4
        for (int i = lane; i < cnt; i += 32) a2 += __ldcg(src + i);
        v = warp_sum(a2);
        if (lane == 0) sc[wid] = v;
      }
      __syncthreads();
    }
    stamp(k, 7);
    const double g = sc[0], d = sc[1];
    double beta = 0.0, pap = d;
    if (k > 0) {
      beta = g / sc[2];
      pap = d - beta * g / alpha_old;
    }
    const double alpha = g / pap;
    if (blockIdx.x == 0 && threadIdx.x == 0) {
      if (pap == 0.0 || !isfinite(pap)) pa.flags[0] = 1;
      pa.alpha2[k & 1] = alpha;
      pa.flags[2] = k + 1;
    }
    alpha_old = alpha;
    double gacc = 0.0;
    for (int64_t j = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; j < pa.n; j += gstride) {
      const double rj0 = pa.r[j], wj = pa.w[j];
      const double pj = k > 0 ? rj0 + beta * pa.p[j] : rj0;
      const double sj = k > 0 ? wj + beta * pa.s[j] : wj;
      const double rj = rj0 - alpha * sj;
      pa.p[j] = pj;
      pa.s[j] = sj;
      pa.z[j] = pa.z[j] + alpha * pj;
      pa.r[j] = rj;
      gacc += rj * rj;
    }
    {
      const double ts = block_sum(gacc, red);
      if (threadIdx.x == 0) pa.part_g[((k + 1) % 3) * pa.pstride + blockIdx.x] = ts;
    }
    stamp(k, 5);
    grid_barrier(pa.gbar, ++gepoch);
    stamp(k, 6);
  }
  // leave together (peers may still be signalling this CTA's barriers)
  cluster_arrive();
  cluster_wait();
}

}  // namespace spmv
