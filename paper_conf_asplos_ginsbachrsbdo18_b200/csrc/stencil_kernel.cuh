// stencil_kernel.cuh -- matrix-free 27-point stencil:
// the paper's Stencil idiom (Fig. 13: a loop nest whose
// store is a kernel function of reads at constant offsets), with the kernel
// function a weighted sum over the 3x3x3 neighbourhood and Dirichlet
// truncation (reading R19): for every grid point p = x + nx*(y + ny*z)
//     y[p] = alpha * sum_{d in {-1,0,1}^3, p+d inside} w[d] * x[p+d] + beta * y[p]
// It is the operator whose CSR form is BJ.cfg[4]; with general weights the
// result equals spmv_csr on the same CSR matrix (same terms, same order);
// with R19's weights (26, -1) the separable box-sum form below is used.
//
// 2.5-D blocking: a CTA owns a TX x TY tile of (x, y) and marches a range of
// z planes.  Each plane (+ a one-point halo) is staged once in shared memory
// (double-buffered, the next plane's loads in flight while the current one is
// consumed); a plane zp contributes its 3x3 in-plane neighbourhood to three
// outputs held in registers: z = zp+1 (weights of dz = -1), z = zp (dz = 0)
// and z = zp-1 (dz = +1), after which output zp-1 is complete and stored.
// Every output therefore receives its 27 terms in ascending linear index
// (dz, dy, dx), exactly the CSR row order (points outside the grid are staged
// as 0 and add an exact zero), accumulated with FMA like the CSR kernels
// (reading R11).  A bit-exact variant (separate round-to-nearest mul and add,
// as the oracle's -ffp-contract=off loop) measured 108 us on 256^3: 54 fp64
// operations per point make it fp64-ALU-bound (~49 us of DMUL/DADD issue at
// 64 per clock per SM) before memory; the FMA form halves that.  HBM traffic:
// x once (+2 halo planes per z range, mostly L2 hits) and y once:
// 2*sizeof(T) bytes per point.
// Measured on 256^3 fp64 (tools/run_stencil_variants.sh): 1 point per thread
// 86 us whatever the prefetch depth (1-4 planes in flight: not latency-bound;
// ncu: issue-bound, ~130 instructions per point incl. the 27 weights held in
// uniform registers); 2 rows per thread 76-78 us (shared loads and loop
// overhead amortised), 4 rows 80 us (register-limited occupancy).
#pragma once
#include <cuda.h>  // CUtensorMap (the TMA form of k_stencil27_box2)
#include "common.cuh"
#include "xstat_kernel.cuh"  // smem_u32 / mbarrier helpers

namespace spmv {

#ifndef ST_RY_DEF
#define ST_RY_DEF 2
#endif
constexpr int ST_RY = ST_RY_DEF;  // outputs per thread along y (register blocking: shared loads and
                                  // loop overhead amortised over ST_RY points)
constexpr int ST_TX = 32, ST_NT = 256, ST_TY = (ST_NT / ST_TX) * ST_RY;
constexpr int ST_PX = ST_TX + 2, ST_PY = ST_TY + 2, ST_PN = ST_PX * ST_PY;
constexpr int ST_LPT = (ST_PN + ST_NT - 1) / ST_NT;  // plane elements staged per thread
#ifndef ST_PF_DEF
#define ST_PF_DEF 1
#endif
constexpr int ST_PF = ST_PF_DEF;  // planes whose loads are in flight (register ring)
#ifndef ST_ASYNC_DEF
#define ST_ASYNC_DEF 1
#endif
#ifndef ST_NS_DEF
#define ST_NS_DEF 3
#endif
// ST_ASYNC: planes are copied global -> shared with cp.async (zero-fill for
// the halo outside the grid) into a ring of ST_NS plane buffers, so ST_NS-1
// planes are in flight per CTA without holding them in registers
constexpr bool ST_ASYNC = ST_ASYNC_DEF != 0;
constexpr int ST_NS = ST_NS_DEF;

template <int BYTES>
__device__ __forceinline__ void cp_async_zfill(void* sdst, const void* gsrc, int src_bytes) {
  const uint32_t d = static_cast<uint32_t>(__cvta_generic_to_shared(sdst));
  asm volatile("cp.async.ca.shared.global [%0], [%1], %2, %3;\n" ::"r"(d), "l"(gsrc), "n"(BYTES), "r"(src_bytes)
               : "memory");
}
__device__ __forceinline__ void cp_async_commit() { asm volatile("cp.async.commit_group;\n" ::: "memory"); }
template <int N>
__device__ __forceinline__ void cp_async_wait() { asm volatile("cp.async.wait_group %0;\n" ::"n"(N) : "memory"); }

struct StencilArgs {
  int64_t nx, ny, nz;
  int zchunk;          // planes per CTA (blockIdx.z)
  double w[27];        // w[(dz+1)*9 + (dy+1)*3 + (dx+1)]
  const void* x;
  void* y;
  double alpha, beta;
  double wd, wn;       // BOX: w[13] - wn and the common neighbour weight wn
};

// BOX = every one of the 26 neighbour weights equals wn (R19's Laplacian:
// wn = -1, centre 26).  Then  y = alpha*((w_c - wn)*x_c + wn*B)  with B the
// 3x3x3 box sum, which is separable: per plane, 3-point row sums then 3-row
// column sums (the in-plane 3x3 box, 4 adds per point for ST_RY = 2), and
// the three plane boxes of an output added in z.  ~11 fp64 operations per
// point instead of 27 FMAs; a different summation order than the CSR row,
// within reading R11's per-row bound (the bound holds |x_j| of all 27 terms).
#ifndef ST_MINB_DEF
#define ST_MINB_DEF 1
#endif
template <typename T, bool BOX>
__global__ void __launch_bounds__(ST_NT, ST_MINB_DEF)
k_stencil27(StencilArgs a) {
  __shared__ __align__(16) T pl[ST_ASYNC ? ST_NS : 2][ST_PN];
  const T* __restrict__ x = static_cast<const T*>(a.x);
  T* __restrict__ y = static_cast<T*>(a.y);
  const int tx = threadIdx.x % ST_TX, ty = (threadIdx.x / ST_TX) * ST_RY;  // first of ST_RY rows
  const int64_t nx = a.nx, ny = a.ny, nz = a.nz, nxy = nx * ny;
  const int64_t x0 = int64_t(blockIdx.x) * ST_TX, y0 = int64_t(blockIdx.y) * ST_TY;
  const int64_t z0 = int64_t(blockIdx.z) * a.zchunk;
  const int64_t z1 = cmin64(nz, z0 + a.zchunk);
  const int64_t gx = x0 + tx, gy = y0 + ty;

  // staging: element e of the haloed plane -> (lx, ly); global offset inside a plane or -1
  int64_t off[ST_LPT];
#pragma unroll
  for (int u = 0; u < ST_LPT; ++u) {
    const int e = threadIdx.x + u * ST_NT;
    off[u] = -1;
    if (e < ST_PN) {
      const int64_t X = x0 + (e % ST_PX) - 1, Y = y0 + (e / ST_PX) - 1;
      if (X >= 0 && X < nx && Y >= 0 && Y < ny) off[u] = X + nx * Y;
    }
  }
  // register ring: v[k] holds plane zp+1+k while plane zp is consumed
  T v[ST_PF][ST_LPT];
  auto fetch = [&](int64_t zp, T* dst) {
    const bool zin = zp >= 0 && zp < nz && zp <= z1;
#pragma unroll
    for (int u = 0; u < ST_LPT; ++u) dst[u] = (zin && off[u] >= 0) ? __ldg(x + zp * nxy + off[u]) : T(0);
  };
  auto stash = [&](int buf, const T* src) {
#pragma unroll
    for (int u = 0; u < ST_LPT; ++u) {
      const int e = threadIdx.x + u * ST_NT;
      if (e < ST_PN) pl[buf][e] = src[u];
    }
  };

  const double alpha = a.alpha, beta = a.beta;
  double acc_m[ST_RY], acc_c[ST_RY], acc_p[ST_RY];  // outputs zp-1, zp, zp+1 of each row
  double cen_m[ST_RY];                               // BOX: centre x of output zp-1
#pragma unroll
  for (int r = 0; r < ST_RY; ++r) acc_m[r] = acc_c[r] = acc_p[r] = cen_m[r] = 0.0;
  // cp.async staging of plane zp into ring slot `slot` (always one commit group)
  auto issue = [&](int64_t zp, int slot) {
    const bool zin = zp >= 0 && zp < nz && zp <= z1;
#pragma unroll
    for (int u = 0; u < ST_LPT; ++u) {
      const int e = threadIdx.x + u * ST_NT;
      if (e < ST_PN) {
        const bool ok = zin && off[u] >= 0;
        cp_async_zfill<sizeof(T)>(&pl[slot][e], ok ? x + zp * nxy + off[u] : x, ok ? int(sizeof(T)) : 0);
      }
    }
    cp_async_commit();
  };
  int cur = 0;
  if (ST_ASYNC) {
#pragma unroll
    for (int k = 0; k < ST_NS - 1; ++k) issue(z0 - 1 + k, k);
  } else {
    {
      T v0[ST_LPT];
      fetch(z0 - 1, v0);
      stash(0, v0);
    }
#pragma unroll
    for (int k = 0; k < ST_PF; ++k) fetch(z0 + k, v[k]);
    __syncthreads();
  }
  for (int64_t zp = z0 - 1; zp <= z1; ++zp) {
    T vf[ST_LPT];
    if (ST_ASYNC) {
      // slot (cur + NS - 1) % NS was consumed in the previous iteration (barrier at its end)
      issue(zp + ST_NS - 1, (cur + ST_NS - 1) % ST_NS);
      cp_async_wait<ST_NS - 1>();  // plane zp has landed (the newest NS-1 groups may be in flight)
      __syncthreads();
    } else {
      fetch(zp + 1 + ST_PF, vf);  // ST_PF planes ahead (zeros past z1: never stashed)
    }
    const T* P = pl[cur];
    if (BOX) {
      double rs[ST_RY + 2];  // 3-point row sums of plane rows ty-1 .. ty+ST_RY
#pragma unroll
      for (int sy = 0; sy < ST_RY + 2; ++sy) {
        const T* q = P + (ty + sy) * ST_PX + tx;
        rs[sy] = (double(q[0]) + double(q[1])) + double(q[2]);
      }
#pragma unroll
      for (int r = 0; r < ST_RY; ++r) {
        const double b2 = (rs[r] + rs[r + 1]) + rs[r + 2];  // in-plane 3x3 box of output row r
        acc_p[r] += b2;
        acc_c[r] += b2;
        acc_m[r] += b2;
      }
    } else {
#pragma unroll
      for (int sy = 0; sy < ST_RY + 2; ++sy)  // plane rows ty-1 .. ty+ST_RY
#pragma unroll
        for (int dx = 0; dx < 3; ++dx) {
          const double xv = double(P[(ty + sy) * ST_PX + tx + dx]);
#pragma unroll
          for (int r = 0; r < ST_RY; ++r) {
            const int dy = sy - r;  // row offset + 1 of this value for output row r
            if (dy < 0 || dy > 2) continue;
            acc_p[r] = fma(a.w[0 * 9 + dy * 3 + dx], xv, acc_p[r]);  // output zp+1, dz = -1
            acc_c[r] = fma(a.w[1 * 9 + dy * 3 + dx], xv, acc_c[r]);  // output zp,   dz =  0
            acc_m[r] = fma(a.w[2 * 9 + dy * 3 + dx], xv, acc_m[r]);  // output zp-1, dz = +1
          }
        }
    }
    const int64_t zo = zp - 1;  // complete now
    if (gx < nx && zo >= z0 && zo < z1) {
#pragma unroll
      for (int r = 0; r < ST_RY; ++r) {
        if (gy + r >= ny) continue;
        const int64_t p = gx + nx * (gy + r) + nxy * zo;
        double res;
        if (BOX) res = alpha * fma(a.wd, cen_m[r], a.wn * acc_m[r]);  // (w_c - wn) x_c + wn B
        else res = alpha * acc_m[r];
        if (beta != 0.0) res += beta * double(y[p]);
        y[p] = T(res);
      }
    }
    if (BOX) {
#pragma unroll
      for (int r = 0; r < ST_RY; ++r)  // centre of plane zp: the output written next iteration
        cen_m[r] = double(P[(ty + 1 + r) * ST_PX + tx + 1]);
    }
#pragma unroll
    for (int r = 0; r < ST_RY; ++r) {
      acc_m[r] = acc_c[r];
      acc_c[r] = acc_p[r];
      acc_p[r] = 0.0;
    }
    if (ST_ASYNC) {
      __syncthreads();  // every thread is done with slot cur before it is refilled
      cur = (cur + 1) % ST_NS;
    } else {
      if (zp + 1 <= z1) stash(cur ^ 1, v[0]);
      __syncthreads();
      cur ^= 1;
#pragma unroll
      for (int k = 0; k + 1 < ST_PF; ++k)
#pragma unroll
        for (int u = 0; u < ST_LPT; ++u) v[k][u] = v[k + 1][u];
#pragma unroll
      for (int u = 0; u < ST_LPT; ++u) v[ST_PF - 1][u] = vf[u];
    }
  }
  if (ST_ASYNC) cp_async_wait<0>();  // no copy may outlive the CTA's shared memory
}

}  // namespace spmv

namespace spmv {

// ---------------------------------------------------------------------------
// BOX form with two adjacent columns per thread (k_stencil27_box2): the
// x-direction row sums of columns 2c and 2c+1 share the plane values
// x[2c-1..2c+2], read as two 16-B (fp64) / 8-B (fp32) shared loads instead
// of six scalar ones, and the two centre values come out of the same loads.
// Same staging (cp.async ring, zero-filled halo), same z marching and
// summation order as the BOX form of k_stencil27.
constexpr int SB_CX = 32;                  // column pairs per CTA row (warp)
constexpr int SB_TX = 2 * SB_CX;           // 64 columns per tile
#ifndef SB_RY_DEF
#define SB_RY_DEF 2
#endif
constexpr int SB_NT = 256, SB_RY = SB_RY_DEF;
constexpr int SB_TY = (SB_NT / SB_CX) * SB_RY;  // 16 rows per tile
constexpr int SB_PY = SB_TY + 2;  // 18 staged rows

template <typename T> struct V2;
template <> struct V2<double> { using t = double2; };
template <> struct V2<float> { using t = float2; };

// TMA: the plane tile (PX x 18, one-point halo) is one cp.async.bulk.tensor.3d
// box at (x0-1, y0-1, zp) issued by one thread; the tensor map's out-of-bound
// fill supplies the zero halo outside the grid (nx, ny); planes zp < 0 or
// zp >= nz are zero-filled by the CTA's threads instead (no copy issued).  The
// box's inner extent must be a multiple of 16 B: 66 fp64 (528 B), 68 fp32,
// and so must its innermost start coordinate (measured on this B200: an
// origin at x = -1 fp64 traps with an illegal instruction, x = -2 zero-fills;
// profiles/r01q_tma3d_origin_check.txt).  The TMA tiles are therefore shifted
// left by SHIFT columns (output columns [64 bx - SHIFT, 64 bx + 64 - SHIFT),
// staged from 64 bx - SHIFT - 1, a multiple of 16 B), which keeps each
// thread's 4 staged values one aligned pair of vector loads.
// ST_TMA_SHFL=1 (measured slower, not the default: 256^3 65.5 vs 61.4 us for the
// shifted tiles, profiles/r01q_stencil_tma_shfl_*): no shift; the box starts HL = 16 B / sizeof(T) columns
// left of the tile (PX = 64 + 2 HL), each thread loads its aligned pair
// x[2c], x[2c+1] as one vector and takes x[2c-1], x[2c+2] from its neighbour
// lanes (warp shuffles; lanes 0 and 31 read the halo column from shared).
#ifndef ST_TMA_SHFL_DEF
#define ST_TMA_SHFL_DEF 0
#endif
constexpr bool ST_TMA_SHFL = ST_TMA_SHFL_DEF != 0;
template <typename T, bool TMA> struct SBL {
  static constexpr bool SHFL = TMA && ST_TMA_SHFL;
  static constexpr int HL = SHFL ? 16 / int(sizeof(T)) : 1;  // staged columns left of the tile
  static constexpr int SHIFT = (TMA && !SHFL) ? (sizeof(T) == 8 ? 1 : 3) : 0;
  static constexpr int PX = SHFL ? SB_TX + 2 * HL : (TMA && sizeof(T) == 4) ? SB_TX + 4 : SB_TX + 2;  // row pitch
  static constexpr int PN = PX * SB_PY;
  static constexpr int SLOT = TMA ? ((PN * int(sizeof(T)) + 127) / 128) * 128 / int(sizeof(T)) : PN;
  static constexpr int LPT = (PN + SB_NT - 1) / SB_NT;
};

__device__ __forceinline__ void tma_load_3d(void* dst, uint64_t tm, int c0, int c1, int c2, uint64_t* bar) {
  asm volatile(
      "cp.async.bulk.tensor.3d.shared::cluster.global.tile.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3, %4}], "
      "[%5];\n" ::"r"(smem_u32(dst)),
      "l"(tm), "r"(c0), "r"(c1), "r"(c2), "r"(smem_u32(bar))
      : "memory");
}

template <typename T, bool TMA>
__global__ void __launch_bounds__(SB_NT)
k_stencil27_box2(StencilArgs a, const __grid_constant__ CUtensorMap tm) {
  using V = typename V2<T>::t;
  using L = SBL<T, TMA>;
  constexpr int SB_PX = L::PX, SB_PN = L::PN, SB_LPT = L::LPT;
  __shared__ __align__(128) T pl[ST_NS][L::SLOT];
  __shared__ __align__(8) uint64_t bar[ST_NS];
  const T* __restrict__ x = static_cast<const T*>(a.x);
  T* __restrict__ y = static_cast<T*>(a.y);
  const int cx = threadIdx.x % SB_CX, ty = (threadIdx.x / SB_CX) * SB_RY;
  const int64_t nx = a.nx, ny = a.ny, nz = a.nz, nxy = nx * ny;
  const int64_t x0 = int64_t(blockIdx.x) * SB_TX - L::SHIFT, y0 = int64_t(blockIdx.y) * SB_TY;
  const int64_t z0 = int64_t(blockIdx.z) * a.zchunk;
  const int64_t z1 = cmin64(nz, z0 + a.zchunk);
  const int64_t gx = x0 + 2 * cx, gy = y0 + ty;

  int off[TMA ? 1 : SB_LPT];  // in-plane offsets (the host guarantees nx*ny < 2^31); -1 = outside
  uint32_t phase = 0;         // TMA: parity bit of each slot's mbarrier
  // generic address of the __grid_constant__ parameter, taken here: a lambda capturing the parameter
  // by reference would see a local copy, which the TMA unit cannot read (illegal instruction)
  const uint64_t tmap = reinterpret_cast<uint64_t>(&tm);
  if (TMA) {
    if (threadIdx.x == 0) {
#pragma unroll
      for (int k = 0; k < ST_NS; ++k) mbar_init(&bar[k], 1);
      asm volatile("fence.mbarrier_init.release.cluster;\n" ::: "memory");
    }
  } else {
#pragma unroll
    for (int u = 0; u < SB_LPT; ++u) {
      const int e = threadIdx.x + u * SB_NT;
      off[u] = -1;
      if (e < SB_PN) {
        const int64_t X = x0 + (e % SB_PX) - 1, Y = y0 + (e / SB_PX) - 1;
        if (X >= 0 && X < nx && Y >= 0 && Y < ny) off[u] = int(X + nx * Y);
      }
    }
  }
  auto issue = [&](int64_t zp, int slot) {
    const bool zin = zp >= 0 && zp < nz && zp <= z1;
    if constexpr (TMA) {
      if (zp > z1) return;  // never consumed
      if (zin) {
        if (threadIdx.x == 0) {
          asm volatile("fence.proxy.async.shared::cta;\n" ::: "memory");  // after generic zero fills / reads
          mbar_expect_tx(&bar[slot], uint32_t(SB_PN * sizeof(T)));
          tma_load_3d(&pl[slot][0], tmap, int(x0 - L::HL), int(y0 - 1), int(zp), &bar[slot]);
        }
      } else {
        for (int e = threadIdx.x; e < SB_PN; e += SB_NT) pl[slot][e] = T(0);
      }
    } else {
#pragma unroll
      for (int u = 0; u < SB_LPT; ++u) {
        const int e = threadIdx.x + u * SB_NT;
        if (e < SB_PN) {
          const bool ok = zin && off[u] >= 0;
          cp_async_zfill<sizeof(T)>(&pl[slot][e], ok ? x + zp * nxy + off[u] : x, ok ? int(sizeof(T)) : 0);
        }
      }
      cp_async_commit();
    }
  };
  const double alpha = a.alpha, beta = a.beta;
  double acc_m[SB_RY][2], acc_c[SB_RY][2], acc_p[SB_RY][2], cen_m[SB_RY][2];
#pragma unroll
  for (int r = 0; r < SB_RY; ++r)
#pragma unroll
    for (int c = 0; c < 2; ++c) acc_m[r][c] = acc_c[r][c] = acc_p[r][c] = cen_m[r][c] = 0.0;
  if (TMA) __syncthreads();  // barriers initialised before the first copy
#pragma unroll
  for (int k = 0; k < ST_NS - 1; ++k) issue(z0 - 1 + k, k);
  if (TMA) __syncthreads();  // zero-filled prologue planes visible
  int cur = 0;
  for (int64_t zp = z0 - 1; zp <= z1; ++zp) {
    issue(zp + ST_NS - 1, (cur + ST_NS - 1) % ST_NS);
    if (TMA) {
      if (zp >= 0 && zp < nz) {  // a copied plane (zero-filled ones were made visible by the last barrier)
        mbar_wait(&bar[cur], (phase >> cur) & 1u, 7);
        phase ^= 1u << cur;
      }
    } else {
      cp_async_wait<ST_NS - 1>();
      __syncthreads();
    }
    const T* P = pl[cur];
    double rs0[SB_RY + 2], rs1[SB_RY + 2], cc0[SB_RY], cc1[SB_RY];
#pragma unroll
    for (int sy = 0; sy < SB_RY + 2; ++sy) {
      double e0, e1, e2, e3;  // x[2c-1], x[2c], x[2c+1], x[2c+2] of plane row ty+sy-1
      if constexpr (L::SHFL) {
        const T* row = P + (ty + sy) * SB_PX + L::HL;  // row[X - x0]
        const V mid = *reinterpret_cast<const V*>(row + 2 * cx);
        T l = __shfl_up_sync(0xffffffffu, mid.y, 1), r = __shfl_down_sync(0xffffffffu, mid.x, 1);
        if (cx == 0) l = row[-1];
        if (cx == SB_CX - 1) r = row[SB_TX];
        e0 = double(l); e1 = double(mid.x); e2 = double(mid.y); e3 = double(r);
      } else {
        const V* q = reinterpret_cast<const V*>(P + (ty + sy) * SB_PX + 2 * cx);
        const V lo = q[0], hi = q[1];
        e0 = double(lo.x); e1 = double(lo.y); e2 = double(hi.x); e3 = double(hi.y);
      }
      rs0[sy] = (e0 + e1) + e2;
      rs1[sy] = (e1 + e2) + e3;
      if (sy >= 1 && sy <= SB_RY) {
        cc0[sy - 1] = e1;
        cc1[sy - 1] = e2;
      }
    }
#pragma unroll
    for (int r = 0; r < SB_RY; ++r) {
      const double b0 = (rs0[r] + rs0[r + 1]) + rs0[r + 2];
      const double b1 = (rs1[r] + rs1[r + 1]) + rs1[r + 2];
      acc_p[r][0] += b0; acc_c[r][0] += b0; acc_m[r][0] += b0;
      acc_p[r][1] += b1; acc_c[r][1] += b1; acc_m[r][1] += b1;
    }
    const int64_t zo = zp - 1;
    if (zo >= z0 && zo < z1) {
#pragma unroll
      for (int r = 0; r < SB_RY; ++r) {
        if (gy + r >= ny) continue;
#pragma unroll
        for (int c = 0; c < 2; ++c) {
          if (gx + c >= nx || gx + c < 0) continue;
          const int64_t p = gx + c + nx * (gy + r) + nxy * zo;
          double res = alpha * fma(a.wd, cen_m[r][c], a.wn * acc_m[r][c]);
          if (beta != 0.0) res += beta * double(y[p]);
          y[p] = T(res);
        }
      }
    }
#pragma unroll
    for (int r = 0; r < SB_RY; ++r) {
      cen_m[r][0] = cc0[r];
      cen_m[r][1] = cc1[r];
#pragma unroll
      for (int c = 0; c < 2; ++c) {
        acc_m[r][c] = acc_c[r][c];
        acc_c[r][c] = acc_p[r][c];
        acc_p[r][c] = 0.0;
      }
    }
    __syncthreads();
    cur = (cur + 1) % ST_NS;
  }
  if (!TMA) cp_async_wait<0>();
}

}  // namespace spmv
