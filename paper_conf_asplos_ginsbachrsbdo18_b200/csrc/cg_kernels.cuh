// cg_kernels.cuh -- fused vector kernels of textbook CG (NPB conj_grad
// [ext:NPB]).  One CG iteration is
//   K1  q = A p  and partial p.q              (k_spmv_vector<..., DOT=true>)
//   K2  d = p.q; alpha = rho/d; z += alpha p; r -= alpha q; partial r.r
//   K3  rho' = r.r; beta = rho'/rho; p = r + beta p
// Scalars never leave the device: every CTA of a consumer kernel sums the
// producer's per-CTA partials in the same fixed order (read_sum), so all CTAs
// (and all runs) see bit-identical alpha/beta.  In distributed mode the
// partials are first finalized into one value and NCCL-all-reduced; the
// consumers then read that single value (SumSrc.count == 1).
#pragma once
#include "common.cuh"

namespace spmv {

constexpr int CG_U = 4;  // elements per thread issued together in the vector kernels

struct CgState {
  int* flags;   // [0] breakdown (sticky), [1] converged, [2] iterations done
};

// z = 0, r = b, p = b, partial r.r
static __global__ void __launch_bounds__(256)
k_cg_init(int64_t n, const double* __restrict__ b, double* __restrict__ z,
          double* __restrict__ r, double* __restrict__ p, double* __restrict__ part_rr) {
  __shared__ double red[8];
  double acc = 0.0;
  for (int64_t j = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; j < n;
       j += int64_t(gridDim.x) * blockDim.x) {
    const double bj = b[j];
    z[j] = 0.0;
    r[j] = bj;
    p[j] = bj;
    acc += bj * bj;
  }
  const double t = block_sum(acc, red);
  if (threadIdx.x == 0) part_rr[blockIdx.x] = t;
}

// K2.  pq: p.q; rr_old: rho.  If tol_check, iterations stop once done.
static __global__ void __launch_bounds__(256)
k_cg_zr(int64_t n, SumSrc pq, SumSrc rr_old, const double* __restrict__ p,
        const double* __restrict__ q, double* __restrict__ z, double* __restrict__ r,
        double* __restrict__ part_rr_new, int* __restrict__ flags, P2PHook hk) {
  __shared__ double red[8];
  __shared__ double sc[2];
  if (flags[1]) return;  // converged (tol mode): no-op
  const int64_t stride = int64_t(gridDim.x) * blockDim.x;
  const int64_t jstart = int64_t(blockIdx.x) * blockDim.x + threadIdx.x;
  double pz[CG_U], pp[CG_U], pr[CG_U], pq_[CG_U];
  auto load_own = [&](int64_t j0) {  // z, p, r: complete before the SpMV passed its pdl_wait
#pragma unroll
    for (int u = 0; u < CG_U; ++u) {
      const int64_t j = j0 + u * stride;
      if (j < n) { pz[u] = z[j]; pp[u] = p[j]; pr[u] = r[j]; }
    }
  };
  auto load_q = [&](int64_t j0) {  // q = A p: the SpMV's output
#pragma unroll
    for (int u = 0; u < CG_U; ++u) {
      const int64_t j = j0 + u * stride;
      if (j < n) pq_[u] = q[j];
    }
  };
  if (jstart < n) load_own(jstart);
  pdl_wait();
  pdl_trigger();
  if (jstart < n) load_q(jstart);
  {  // both scalar sources at once, one warp each (bit-identical to read_sum)
    const int wid = threadIdx.x >> 5;
    double v = 0.0;
    if (wid == 0) v = warp_read_sum(pq);
    else if (wid == 1) v = warp_read_sum(rr_old);
    if (wid < 2 && (threadIdx.x & 31) == 0) sc[wid] = v;
    __syncthreads();
  }
  const double d = sc[0], rho = sc[1];
  if (d == 0.0 || !isfinite(d)) {
    if (blockIdx.x == 0 && threadIdx.x == 0) flags[0] = 1;
  }
  const double alpha = rho / d;
  double acc = 0.0;
  // CG_U consecutive-stride elements per thread with all loads issued first
  for (int64_t j0 = jstart; j0 < n; j0 += CG_U * stride) {
    if (j0 != jstart) {
      load_own(j0);
      load_q(j0);
    }
#pragma unroll
    for (int u = 0; u < CG_U; ++u) {
      const int64_t j = j0 + u * stride;
      if (j < n) {
        const double zj = pz[u] + alpha * pp[u];
        const double rj = pr[u] - alpha * pq_[u];
        z[j] = zj;
        r[j] = rj;
        acc += rj * rj;
      }
    }
  }
  const double t = block_sum(acc, red);
  if (threadIdx.x == 0) part_rr_new[blockIdx.x] = t;
  p2p_push_partials_last(hk, part_rr_new, gridDim.x);
}

// K3.  rr_new: rho', rr_old: rho.  tol > 0: after the update, mark converged
// once sqrt(rho') <= tol * ||b|| (rr_b: ||b||^2 source), recording `it`+1.
static __global__ void __launch_bounds__(256)
k_cg_p(int64_t n, SumSrc rr_new, SumSrc rr_old, const double* __restrict__ r,
       double* __restrict__ p, int* __restrict__ flags, double tol, SumSrc rr_b, int it, P2PHook hk,
       int64_t xoff) {
  __shared__ double s_b;
  __shared__ double sc[2];
  if (flags[1]) return;
  const int64_t stride = int64_t(gridDim.x) * blockDim.x;
  const int64_t jstart = int64_t(blockIdx.x) * blockDim.x + threadIdx.x;
  double pr[CG_U], pp[CG_U];
  auto load_p = [&](int64_t j0) {  // p: last written by the previous k_cg_p
#pragma unroll
    for (int u = 0; u < CG_U; ++u) {
      const int64_t j = j0 + u * stride;
      if (j < n) pp[u] = p[j];
    }
  };
  auto load_r = [&](int64_t j0) {  // r: k_cg_zr's output
#pragma unroll
    for (int u = 0; u < CG_U; ++u) {
      const int64_t j = j0 + u * stride;
      if (j < n) pr[u] = r[j];
    }
  };
  if (jstart < n) load_p(jstart);
  pdl_wait();
  pdl_trigger();
  if (jstart < n) load_r(jstart);
  {  // both scalar sources at once, one warp each (bit-identical to read_sum)
    const int wid = threadIdx.x >> 5;
    double v = 0.0;
    if (wid == 0) v = warp_read_sum(rr_new);
    else if (wid == 1) v = warp_read_sum(rr_old);
    if (wid < 2 && (threadIdx.x & 31) == 0) sc[wid] = v;
    __syncthreads();
  }
  const double rho1 = sc[0], rho0 = sc[1];
  const double beta = rho1 / rho0;
  for (int64_t j0 = jstart; j0 < n; j0 += CG_U * stride) {
    if (j0 != jstart) {
      load_p(j0);
      load_r(j0);
    }
#pragma unroll
    for (int u = 0; u < CG_U; ++u) {
      const int64_t j = j0 + u * stride;
      if (j < n) {
        const double pj = pr[u] + beta * pp[u];
        p[j] = pj;
        if (hk.enabled)  // fused all-gather: the slice goes straight into every peer's xpad
          for (int q = 0; q < hk.c.P; ++q)
            if (q != hk.c.me && p2p_sends(hk.c, q, j)) reinterpret_cast<double*>(hk.c.peer[q])[xoff + j] = pj;
      }
    }
  }
  if (hk.enabled) {
    // the CTA's peer stores happen-before thread 0's acq_rel ticket (bar.sync);
    // the last CTA fences at system scope and publishes (p2p_signal)
    __syncthreads();
    if (threadIdx.x == 0 && ticket_acq_rel_gpu(hk.c.ticket) == int(gridDim.x) - 1) {
      *hk.c.ticket = 0;
      p2p_signal(hk.c, P2P_XSLOT);
    }
  }
  if (tol > 0.0) {
    const double bb = read_sum(rr_b, &s_b);
    if (blockIdx.x == 0 && threadIdx.x == 0) {
      flags[2] = it + 1;
      if (sqrt(rho1) <= tol * sqrt(bb)) flags[1] = 1;
    }
  } else if (blockIdx.x == 0 && threadIdx.x == 0) {
    flags[2] = it + 1;
  }
}

// ------------------------------------------------------------ NEXT-1
// Single-reduction CG (Chronopoulos & Gear).  In exact
// arithmetic it produces the iterates z_k of NPB conj_grad, with one
// reduction point per iteration instead of two.  Iteration k:
//   K1  w = A r  and partial d = w.r        (the SpMV with x = r, DOT fused)
//   K2  (this kernel)  g = r.r (from the previous K2), d:
//        k == 0: beta = 0, alpha = g/d
//        else  : beta = g/g_old, alpha = g/(d - beta*g/alpha_old)
//       p = r + beta p;  s = w + beta s;  z += alpha p;  r -= alpha s;
//       partial r.r of the new r.
// (s = A p is carried by recurrence, so p.Ap = d - beta*g/alpha_old.)
// alpha is handed to the next K2 through alpha2[k & 1] (written by CTA 0;
// every CTA computes the same value from the same partials in the same
// order).  tol > 0: the check sqrt(g) <= tol*||b|| is made on entry, before
// the update, so the solve stops with the same z_k as the textbook loop.
static __global__ void __launch_bounds__(256)
k_cgcg(int64_t n, int k, SumSrc gam, SumSrc gam_old, SumSrc del, double* __restrict__ alpha2,
       double* __restrict__ p, double* __restrict__ sv, const double* __restrict__ w,
       double* __restrict__ z, double* __restrict__ r, double* __restrict__ part_rr_new,
       int* __restrict__ flags, double tol, SumSrc rr_b, P2PHook hk, int64_t xoff) {
  __shared__ double red[8];
  __shared__ double sc[4];
  if (flags[1]) return;  // converged (tol mode): no-op
  const int64_t stride = int64_t(gridDim.x) * blockDim.x;
  const int64_t jstart = int64_t(blockIdx.x) * blockDim.x + threadIdx.x;
  double pr[CG_U], pw[CG_U], pp[CG_U], ps[CG_U], pz[CG_U];
  auto load_own = [&](int64_t j0) {  // r, z, p, s: written only by the previous update
#pragma unroll
    for (int u = 0; u < CG_U; ++u) {
      const int64_t j = j0 + u * stride;
      if (j < n) {
        pr[u] = r[j]; pz[u] = z[j];
        if (k > 0) { pp[u] = p[j]; ps[u] = sv[j]; }
      }
    }
  };
  auto load_w = [&](int64_t j0) {  // w: the SpMV's output
#pragma unroll
    for (int u = 0; u < CG_U; ++u) {
      const int64_t j = j0 + u * stride;
      if (j < n) pw[u] = w[j];
    }
  };
  // the first batch of vector loads does not depend on the scalars: issue it,
  // then read the (up to four) scalar sources concurrently, one warp each.
  // Under PDL the SpMV may still be running: r, z, p, s (complete since the
  // SpMV passed its own pdl_wait) are loaded before pdl_wait, w after it.
  if (jstart < n) load_own(jstart);
  pdl_wait();
  pdl_trigger();
  if (jstart < n) load_w(jstart);
  {
    const int wid = threadIdx.x >> 5, lane = threadIdx.x & 31;
    double v = 0.0;
    if (wid == 0) v = warp_read_sum(gam);
    else if (wid == 1) v = warp_read_sum(del);
    else if (wid == 2 && k > 0) v = warp_read_sum(gam_old);
    else if (wid == 3 && tol > 0.0) v = warp_read_sum(rr_b);
    if (wid < 4 && lane == 0) sc[wid] = v;
    __syncthreads();
  }
  const double g = sc[0], d = sc[1];
  if (tol > 0.0 && sqrt(g) <= tol * sqrt(sc[3])) {
    if (blockIdx.x == 0 && threadIdx.x == 0) flags[1] = 1;
    return;
  }
  double beta = 0.0, alpha, pap;
  if (k == 0) {
    pap = d;
  } else {
    const double go = sc[2];
    beta = g / go;
    pap = d - beta * g / __ldcg(alpha2 + ((k - 1) & 1));
  }
  alpha = g / pap;
  if (blockIdx.x == 0 && threadIdx.x == 0) {
    if (pap == 0.0 || !isfinite(pap)) flags[0] = 1;
    alpha2[k & 1] = alpha;
    flags[2] = k + 1;
  }
  double acc = 0.0;
  for (int64_t j0 = jstart; j0 < n; j0 += CG_U * stride) {
    if (j0 != jstart) {
      load_own(j0);
      load_w(j0);
    }
#pragma unroll
    for (int u = 0; u < CG_U; ++u) {
      const int64_t j = j0 + u * stride;
      if (j < n) {
        const double pj = k > 0 ? pr[u] + beta * pp[u] : pr[u];
        const double sj = k > 0 ? pw[u] + beta * ps[u] : pw[u];
        const double rj = pr[u] - alpha * sj;
        p[j] = pj;
        sv[j] = sj;
        z[j] = pz[u] + alpha * pj;
        r[j] = rj;
        acc += rj * rj;
        if (hk.enabled)  // fused all-gather of the next SpMV's x (= r)
          for (int q = 0; q < hk.c.P; ++q)
            if (q != hk.c.me && p2p_sends(hk.c, q, j)) reinterpret_cast<double*>(hk.c.peer[q])[xoff + j] = rj;
      }
    }
  }
  const double t = block_sum(acc, red);
  if (threadIdx.x == 0) part_rr_new[blockIdx.x] = t;
  if (hk.enabled && hk.push_slot >= 0) {
    // one ticket publishes both the r.r partials and this rank's x slice (the
    // peer stores above precede every CTA's ticket like the partials do)
    p2p_push_partials_last(hk, part_rr_new, gridDim.x, P2P_XSLOT);
  } else if (hk.enabled) {
    // x only: its own ticket (the next u64 slot)
    int* tk2 = hk.c.ticket + 2;
    __syncthreads();
    if (threadIdx.x == 0 && ticket_acq_rel_gpu(tk2) == int(gridDim.x) - 1) {
      *tk2 = 0;
      p2p_signal(hk.c, P2P_XSLOT);
    }
  }
}

// Residual / NPB norms: partials of ||b - Az||^2 and (NPB) x.z, z.z.
// b is the right-hand side (NPB: x), az = A z.
template <bool NPB>
__global__ void __launch_bounds__(256)
k_cg_resid(int64_t n, const double* __restrict__ b, const double* __restrict__ az,
           const double* __restrict__ z, double* __restrict__ part_res,
           double* __restrict__ part_xz, double* __restrict__ part_zz) {
  __shared__ double red[8];
  double a0 = 0.0, a1 = 0.0, a2 = 0.0;
  for (int64_t j = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; j < n;
       j += int64_t(gridDim.x) * blockDim.x) {
    const double bj = b[j];
    const double d = bj - az[j];
    a0 += d * d;
    if (NPB) {
      const double zj = z[j];
      a1 += bj * zj;
      a2 += zj * zj;
    }
  }
  double t = block_sum(a0, red);
  if (threadIdx.x == 0) part_res[blockIdx.x] = t;
  if (NPB) {
    t = block_sum(a1, red);
    if (threadIdx.x == 0) part_xz[blockIdx.x] = t;
    t = block_sum(a2, red);
    if (threadIdx.x == 0) part_zz[blockIdx.x] = t;
  }
}

// NAS outer iteration, split so the new x exists before the residual SpMV
// (its host copy then overlaps the residual): partials of x.z and z.z (the
// same accumulation and block sums as k_cg_resid<true>), then zeta and
// x_new = z / ||z|| into a separate buffer (the residual still reads the old x).
static __global__ void __launch_bounds__(256)
k_npb_xz(int64_t n, const double* __restrict__ x, const double* __restrict__ z, double* __restrict__ part_xz,
         double* __restrict__ part_zz) {
  __shared__ double red[8];
  double a1 = 0.0, a2 = 0.0;
  for (int64_t j = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; j < n; j += int64_t(gridDim.x) * blockDim.x) {
    const double zj = z[j];
    a1 += x[j] * zj;
    a2 += zj * zj;
  }
  double t = block_sum(a1, red);
  if (threadIdx.x == 0) part_xz[blockIdx.x] = t;
  t = block_sum(a2, red);
  if (threadIdx.x == 0) part_zz[blockIdx.x] = t;
}

static __global__ void __launch_bounds__(256)
k_npb_xnew(int64_t n, SumSrc xz, SumSrc zz, const double* __restrict__ z, double* __restrict__ xn, double shift,
           double* __restrict__ out2) {
  __shared__ double s1, s2;
  const double nt1 = read_sum(xz, &s1);
  double nt2 = read_sum(zz, &s2);
  nt2 = 1.0 / sqrt(nt2);
  for (int64_t j = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; j < n; j += int64_t(gridDim.x) * blockDim.x)
    xn[j] = nt2 * z[j];
  if (blockIdx.x == 0 && threadIdx.x == 0) out2[0] = shift + 1.0 / nt1;
}

// cg_solve tail: rnorm = sqrt(sum).
static __global__ void k_finish_norm(SumSrc res, double* out) {
  __shared__ double s0;
  const double rr = read_sum(res, &s0);
  if (threadIdx.x == 0) *out = sqrt(rr);
}

// Per-CTA partials of w.y (used after SpMV kernels without a fused dot).
static __global__ void __launch_bounds__(256)
k_dot_partials(int64_t n, const double* __restrict__ w, const double* __restrict__ y, double* __restrict__ part,
               P2PHook hk) {
  __shared__ double red[8];
  double acc = 0.0;
  for (int64_t j = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; j < n; j += int64_t(gridDim.x) * blockDim.x)
    acc += w[j] * y[j];
  const double t = block_sum(acc, red);
  if (threadIdx.x == 0) part[blockIdx.x] = t;
  p2p_push_partials_last(hk, part, gridDim.x);
}

// Distributed mode: sum `count` partials into one value (then all-reduced).
static __global__ void k_finalize(SumSrc s, double* out) {
  __shared__ double s0;
  const double v = read_sum(s, &s0);
  if (threadIdx.x == 0) *out = v;
}

}  // namespace spmv
