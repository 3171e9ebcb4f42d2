// cg_driver.cu -- CG (textbook NPB conj_grad, and the
// single-reduction CG of NEXT-1) and the NAS outer iteration (a4), enqueued
// without host round trips and replayed as a CUDA graph.  Kernels in
// cg_kernels.cuh; the SpMV through run_spmv (plans.cu); exchanges through
// dist.cu.
#include "abi_common.h"
#include "cg_kernels.cuh"

// ------------------------------------------------------------------ CG
static spmv_status cg_alloc(spmv_csr_s* h) {
  if (h->z) return SPMV_OK;
  const size_t nb = sizeof(double) * (size_t)std::max<int64_t>(h->m_loc, 1);
  const size_t pb = sizeof(double) * (size_t)std::max<int64_t>(std::max(std::max(h->grid, h->grid_vec), h->vgrid), 1);
  {
    // z | r | q | s | p_single: one allocation (see cgws in abi_common.h)
    const size_t nba = (nb + 255) & ~size_t(255);
    h->cgws_bytes = nba * (h->dist ? 4 : 5);
    CK(cudaMalloc(&h->cgws, h->cgws_bytes));
    h->z = reinterpret_cast<double*>(h->cgws);
    h->r = reinterpret_cast<double*>(h->cgws + nba);
    h->q = reinterpret_cast<double*>(h->cgws + 2 * nba);
    h->s_vec = reinterpret_cast<double*>(h->cgws + 3 * nba);
    if (!h->dist) h->p_single = reinterpret_cast<double*>(h->cgws + 4 * nba);
    // a persisting-L2 window over the CG vectors on every CG launch, so the plan's stream (larger
    // than L2) does not evict them between the update and the SpMV (SPMV_CG_L2WIN=0: off).
    // Measured, class C (profiles/r02ae_*): 12,956 / 12,961 -> 13,055 / 13,048 CG it/s
    int cw = 1;
    env_int("SPMV_CG_L2WIN", &cw);
    int maxwin = 0, maxpersist = 0;
    cudaDeviceGetAttribute(&maxwin, cudaDevAttrMaxAccessPolicyWindowSize, h->device);
    cudaDeviceGetAttribute(&maxpersist, cudaDevAttrMaxPersistingL2CacheSize, h->device);
    if (cw && maxwin > 0 && maxpersist > 0) {
      size_t cur = 0;
      cudaDeviceGetLimit(&cur, cudaLimitPersistingL2CacheSize);
      const size_t want = std::min<size_t>(h->cgws_bytes + h->xp.win_bytes, (size_t)maxpersist);
      if (want > cur && cudaDeviceSetLimit(cudaLimitPersistingL2CacheSize, want) != cudaSuccess) cudaGetLastError();
      cudaDeviceGetLimit(&cur, cudaLimitPersistingL2CacheSize);
      if (cur > 0) {
        h->cgwin_bytes = std::min<size_t>(h->cgws_bytes, (size_t)maxwin);
        h->cgwin_ratio = (float)std::min(1.0, (double)cur / (double)h->cgwin_bytes);
      }
    }
  }
  ST(ensure_buf((void**)&h->part_pq, pb));
  // [0],[1]: parity slots; [2]: ||b||^2 (init); [3..5]: rotating r.r of the single-reduction CG
  ST(ensure_buf((void**)&h->part_rr, 6 * pb));
  ST(ensure_buf((void**)&h->alpha2, sizeof(double) * 2));
  ST(ensure_buf((void**)&h->part_res, pb));
  ST(ensure_buf((void**)&h->part_xz, pb));
  ST(ensure_buf((void**)&h->part_zz, pb));
  ST(ensure_buf((void**)&h->scal, sizeof(double) * 16));
  ST(ensure_buf((void**)&h->out2, sizeof(double) * 2));
  ST(ensure_buf((void**)&h->flags, sizeof(int) * 4));
  ST(ensure_buf((void**)&h->gbar, sizeof(unsigned int)));  // persistent CG (allocated outside graph capture)
  CK(cudaMemset(h->flags, 0, sizeof(int) * 4));
  return SPMV_OK;
}

static double* cg_p(spmv_csr_s* h) {
  if (!h->dist) return h->p_single;
  return (double*)h->xpad + h->dist->rank * h->maxlen;
}

static spmv_status gather_p(spmv_csr_s* h, cudaStream_t s) {
  if (!h->dist) return SPMV_OK;
  return exchange_x(h, s);
}

// CG enqueue state: the scalar sources carried between iterations.
struct CgRun {
  SumSrc rr_b, rr_old, rr_prev;  // rr_prev: gamma_{k-1} of the single-reduction CG
  int it = 0;
};

// Enqueue CG init (x0 = 0): z = 0, r = b, p = b, rho = r.r (no host sync).
static spmv_status cg_enqueue_init(spmv_csr_s* h, cudaStream_t s, const double* b, double* z,
                                   CgRun* run) {
  const int vg = (int)h->vgrid;
  double* prb = h->part_rr + 2 * std::max(std::max(h->grid, h->grid_vec), h->vgrid);
  // textbook: r = h->r, p = the SpMV input (cg_p); single-reduction: the SpMV
  // input is r (cg_p) and h->r holds p (overwritten before it is read)
  if (h->cg_variant >= 1) k_cg_init<<<vg, 256, 0, s>>>(h->m_loc, b, z, cg_p(h), h->r, prb);
  else k_cg_init<<<vg, 256, 0, s>>>(h->m_loc, b, z, h->r, cg_p(h), prb);
  LAUNCHED();
  ST(reduce_src(h, s, SumSrc{prb, vg}, 0, &run->rr_b));
  run->rr_old = run->rr_b;
  run->rr_prev = run->rr_b;
  run->it = 0;
  if (use_p2p(h)) ST(exchange_x(h, s));  // p = b to every peer; later rounds are fused into k_cg_p
  return SPMV_OK;
}

// Enqueue `iters` CG iterations (no host sync).  tol > 0: kernels become
// no-ops once sqrt(rho) <= tol*||b|| (flags[1]).
static spmv_status cg_enqueue_iters(spmv_csr_s* h, cudaStream_t s, double* z, int iters, double tol,
                                    CgRun* run) {
  const int64_t n = h->m_loc;
  double* p = cg_p(h);
  const void* xg = h->dist ? h->xpad : (const void*)p;
  const int vg = (int)h->vgrid, sg = (int)h->grid;
  const int64_t pstride = std::max(std::max(h->grid, h->grid_vec), h->vgrid);
  const bool p2p = use_p2p(h);
  P2PHook base;
  if (p2p) {
    base.c = p2p_ctx(h);
    base.enabled = 1;
  }
  if (h->cg_variant == 2 && tol == 0.0 && iters > 0 && persist_eligible(h)) {
    // NEXT-1: the persistent single-reduction CG -- all `iters` iterations in ONE
    // launch (persist_kernel.cuh); the scalars of the last iteration stay in
    // the kernel, so the run's sources are not used afterwards
    ST(launch_cg_persist(h, s, xg, p, h->r, h->s_vec, h->q, z, h->part_pq, h->part_rr + 3 * pstride, pstride,
                         run->rr_b.p, run->rr_b.count, iters));
    run->it += iters;
    return SPMV_OK;
  }
  if (h->cg_variant >= 1) {
    // single-reduction CG (cg_kernels.cuh k_cgcg): SpMV w = A r with w.r fused, then one update
    // (variant 2 when the persistent kernel is not eligible: tol > 0, a non-XPLAN kernel, >1 GPU)
    double* rv = p;  // the SpMV input slice holds r
    static const int kGamSlot[3] = {2, 3, 7};
    for (int c = 0; c < iters; ++c) {
      const int k = run->it++;
      SumSrc del;
      if (p2p) {
        P2PHook hs = base;
        hs.wait_x = 1;
        hs.push_slot = 1;
        hs.push_per = p2p_spmv_push_per(h);
        ST(run_spmv(h, s, h->vals, xg, h->q, 1.0, 0.0, rv, h->part_pq, &hs));
        del = p2p_src(h, 1, std::max(hs.push_per, 1));
      } else {
        ST(gather_p(h, s));
        ST(run_spmv(h, s, h->vals, xg, h->q, 1.0, 0.0, rv, h->part_pq));
        ST(reduce_src(h, s, SumSrc{h->part_pq, sg}, 1, &del));
      }
      double* gnew = h->part_rr + (3 + (k + 1) % 3) * pstride;
      const int gslot = kGamSlot[(k + 1) % 3];
      P2PHook hz = base;
      hz.push_slot = p2p ? gslot : -1;
      hz.push_per = p2p_push_per(h, vg);
      const int64_t xoff = h->dist ? (int64_t)h->dist->rank * h->maxlen : 0;
      cudaAccessPolicyWindow cwv;
      CK(launch_maybe_pdl(k_cgcg, dim3(vg), dim3(256), 0, s, h->pdl, cg_window(h, &cwv), n, k, run->rr_old, run->rr_prev, del,
                          h->alpha2, h->r, h->s_vec, (const double*)h->q, z, rv, gnew, h->flags, tol, run->rr_b, hz,
                          xoff));
      LAUNCHED();
      SumSrc g1;
      if (p2p) g1 = p2p_src(h, gslot, std::max(hz.push_per, 1));
      else ST(reduce_src(h, s, SumSrc{gnew, vg}, gslot, &g1));
      run->rr_prev = run->rr_old;
      run->rr_old = g1;
    }
    return SPMV_OK;
  }
  for (int c = 0; c < iters; ++c) {
    const int it = run->it++;
    SumSrc pq;
    if (p2p) {
      // fused exchange: the SpMV waits for the peers' p slices (pushed by
      // k_cg_p / the init exchange) and its last CTA pushes p.q (slot 1)
      P2PHook hs = base;
      hs.wait_x = 1;
      hs.push_slot = 1;
      hs.push_per = p2p_spmv_push_per(h);
      ST(run_spmv(h, s, h->vals, xg, h->q, 1.0, 0.0, p, h->part_pq, &hs));
      pq = p2p_src(h, 1, std::max(hs.push_per, 1));
    } else {
      ST(gather_p(h, s));
      ST(run_spmv(h, s, h->vals, xg, h->q, 1.0, 0.0, p, h->part_pq));
      ST(reduce_src(h, s, SumSrc{h->part_pq, sg}, 1, &pq));
    }
    double* pnew = h->part_rr + ((it + 1) & 1) * pstride;
    const int rslot = 2 + ((it + 1) & 1);
    P2PHook hz = base;
    hz.push_slot = p2p ? rslot : -1;
    hz.push_per = p2p_push_per(h, vg);
    cudaAccessPolicyWindow cwv;
    CK(launch_maybe_pdl(k_cg_zr, dim3(vg), dim3(256), 0, s, h->pdl, cg_window(h, &cwv), n, pq, run->rr_old, (const double*)p,
                        (const double*)h->q, z, h->r, pnew, h->flags, hz));
    LAUNCHED();
    SumSrc rr_new;
    if (p2p) rr_new = p2p_src(h, rslot, std::max(hz.push_per, 1));
    else ST(reduce_src(h, s, SumSrc{pnew, vg}, rslot, &rr_new));
    // p2p: the p update stores its slice into every peer's x buffer and publishes it
    const int64_t xoff = h->dist ? (int64_t)h->dist->rank * h->maxlen : 0;
    CK(launch_maybe_pdl(k_cg_p, dim3(vg), dim3(256), 0, s, h->pdl, cg_window(h, &cwv), n, rr_new, run->rr_old,
                        (const double*)h->r, p, h->flags, tol, run->rr_b, it, base, xoff));
    LAUNCHED();
    run->rr_old = rr_new;
  }
  return SPMV_OK;
}

// Residual SpMV (Fig. 4 verbatim: r = A z) into q and the norm partials.
template <bool NPB>
static spmv_status cg_resid(spmv_csr_s* h, cudaStream_t s, const double* b, const double* z) {
  const void* zg = z;
  if (h->dist) {
    double* mine = (double*)h->xpad + h->dist->rank * h->maxlen;
    if (h->m_loc > 0) CK(cudaMemcpyAsync(mine, z, sizeof(double) * h->m_loc, cudaMemcpyDeviceToDevice, s));
    ST(gather_p(h, s));
    zg = h->xpad;
  }
  ST(run_spmv(h, s, h->vals, zg, h->q, 1.0, 0.0, nullptr, nullptr));
  k_cg_resid<NPB><<<(int)h->vgrid, 256, 0, s>>>(h->m_loc, b, h->q, z, h->part_res, h->part_xz,
                                               h->part_zz);
  LAUNCHED();
  return SPMV_OK;
}

static spmv_status stage_in(spmv_csr_s* h, cudaStream_t s, const void* src, double** dev_stage,
                            const double** use, bool copy) {
  const int k = mem_kind(src, h->device);
  if (k == 1 || (src == nullptr && h->m_loc == 0)) { *use = (const double*)src; return SPMV_OK; }
  if (k < 0) return arg_fail("vector is device memory of another GPU");
  ST(ensure_buf((void**)dev_stage, sizeof(double) * std::max<int64_t>(h->m_loc, 1)));
  if (copy && h->m_loc > 0)
    CK(cudaMemcpyAsync(*dev_stage, src, sizeof(double) * h->m_loc, cudaMemcpyHostToDevice, s));
  *use = *dev_stage;
  return SPMV_OK;
}

extern "C" spmv_status cg_solve(spmv_csr_t h, const void* b, void* x, int32_t max_iter, double tol,
                                int32_t* iters_out, double* rnorm_out) {
  if (!h) return arg_fail("handle is NULL");
  if (h->dt != SPMV_F64) { g_err = "cg_solve is fp64 only"; return SPMV_ERR_UNSUPPORTED; }
  if (h->m != h->n) return arg_fail("cg_solve needs a square matrix");
  if (max_iter < 0 || !(tol >= 0.0)) return arg_fail("max_iter >= 0, tol >= 0");
  if ((!b || !x) && h->m_loc > 0) return arg_fail("b and x must not be NULL");
  CK(cudaSetDevice(h->device));
  ST(cg_alloc(h));
  cudaStream_t s = h->stream;
  const double* bd;
  const double* xd;
  ST(stage_in(h, s, b, &h->stage_x, &bd, true));
  ST(stage_in(h, s, x, &h->stage_z, &xd, false));
  double* xw = const_cast<double*>(xd);
  CK(cudaMemsetAsync(h->flags, 0, sizeof(int) * 4, s));
  CgRun run;
  ST(cg_enqueue_init(h, s, bd, xw, &run));
  if (tol == 0.0) {
    ST(cg_enqueue_iters(h, s, xw, max_iter, 0.0, &run));
  } else {
    // chunks of iterations; the kernels are no-ops once converged, the host
    // polls the converged flag between chunks
    const int chunk = 8;
    for (int done = 0; done < max_iter; done += chunk) {
      ST(cg_enqueue_iters(h, s, xw, std::min(chunk, max_iter - done), tol, &run));
      int hf[4];
      CK(cudaMemcpyAsync(hf, h->flags, sizeof(int) * 4, cudaMemcpyDeviceToHost, s));
      CK(cudaStreamSynchronize(s));
      if (hf[1] || hf[0]) break;
    }
  }
  ST(cg_resid<false>(h, s, bd, xw));
  SumSrc res;
  ST(reduce_src(h, s, SumSrc{h->part_res, (int)h->vgrid}, 4, &res));
  k_finish_norm<<<1, 32, 0, s>>>(res, h->out2 + 1);
  LAUNCHED();
  int hf[4];
  double rn = 0;
  CK(cudaMemcpyAsync(hf, h->flags, sizeof(int) * 4, cudaMemcpyDeviceToHost, s));
  CK(cudaMemcpyAsync(&rn, h->out2 + 1, sizeof(double), cudaMemcpyDeviceToHost, s));
  if (xd != x && h->m_loc > 0)
    CK(cudaMemcpyAsync(x, xd, sizeof(double) * h->m_loc, cudaMemcpyDeviceToHost, s));
  CK(cudaStreamSynchronize(s));
  if (iters_out) *iters_out = hf[0] ? 0 : hf[2];
  if (rnorm_out) *rnorm_out = rn;
  if (hf[0]) { g_err = "CG breakdown: p.Ap == 0 or not finite"; return SPMV_ERR_BREAKDOWN; }
  return SPMV_OK;
}

// The whole NAS outer iteration enqueued on stream s (used for capture).
static spmv_status npb_enqueue(spmv_csr_s* h, cudaStream_t s, double* x, double* z, int cgitmax,
                               double shift, double* out2) {
  CgRun run;
  ST(cg_enqueue_init(h, s, x, z, &run));
  ST(cg_enqueue_iters(h, s, z, cgitmax, 0.0, &run));
  // z is final here: an external event lets the host copy of z overlap the rest
  cudaStreamCaptureStatus cst = cudaStreamCaptureStatusNone;
  CK(cudaStreamIsCapturing(s, &cst));
  auto mark = [&](cudaEvent_t ev) -> spmv_status {
    if (cst == cudaStreamCaptureStatusActive) CK(cudaEventRecordWithFlags(ev, s, cudaEventRecordExternal));
    else CK(cudaEventRecord(ev, s));
    return SPMV_OK;
  };
  ST(mark(h->ev_a));
  // zeta and x_new = z/||z|| first (they do not need the residual), x_new into a free CG
  // vector (s), so its host copy overlaps the residual SpMV, which still reads the old x
  const int vg = (int)h->vgrid;
  k_npb_xz<<<vg, 256, 0, s>>>(h->m_loc, x, z, h->part_xz, h->part_zz);
  LAUNCHED();
  SumSrc res, xz, zz;
  ST(reduce_src(h, s, SumSrc{h->part_xz, vg}, 5, &xz));
  ST(reduce_src(h, s, SumSrc{h->part_zz, vg}, 6, &zz));
  double* xn = h->s_vec;
  k_npb_xnew<<<vg, 256, 0, s>>>(h->m_loc, xz, zz, z, xn, shift, out2);
  LAUNCHED();
  ST(mark(h->ev_b));
  ST(cg_resid<false>(h, s, x, z));
  ST(reduce_src(h, s, SumSrc{h->part_res, vg}, 4, &res));
  k_finish_norm<<<1, 32, 0, s>>>(res, out2 + 1);
  LAUNCHED();
  if (h->m_loc > 0) CK(cudaMemcpyAsync(x, xn, sizeof(double) * h->m_loc, cudaMemcpyDeviceToDevice, s));
  return SPMV_OK;
}

static bool use_graphs() {
  int v = 1;
  env_int("SPMV_GRAPH", &v);
  return v != 0;
}

extern "C" spmv_status cg_npb_outer(spmv_csr_t h, void* x, void* z, int32_t cgitmax, double shift,
                                    double* out2) {
  if (!h) return arg_fail("handle is NULL");
  if (h->dt != SPMV_F64) { g_err = "cg_npb_outer is fp64 only"; return SPMV_ERR_UNSUPPORTED; }
  if (h->m != h->n) return arg_fail("needs a square matrix");
  if (cgitmax < 0) return arg_fail("cgitmax >= 0");
  if (!out2) return arg_fail("out2 is NULL");
  if ((!x || !z) && h->m_loc > 0) return arg_fail("x and z must not be NULL");
  CK(cudaSetDevice(h->device));
  ST(cg_alloc(h));
  cudaStream_t s = h->stream;
  const double *xd, *zd;
  ST(stage_in(h, s, x, &h->stage_x, &xd, true));
  ST(stage_in(h, s, z, &h->stage_z, &zd, false));
  const int ok = mem_kind(out2, h->device);
  double* o2 = h->out2;  // the graph writes here; copied to out2 after the launch
  double* xw = const_cast<double*>(xd);
  double* zw = const_cast<double*>(zd);
  if (use_graphs()) {
    Graph& g = h->g_npb;
    if (!g.exec || g.k0 != xw || g.k1 != zw || g.ki != cgitmax || g.kd != shift) {
      g.reset();
      const uint64_t before = g_launches.load();
      CK(cudaStreamBeginCapture(h->cap, cudaStreamCaptureModeThreadLocal));
      spmv_status st = npb_enqueue(h, h->cap, xw, zw, cgitmax, shift, o2);
      cudaGraph_t graph = nullptr;
      cudaError_t e = cudaStreamEndCapture(h->cap, &graph);
      if (st != SPMV_OK) { if (graph) cudaGraphDestroy(graph); return st; }
      if (e != cudaSuccess) return cuda_fail(e, "graph capture", __LINE__);
      e = cudaGraphInstantiate(&g.exec, graph, 0);
      cudaGraphDestroy(graph);
      if (e != cudaSuccess) { g.exec = nullptr; return cuda_fail(e, "graph instantiate", __LINE__); }
      g.nodes = g_launches.load() - before;
      g_launches.fetch_sub(g.nodes);  // counted when replayed
      g.k0 = xw; g.k1 = zw; g.ki = cgitmax; g.kd = shift;
    }
    CK(cudaGraphLaunch(g.exec, s));
    g_launches.fetch_add(g.nodes);
  } else {
    ST(npb_enqueue(h, s, xw, zw, cgitmax, shift, o2));
  }
  bool sync = false;
  if (ok == 1) CK(cudaMemcpyAsync(out2, o2, sizeof(double) * 2, cudaMemcpyDeviceToDevice, s));
  bool copy_used = false;
  if ((zd != z || xd != x) && h->m_loc > 0 && !h->copy)
    CK(cudaStreamCreateWithFlags(&h->copy, cudaStreamNonBlocking));
  if (zd != z && h->m_loc > 0) {
    // z (host) is copied on a side stream as soon as the CG loop wrote it,
    // overlapping the residual SpMV and the finishing kernels
    CK(cudaStreamWaitEvent(h->copy, h->ev_a, 0));
    CK(cudaMemcpyAsync(z, zd, sizeof(double) * h->m_loc, cudaMemcpyDeviceToHost, h->copy));
    copy_used = true;
    sync = true;
  }
  if (xd != x && h->m_loc > 0) {
    // x_new (host) likewise, from the buffer it is computed into before the residual
    CK(cudaStreamWaitEvent(h->copy, h->ev_b, 0));
    CK(cudaMemcpyAsync(x, h->s_vec, sizeof(double) * h->m_loc, cudaMemcpyDeviceToHost, h->copy));
    copy_used = true;
    sync = true;
  }
  if (ok != 1) {
    CK(cudaMemcpyAsync(out2, o2, sizeof(double) * 2, cudaMemcpyDeviceToHost, s));
    sync = true;
  }
  if (sync) {
    int hf[4];
    CK(cudaMemcpyAsync(hf, h->flags, sizeof(int) * 4, cudaMemcpyDeviceToHost, s));
    CK(cudaStreamSynchronize(s));
    if (copy_used) CK(cudaStreamSynchronize(h->copy));
    if (hf[0]) { g_err = "CG breakdown"; return SPMV_ERR_BREAKDOWN; }
  }
  return SPMV_OK;
}


extern "C" spmv_status spmv_csr_set_cg_variant(spmv_csr_t h, int32_t variant) {
  if (!h) return arg_fail("handle is NULL");
  if (variant < 0 || variant > 2)
    return arg_fail("variant must be 0 (textbook), 1 (single reduction) or 2 (persistent single reduction)");
  if (h->cg_variant != variant) {
    h->cg_variant = variant;
    h->g_npb.reset();  // the captured NPB graph belongs to the other variant
  }
  return SPMV_OK;
}

extern "C" spmv_status spmv_cg_status(spmv_csr_t h) {
  if (!h) return arg_fail("handle is NULL");
  if (!h->flags) return SPMV_OK;
  CK(cudaSetDevice(h->device));
  int hf[4];
  CK(cudaMemcpyAsync(hf, h->flags, sizeof(int) * 4, cudaMemcpyDeviceToHost, h->stream));
  CK(cudaStreamSynchronize(h->stream));
  if (hf[0]) { g_err = "CG breakdown"; return SPMV_ERR_BREAKDOWN; }
  return SPMV_OK;
}
