// spmv_abi.cu -- the C ABI of include/spmv.h, core: handle creation (ingest +
// analyse: validation, row statistics, kernel choice, the
// distributed partition), spmv_csr (a2), destruction and introspection.  The
// plans, CG drivers, transports and the stencil are in their own units (see
// abi_common.h); all arithmetic of the hot path runs in the kernels.
#include "abi_common.h"
#include "analysis_kernels.cuh"

thread_local std::string g_err = "no error";
std::atomic<uint64_t> g_launches{0};

// Kernel selection from row statistics (the paper's "try every API, keep the
// fastest", becomes a rule fitted by the bench sweep).
static void choose_kernel(spmv_csr_s* h, int req_kernel, int req_lanes) {
  int lanes;
  const double mean = h->row_mean;
  if (mean < 2.0) lanes = 1;
  else if (mean < 6.0) lanes = 2;
  else if (mean < 12.0) lanes = 4;
  else if (mean < 24.0) lanes = 8;
  else if (mean < 48.0) lanes = 16;
  else lanes = 32;
  h->kernel = SPMV_KERNEL_VECTOR;
  if (req_kernel == SPMV_KERNEL_SCALAR) lanes = 1;
  if (req_lanes == 1 || req_lanes == 2 || req_lanes == 4 || req_lanes == 8 || req_lanes == 16 ||
      req_lanes == 32)
    lanes = req_lanes;
  h->lanes = lanes;
  h->unroll = 4;
  int u;
  if (env_int("SPMV_UNROLL", &u) && (u == 2 || u == 4 || u == 8)) h->unroll = u;
  const int sms = num_sms(h->device);
  // fixed grid-stride grid (deterministic CTA partials): 8 CTAs of 256 per SM
  const int64_t groups_per_cta = 256 / lanes;
  h->grid = std::max<int64_t>(1, std::min<int64_t>(cdiv(h->m_loc, groups_per_cta), 8LL * sms));
  h->grid_vec = h->grid;
  // CG vector kernels: elements per CTA (SPMV_VGRID_ELEMS overrides, for sweeps)
  int vel = 1024;
  tuning_env("SPMV_VGRID_ELEMS", &vel);
  vel = std::max(vel, 32);
  h->vgrid = std::max<int64_t>(1, std::min<int64_t>(cdiv(h->m_loc, vel), 4LL * sms));
}

// ----------------------------------------------------------------- create
extern "C" spmv_status spmv_csr_create(spmv_csr_t* out, spmv_dtype dt, int64_t m, int64_t n,
                                       int64_t nnz, const int32_t* rowptr, const int32_t* colidx,
                                       const void* vals, const spmv_opts* opts) {
  if (!out) return arg_fail("out is NULL");
  *out = nullptr;
  if (dt != SPMV_F64 && dt != SPMV_F32) return arg_fail("dtype must be SPMV_F64 or SPMV_F32");
  if (m < 0 || n < 0 || nnz < 0 || nnz > 2147483647LL || m > 2147483646LL || n > 2147483647LL)
    return arg_fail("sizes out of range (m, n, nnz >= 0; nnz < 2^31)");
  if (!rowptr) return arg_fail("rowptr is NULL");
  spmv_opts o{};
  if (opts) o = *opts;
  int dev = 0;
  CK(cudaGetDevice(&dev));
  if (o.dist) dev = o.dist->device;
  CK(cudaSetDevice(dev));
  ST(need_device(rowptr, dev, "rowptr must be a device pointer on the current device", false));
  ST(need_device(colidx, dev, "colidx must be a device pointer", nnz == 0));
  ST(need_device(vals, dev, "vals must be a device pointer", nnz == 0));
  if (o.dist && m != n) return arg_fail("distributed mode needs a square matrix (R25)");

  // rowptr[0], rowptr[m] -> nnz check (R1)
  int32_t ends[2];
  CK(cudaMemcpy(&ends[0], rowptr, 4, cudaMemcpyDeviceToHost));
  CK(cudaMemcpy(&ends[1], rowptr + m, 4, cudaMemcpyDeviceToHost));
  if ((int64_t)ends[1] - (int64_t)ends[0] != nnz)
    return arg_fail("nnz != rowptr[m] - rowptr[0] (reading R1)");

  spmv_csr_s* h = new spmv_csr_s();
  h->device = dev;
  h->stream = (cudaStream_t)o.stream;
  h->dt = dt;
  h->ts = dt == SPMV_F64 ? 8 : 4;
  h->m = m;
  h->n = n;
  h->nnz = nnz;
  h->base = ends[0];
  h->rowptr = rowptr;
  h->colidx = colidx;
  h->vals = vals;
  h->dist = o.dist;
  auto fail = [&](spmv_status s) {
    spmv_csr_destroy(h);
    return s;
  };
  cudaStream_t s = h->stream;
  const int sms = num_sms(dev);

  // validation (device pass, synchronous)
  if (o.validate && m > 0) {
    int* fl = nullptr;
    if (cudaMalloc(&fl, sizeof(int)) != cudaSuccess) return fail(cuda_fail(cudaErrorMemoryAllocation, "cudaMalloc", __LINE__));
    cudaMemsetAsync(fl, 0, sizeof(int), s);
    k_validate<<<std::min<int64_t>(cdiv(std::max(m, nnz), 256), 8LL * sms), 256, 0, s>>>(m, n, rowptr, colidx, fl);
    g_launches.fetch_add(1);
    int hv = 0;
    cudaError_t e = cudaMemcpyAsync(&hv, fl, sizeof(int), cudaMemcpyDeviceToHost, s);
    if (e == cudaSuccess) e = cudaStreamSynchronize(s);
    cudaFree(fl);
    if (e != cudaSuccess) return fail(cuda_fail(e, "validate", __LINE__));
    if (hv) {
      g_err = (hv & 1) ? "rowptr is decreasing" : "colidx outside [0, n)";
      return fail(SPMV_ERR_INDEX);
    }
  }

  // row statistics (device pass over rowptr [+ colidx sortedness]; host reduce in CTA order)
  if (m > 0) {
    const int64_t g = std::min<int64_t>(cdiv(m, 256), 2LL * sms);
    double* dpart = nullptr;
    if (cudaMalloc(&dpart, sizeof(double) * 5 * g) != cudaSuccess)
      return fail(cuda_fail(cudaErrorMemoryAllocation, "cudaMalloc", __LINE__));
    k_row_stats<<<g, 256, 0, s>>>(m, rowptr, colidx, nnz > 0 ? 1 : 0, dpart);
    g_launches.fetch_add(1);
    std::vector<double> hp(5 * g);
    cudaError_t e = cudaMemcpyAsync(hp.data(), dpart, sizeof(double) * 5 * g, cudaMemcpyDeviceToHost, s);
    if (e == cudaSuccess) e = cudaStreamSynchronize(s);
    cudaFree(dpart);
    if (e != cudaSuccess) return fail(cuda_fail(e, "row stats", __LINE__));
    double mn = 1e300, mx = -1e300, sum = 0, sq = 0, uns = 0;
    for (int64_t b = 0; b < g; ++b) {
      uns += hp[5 * b + 4];
      mn = std::min(mn, hp[5 * b]);
      mx = std::max(mx, hp[5 * b + 1]);
      sum += hp[5 * b + 2];
      sq += hp[5 * b + 3];
    }
    h->sorted = (uns == 0.0) ? 1 : 0;
    h->row_min = (int64_t)mn;
    h->row_max = (int64_t)mx;
    h->row_mean = sum / (double)m;
    const double var = std::max(0.0, sq / (double)m - h->row_mean * h->row_mean);
    h->row_cv = h->row_mean > 0 ? std::sqrt(var) / h->row_mean : 0.0;
  }

  // execution view
  if (!o.dist) {
    h->m_loc = m;
    h->row0 = 0;
    h->k0 = ends[0];
    h->k1 = ends[1];
    h->rp_loc = rowptr;
    h->ci_loc = colidx;
  } else {
    spmv_dist_s* d = o.dist;
    const int P = d->nranks;
    long long* dbounds = nullptr;
    if (cudaMalloc(&dbounds, sizeof(long long) * (P + 1)) != cudaSuccess)
      return fail(cuda_fail(cudaErrorMemoryAllocation, "cudaMalloc", __LINE__));
    k_partition<<<cdiv(P + 1, 128), 128, 0, s>>>(m, rowptr, P, dbounds);
    g_launches.fetch_add(1);
    h->bounds.assign(P + 1, 0);
    cudaError_t e = cudaMemcpyAsync(h->bounds.data(), dbounds, sizeof(long long) * (P + 1),
                                    cudaMemcpyDeviceToHost, s);
    if (e == cudaSuccess) e = cudaStreamSynchronize(s);
    if (e != cudaSuccess) { cudaFree(dbounds); return fail(cuda_fail(e, "partition", __LINE__)); }
    long long maxlen = 1;
    for (int r = 0; r < P; ++r) maxlen = std::max(maxlen, h->bounds[r + 1] - h->bounds[r]);
    h->maxlen = maxlen;
    const int r = d->rank;
    h->row0 = h->bounds[r];
    h->m_loc = h->bounds[r + 1] - h->bounds[r];
    int32_t kk[2] = {0, 0};
    e = cudaMemcpy(&kk[0], rowptr + h->row0, 4, cudaMemcpyDeviceToHost);
    if (e == cudaSuccess) e = cudaMemcpy(&kk[1], rowptr + h->row0 + h->m_loc, 4, cudaMemcpyDeviceToHost);
    if (e != cudaSuccess) { cudaFree(dbounds); return fail(cuda_fail(e, "rowptr", __LINE__)); }
    h->k0 = kk[0];
    h->k1 = kk[1];
    const int64_t nloc = h->k1 - h->k0;
    bool okm = cudaMalloc(&h->ci_own, sizeof(int32_t) * std::max<int64_t>(nloc, 1)) == cudaSuccess;
    if (okm && !d->p2p) {
      okm = cudaMalloc(&h->xpad, h->ts * (size_t)(maxlen * P)) == cudaSuccess;
      if (okm) cudaMemsetAsync(h->xpad, 0, h->ts * (size_t)(maxlen * P), s);
    } else if (okm) {
      // fabric: xpad | exch [NSLOT][P][PMAX] double | flags [P] u64, one IPC-exportable allocation
      const size_t xb = (h->ts * (size_t)(maxlen * P) + 255) & ~size_t(255);
      h->off_exch = xb;
      h->off_flags = xb + ((sizeof(double) * P2P_NSLOT * P * P2P_PMAX + 255) & ~size_t(255));
      h->fab_bytes = h->off_flags + ((sizeof(unsigned long long) * P + 255) & ~size_t(255));
      okm = cudaMalloc(&h->fabric, h->fab_bytes) == cudaSuccess &&
            cudaMalloc(&h->p2p_local, sizeof(unsigned long long) * (P2P_NSLOT + 4)) == cudaSuccess &&
            cudaMalloc(&h->peer_table, sizeof(unsigned char*) * P) == cudaSuccess;
      if (okm) {
        cudaMemsetAsync(h->fabric, 0, h->fab_bytes, s);
        cudaMemsetAsync(h->p2p_local, 0, sizeof(unsigned long long) * (P2P_NSLOT + 4), s);
        h->xpad = h->fabric;
        h->peers.assign(P, nullptr);
        h->peers[d->rank] = h->fabric;
      }
    }
    if (!okm) {
      cudaFree(dbounds);
      return fail(cuda_fail(cudaErrorMemoryAllocation, "cudaMalloc", __LINE__));
    }
    if (nloc > 0) {
      k_renumber<<<std::min<int64_t>(cdiv(nloc, 256), 8LL * sms), 256, sizeof(long long) * (P + 1), s>>>(
          h->k0, h->k1, colidx, dbounds, P, maxlen, h->ci_own);
      g_launches.fetch_add(1);
    }
    // halo intervals of every (reader, owner) pair from the GLOBAL matrix (identical on all ranks)
    int* dtab = nullptr;
    if (P > 1 && m > 0) {
      const size_t tb = sizeof(int) * 2 * (size_t)P * P;
      okm = cudaMalloc(&dtab, tb) == cudaSuccess;
      if (!okm) { cudaFree(dbounds); return fail(cuda_fail(cudaErrorMemoryAllocation, "cudaMalloc", __LINE__)); }
      std::vector<int> init(2 * (size_t)P * P);
      for (size_t i = 0; i < init.size(); i += 2) { init[i] = 0x7fffffff; init[i + 1] = -1; }
      cudaMemcpyAsync(dtab, init.data(), tb, cudaMemcpyHostToDevice, s);
      const size_t sm = sizeof(long long) * (P + 1) + tb;
      k_halo_bounds<<<(unsigned)std::min<int64_t>(cdiv(m * 32, 256), 8LL * sms), 256, sm, s>>>(m, rowptr, colidx,
                                                                                                 dbounds, P, dtab);
      g_launches.fetch_add(1);
    }
    e = cudaStreamSynchronize(s);
    cudaFree(dbounds);
    if (e != cudaSuccess) { cudaFree(dtab); return fail(cuda_fail(e, "renumber", __LINE__)); }
    h->halo.assign(2 * (size_t)P * P, 0);
    if (dtab) {
      std::vector<int> tab(2 * (size_t)P * P);
      e = cudaMemcpy(tab.data(), dtab, sizeof(int) * tab.size(), cudaMemcpyDeviceToHost);
      cudaFree(dtab);
      if (e != cudaSuccess) return fail(cuda_fail(e, "halo", __LINE__));
      long long vol = 0;
      for (size_t i = 0; i < tab.size(); i += 2)
        if (tab[i + 1] >= 0) {
          h->halo[i] = tab[i];
          h->halo[i + 1] = (long long)tab[i + 1] + 1;
          vol += h->halo[i + 1] - h->halo[i];
        }
      // exchange only the intervals when they move less than half of the padded all-gather
      // (a decision every rank takes from the same global table)
      int hv = 1;
      env_int("SPMV_HALO", &hv);
      h->use_halo = hv != 0 && 2 * vol < (long long)P * (P - 1) * maxlen;
      std::vector<int2> siv(P);
      for (int q = 0; q < P; ++q) {
        const size_t i = 2 * ((size_t)q * P + r);  // reader q, owner r (this rank)
        siv[q] = make_int2((int)h->halo[i], (int)h->halo[i + 1]);
      }
      if (cudaMalloc(&h->send_iv, sizeof(int2) * P) != cudaSuccess)
        return fail(cuda_fail(cudaErrorMemoryAllocation, "cudaMalloc", __LINE__));
      CK(cudaMemcpy(h->send_iv, siv.data(), sizeof(int2) * P, cudaMemcpyHostToDevice));
    }
    h->rp_loc = rowptr + h->row0;
    h->ci_loc = h->ci_own - h->k0;  // absolute k addressing
  }

  h->pdl = 1;
  env_int("SPMV_PDL", &h->pdl);  // programmatic dependent launch of the SpMV / k_cgcg chain (A/B: 0 = off)
  int rk = 0, rl = 0;
  if (!env_int("SPMV_KERNEL", &rk)) rk = o.kernel;
  if (!env_int("SPMV_LANES", &rl)) rl = o.vec_lanes;
  h->nx = o.dist ? (int64_t)h->maxlen * o.dist->nranks : n;
  choose_kernel(h, rk, rl);
  int plan = o.plan;
  env_int("SPMV_PLAN", &plan);
  if (rk == SPMV_KERNEL_XT) {
    // the TMA-streamed column-parted plan: on request only --
    // measured slower than XPLAN on the NAS shapes, so auto keeps XPLAN
    {
      bool ok = false;
      spmv_status st = xt_build(h, &ok);
      if (st != SPMV_OK) return fail(st);
      if (ok) {
        h->kernel = SPMV_KERNEL_XT;
        h->grid = (int64_t)h->xt.ncl * h->xt.B;
      }
    }
  }
  if (h->kernel != SPMV_KERNEL_XT && (rk == SPMV_KERNEL_XPLAN || (rk == SPMV_KERNEL_AUTO && plan))) {
    // auto + plan: the column-blocked x-stationary plan whenever x fits the
    // shared memory of a cluster and rows are long enough
    if (rk == SPMV_KERNEL_XPLAN || h->row_mean >= 16.0) {
      bool ok = false;
      spmv_status st = xplan_build(h, &ok);
      if (st != SPMV_OK) return fail(st);
      if (ok) {
        h->kernel = SPMV_KERNEL_XPLAN;
        // dot partials: one per (tile, owner CTA) with dynamic tiles, else one per CTA
        h->grid = h->xp.dyn ? (int64_t)h->xp.ntiles * h->xp.B : (int64_t)h->xp.ncl * h->xp.B;
        if (h->xp.mplan < h->m_loc) h->grid += h->xp.g2;  // dot partials: clusters, then the side kernel
      }
    }
  }
  const bool skewed = (double)h->row_max > 32.0 * std::max(h->row_mean, 1.0);
  if (h->kernel != SPMV_KERNEL_XPLAN && h->kernel != SPMV_KERNEL_XT && (rk == SPMV_KERNEL_SELL || rk == SPMV_KERNEL_SELL_SORTED ||
                                         (rk == SPMV_KERNEL_AUTO && plan))) {
    // auto + plan, x too large for the clusters (or short rows): a SELL-32 plan
    // with global x gathers -- chunks of consecutive rows when they pad by
    // <= 20 % (the 27-point stencil), else (skewed rows: the power law) the
    // length-sorted chunks with the long rows warp-per-row; forced: any padding
    const int sorted = rk == SPMV_KERNEL_SELL_SORTED || (rk == SPMV_KERNEL_AUTO && skewed);
    bool ok = false;
    spmv_status st = sell_build(h, rk == SPMV_KERNEL_AUTO ? 1.2 : 1e30, sorted, &ok);
    if (st != SPMV_OK) return fail(st);
    if (ok) {
      h->kernel = sorted ? SPMV_KERNEL_SELL_SORTED : SPMV_KERNEL_SELL;
      h->grid = h->sl.nmulti > 0 ? h->vgrid : h->sl.grid;  // dot partials: k_dot_partials or fused
    }
  }
  if (h->kernel != SPMV_KERNEL_XPLAN && h->kernel != SPMV_KERNEL_XT && h->kernel != SPMV_KERNEL_SELL &&
      h->kernel != SPMV_KERNEL_SELL_SORTED &&
      rk != SPMV_KERNEL_VECTOR && rk != SPMV_KERNEL_SCALAR && rk != SPMV_KERNEL_XSTAT && h->m_loc > 0 &&
      (rk == SPMV_KERNEL_MERGE || skewed)) {
    // skewed rows without a plan (a long row would pin one warp of the vector kernel): merge path
    spmv_status st = merge_setup(h);
    if (st != SPMV_OK) return fail(st);
    h->kernel = SPMV_KERNEL_MERGE;
    h->grid = h->vgrid;  // dot partials come from k_dot_partials
  }
  if (h->kernel == SPMV_KERNEL_XPLAN || h->kernel == SPMV_KERNEL_XT || h->kernel == SPMV_KERNEL_MERGE ||
      h->kernel == SPMV_KERNEL_SELL ||
      h->kernel == SPMV_KERNEL_SELL_SORTED) {
  } else if (rk == SPMV_KERNEL_XSTAT) {
    bool ok = false;
    spmv_status st = xstat_setup(h, &ok);
    if (st != SPMV_OK) return fail(st);
    if (ok) {
      h->kernel = SPMV_KERNEL_XSTAT;
      h->grid = (int64_t)h->nclusters * h->xB;
    }
  }
  if (o.l2_window) {
    // BJ.ns: "an L2 persisting-access window on x" -- reserve the persisting
    // L2 carve-out for x (device-wide limit, raised only) and record the window
    int maxwin = 0, maxpersist = 0;
    cudaDeviceGetAttribute(&maxwin, cudaDevAttrMaxAccessPolicyWindowSize, dev);
    cudaDeviceGetAttribute(&maxpersist, cudaDevAttrMaxPersistingL2CacheSize, dev);
    const size_t xb = h->ts * (size_t)std::max<int64_t>(h->nx, 1);
    size_t cur = 0;
    cudaDeviceGetLimit(&cur, cudaLimitPersistingL2CacheSize);
    const size_t want = std::min<size_t>(xb, (size_t)std::max(maxpersist, 0));
    if (want > cur && cudaDeviceSetLimit(cudaLimitPersistingL2CacheSize, want) != cudaSuccess) cudaGetLastError();
    cudaDeviceGetLimit(&cur, cudaLimitPersistingL2CacheSize);
    if (maxwin > 0 && cur > 0) {
      h->l2win_bytes = std::min<size_t>(xb, (size_t)maxwin);
      h->l2persist_bytes = cur;
    }
  }
  CK(cudaStreamCreateWithFlags(&h->cap, cudaStreamNonBlocking));
  CK(cudaEventCreateWithFlags(&h->ev_a, cudaEventDisableTiming));
  CK(cudaEventCreateWithFlags(&h->ev_b, cudaEventDisableTiming));
  *out = h;
  return SPMV_OK;
}

extern "C" spmv_status spmv_csr_destroy(spmv_csr_t h) {
  if (!h) return SPMV_OK;
  cudaSetDevice(h->device);
  spmv_status st = SPMV_OK;
  cudaError_t e = h->stream ? cudaStreamSynchronize(h->stream) : cudaDeviceSynchronize();
  if (e != cudaSuccess) st = cuda_fail(e, "pending asynchronous error", __LINE__);
  h->g_npb.reset();
  h->xt.release();
  for (size_t q = 0; q < h->peers.size(); ++q)
    if (h->peers[q] && h->peers[q] != h->fabric) cudaIpcCloseMemHandle(h->peers[q]);
  if (h->fabric) {
    cudaFree(h->fabric);
    if (h->xpad == h->fabric) h->xpad = nullptr;
  }
  void* bufs[] = {h->p2p_local, h->peer_table, h->mg.split_row, h->mg.split_nz, h->mg.head, h->mg.carry, h->mg.head_flag, h->xp.crow, h->xp.chunk_off, h->xp.tile0, h->xp.chunk_len, h->xp.seg, h->xp.row_slot,
                  h->xp.chunk_row, h->xp.plan, h->xp.tq, h->xp.cta_range, h->sl.pair_off, h->sl.vals, h->sl.cols, h->sl.perm, h->sl.seg, h->sl.seg_part, h->sl.seg_cnt,
                  h->seg, h->crow, h->ci_own, h->send_iv, h->xpad, h->cgws, h->part_pq, h->part_rr,
                  h->part_res, h->part_xz, h->part_zz, h->scal, h->out2, h->flags, h->alpha2,
                  h->stage_x, h->stage_z, h->gbar};
  // lines pinned by a persisting window over the plan go back to normal (device-wide; other
  // handles' windows re-pin theirs on their next launch)
  if (h->xp.win_bytes || h->cgwin_bytes) cudaCtxResetPersistingL2Cache();
  for (void* b : bufs)
    if (b) cudaFree(b);
  if (h->cap) cudaStreamDestroy(h->cap);
  if (h->side) cudaStreamDestroy(h->side);
  if (h->ev_fork) cudaEventDestroy(h->ev_fork);
  if (h->ev_join) cudaEventDestroy(h->ev_join);
  if (h->ev_a) cudaEventDestroy(h->ev_a);
  if (h->copy) cudaStreamDestroy(h->copy);
  if (h->ev_b) cudaEventDestroy(h->ev_b);
  delete h;
  return st;
}

// ------------------------------------------------------------------ spmv

extern "C" spmv_status spmv_csr(spmv_csr_t h, int64_t m, int64_t n, int64_t nnz,
                                const int32_t* rowptr, const int32_t* colidx, const void* vals,
                                const void* x, void* y, double alpha, double beta) {
  if (!h) return arg_fail("handle is NULL");
  if (m != h->m || n != h->n || nnz != h->nnz || rowptr != h->rowptr || colidx != h->colidx)
    return arg_fail("m, n, nnz, rowptr, colidx must equal those bound at create");
  CK(cudaSetDevice(h->device));
  const int64_t ml = h->m_loc;
  const int64_t xl = h->dist ? h->m_loc : n;  // local slice length of x in dist mode
  if (ml > 0) ST(need_device(y, h->device, "y must be a device pointer", false));
  if (alpha != 0.0) {
    ST(need_device(x, h->device, "x must be a device pointer", xl == 0));
    ST(need_device(vals, h->device, "vals must be a device pointer", nnz == 0));
  }
  const size_t ts = h->ts;
  // aliasing check (reading R13)
  const size_t ybytes = ts * (size_t)ml;
  if (overlap(y, ybytes, x, ts * (size_t)xl) ||
      overlap(y, ybytes, (const char*)vals + ts * (size_t)h->base, ts * (size_t)nnz) ||
      overlap(y, ybytes, colidx + h->base, 4 * (size_t)nnz) ||
      overlap(y, ybytes, rowptr, 4 * (size_t)(m + 1))) {
    g_err = "y overlaps x, vals, colidx or rowptr";
    return SPMV_ERR_ALIAS;
  }
  cudaStream_t s = h->stream;
  const void* xin = x;
  if (h->dist && alpha != 0.0) {
    spmv_dist_s* d = h->dist;
    char* mine = (char*)h->xpad + ts * (size_t)(d->rank * h->maxlen);
    if (ml > 0 && x != mine) CK(cudaMemcpyAsync(mine, x, ts * (size_t)ml, cudaMemcpyDeviceToDevice, s));
    ST(exchange_x(h, s));
    xin = h->xpad;
  }
  return run_spmv(h, s, vals, xin, y, alpha, beta, nullptr, nullptr);
}

extern "C" spmv_status spmv_csr_update_values(spmv_csr_t h, const void* vals) {
  if (!h) return arg_fail("handle is NULL");
  CK(cudaSetDevice(h->device));
  ST(need_device(vals, h->device, "vals must be a device pointer", h->nnz == 0));
  h->vals = vals;
  if (h->xp.built) ST(xplan_pack(h, vals, 1));
  if (h->xt.built) ST(xt_pack(h, vals, 1));
  if (h->sl.built) ST(sell_pack(h, vals, 1));
  h->g_npb.reset();
  return SPMV_OK;
}

// ---------------------------------------------------------- introspection
extern "C" spmv_status spmv_csr_partition(const int32_t* rowptr, int64_t m, int32_t P,
                                          int64_t* bounds) {
  if (!rowptr || !bounds || m < 0 || P < 1) return arg_fail("bad partition arguments");
  const int64_t base = rowptr[0];
  const int64_t nnz = (int64_t)rowptr[m] - base;
  bounds[0] = 0;
  for (int32_t r = 1; r < P; ++r) {
    const int64_t t = ((int64_t)r * nnz) / P;
    int64_t lo = 0, hi = m;
    while (lo < hi) {
      const int64_t mid = lo + ((hi - lo) >> 1);
      if ((int64_t)rowptr[mid] - base >= t) hi = mid; else lo = mid + 1;
    }
    bounds[r] = lo;
  }
  bounds[P] = m;
  return SPMV_OK;
}

extern "C" spmv_status spmv_csr_merge_splits(const int32_t* rowptr, int64_t m, int64_t C,
                                             int64_t* split_row, int64_t* split_nz) {
  if (!rowptr || !split_row || !split_nz || m < 0 || C < 1) return arg_fail("bad merge-split arguments");
  const int64_t base = rowptr[0];
  const int64_t nnz = (int64_t)rowptr[m] - base;
  for (int64_t c = 0; c <= C; ++c) {
    const int64_t d = (c * (m + nnz)) / C;
    // largest i in [max(0,d-nnz), min(d,m)] with row_end(i-1) <= d - i  (i rows consumed)
    int64_t lo = std::max<int64_t>(0, d - nnz), hi = std::min<int64_t>(d, m);
    while (lo < hi) {
      const int64_t i = lo + ((hi - lo + 1) >> 1);
      // consuming i rows needs row end i-1 (value rowptr[i]-base) <= j = d - i
      if ((int64_t)rowptr[i] - base <= d - i) lo = i; else hi = i - 1;
    }
    split_row[c] = lo;
    split_nz[c] = d - lo;
  }
  return SPMV_OK;
}

extern "C" spmv_status spmv_dist_plan_host(const int32_t* rowptr, const int32_t* colidx, int64_t m,
                                           int32_t nranks, int32_t rank, int64_t* bounds,
                                           int64_t* maxlen, int32_t* colidx_local) {
  if (!rowptr || !bounds || !maxlen || nranks < 1 || rank < 0 || rank >= nranks)
    return arg_fail("bad dist plan arguments");
  ST(spmv_csr_partition(rowptr, m, nranks, bounds));
  int64_t ml = 1;
  for (int r = 0; r < nranks; ++r) ml = std::max<int64_t>(ml, bounds[r + 1] - bounds[r]);
  *maxlen = ml;
  if (!colidx_local) return SPMV_OK;
  const int64_t k0 = rowptr[bounds[rank]], k1 = rowptr[bounds[rank + 1]];
  for (int64_t k = k0; k < k1; ++k) {
    const int64_t c = colidx[k];
    // owner: the last rank whose block starts at or before c
    const int64_t* it = std::upper_bound(bounds, bounds + nranks, c);
    const int64_t s = (it - bounds) - 1;
    colidx_local[k - k0] = (int32_t)(s * ml + (c - bounds[s]));
  }
  return SPMV_OK;
}

extern "C" spmv_status spmv_csr_merge_splits_device(spmv_csr_t h, int64_t* split_row, int64_t* split_nz,
                                                    int64_t cap, int64_t* count) {
  if (!h || !count) return arg_fail("NULL argument");
  *count = h->kernel == SPMV_KERNEL_MERGE ? (int64_t)h->mg.ntiles + 1 : 0;
  if (*count == 0 || !split_row || !split_nz) return SPMV_OK;
  if (cap < *count) return arg_fail("cap too small");
  CK(cudaSetDevice(h->device));
  CK(cudaMemcpy(split_row, h->mg.split_row, sizeof(long long) * (size_t)*count, cudaMemcpyDeviceToHost));
  CK(cudaMemcpy(split_nz, h->mg.split_nz, sizeof(long long) * (size_t)*count, cudaMemcpyDeviceToHost));
  return SPMV_OK;
}

extern "C" spmv_status spmv_csr_info(spmv_csr_t h, spmv_info_t* info) {
  if (!h || !info) return arg_fail("NULL argument");
  memset(info, 0, sizeof *info);
  info->kernel = h->kernel;
  info->vec_lanes = h->lanes;
  info->row_min = h->row_min;
  info->row_max = h->row_max;
  info->row_mean = h->row_mean;
  info->row_cv = h->row_cv;
  info->m_local = h->m_loc;
  info->row_begin = h->row0;
  info->row_end = h->row0 + h->m_loc;
  info->nnz_local = h->k1 - h->k0;
  info->rank = h->dist ? h->dist->rank : 0;
  info->transport = h->dist ? (h->dist->p2p ? 2 : h->dist->proxy ? 3 : 1) : 0;
  info->nranks = h->dist ? h->dist->nranks : 1;
  info->sorted_cols = h->sorted;
  info->grid = h->grid;
  info->cluster = h->kernel == SPMV_KERNEL_XPLAN ? h->xp.B
                : h->kernel == SPMV_KERNEL_XT    ? h->xt.B
                : h->kernel == SPMV_KERNEL_XSTAT ? h->xB
                                                 : 0;
  info->plan_bytes = h->xt.built ? (int64_t)h->xt.bytes
                   : h->xp.built ? (int64_t)h->xp.bytes
                   : h->sl.built  ? (int64_t)h->sl.pairs * 64 * (int64_t)(h->ts + 4)
                                  : 0;
  return SPMV_OK;
}

extern "C" uint64_t spmv_launch_count(void) { return g_launches.load(); }

extern "C" const char* spmv_status_string(spmv_status s) {
  switch (s) {
    case SPMV_OK: return "SPMV_OK";
    case SPMV_ERR_ARG: return "SPMV_ERR_ARG";
    case SPMV_ERR_INDEX: return "SPMV_ERR_INDEX";
    case SPMV_ERR_ALIAS: return "SPMV_ERR_ALIAS";
    case SPMV_ERR_CUDA: return "SPMV_ERR_CUDA";
    case SPMV_ERR_NCCL: return "SPMV_ERR_NCCL";
    case SPMV_ERR_NOMEM: return "SPMV_ERR_NOMEM";
    case SPMV_ERR_BREAKDOWN: return "SPMV_ERR_BREAKDOWN";
    case SPMV_ERR_UNSUPPORTED: return "SPMV_ERR_UNSUPPORTED";
  }
  return "unknown spmv_status";
}

extern "C" const char* spmv_last_error_string(void) { return g_err.c_str(); }
