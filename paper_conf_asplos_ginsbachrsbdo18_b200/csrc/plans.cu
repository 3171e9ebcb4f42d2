// plans.cu -- kernel plans of a handle and the local SpMV launch (SURVEY 8(a)
// a1/a2): the x-stationary XPLAN plan, the zero-copy XSTAT
// cluster kernel, the SELL-32 plans (5.3a/5.3c), merge-path tiles (5.3b) and
// run_spmv, which picks among them.  Validation and choice live in
// spmv_abi.cu; arithmetic in the *_kernel.cuh headers.
#include <cub/device/device_radix_sort.cuh>

#include "abi_common.h"
#include "analysis_kernels.cuh"
#include "cg_kernels.cuh"  // k_dot_partials
#include "persist_kernel.cuh"

// ------------------------------------------------------- kernel dispatch
// Launch with the handle's L2 persisting-access window on x (opts.l2_window,
// BJ.ns "an L2 persisting-access window on x") as a per-launch attribute, so
// it is captured into CUDA graphs and leaves the caller's stream unchanged.
// Errors surface through cudaGetLastError (LAUNCHED()).
template <typename... P, typename... A>
static void klaunch(const cudaAccessPolicyWindow* win, void (*k)(P...), dim3 g, dim3 b, cudaStream_t s, A... args) {
  if (!win) {
    k<<<g, b, 0, s>>>(args...);
    return;
  }
  cudaLaunchConfig_t cfg = {};
  cfg.gridDim = g;
  cfg.blockDim = b;
  cfg.stream = s;
  cudaLaunchAttribute at[1];
  at[0].id = cudaLaunchAttributeAccessPolicyWindow;
  at[0].val.accessPolicyWindow = *win;
  cfg.attrs = at;
  cfg.numAttrs = 1;
  cudaLaunchKernelEx(&cfg, k, args...);
}

template <typename T, int G, bool DOT>
static void launch_vec_u(int unroll, int64_t grid, cudaStream_t s, const SpmvArgs& a, const cudaAccessPolicyWindow* w) {
  switch (unroll) {
    case 2: klaunch(w, k_spmv_vector<T, G, 2, DOT>, dim3((unsigned)grid), dim3(256), s, a); break;
    case 8: klaunch(w, k_spmv_vector<T, G, 8, DOT>, dim3((unsigned)grid), dim3(256), s, a); break;
    default: klaunch(w, k_spmv_vector<T, G, 4, DOT>, dim3((unsigned)grid), dim3(256), s, a); break;
  }
}

template <typename T, bool DOT>
static void launch_vec(int lanes, int unroll, int64_t grid, cudaStream_t s, const SpmvArgs& a,
                       const cudaAccessPolicyWindow* w = nullptr) {
  switch (lanes) {
    case 1: launch_vec_u<T, 1, DOT>(unroll, grid, s, a, w); break;
    case 2: launch_vec_u<T, 2, DOT>(unroll, grid, s, a, w); break;
    case 4: launch_vec_u<T, 4, DOT>(unroll, grid, s, a, w); break;
    case 8: launch_vec_u<T, 8, DOT>(unroll, grid, s, a, w); break;
    case 16: launch_vec_u<T, 16, DOT>(unroll, grid, s, a, w); break;
    default: launch_vec_u<T, 32, DOT>(unroll, grid, s, a, w); break;
  }
}

template <typename T, bool DOT, int U>
static void (*xstat_fn_u(int G))(XstatArgs) {
  switch (G) {
    case 4: return k_spmv_xstat<T, 4, U, DOT>;
    case 16: return k_spmv_xstat<T, 16, U, DOT>;
    case 32: return k_spmv_xstat<T, 32, U, DOT>;
    default: return k_spmv_xstat<T, 8, U, DOT>;
  }
}
template <typename T, bool DOT>
static void (*xstat_fn(int G, int U))(XstatArgs) {
  return U == 8 ? xstat_fn_u<T, DOT, 8>(G) : xstat_fn_u<T, DOT, 4>(G);
}

static spmv_status launch_xstat(spmv_csr_s* h, cudaStream_t s, const void* vals, const void* x, void* y,
                                double alpha, double beta, const double* w, double* part, const P2PHook& hook) {
  XstatArgs a;
  a.m = h->m_loc;
  a.nx = h->nx;
  a.W = h->xW;
  a.R = h->xR;
  a.rowptr = h->rp_loc;
  a.colidx = h->ci_loc;
  a.vals = vals;
  a.seg = h->seg;
  a.crow = h->crow;
  a.x = x;
  a.y = y;
  a.alpha = alpha;
  a.beta = beta;
  a.w = w;
  a.part = part;
  a.hk = hook;
  if (h->dt == SPMV_F32) {
    a.alpha = (double)(float)alpha;
    a.beta = (double)(float)beta;
  }
  cudaLaunchConfig_t cfg = {};
  cfg.gridDim = dim3((unsigned)(h->nclusters * h->xB), 1, 1);
  cfg.blockDim = dim3(1024, 1, 1);
  cfg.dynamicSmemBytes = h->xsmem;
  cfg.stream = s;
  cudaLaunchAttribute at[1];
  at[0].id = cudaLaunchAttributeClusterDimension;
  at[0].val.clusterDim.x = (unsigned)h->xB;
  at[0].val.clusterDim.y = 1;
  at[0].val.clusterDim.z = 1;
  cfg.attrs = at;
  cfg.numAttrs = 1;
  CK(cudaLaunchKernelEx(&cfg, part ? h->xk_dot : h->xk, a));
  LAUNCHED();
  return SPMV_OK;
}

// XSTAT set-up (create): column-block width, cluster size, split points,
// static nnz-balanced cluster row ranges.  Returns false if not eligible.
spmv_status xstat_setup(spmv_csr_s* h, bool* ok) {
  *ok = false;
  if (!h->sorted || h->m_loc == 0 || h->nx == 0) return SPMV_OK;
  const size_t budget = 200 * 1024;  // of the 227 KB a CTA may use
  const size_t pb = 3 * (size_t)h->xR * sizeof(double) + 4 * (size_t)h->xR * sizeof(int) + 16;
  if (budget <= pb) return SPMV_OK;
  int B = (int)cdiv((int64_t)h->ts * h->nx, (int64_t)(budget - pb));
  if (B < 1) B = 1;
  // cluster sizes that tile the GPCs well: 1, 2, 4, 8
  B = B <= 1 ? 1 : B <= 2 ? 2 : B <= 4 ? 4 : B <= 8 ? 8 : B;
  int forced = 0;
  if (env_int("SPMV_XSTAT_B", &forced) && forced >= B && forced <= 8) B = forced;
  if (B > 8) return SPMV_OK;
  int W = (int)cdiv(h->nx, B);
  W = (W + 3) & ~3;
  const size_t xbytes = ((size_t)W * h->ts + 15) & ~size_t(15);
  const size_t smem = xbytes + 3 * (size_t)h->xR * sizeof(double) + 4 * (size_t)h->xR * sizeof(int);
  const double seg_mean = h->row_mean / B;
  // lanes x unroll ~ the mean segment length, unroll 8 for memory-level parallelism
  int G = seg_mean < 48 ? 4 : seg_mean < 96 ? 8 : seg_mean < 192 ? 16 : 32;
  int U = 8;
  int g2 = 0;
  if (env_int("SPMV_XSTAT_G", &g2) && (g2 == 4 || g2 == 8 || g2 == 16 || g2 == 32)) G = g2;
  if (tuning_env("SPMV_XSTAT_U", &g2) && (g2 == 4 || g2 == 8)) U = g2;
  void (*fn)(XstatArgs) = h->dt == SPMV_F64 ? xstat_fn<double, false>(G, U) : xstat_fn<float, false>(G, U);
  void (*fnd)(XstatArgs) = h->dt == SPMV_F64 ? xstat_fn<double, true>(G, U) : nullptr;
  CK(cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem));
  if (fnd) CK(cudaFuncSetAttribute(fnd, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem));
  cudaLaunchConfig_t cfg = {};
  cfg.gridDim = dim3((unsigned)B, 1, 1);
  cfg.blockDim = dim3(1024, 1, 1);
  cfg.dynamicSmemBytes = smem;
  cudaLaunchAttribute at[1];
  at[0].id = cudaLaunchAttributeClusterDimension;
  at[0].val.clusterDim.x = (unsigned)B;
  at[0].val.clusterDim.y = 1;
  at[0].val.clusterDim.z = 1;
  cfg.attrs = at;
  cfg.numAttrs = 1;
  int ncl = 0;
  cudaError_t e = cudaOccupancyMaxActiveClusters(&ncl, fn, &cfg);
  if (e != cudaSuccess || ncl < 1) { cudaGetLastError(); return SPMV_OK; }
  int nc_env = 0;
  if (env_int("SPMV_XSTAT_CLUSTERS", &nc_env) && nc_env >= 1 && nc_env <= ncl) ncl = nc_env;
  cudaStream_t s = h->stream;
  if (B > 1) {
    CK(cudaMalloc(&h->seg, sizeof(int) * (size_t)(B - 1) * (size_t)h->m_loc));
    k_xstat_splits<<<std::min<int64_t>(cdiv(h->m_loc, 256), 8LL * num_sms(h->device)), 256, 0, s>>>(
        h->m_loc, h->rp_loc, h->ci_loc, B, W, h->seg);
    LAUNCHED();
  }
  CK(cudaMalloc(&h->crow, sizeof(long long) * (ncl + 1)));
  k_partition<<<cdiv(ncl + 1, 128), 128, 0, s>>>(h->m_loc, h->rp_loc, ncl, h->crow);
  LAUNCHED();
  CK(cudaStreamSynchronize(s));
  h->xB = B;
  h->xW = W;
  h->xG = G;
  h->xsmem = smem;
  h->nclusters = ncl;
  h->xk = fn;
  h->xk_dot = fnd;
  *ok = true;
  return SPMV_OK;
}

static XplanArgs xplan_args(spmv_csr_s* h, const void* x, void* y, double alpha, double beta, const double* w,
                            double* part, const P2PHook& hook) {
  XplanArgs a;
  a.nx = h->nx;
  a.W = h->xp.W;
  a.plan = h->xp.plan;
  a.chunk_off = h->xp.chunk_off;
  a.chunk_len = h->xp.chunk_len;
  a.chunk_row = h->xp.chunk_row;
  a.dbg = dbg() ? 1 : 0;
  a.prefetch = 0;
  tuning_env("SPMV_XPLAN_PF", &a.prefetch);
  a.cta_range = h->xp.cta_range;  // set at build for small plans (whole-range L2 prefetch)
  a.hk = hook;
  a.crow = h->xp.crow;
  a.tile0 = h->xp.tile0;
  a.x = x;
  a.y = y;
  a.alpha = alpha;
  a.beta = beta;
  a.w = w;
  a.part = part;
  if (h->dt == SPMV_F32) {
    a.alpha = (double)(float)alpha;
    a.beta = (double)(float)beta;
  }
  a.tq = h->xp.tq;
  a.tq_done = h->xp.tq ? h->xp.tq + 1 : nullptr;
  a.ntiles_total = h->xp.ntiles;
  a.tstamp = nullptr;
  return a;
}

static spmv_status launch_xplan(spmv_csr_s* h, cudaStream_t s, const void* x, void* y, double alpha,
                                double beta, const double* w, double* part, const P2PHook& hook) {
  XplanArgs a = xplan_args(h, x, y, alpha, beta, w, part, hook);
  cudaLaunchConfig_t cfg = {};
  cfg.gridDim = dim3((unsigned)(h->xp.ncl * h->xp.B), 1, 1);
  cfg.blockDim = dim3(XP_THREADS, 1, 1);
  cfg.dynamicSmemBytes = h->xp.smem;
  cfg.stream = s;
  cudaLaunchAttribute at[3];
  at[0].id = cudaLaunchAttributeClusterDimension;
  at[0].val.clusterDim.x = (unsigned)h->xp.B;
  at[0].val.clusterDim.y = 1;
  at[0].val.clusterDim.z = 1;
  // PDL (programmatic dependent launch): the barrier set-up overlaps the previous
  // kernel's tail (the p2p hooks wait on their peers' flags after pdl_wait)
  at[1].id = cudaLaunchAttributeProgrammaticStreamSerialization;
  at[1].val.programmaticStreamSerializationAllowed = 1;
  cfg.attrs = at;
  cfg.numAttrs = (h->pdl && !h->xp.dyn) ? 2 : 1;
  cudaAccessPolicyWindow cwv;
  if (!h->xp.win_bytes && cg_window(h, &cwv) && (y == h->q || x == (const void*)h->p_single || x == (const void*)h->r)) {
    // a CG SpMV on a plan without its own window: the CG vectors' window (SPMV_CG_L2WIN)
    at[cfg.numAttrs].id = cudaLaunchAttributeAccessPolicyWindow;
    at[cfg.numAttrs].val.accessPolicyWindow = cwv;
    ++cfg.numAttrs;
  }
  if (h->xp.win_bytes) {
    at[cfg.numAttrs].id = cudaLaunchAttributeAccessPolicyWindow;
    at[cfg.numAttrs].val.accessPolicyWindow.base_ptr = h->xp.plan;
    at[cfg.numAttrs].val.accessPolicyWindow.num_bytes = h->xp.win_bytes;
    at[cfg.numAttrs].val.accessPolicyWindow.hitRatio = h->xp.win_ratio;
    at[cfg.numAttrs].val.accessPolicyWindow.hitProp = cudaAccessPropertyPersisting;
    at[cfg.numAttrs].val.accessPolicyWindow.missProp = cudaAccessPropertyStreaming;
    ++cfg.numAttrs;
  }
  int times = 0;
  if (tuning_env("SPMV_XPLAN_TIMES", &times) && times) {
    // diagnostics: per-CTA {start, x ready, streaming done, end} (globaltimer, ns), summarised on stderr
    const size_t nb = sizeof(unsigned long long) * 4 * cfg.gridDim.x;
    CK(cudaMalloc(&a.tstamp, nb));
    CK(cudaMemsetAsync(a.tstamp, 0, nb, s));
  }
  const bool side = h->xp.mplan >= 0 && h->xp.mplan < h->m_loc;
  if (side) {
    if (!h->side) {
      CK(cudaStreamCreateWithFlags(&h->side, cudaStreamNonBlocking));
      CK(cudaEventCreateWithFlags(&h->ev_fork, cudaEventDisableTiming));
      CK(cudaEventCreateWithFlags(&h->ev_join, cudaEventDisableTiming));
    }
    CK(cudaEventRecord(h->ev_fork, s));
    CK(cudaStreamWaitEvent(h->side, h->ev_fork, 0));
  }
  CK(cudaLaunchKernelEx(&cfg, part ? h->xp.kdot : h->xp.k, a));
  LAUNCHED();
  if (side) {
    // rows [mplan, m) in the vector kernel, launched after the clusters so it
    // takes the SMs they leave idle; its dot partials follow the clusters'
    const int64_t ms = h->m_loc - h->xp.mplan;
    SpmvArgs sa;
    sa.m = ms;
    sa.rowptr = h->rp_loc + h->xp.mplan;
    sa.colidx = h->ci_loc;
    sa.vals = h->vals;
    sa.x = x;
    sa.y = (char*)y + h->ts * (size_t)h->xp.mplan;
    sa.alpha = a.alpha;
    sa.beta = a.beta;
    sa.w = w ? (const void*)(w + h->xp.mplan) : nullptr;
    sa.part = part ? part + (h->xp.dyn ? (int64_t)h->xp.ntiles * h->xp.B : (int64_t)cfg.gridDim.x) : nullptr;
    sa.hk = P2PHook();
    if (h->dt == SPMV_F64) {
      if (part) launch_vec<double, true>(h->lanes, h->unroll, h->xp.g2, h->side, sa);
      else launch_vec<double, false>(h->lanes, h->unroll, h->xp.g2, h->side, sa);
    } else {
      launch_vec<float, false>(h->lanes, h->unroll, h->xp.g2, h->side, sa);
    }
    LAUNCHED();
    CK(cudaEventRecord(h->ev_join, h->side));
    CK(cudaStreamWaitEvent(s, h->ev_join, 0));
  }
  if (a.tstamp) {
    std::vector<unsigned long long> t(4 * cfg.gridDim.x);
    CK(cudaMemcpyAsync(t.data(), a.tstamp, sizeof(unsigned long long) * t.size(), cudaMemcpyDeviceToHost, s));
    CK(cudaStreamSynchronize(s));
    cudaFree(a.tstamp);
    unsigned long long t0 = ~0ull, tend = 0;
    for (unsigned i = 0; i < cfg.gridDim.x; ++i) { t0 = std::min(t0, t[4 * i] & ~0xffull); tend = std::max(tend, t[4 * i + 3]); }
    fprintf(stderr, "[xplan times] kernel span %.2f us; per CTA (us from first start): start/xready/streamed/end\n",
            (tend - t0) / 1e3);
    for (unsigned i = 0; i < cfg.gridDim.x; ++i)
      fprintf(stderr, "  cta %3u cl %2u  %6.2f %6.2f %6.2f %6.2f sm %3u\n", i, i / (unsigned)h->xp.B,
              ((t[4 * i] & ~0xffull) - t0) / 1e3, (t[4 * i + 1] - t0) / 1e3, (t[4 * i + 2] - t0) / 1e3,
              (t[4 * i + 3] - t0) / 1e3, unsigned(t[4 * i] & 0xff));
  }
  return SPMV_OK;
}

// Pack (or re-pack, values_only) the nonzeros into the plan chunks, then
// spread each step's x gathers over the shared-memory banks (k_xplan_bankperm;
// a re-pack rewrites the columns in CSR order too, so the deterministic
// permutation is reproduced).
spmv_status xplan_pack(spmv_csr_s* h, const void* vals, int values_only) {
  cudaStream_t s = h->stream;
  auto& P = h->xp;
  const bool perm = P.bankperm && !XP_ODD && P.nchunks > 0;
  if (perm && values_only) {
    // the permuted chunks hold real entries where the CSR order has pads: restore
    // the create-time state (pads everywhere, then every entry in CSR order)
    k_xplan_fill<<<(unsigned)std::min<int64_t>(P.nchunks, 16LL * num_sms(h->device)), 256, 0, s>>>(
        P.plan, P.chunk_off, P.chunk_len, P.nchunks, (int)h->ts, (uint16_t)P.W);
    LAUNCHED();
    values_only = 0;
  }
  const int64_t g = std::min<int64_t>(cdiv(h->m_loc * 32, 256), 16LL * num_sms(h->device));
  if (h->dt == SPMV_F64)
    k_xplan_pack<double><<<g, 256, 0, s>>>(h->rp_loc, h->ci_loc, (const double*)vals, P.seg, h->m_loc, P.B, P.W,
                                          P.crow, P.tile0, P.ncl_plan, P.chunk_off, P.chunk_len, P.row_slot, P.plan,
                                          values_only, P.mplan);
  else
    k_xplan_pack<float><<<g, 256, 0, s>>>(h->rp_loc, h->ci_loc, (const float*)vals, P.seg, h->m_loc, P.B, P.W,
                                         P.crow, P.tile0, P.ncl_plan, P.chunk_off, P.chunk_len, P.row_slot, P.plan,
                                         values_only, P.mplan);
  LAUNCHED();
  if (perm) {
    const unsigned gp = (unsigned)std::min<int64_t>(cdiv(P.nchunks, 8), 64LL * num_sms(h->device));
    if (h->dt == SPMV_F64) k_xplan_bankperm<double><<<gp, 256, 0, s>>>(P.plan, P.chunk_off, P.chunk_len, P.nchunks, P.W);
    else k_xplan_bankperm<float><<<gp, 256, 0, s>>>(P.plan, P.chunk_off, P.chunk_len, P.nchunks, P.W);
    LAUNCHED();
  }
  return SPMV_OK;
}

// Build the column-blocked SELL-32 plan (create).  *ok = false if not eligible.
spmv_status xplan_build(spmv_csr_s* h, bool* ok) {
  *ok = false;
  if (!h->sorted || h->m_loc == 0 || h->nx == 0 || h->k1 - h->k0 == 0) return SPMV_OK;
  const int ts = (int)h->ts;
  const size_t smem_cap = 227 * 1024 - 1024;  // dynamic smem a CTA may use (static < 1 KB)
  const size_t recv = (size_t)XP_K * XP_R * 8;
  if (smem_cap <= recv + 1024) return SPMV_OK;
  const size_t xbudget = smem_cap - recv - 64;
  const int64_t Bneed = cdiv((int64_t)(ts * h->nx), (int64_t)xbudget);
  if (Bneed > 16) return SPMV_OK;  // x does not fit the shared memory of a 16-CTA cluster
  // dynamic tile scheduling (SPMV_XPLAN_DYN=1; measured slower: 85.3 vs 79.9 us on class C,
  // 55.3 vs 45.1 us on B) -- static nnz-balanced cluster row ranges by default
  int dyn = 0;
  env_int("SPMV_XPLAN_DYN", &dyn);
  // bank spreading of each chunk's steps (k_xplan_bankperm; SPMV_XPLAN_PERM=0: CSR order)
  h->xp.bankperm = 1;
  env_int("SPMV_XPLAN_PERM", &h->xp.bankperm);
  void (*fn)(XplanArgs) = h->dt == SPMV_F64 ? (dyn ? k_spmv_xplan<double, false, true> : k_spmv_xplan<double, false, false>)
                                            : (dyn ? k_spmv_xplan<float, false, true> : k_spmv_xplan<float, false, false>);
  void (*fnd)(XplanArgs) =
      h->dt == SPMV_F64 ? (dyn ? k_spmv_xplan<double, true, true> : k_spmv_xplan<double, true, false>) : nullptr;
  // cluster size: any B >= Bneed that divides the tile height R (rows are
  // owned in R/B blocks); among those, the one whose resident clusters cover
  // the most SMs (ties: the smaller B, whose x blocks are larger); clusters of
  // 16 only when nothing smaller fits.  SPMV_XPLAN_B forces a size.
  int forced = 0;
  env_int("SPMV_XPLAN_B", &forced);
  if (forced < Bneed || forced < 2 || forced > 16 || XP_R % std::max(forced, 1)) forced = 0;  // infeasible request: ignored
  int B = 0, W = 0, ncl = 0;
  size_t smem = 0;
  // clusters of >= 2 CTAs: st.async / remote mbarrier completion need a real
  // cluster (compute-sanitizer memcheck rejects them in a 1-CTA "cluster")
  for (int cand = (int)std::max<int64_t>(2, Bneed); cand <= 16; ++cand) {
    if (XP_R % cand) continue;
    if (forced && cand != forced) continue;
    if (cand > 8 && B > 0) break;  // non-portable sizes only as the last resort
    int Wc = (int)cdiv(h->nx, cand);
    Wc = (Wc + 7) & ~7;
    if (Wc > 65534) continue;  // 16-bit column offsets, pad column W
    const size_t sm = (((size_t)(Wc + 1) * ts + 15) & ~size_t(15)) + recv;
    if (sm > smem_cap) continue;
    CK(cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)sm));
    if (cand > 8) CK(cudaFuncSetAttribute(fn, cudaFuncAttributeNonPortableClusterSizeAllowed, 1));
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = dim3((unsigned)cand, 1, 1);
    cfg.blockDim = dim3(XP_THREADS, 1, 1);
    cfg.dynamicSmemBytes = sm;
    cudaLaunchAttribute at[1];
    at[0].id = cudaLaunchAttributeClusterDimension;
    at[0].val.clusterDim.x = (unsigned)cand;
    at[0].val.clusterDim.y = 1;
    at[0].val.clusterDim.z = 1;
    cfg.attrs = at;
    cfg.numAttrs = 1;
    int nc = 0;
    cudaError_t e = cudaOccupancyMaxActiveClusters(&nc, fn, &cfg);
    if (e != cudaSuccess || nc < 1) { cudaGetLastError(); continue; }
    DBG("candidate B=%d W=%d clusters=%d SMs=%d", cand, Wc, nc, nc * cand);
    // prefer >= 2 tiles per cluster (the split tile barrier then overlaps one tile's exchange with
    // the next tile's streaming: class B 35.6 us with B = 8 / 2.4 tiles vs 37.2 us with B = 4 /
    // 1.1 tiles, steady state), then the most SMs
    const bool two = h->m_loc >= 2LL * XP_R * nc, two_best = B > 0 && h->m_loc >= 2LL * XP_R * ncl;
    if (B == 0 || (two && !two_best) || (two == two_best && nc * cand > ncl * B)) {
      B = cand; W = Wc; ncl = nc; smem = sm;
    }
  }
  if (B == 0) return SPMV_OK;
  CK(cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem));
  if (fnd) CK(cudaFuncSetAttribute(fnd, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem));
  if (B > 8) {  // clusters of 16 need the non-portable size
    CK(cudaFuncSetAttribute(fn, cudaFuncAttributeNonPortableClusterSizeAllowed, 1));
    if (fnd) CK(cudaFuncSetAttribute(fnd, cudaFuncAttributeNonPortableClusterSizeAllowed, 1));
  }
  int nc_env = 0;
  if (env_int("SPMV_XPLAN_CLUSTERS", &nc_env) && nc_env >= 1 && nc_env <= ncl) ncl = nc_env;
  cudaStream_t s = h->stream;
  auto& P = h->xp;
  auto cleanup = [&]() {
    void* bufs[] = {P.crow, P.chunk_off, P.tile0, P.chunk_len, P.seg, P.row_slot, P.chunk_row, P.plan, P.tq,
                    P.cta_range};
    for (void* q : bufs)
      if (q) cudaFree(q);
    P = spmv_csr_s::XPlan();
  };
  P.B = B; P.W = W; P.ncl = ncl; P.smem = smem; P.k = fn; P.kdot = fnd; P.dyn = dyn;
  // DYN: the plan is one row range cut into tiles the clusters pop at run time
  const int ncl_plan = dyn ? 1 : ncl;
  DBG("B=%d W=%d ncl=%d smem=%zu", B, W, ncl, smem);
  const int64_t m = h->m_loc;
  // side split: the last SPMV_XPLAN_SIDE per mille of the nonzeros go to the
  // vector kernel on the idle SMs (single GPU only)
  P.mplan = m;
  {
    int side_pm = 0;
    tuning_env("SPMV_XPLAN_SIDE", &side_pm);
    const int idle = num_sms(h->device) - ncl * B;
    if (side_pm > 0 && side_pm < 500 && !h->dist && idle > 0) {
      std::vector<int> rph((size_t)m + 1);
      CK(cudaMemcpyAsync(rph.data(), h->rp_loc, sizeof(int) * (m + 1), cudaMemcpyDeviceToHost, s));
      CK(cudaStreamSynchronize(s));
      const long long nz = (long long)rph[m] - rph[0];
      const long long target = rph[0] + nz - nz * side_pm / 1000;
      P.mplan = std::lower_bound(rph.begin(), rph.end(), (int)target) - rph.begin();
      P.mplan = std::min<int64_t>(std::max<int64_t>(P.mplan, 1), m);
      P.g2 = idle * 8;
      DBG("side split: plan rows %lld of %lld, side grid %d", (long long)P.mplan, (long long)m, P.g2);
    }
  }
  CK(cudaMalloc(&P.crow, sizeof(long long) * (ncl_plan + 1)));
  k_partition<<<cdiv(ncl_plan + 1, 128), 128, 0, s>>>(P.mplan, h->rp_loc, ncl_plan, P.crow);
  LAUNCHED();
  std::vector<long long> crow(ncl_plan + 1);
  CK(cudaMemcpyAsync(crow.data(), P.crow, sizeof(long long) * (ncl_plan + 1), cudaMemcpyDeviceToHost, s));
  CK(cudaStreamSynchronize(s));
  std::vector<int> tile0(ncl_plan + 1, 0);
  for (int c = 0; c < ncl_plan; ++c) tile0[c + 1] = tile0[c] + (int)cdiv(crow[c + 1] - crow[c], XP_R);
  const int ntiles = tile0[ncl_plan];
  P.ntiles = ntiles;
  DBG("ntiles=%d", ntiles);
  CK(cudaMalloc(&P.tile0, sizeof(int) * (ncl_plan + 1)));
  CK(cudaMemcpyAsync(P.tile0, tile0.data(), sizeof(int) * (ncl_plan + 1), cudaMemcpyHostToDevice, s));
  if (B > 1) {
    CK(cudaMalloc(&P.seg, sizeof(int) * (size_t)(B - 1) * (size_t)m));
    k_xstat_splits<<<std::min<int64_t>(cdiv(m, 256), 8LL * num_sms(h->device)), 256, 0, s>>>(
        m, h->rp_loc, h->ci_loc, B, W, P.seg);
    LAUNCHED();
  }
  DBG("splits done");
  const int64_t nch = (int64_t)ntiles * B * XP_CPT;
  P.nchunks = nch;
  CK(cudaMalloc(&P.chunk_len, sizeof(int) * std::max<int64_t>(nch, 1)));
  CK(cudaMalloc(&P.chunk_off, sizeof(long long) * std::max<int64_t>(nch, 1)));
  CK(cudaMalloc(&P.chunk_row, sizeof(uint16_t) * 32 * std::max<int64_t>(nch, 1)));
  CK(cudaMalloc(&P.row_slot, sizeof(int) * (size_t)B * (size_t)m));
  if (ntiles > 0) {
    k_xplan_sell<<<(unsigned)(ntiles * B), XP_THREADS, 0, s>>>(h->rp_loc, P.seg, m, B, P.crow, P.tile0, ncl_plan, P.chunk_len,
                                                          P.chunk_row, P.row_slot);
    LAUNCHED();
  }
  DBG("sell done nch=%lld", (long long)nch);
  std::vector<int> len(std::max<int64_t>(nch, 1), 0);
  CK(cudaMemcpyAsync(len.data(), P.chunk_len, sizeof(int) * nch, cudaMemcpyDeviceToHost, s));
  CK(cudaStreamSynchronize(s));
  // padding check: SELL must not blow up the stream (skewed segments)
  long long steps = 0;
  for (int64_t i = 0; i < nch; ++i) steps += len[i];
  const long long padded = steps * 32;
  const long long real = h->k1 - h->k0;
  double maxpad = 1.5;
  if (padded > (long long)(maxpad * (double)real) + 64LL * nch) {
    cleanup();
    return SPMV_OK;
  }
  // chunk offsets in stream order [c][b][t][w]: the chunks of one CTA are contiguous
  std::vector<long long> off(std::max<int64_t>(nch, 1), 0);
  long long pos = 0;
  for (int c = 0; c < ncl_plan; ++c)
    for (int bb = 0; bb < B; ++bb)
      for (int t = tile0[c]; t < tile0[c + 1]; ++t)
        for (int w = 0; w < XP_CPT; ++w) {
          const size_t id = ((size_t)t * B + bb) * XP_CPT + w;
          off[id] = pos;
          pos += (long long)len[id] * 32 * (ts + 2);
        }
  P.bytes = pos;
  P.ncl_plan = ncl_plan;
  // small plans: each CTA prefetches its whole contiguous chunk range into L2 at
  // kernel start; SPMV_XPLAN_L2PF=0/1 forces it off/on
  {
    // plans that stay L2-resident across CG iterations (<= 96 MB of the 126 MB L2; measured on the
    // class-C rank blocks: P = 4 (94 MB) 38.1 -> 32.2 us, P = 8 (47 MB) 24.4 -> 21.4 us per CG
    // iteration; P = 2 (188 MB) and the whole matrix lose: the prefetch thrashes L2)
    // plans that fit the device's persisting-L2 carve-out (B200: 79 MB; the P = 8 rank block's 47 MB)
    // are pinned there instead: a persisting access window over the plan on every launch
    // (SPMV_XPLAN_PLANWIN=0/1 forces it).  Measured, class-C P = 8 block (profiles/r02u_*): CG
    // iteration 16.67 vs 16.86 us (graph path), 17.15 vs 17.48 us (persistent), SpMV back to back
    // 0.664 vs 0.585 of the copy peak; the P = 4 block (94 MB) only fits partly and keeps the prefetch
    // (31.7 us with the window vs 25.7 us with the prefetch).
    {
      int maxwin = 0, maxpersist = 0;
      cudaDeviceGetAttribute(&maxwin, cudaDevAttrMaxAccessPolicyWindowSize, h->device);
      cudaDeviceGetAttribute(&maxpersist, cudaDevAttrMaxPersistingL2CacheSize, h->device);
      int pw = (!dyn && maxwin > 0 && maxpersist > 0 && pos <= (long long)maxpersist && pos <= (long long)maxwin) ? 1 : 0;
      env_int("SPMV_XPLAN_PLANWIN", &pw);
      if (pw && maxwin > 0 && maxpersist > 0) {
        size_t cur = 0;
        cudaDeviceGetLimit(&cur, cudaLimitPersistingL2CacheSize);
        const size_t want = std::min<size_t>((size_t)pos, (size_t)maxpersist);
        if (want > cur && cudaDeviceSetLimit(cudaLimitPersistingL2CacheSize, want) != cudaSuccess) cudaGetLastError();
        cudaDeviceGetLimit(&cur, cudaLimitPersistingL2CacheSize);
        if (cur > 0) {
          P.win_bytes = std::min<size_t>((size_t)pos, (size_t)maxwin);
          P.win_ratio = (float)std::min(1.0, (double)cur / (double)P.win_bytes);
        }
      }
    }
    int pf = (!dyn && !P.win_bytes && pos <= (long long)(96) << 20) ? 1 : 0;
    env_int("SPMV_XPLAN_L2PF", &pf);
    if (pf && !dyn) {
      std::vector<long long> rng(2 * (size_t)ncl * B, 0);
      for (int c = 0; c < ncl; ++c)
        for (int bb = 0; bb < B; ++bb) {
          long long lo = 0, hi = 0;
          if (tile0[c + 1] > tile0[c]) {
            const size_t first = ((size_t)tile0[c] * B + bb) * XP_CPT;
            const size_t last = ((size_t)(tile0[c + 1] - 1) * B + bb) * XP_CPT + XP_CPT - 1;
            lo = off[first];
            hi = off[last] + (long long)len[last] * 32 * (ts + 2);
          }
          rng[2 * ((size_t)c * B + bb)] = lo;
          rng[2 * ((size_t)c * B + bb) + 1] = hi;
        }
      CK(cudaMalloc(&P.cta_range, sizeof(long long) * rng.size()));
      CK(cudaMemcpyAsync(P.cta_range, rng.data(), sizeof(long long) * rng.size(), cudaMemcpyHostToDevice, s));
    }
  }
  if (dyn) {
    CK(cudaMalloc(&P.tq, sizeof(int) * 2));
    CK(cudaMemsetAsync(P.tq, 0, sizeof(int) * 2, s));
  }
  CK(cudaMemcpyAsync(P.chunk_off, off.data(), sizeof(long long) * nch, cudaMemcpyHostToDevice, s));
  CK(cudaMalloc(&P.plan, (size_t)std::max<long long>(pos, 16)));
  if (nch > 0) {
    k_xplan_fill<<<(unsigned)std::min<int64_t>(nch, 16LL * num_sms(h->device)), 256, 0, s>>>(
        P.plan, P.chunk_off, P.chunk_len, nch, ts, (uint16_t)W);
    LAUNCHED();
  }
  DBG("fill done bytes=%lld", (long long)pos);
  ST(xplan_pack(h, h->vals, 0));
  DBG("pack done");
  CK(cudaStreamSynchronize(s));
  P.built = true;
  *ok = true;
  return SPMV_OK;
}

// ------------------------------------------------------------------ SELL
spmv_status sell_pack(spmv_csr_s* h, const void* vals, int values_only) {
  cudaStream_t s = h->stream;
  const auto& S = h->sl;
  const int64_t g = std::max<int64_t>(1, std::min<int64_t>(cdiv(h->m_loc - S.nlong, 256), 16LL * num_sms(h->device)));
  if (h->dt == SPMV_F64)
    k_sell_pack<double><<<g, 256, 0, s>>>(h->m_loc, h->rp_loc, h->ci_loc, (const double*)vals, S.pair_off, S.perm,
                                          S.nlong, (double*)S.vals, S.cols, values_only);
  else
    k_sell_pack<float><<<g, 256, 0, s>>>(h->m_loc, h->rp_loc, h->ci_loc, (const float*)vals, S.pair_off, S.perm,
                                         S.nlong, (float*)S.vals, S.cols, values_only);
  LAUNCHED();
  return SPMV_OK;
}

// Build the SELL-32 plan (create).  sorted = 0: chunks of consecutive rows;
// sorted = 1: rows ordered by length (descending, stable device radix sort),
// rows longer than SELL_LONG kept in the CSR and processed warp-per-row.
// Not eligible (*ok = false) when the padding exceeds max_pad x nnz.
spmv_status sell_build(spmv_csr_s* h, double max_pad, int sorted, bool* ok) {
  *ok = false;
  const int64_t m = h->m_loc, nnz = h->k1 - h->k0;
  if (m == 0 || nnz == 0) return SPMV_OK;
  if (sorted && m > 2147483647LL) return SPMV_OK;
  cudaStream_t s = h->stream;
  auto& S = h->sl;
  auto cleanup = [&]() {
    void* bufs[] = {S.pair_off, S.vals, S.cols, S.perm, S.seg, S.seg_part, S.seg_cnt};
    for (void* q : bufs)
      if (q) cudaFree(q);
    S = spmv_csr_s::Sell();
  };
  const int sms = num_sms(h->device);
  if (sorted) {
    int *keys = nullptr, *keys_out = nullptr, *ids = nullptr;
    void* tmp = nullptr;
    size_t tmp_bytes = 0;
    CK(cudaMalloc(&keys, sizeof(int) * m));
    CK(cudaMalloc(&keys_out, sizeof(int) * m));
    CK(cudaMalloc(&ids, sizeof(int) * m));
    CK(cudaMalloc(&S.perm, sizeof(int) * m));
    k_row_len_ids<<<(unsigned)std::min<int64_t>(cdiv(m, 256), 8LL * sms), 256, 0, s>>>(m, h->rp_loc, keys, ids);
    LAUNCHED();
    CK(cub::DeviceRadixSort::SortPairsDescending(nullptr, tmp_bytes, keys, keys_out, ids, S.perm, (int)m, 0, 32, s));
    CK(cudaMalloc(&tmp, tmp_bytes));
    CK(cub::DeviceRadixSort::SortPairsDescending(tmp, tmp_bytes, keys, keys_out, ids, S.perm, (int)m, 0, 32, s));
    std::vector<int> sk(m);
    CK(cudaMemcpyAsync(sk.data(), keys_out, sizeof(int) * m, cudaMemcpyDeviceToHost, s));
    CK(cudaStreamSynchronize(s));
    cudaFree(tmp);
    cudaFree(keys);
    cudaFree(keys_out);
    cudaFree(ids);
    // long rows: the prefix with length > SELL_LONG, cut into segments of <= SELL_SEG entries
    S.nlong = std::lower_bound(sk.begin(), sk.end(), SELL_LONG, std::greater<int>()) - sk.begin();
    if (S.nlong > 0) {
      std::vector<int> lp(S.nlong), rp(m + 1);
      CK(cudaMemcpy(lp.data(), S.perm, sizeof(int) * S.nlong, cudaMemcpyDeviceToHost));
      CK(cudaMemcpy(rp.data(), h->rp_loc, sizeof(int) * (m + 1), cudaMemcpyDeviceToHost));
      std::vector<SellSeg> segs;
      int npart = 0, ncnt = 0;
      for (int64_t j = 0; j < S.nlong; ++j) {
        const int i = lp[j], k0 = rp[i], k1 = rp[i + 1];
        const int ns = (int)cdiv(k1 - k0, SELL_SEG);
        for (int q = 0; q < ns; ++q) {
          SellSeg g{};
          g.row = i;
          g.k0 = k0 + q * SELL_SEG;
          g.k1 = std::min(k1, g.k0 + SELL_SEG);
          g.pbase = ns > 1 ? npart : -1;
          g.sidx = q;
          g.nseg = ns;
          g.cslot = ns > 1 ? ncnt : -1;
          segs.push_back(g);
        }
        if (ns > 1) { npart += ns; ++ncnt; }
      }
      S.nseg = (int64_t)segs.size();
      S.nmulti = ncnt;
      CK(cudaMalloc(&S.seg, sizeof(SellSeg) * segs.size()));
      CK(cudaMemcpy(S.seg, segs.data(), sizeof(SellSeg) * segs.size(), cudaMemcpyHostToDevice));
      CK(cudaMalloc(&S.seg_part, sizeof(double) * std::max(npart, 1)));
      CK(cudaMalloc(&S.seg_cnt, sizeof(int) * std::max(ncnt, 1)));
      CK(cudaMemset(S.seg_cnt, 0, sizeof(int) * std::max(ncnt, 1)));
    }
  }
  const int64_t nch = cdiv(m - S.nlong, 32);
  CK(cudaMalloc(&S.pair_off, sizeof(long long) * (nch + 1)));
  if (nch > 0) {
    const unsigned g = (unsigned)std::max<int64_t>(1, std::min<int64_t>(cdiv(nch, 256), 8LL * sms));
    if (sorted) k_sell_pairs_sorted<<<g, 256, 0, s>>>(m, h->rp_loc, S.perm, S.nlong, nch, S.pair_off);
    else k_sell_pairs<<<g, 256, 0, s>>>(m, h->rp_loc, nch, S.pair_off);
    LAUNCHED();
  }
  std::vector<long long> off(nch + 1);
  CK(cudaMemcpyAsync(off.data(), S.pair_off, sizeof(long long) * nch, cudaMemcpyDeviceToHost, s));
  CK(cudaStreamSynchronize(s));
  long long pos = 0;
  for (int64_t c = 0; c < nch; ++c) {
    const long long np = off[c];
    off[c] = pos;
    pos += np;
  }
  off[nch] = pos;
  if ((double)pos * 64.0 > max_pad * (double)nnz + 64.0) {
    cleanup();
    return SPMV_OK;
  }
  S.nchunks = nch;
  S.pairs = pos;
  const size_t slots = (size_t)std::max<long long>(pos, 1) * 64;  // 32 lanes x 2 steps
  CK(cudaMemcpyAsync(S.pair_off, off.data(), sizeof(long long) * (nch + 1), cudaMemcpyHostToDevice, s));
  CK(cudaMalloc(&S.vals, slots * h->ts));
  CK(cudaMalloc(&S.cols, slots * sizeof(int)));
  CK(cudaMemsetAsync(S.vals, 0, slots * h->ts, s));
  CK(cudaMemsetAsync(S.cols, 0xff, slots * sizeof(int), s));  // -1: padding
  ST(sell_pack(h, h->vals, 0));
  CK(cudaStreamSynchronize(s));
  // grid: 8 CTAs of SELL_NT per SM, never more warps than work items
  S.grid = std::max<int64_t>(1, std::min<int64_t>(cdiv(nch + S.nseg, SELL_NT / 32), 8LL * sms));
  S.sorted = sorted;
  S.built = true;
  *ok = true;
  return SPMV_OK;
}

static spmv_status launch_sell(spmv_csr_s* h, cudaStream_t s, const void* x, void* y, double alpha, double beta,
                               const double* w, double* part, const P2PHook& hook, const cudaAccessPolicyWindow* win) {
  SellArgs a;
  a.m = h->m_loc;
  a.nchunks = h->sl.nchunks;
  a.perm = h->sl.perm;
  a.nlong = h->sl.nlong;
  a.nseg = h->sl.nseg;
  a.seg = h->sl.seg;
  a.seg_part = h->sl.seg_part;
  a.seg_cnt = h->sl.seg_cnt;
  a.colidx = h->ci_loc;
  a.csr_vals = h->vals;
  a.vals = h->sl.vals;
  a.cols = reinterpret_cast<const int2*>(h->sl.cols);
  a.pair_off = h->sl.pair_off;
  a.x = x;
  a.y = y;
  a.alpha = alpha;
  a.beta = beta;
  a.w = w;
  a.part = part;
  a.hk = hook;
  const unsigned g = (unsigned)h->sl.grid;
  if (h->dt == SPMV_F64) {
    if (part && h->sl.nmulti > 0) {
      // multi-segment rows are finished by whichever warp completes them: the dot
      // runs as a separate pass so its per-CTA partials stay deterministic
      P2PHook wait_only = hook;
      wait_only.push_slot = -1;
      a.hk = wait_only;
      klaunch(win, k_spmv_sell<double, false>, dim3(g), dim3(SELL_NT), s, a);
      LAUNCHED();
      P2PHook push_only = hook;
      push_only.wait_x = 0;
      k_dot_partials<<<(int)h->vgrid, 256, 0, s>>>(h->m_loc, w, (const double*)y, part, push_only);
    } else if (part) {
      klaunch(win, k_spmv_sell<double, true>, dim3(g), dim3(SELL_NT), s, a);
    } else {
      klaunch(win, k_spmv_sell<double, false>, dim3(g), dim3(SELL_NT), s, a);
    }
  } else {
    a.alpha = (double)(float)alpha;
    a.beta = (double)(float)beta;
    klaunch(win, k_spmv_sell<float, false>, dim3(g), dim3(SELL_NT), s, a);
  }
  LAUNCHED();
  return SPMV_OK;
}

spmv_status merge_setup(spmv_csr_s* h) {
  const int64_t items = h->m_loc + (h->k1 - h->k0);
  const int64_t C = std::max<int64_t>(1, cdiv(items, MG_D));
  if (C > 2147483647LL) return arg_fail("matrix too large for the merge kernel");
  auto& G = h->mg;
  G.ntiles = (int)C;
  CK(cudaMalloc(&G.split_row, sizeof(long long) * (C + 1)));
  CK(cudaMalloc(&G.split_nz, sizeof(long long) * (C + 1)));
  CK(cudaMalloc(&G.head, sizeof(double) * C));
  CK(cudaMalloc(&G.carry, sizeof(double) * C));
  CK(cudaMalloc(&G.head_flag, sizeof(int) * C));
  k_merge_splits<<<(unsigned)cdiv(C + 1, 256), 256, 0, h->stream>>>(h->m_loc, h->rp_loc, C, G.split_row, G.split_nz);
  LAUNCHED();
  CK(cudaStreamSynchronize(h->stream));
  return SPMV_OK;
}

static spmv_status launch_merge(spmv_csr_s* h, cudaStream_t s, const void* vals, const void* x, void* y,
                                double alpha, double beta, const P2PHook& hook, const cudaAccessPolicyWindow* win) {
  MergeArgs a;
  a.m = h->m_loc;
  a.ntiles = h->mg.ntiles;
  a.rowptr = h->rp_loc;
  a.colidx = h->ci_loc;
  a.vals = vals;
  a.split_row = h->mg.split_row;
  a.split_nz = h->mg.split_nz;
  a.x = x;
  a.y = y;
  a.alpha = alpha;
  a.beta = beta;
  a.head = h->mg.head;
  a.carry = h->mg.carry;
  a.head_flag = h->mg.head_flag;
  a.hk = hook;
  if (h->dt == SPMV_F64) {
    klaunch(win, k_spmv_merge<double>, dim3((unsigned)a.ntiles), dim3(MG_NT), s, a);
    LAUNCHED();
    k_merge_fixup<double><<<(unsigned)cdiv(a.ntiles, 256), 256, 0, s>>>(a);
    LAUNCHED();
  } else {
    a.alpha = (double)(float)alpha;
    a.beta = (double)(float)beta;
    klaunch(win, k_spmv_merge<float>, dim3((unsigned)a.ntiles), dim3(MG_NT), s, a);
    LAUNCHED();
    k_merge_fixup<float><<<(unsigned)cdiv(a.ntiles, 256), 256, 0, s>>>(a);
    LAUNCHED();
  }
  return SPMV_OK;
}

spmv_status run_spmv(spmv_csr_s* h, cudaStream_t s, const void* vals, const void* x, void* y, double alpha,
                     double beta, const double* w, double* part, const P2PHook* hk) {
  const P2PHook hook = hk ? *hk : P2PHook();
  if (h->m_loc == 0) {
    if (part) {
      CK(cudaMemsetAsync(part, 0, sizeof(double) * h->grid, s));
    }
    return SPMV_OK;
  }
  if (alpha == 0.0 && !part) {
    const int64_t g = std::min<int64_t>(cdiv(h->m_loc, 256), 4 * num_sms(h->device));
    if (h->dt == SPMV_F64) k_scale<double><<<g, 256, 0, s>>>(h->m_loc, (double*)y, beta);
    else k_scale<float><<<g, 256, 0, s>>>(h->m_loc, (float*)y, (double)(float)beta);
    LAUNCHED();
    return SPMV_OK;
  }
  if (h->kernel == SPMV_KERNEL_XT && vals == h->vals) return launch_xt(h, s, x, y, alpha, beta, w, part, hook);
  if (h->kernel == SPMV_KERNEL_XPLAN && vals == h->vals) return launch_xplan(h, s, x, y, alpha, beta, w, part, hook);
  const bool sell = h->kernel == SPMV_KERNEL_SELL || h->kernel == SPMV_KERNEL_SELL_SORTED;
  // opts.l2_window: persisting L2 window over x for the kernels that gather x through L1/L2
  cudaAccessPolicyWindow win_v = {};
  const cudaAccessPolicyWindow* win = nullptr;
  if (h->l2win_bytes > 0 && x) {
    win_v.base_ptr = const_cast<void*>(x);
    win_v.num_bytes = std::min<size_t>(h->ts * (size_t)h->nx, h->l2win_bytes);
    win_v.hitRatio = (float)std::min(1.0, (double)h->l2persist_bytes / (double)std::max<size_t>(win_v.num_bytes, 1));
    win_v.hitProp = cudaAccessPropertyPersisting;
    win_v.missProp = cudaAccessPropertyStreaming;
    win = &win_v;
  }
  if (sell && vals == h->vals) return launch_sell(h, s, x, y, alpha, beta, w, part, hook, win);
  const int64_t vgrid_spmv = (h->kernel == SPMV_KERNEL_XPLAN || h->kernel == SPMV_KERNEL_XT || sell) ? h->grid_vec : h->grid;
  if (h->kernel == SPMV_KERNEL_XSTAT) return launch_xstat(h, s, vals, x, y, alpha, beta, w, part, hook);
  if (h->kernel == SPMV_KERNEL_MERGE) {
    P2PHook wait_only = hook;
    wait_only.push_slot = -1;
    ST(launch_merge(h, s, vals, x, y, alpha, beta, wait_only, win));
    if (part) {  // no fused dot in the merge kernel: one pass over w, y
      P2PHook push_only = hook;
      push_only.wait_x = 0;
      k_dot_partials<<<(int)h->vgrid, 256, 0, s>>>(h->m_loc, w, (const double*)y, part, push_only);
      LAUNCHED();
    }
    return SPMV_OK;
  }
  SpmvArgs a;
  a.m = h->m_loc;
  a.rowptr = h->rp_loc;
  a.colidx = h->ci_loc;
  a.vals = vals;
  a.x = x;
  a.y = y;
  a.alpha = alpha;
  a.beta = beta;
  a.w = w;
  a.part = part;
  a.hk = hook;
  if (h->dt == SPMV_F64) {
    if (part) launch_vec<double, true>(h->lanes, h->unroll, vgrid_spmv, s, a, win);
    else launch_vec<double, false>(h->lanes, h->unroll, vgrid_spmv, s, a, win);
  } else {
    a.alpha = (double)(float)alpha;
    a.beta = (double)(float)beta;
    launch_vec<float, false>(h->lanes, h->unroll, vgrid_spmv, s, a, win);
  }
  LAUNCHED();
  return SPMV_OK;
}

// ------------------------------------------------------------- NEXT-1
// Persistent single-reduction CG over the XPLAN plan (persist_kernel.cuh):
// eligible with the static XPLAN plan whose co-resident clusters fit the grid.
bool persist_eligible(const spmv_csr_s* h) {
  if (h->kernel != SPMV_KERNEL_XPLAN || !h->xp.built || h->xp.dyn || h->dt != SPMV_F64) return false;
  if (h->xp.mplan >= 0 && h->xp.mplan < h->m_loc) return false;  // side split
  // real transports exchange x and the scalars between iterations: not inside this kernel
  // (no cross-GPU grid barrier); the proxy transport has no exchanges
  if (h->dist && !h->dist->proxy) return false;
  return true;
}

spmv_status launch_cg_persist(spmv_csr_s* h, cudaStream_t s, const void* x_input, double* r, double* p, double* sv,
                              double* w, double* z, double* part_d, double* part_g, int64_t pstride,
                              const double* gam0, int gam0_count, int iters) {
  void (*kfn)(PersistArgs) = k_cg_persist;
  static std::atomic<size_t> attr_smem{0};  // largest dynamic smem requested so far
  if (h->xp.smem > attr_smem.load()) {
    CK(cudaFuncSetAttribute(kfn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)h->xp.smem));
    attr_smem.store(h->xp.smem);
  }
  if (!h->gbar) return arg_fail("internal: persistent CG without its barrier counter (cg_alloc)");
  CK(cudaMemsetAsync(h->gbar, 0, sizeof(unsigned int), s));
  PersistArgs pa;
  pa.sp = xplan_args(h, x_input, w, 1.0, 0.0, r, part_d, P2PHook());
  pa.n = h->m_loc;
  pa.iters = iters;
  pa.r = r;
  pa.p = p;
  pa.s = sv;
  pa.w = w;
  pa.z = z;
  pa.part_d = part_d;
  pa.part_g = part_g;
  pa.pstride = pstride;
  pa.gam0 = gam0;
  pa.gam0_count = gam0_count;
  pa.alpha2 = h->alpha2;
  pa.flags = h->flags;
  pa.gbar = h->gbar;
  cudaLaunchConfig_t cfg = {};
  cfg.gridDim = dim3((unsigned)(h->xp.ncl * h->xp.B), 1, 1);
  cfg.blockDim = dim3(XP_THREADS, 1, 1);
  cfg.dynamicSmemBytes = h->xp.smem;
  cfg.stream = s;
  cudaLaunchAttribute at[2];
  at[0].id = cudaLaunchAttributeClusterDimension;
  at[0].val.clusterDim.x = (unsigned)h->xp.B;
  at[0].val.clusterDim.y = 1;
  at[0].val.clusterDim.z = 1;
  cfg.attrs = at;
  cfg.numAttrs = 1;
  if (h->xp.win_bytes) {  // the plan pinned in the persisting L2 carve-out (see xplan_build)
    at[1].id = cudaLaunchAttributeAccessPolicyWindow;
    at[1].val.accessPolicyWindow.base_ptr = h->xp.plan;
    at[1].val.accessPolicyWindow.num_bytes = h->xp.win_bytes;
    at[1].val.accessPolicyWindow.hitRatio = h->xp.win_ratio;
    at[1].val.accessPolicyWindow.hitProp = cudaAccessPropertyPersisting;
    at[1].val.accessPolicyWindow.missProp = cudaAccessPropertyStreaming;
    cfg.numAttrs = 2;
  } else {
    cudaAccessPolicyWindow cwv;  // no plan window: the CG vectors' (see cg_alloc)
    if (cg_window(h, &cwv)) {
      at[1].id = cudaLaunchAttributeAccessPolicyWindow;
      at[1].val.accessPolicyWindow = cwv;
      cfg.numAttrs = 2;
    }
  }
  int times = 0;
  if (tuning_env("SPMV_PERSIST_TIMES", &times) && times) {
    // diagnostics (cg_solve only: synchronises): per-CTA phase stamps of iteration iters/2
    const size_t nb = sizeof(unsigned long long) * 8 * cfg.gridDim.x;
    CK(cudaMalloc(&pa.sp.tstamp, nb));
    CK(cudaMemsetAsync(pa.sp.tstamp, 0, nb, s));
  }
  CK(cudaLaunchKernelEx(&cfg, kfn, pa));
  LAUNCHED();
  if (pa.sp.tstamp) {
    const unsigned G = cfg.gridDim.x;
    std::vector<unsigned long long> t(8 * G);
    CK(cudaMemcpyAsync(t.data(), pa.sp.tstamp, sizeof(unsigned long long) * t.size(), cudaMemcpyDeviceToHost, s));
    CK(cudaStreamSynchronize(s));
    cudaFree(pa.sp.tstamp);
    unsigned long long t0 = ~0ull;
    for (unsigned i = 0; i < G; ++i) t0 = std::min(t0, t[8 * i]);
    const char* nm[8] = {"start", "xready", "streamed", "spmv_done", "bar1", "update_done", "bar2", "scalars"};
    fprintf(stderr, "[persist times] iteration %d, us from the first CTA's start: median / max over %u CTAs\n",
            iters / 2, G);
    for (int ph : {0, 1, 2, 3, 4, 7, 5, 6}) {
      std::vector<double> v(G);
      for (unsigned i = 0; i < G; ++i) v[i] = (double)(t[8 * i + ph] - t0) / 1e3;
      std::sort(v.begin(), v.end());
      fprintf(stderr, "  %-12s med %7.2f  min %7.2f  max %7.2f\n", nm[ph], v[G / 2], v[0], v[G - 1]);
    }
  }
  return SPMV_OK;
}
