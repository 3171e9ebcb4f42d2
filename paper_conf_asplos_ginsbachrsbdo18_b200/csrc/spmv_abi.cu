// spmv_abi.cu -- the C ABI of include/spmv.h: handle management, argument and
// alias checks, kernel selection, the CG drivers (CUDA-graph captured) and the
// NCCL row-sharded mode.  All arithmetic of the hot path runs in the kernels of
// spmv_kernels.cuh / cg_kernels.cuh; this file only validates, chooses and
// launches.  P:a-b = /root/reference/PAPER.md lines; Rn = DESIGN.md reading n.
#include <algorithm>
#include <atomic>
#include <cmath>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <string>
#include <vector>

#include <cub/device/device_radix_sort.cuh>
#include <cuda_runtime.h>
#include <nccl.h>
#include <functional>

#include "../../include/spmv.h"
#include "analysis_kernels.cuh"
#include "cg_kernels.cuh"
#include "spmv_kernels.cuh"
#include "xstat_kernel.cuh"
#include "xplan_kernel.cuh"
#include "merge_kernel.cuh"
#include "sell_kernel.cuh"
#include "stencil_kernel.cuh"
#include "p2p_kernels.cuh"

using namespace spmv;

// ------------------------------------------------------------------ errors
static thread_local std::string g_err = "no error";
static std::atomic<uint64_t> g_launches{0};

static spmv_status cuda_fail(cudaError_t e, const char* what, int line) {
  char buf[512];
  snprintf(buf, sizeof buf, "%s (line %d): %s", what, line, cudaGetErrorString(e));
  g_err = buf;
  return e == cudaErrorMemoryAllocation ? SPMV_ERR_NOMEM : SPMV_ERR_CUDA;
}
static spmv_status arg_fail(const char* why) {
  g_err = why;
  return SPMV_ERR_ARG;
}
#define CK(call)                                                   \
  do {                                                             \
    cudaError_t e__ = (call);                                      \
    if (e__ != cudaSuccess) return cuda_fail(e__, #call, __LINE__); \
  } while (0)
#define NK(call)                                                   \
  do {                                                             \
    ncclResult_t r__ = (call);                                     \
    if (r__ != ncclSuccess) {                                      \
      g_err = std::string(#call ": ") + ncclGetErrorString(r__);   \
      return SPMV_ERR_NCCL;                                        \
    }                                                              \
  } while (0)
#define ST(call)                         \
  do {                                   \
    spmv_status s__ = (call);            \
    if (s__ != SPMV_OK) return s__;      \
  } while (0)
// after each kernel launch: count it and surface launch-configuration errors
#define LAUNCHED()                                                        \
  do {                                                                    \
    g_launches.fetch_add(1, std::memory_order_relaxed);                   \
    cudaError_t e__ = cudaGetLastError();                                 \
    if (e__ != cudaSuccess) return cuda_fail(e__, "kernel launch", __LINE__); \
  } while (0)

// ------------------------------------------------------------------ types
struct spmv_dist_s {
  ncclComm_t comm = nullptr;  // NCCL transport (nullptr for p2p)
  int rank = 0, nranks = 1, device = 0;
  int p2p = 0;                // 1: exchanges over CUDA-IPC peer memory (p2p_kernels.cuh)
};

struct Graph {
  cudaGraphExec_t exec = nullptr;
  uint64_t nodes = 0;
  const void *k0 = nullptr, *k1 = nullptr, *k2 = nullptr;
  int32_t ki = 0;
  double kd = 0.0;
  void reset() {
    if (exec) cudaGraphExecDestroy(exec);
    exec = nullptr;
    nodes = 0;
  }
};

struct spmv_csr_s {
  int device = 0;
  cudaStream_t stream = nullptr;      // user stream (may be the legacy stream 0)
  cudaStream_t cap = nullptr;         // private stream used for graph capture
  cudaEvent_t ev_a = nullptr, ev_b = nullptr;  // ev_a: z final inside the NPB graph (external event)
  cudaStream_t copy = nullptr;                 // D2H of z overlapping the residual SpMV
  spmv_dtype dt = SPMV_F64;
  size_t ts = 8;
  int64_t m = 0, n = 0, nnz = 0;
  int32_t base = 0;
  const int32_t* rowptr = nullptr;
  const int32_t* colidx = nullptr;
  const void* vals = nullptr;
  // execution view: local rows (all rows on a single GPU)
  int64_t m_loc = 0, row0 = 0, k0 = 0, k1 = 0;
  const int32_t* rp_loc = nullptr;   // rowptr + row0 (absolute k)
  const int32_t* ci_loc = nullptr;   // colidx (single) or renumbered copy - k0 (dist)
  // kernel choice
  int32_t kernel = SPMV_KERNEL_VECTOR, lanes = 32, unroll = 4;
  int64_t grid = 1, vgrid = 1, grid_vec = 1;
  int64_t row_min = 0, row_max = 0;
  double row_mean = 0, row_cv = 0;
  int32_t sorted = 0;
  // XSTAT (x-stationary cluster kernel)
  int xB = 0, xW = 0, xR = 1024, xG = 8, nclusters = 0;
  size_t xsmem = 0;
  int64_t nx = 0;                     // length of the x the kernels read
  int* seg = nullptr;
  long long* crow = nullptr;
  void (*xk)(XstatArgs) = nullptr;
  void (*xk_dot)(XstatArgs) = nullptr;
  // XPLAN (column-blocked SELL-32 device plan of A)
  struct XPlan {
    bool built = false;
    int B = 0, W = 0, ncl = 0, ntiles = 0;
    size_t smem = 0;
    int64_t bytes = 0, nchunks = 0;
    long long *crow = nullptr, *chunk_off = nullptr;
    int *tile0 = nullptr, *chunk_len = nullptr, *seg = nullptr, *row_slot = nullptr;
    uint16_t* chunk_row = nullptr;
    unsigned char* plan = nullptr;
    void (*k)(XplanArgs) = nullptr;
    void (*kdot)(XplanArgs) = nullptr;
    // side split (SPMV_XPLAN_SIDE): rows [mplan, m) run concurrently in the
    // vector kernel on the SMs the clusters leave idle
    int64_t mplan = -1;
    int g2 = 0;
  } xp;
  cudaStream_t side = nullptr;
  cudaEvent_t ev_fork = nullptr, ev_join = nullptr;
  // SELL (SELL-32 device plan, x gathered from global memory)
  struct Sell {
    bool built = false;
    int sorted = 0;
    int64_t nchunks = 0, pairs = 0, grid = 0, nlong = 0, nseg = 0, nmulti = 0;
    int* perm = nullptr;
    SellSeg* seg = nullptr;     // long-row segments
    double* seg_part = nullptr;
    int* seg_cnt = nullptr;
    long long* pair_off = nullptr;
    unsigned char* vals = nullptr;
    int* cols = nullptr;
  } sl;
  // MERGE (merge-path tiles)
  struct {
    int ntiles = 0;
    long long *split_row = nullptr, *split_nz = nullptr;
    double *head = nullptr, *carry = nullptr;
    int* head_flag = nullptr;
  } mg;
  // dist
  spmv_dist_s* dist = nullptr;
  std::vector<long long> bounds;
  long long maxlen = 0;
  // halo intervals (NEXT-2, R27): halo[(r*P+s)*2 .. +1] = [lo, hi) of rank s's slice that rank r reads
  std::vector<long long> halo;
  int2* send_iv = nullptr;            // device [P]: what this rank sends to each rank
  bool use_halo = false;              // exchange only the halo intervals (else the whole slices)
  int32_t* ci_own = nullptr;
  void* xpad = nullptr;               // nranks*maxlen, the gathered x / p
  // p2p transport: the IPC-exported fabric (xpad | exch | flags) and local counters
  unsigned char* fabric = nullptr;
  size_t fab_bytes = 0, off_exch = 0, off_flags = 0;
  unsigned long long* p2p_local = nullptr;  // [0] epoch, [1..NSLOT+1] slot_epoch, then ticket
  unsigned char** peer_table = nullptr;     // device [P]
  std::vector<unsigned char*> peers;        // host copy (opened IPC mappings)
  bool p2p_connected = false;
  // CG workspace (lazy)
  double *z = nullptr, *r = nullptr, *q = nullptr, *p_single = nullptr;
  double *s_vec = nullptr, *alpha2 = nullptr;  // single-reduction CG (NEXT-1): s = A p, alpha_{k-1}
  int cg_variant = 0;                          // 0 textbook (NPB conj_grad), 1 Chronopoulos-Gear
  double *part_pq = nullptr, *part_rr = nullptr, *part_res = nullptr, *part_xz = nullptr,
         *part_zz = nullptr, *scal = nullptr, *out2 = nullptr;
  int* flags = nullptr;
  double *stage_x = nullptr, *stage_z = nullptr;
  Graph g_npb;
};

// --------------------------------------------------------------- helpers
static bool env_int(const char* name, int* v) {
  const char* s = getenv(name);
  if (!s || !*s) return false;
  *v = atoi(s);
  return true;
}

static int num_sms(int dev) {
  int v = kNumSMs;
  cudaDeviceGetAttribute(&v, cudaDevAttrMultiProcessorCount, dev);
  return v > 0 ? v : kNumSMs;
}

// 1 = device (or managed) memory of `dev`, 0 = host (pinned, pageable), -1 = error
static int mem_kind(const void* p, int dev) {
  cudaPointerAttributes a;
  cudaError_t e = cudaPointerGetAttributes(&a, p);
  if (e != cudaSuccess) { cudaGetLastError(); return 0; }
  if (a.type == cudaMemoryTypeDevice || a.type == cudaMemoryTypeManaged)
    return a.device == dev ? 1 : -1;
  return 0;
}

static spmv_status need_device(const void* p, int dev, const char* what, bool may_be_null) {
  if (!p) return may_be_null ? SPMV_OK : arg_fail(what);
  return mem_kind(p, dev) == 1 ? SPMV_OK : arg_fail(what);
}

static bool overlap(const void* a, size_t na, const void* b, size_t nb) {
  if (!a || !b || na == 0 || nb == 0) return false;
  const uintptr_t a0 = (uintptr_t)a, b0 = (uintptr_t)b;
  return a0 < b0 + nb && b0 < a0 + na;
}

static int64_t cdiv(int64_t a, int64_t b) { return (a + b - 1) / b; }

// SPMV_DEBUG=1: trace the create-time plan build on stderr (synchronising).
static bool dbg() {
  static int v = -1;
  if (v < 0) { v = 0; env_int("SPMV_DEBUG", &v); }
  return v != 0;
}
#define DBG(...)                                                                    \
  do {                                                                              \
    if (dbg()) {                                                                    \
      cudaError_t e__ = cudaDeviceSynchronize();                                    \
      fprintf(stderr, "[spmv] %s:%d (%s) ", __func__, __LINE__, cudaGetErrorString(e__)); \
      fprintf(stderr, __VA_ARGS__);                                                 \
      fprintf(stderr, "\n");                                                        \
    }                                                                               \
  } while (0)

static spmv_status ensure_buf(void** p, size_t bytes) {
  if (*p) return SPMV_OK;
  CK(cudaMalloc(p, bytes > 0 ? bytes : 8));
  return SPMV_OK;
}

// ------------------------------------------------------- kernel dispatch
template <typename T, int G, bool DOT>
static void launch_vec_u(int unroll, int64_t grid, cudaStream_t s, const SpmvArgs& a) {
  switch (unroll) {
    case 2: k_spmv_vector<T, G, 2, DOT><<<grid, 256, 0, s>>>(a); break;
    case 8: k_spmv_vector<T, G, 8, DOT><<<grid, 256, 0, s>>>(a); break;
    default: k_spmv_vector<T, G, 4, DOT><<<grid, 256, 0, s>>>(a); break;
  }
}

template <typename T, bool DOT>
static void launch_vec(int lanes, int unroll, int64_t grid, cudaStream_t s, const SpmvArgs& a) {
  switch (lanes) {
    case 1: launch_vec_u<T, 1, DOT>(unroll, grid, s, a); break;
    case 2: launch_vec_u<T, 2, DOT>(unroll, grid, s, a); break;
    case 4: launch_vec_u<T, 4, DOT>(unroll, grid, s, a); break;
    case 8: launch_vec_u<T, 8, DOT>(unroll, grid, s, a); break;
    case 16: launch_vec_u<T, 16, DOT>(unroll, grid, s, a); break;
    default: launch_vec_u<T, 32, DOT>(unroll, grid, s, a); break;
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
static spmv_status xstat_setup(spmv_csr_s* h, bool* ok) {
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
  if (env_int("SPMV_XSTAT_U", &g2) && (g2 == 4 || g2 == 8)) U = g2;
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

static spmv_status launch_xplan(spmv_csr_s* h, cudaStream_t s, const void* x, void* y, double alpha,
                                double beta, const double* w, double* part, const P2PHook& hook) {
  XplanArgs a;
  a.nx = h->nx;
  a.W = h->xp.W;
  a.plan = h->xp.plan;
  a.chunk_off = h->xp.chunk_off;
  a.chunk_len = h->xp.chunk_len;
  a.chunk_row = h->xp.chunk_row;
  a.dbg = dbg() ? 1 : 0;
  a.prefetch = 0;
  env_int("SPMV_XPLAN_PF", &a.prefetch);
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
  cudaLaunchConfig_t cfg = {};
  cfg.gridDim = dim3((unsigned)(h->xp.ncl * h->xp.B), 1, 1);
  cfg.blockDim = dim3(XP_THREADS, 1, 1);
  cfg.dynamicSmemBytes = h->xp.smem;
  cfg.stream = s;
  cudaLaunchAttribute at[1];
  at[0].id = cudaLaunchAttributeClusterDimension;
  at[0].val.clusterDim.x = (unsigned)h->xp.B;
  at[0].val.clusterDim.y = 1;
  at[0].val.clusterDim.z = 1;
  cfg.attrs = at;
  cfg.numAttrs = 1;
  a.tstamp = nullptr;
  int times = 0;
  if (env_int("SPMV_XPLAN_TIMES", &times) && times) {
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
    sa.part = part ? part + cfg.gridDim.x : nullptr;
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
    for (unsigned i = 0; i < cfg.gridDim.x; ++i) { t0 = std::min(t0, t[4 * i]); tend = std::max(tend, t[4 * i + 3]); }
    fprintf(stderr, "[xplan times] kernel span %.2f us; per CTA (us from first start): start/xready/streamed/end\n",
            (tend - t0) / 1e3);
    for (unsigned i = 0; i < cfg.gridDim.x; ++i)
      fprintf(stderr, "  cta %3u cl %2u  %6.2f %6.2f %6.2f %6.2f\n", i, i / (unsigned)h->xp.B, (t[4 * i] - t0) / 1e3,
              (t[4 * i + 1] - t0) / 1e3, (t[4 * i + 2] - t0) / 1e3, (t[4 * i + 3] - t0) / 1e3);
  }
  return SPMV_OK;
}

// Pack (or re-pack, values_only) the nonzeros into the plan chunks.
static spmv_status xplan_pack(spmv_csr_s* h, const void* vals, int values_only) {
  cudaStream_t s = h->stream;
  auto& P = h->xp;
  const int64_t g = std::min<int64_t>(cdiv(h->m_loc * 32, 256), 16LL * num_sms(h->device));
  if (h->dt == SPMV_F64)
    k_xplan_pack<double><<<g, 256, 0, s>>>(h->rp_loc, h->ci_loc, (const double*)vals, P.seg, h->m_loc, P.B, P.W,
                                          P.crow, P.tile0, P.ncl, P.chunk_off, P.chunk_len, P.row_slot, P.plan,
                                          values_only, P.mplan);
  else
    k_xplan_pack<float><<<g, 256, 0, s>>>(h->rp_loc, h->ci_loc, (const float*)vals, P.seg, h->m_loc, P.B, P.W,
                                         P.crow, P.tile0, P.ncl, P.chunk_off, P.chunk_len, P.row_slot, P.plan,
                                         values_only, P.mplan);
  LAUNCHED();
  return SPMV_OK;
}

// Build the column-blocked SELL-32 plan (create).  *ok = false if not eligible.
static spmv_status xplan_build(spmv_csr_s* h, bool* ok) {
  *ok = false;
  if (!h->sorted || h->m_loc == 0 || h->nx == 0 || h->k1 - h->k0 == 0) return SPMV_OK;
  const int ts = (int)h->ts;
  const size_t smem_cap = 227 * 1024 - 1024;  // dynamic smem a CTA may use (static < 1 KB)
  const size_t recv = (size_t)XP_K * XP_R * 8;
  if (smem_cap <= recv + 1024) return SPMV_OK;
  const size_t xbudget = smem_cap - recv - 64;
  const int64_t Bneed = cdiv((int64_t)(ts * h->nx), (int64_t)xbudget);
  if (Bneed > 16) return SPMV_OK;  // x does not fit the shared memory of a 16-CTA cluster
  void (*fn)(XplanArgs) = h->dt == SPMV_F64 ? k_spmv_xplan<double, false> : k_spmv_xplan<float, false>;
  void (*fnd)(XplanArgs) = h->dt == SPMV_F64 ? k_spmv_xplan<double, true> : nullptr;
  // cluster size: any B >= Bneed that divides the tile height R (rows are
  // owned in R/B blocks); among those, the one whose resident clusters cover
  // the most SMs (ties: the smaller B, whose x blocks are larger); clusters of
  // 16 only when nothing smaller fits.  SPMV_XPLAN_B forces a size.
  int forced = 0;
  env_int("SPMV_XPLAN_B", &forced);
  if (forced < Bneed || forced > 16 || XP_R % std::max(forced, 1)) forced = 0;  // infeasible request: ignored
  int B = 0, W = 0, ncl = 0;
  size_t smem = 0;
  for (int cand = (int)std::max<int64_t>(1, Bneed); cand <= 16; ++cand) {
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
    if (B == 0 || nc * cand > ncl * B) { B = cand; W = Wc; ncl = nc; smem = sm; }
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
    void* bufs[] = {P.crow, P.chunk_off, P.tile0, P.chunk_len, P.seg, P.row_slot, P.chunk_row, P.plan};
    for (void* q : bufs)
      if (q) cudaFree(q);
    P = spmv_csr_s::XPlan();
  };
  P.B = B; P.W = W; P.ncl = ncl; P.smem = smem; P.k = fn; P.kdot = fnd;
  DBG("B=%d W=%d ncl=%d smem=%zu", B, W, ncl, smem);
  const int64_t m = h->m_loc;
  // side split: the last SPMV_XPLAN_SIDE per mille of the nonzeros go to the
  // vector kernel on the idle SMs (single GPU only)
  P.mplan = m;
  {
    int side_pm = 0;
    env_int("SPMV_XPLAN_SIDE", &side_pm);
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
  CK(cudaMalloc(&P.crow, sizeof(long long) * (ncl + 1)));
  k_partition<<<cdiv(ncl + 1, 128), 128, 0, s>>>(P.mplan, h->rp_loc, ncl, P.crow);
  LAUNCHED();
  std::vector<long long> crow(ncl + 1);
  CK(cudaMemcpyAsync(crow.data(), P.crow, sizeof(long long) * (ncl + 1), cudaMemcpyDeviceToHost, s));
  CK(cudaStreamSynchronize(s));
  std::vector<int> tile0(ncl + 1, 0);
  for (int c = 0; c < ncl; ++c) tile0[c + 1] = tile0[c] + (int)cdiv(crow[c + 1] - crow[c], XP_R);
  const int ntiles = tile0[ncl];
  P.ntiles = ntiles;
  DBG("ntiles=%d", ntiles);
  CK(cudaMalloc(&P.tile0, sizeof(int) * (ncl + 1)));
  CK(cudaMemcpyAsync(P.tile0, tile0.data(), sizeof(int) * (ncl + 1), cudaMemcpyHostToDevice, s));
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
    k_xplan_sell<<<(unsigned)(ntiles * B), XP_THREADS, 0, s>>>(h->rp_loc, P.seg, m, B, P.crow, P.tile0, ncl, P.chunk_len,
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
  for (int c = 0; c < ncl; ++c)
    for (int bb = 0; bb < B; ++bb)
      for (int t = tile0[c]; t < tile0[c + 1]; ++t)
        for (int w = 0; w < XP_CPT; ++w) {
          const size_t id = ((size_t)t * B + bb) * XP_CPT + w;
          off[id] = pos;
          pos += (long long)len[id] * 32 * (ts + 2);
        }
  P.bytes = pos;
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
static spmv_status sell_pack(spmv_csr_s* h, const void* vals, int values_only) {
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
static spmv_status sell_build(spmv_csr_s* h, double max_pad, int sorted, bool* ok) {
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
                               const double* w, double* part, const P2PHook& hook) {
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
      k_spmv_sell<double, false><<<g, SELL_NT, 0, s>>>(a);
      LAUNCHED();
      P2PHook push_only = hook;
      push_only.wait_x = 0;
      k_dot_partials<<<(int)h->vgrid, 256, 0, s>>>(h->m_loc, w, (const double*)y, part, push_only);
    } else if (part) {
      k_spmv_sell<double, true><<<g, SELL_NT, 0, s>>>(a);
    } else {
      k_spmv_sell<double, false><<<g, SELL_NT, 0, s>>>(a);
    }
  } else {
    a.alpha = (double)(float)alpha;
    a.beta = (double)(float)beta;
    k_spmv_sell<float, false><<<g, SELL_NT, 0, s>>>(a);
  }
  LAUNCHED();
  return SPMV_OK;
}

static spmv_status merge_setup(spmv_csr_s* h) {
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
                                double alpha, double beta, const P2PHook& hook) {
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
    k_spmv_merge<double><<<a.ntiles, MG_NT, 0, s>>>(a);
    LAUNCHED();
    k_merge_fixup<double><<<(unsigned)cdiv(a.ntiles, 256), 256, 0, s>>>(a);
    LAUNCHED();
  } else {
    a.alpha = (double)(float)alpha;
    a.beta = (double)(float)beta;
    k_spmv_merge<float><<<a.ntiles, MG_NT, 0, s>>>(a);
    LAUNCHED();
    k_merge_fixup<float><<<(unsigned)cdiv(a.ntiles, 256), 256, 0, s>>>(a);
    LAUNCHED();
  }
  return SPMV_OK;
}

// Local SpMV of the handle: y = alpha*A_loc*x + beta*y (+ partial w.y per CTA).
static spmv_status run_spmv(spmv_csr_s* h, cudaStream_t s, const void* vals, const void* x, void* y,
                            double alpha, double beta, const double* w, double* part,
                            const P2PHook* hk = nullptr) {
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
  if (h->kernel == SPMV_KERNEL_XPLAN && vals == h->vals) return launch_xplan(h, s, x, y, alpha, beta, w, part, hook);
  const bool sell = h->kernel == SPMV_KERNEL_SELL || h->kernel == SPMV_KERNEL_SELL_SORTED;
  if (sell && vals == h->vals) return launch_sell(h, s, x, y, alpha, beta, w, part, hook);
  const int64_t vgrid_spmv = (h->kernel == SPMV_KERNEL_XPLAN || sell) ? h->grid_vec : h->grid;
  if (h->kernel == SPMV_KERNEL_XSTAT) return launch_xstat(h, s, vals, x, y, alpha, beta, w, part, hook);
  if (h->kernel == SPMV_KERNEL_MERGE) {
    P2PHook wait_only = hook;
    wait_only.push_slot = -1;
    ST(launch_merge(h, s, vals, x, y, alpha, beta, wait_only));
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
    if (part) launch_vec<double, true>(h->lanes, h->unroll, vgrid_spmv, s, a);
    else launch_vec<double, false>(h->lanes, h->unroll, vgrid_spmv, s, a);
  } else {
    a.alpha = (double)(float)alpha;
    a.beta = (double)(float)beta;
    launch_vec<float, false>(h->lanes, h->unroll, vgrid_spmv, s, a);
  }
  LAUNCHED();
  return SPMV_OK;
}

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
  env_int("SPMV_VGRID_ELEMS", &vel);
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
      // fabric: xpad | exch [NSLOT][P] double | flags [P] u64, one IPC-exportable allocation
      const size_t xb = (h->ts * (size_t)(maxlen * P) + 255) & ~size_t(255);
      h->off_exch = xb;
      h->off_flags = xb + ((sizeof(double) * P2P_NSLOT * P + 255) & ~size_t(255));
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

  int rk = 0, rl = 0;
  if (!env_int("SPMV_KERNEL", &rk)) rk = o.kernel;
  if (!env_int("SPMV_LANES", &rl)) rl = o.vec_lanes;
  h->nx = o.dist ? (int64_t)h->maxlen * o.dist->nranks : n;
  choose_kernel(h, rk, rl);
  int plan = o.plan;
  env_int("SPMV_PLAN", &plan);
  if (rk == SPMV_KERNEL_XPLAN || (rk == SPMV_KERNEL_AUTO && plan)) {
    // auto + plan: the column-blocked x-stationary plan whenever x fits the
    // shared memory of a cluster and rows are long enough
    if (rk == SPMV_KERNEL_XPLAN || h->row_mean >= 16.0) {
      bool ok = false;
      spmv_status st = xplan_build(h, &ok);
      if (st != SPMV_OK) return fail(st);
      if (ok) {
        h->kernel = SPMV_KERNEL_XPLAN;
        h->grid = (int64_t)h->xp.ncl * h->xp.B;
        if (h->xp.mplan < h->m_loc) h->grid += h->xp.g2;  // dot partials: clusters, then the side kernel
      }
    }
  }
  const bool skewed = (double)h->row_max > 32.0 * std::max(h->row_mean, 1.0);
  if (h->kernel != SPMV_KERNEL_XPLAN && (rk == SPMV_KERNEL_SELL || rk == SPMV_KERNEL_SELL_SORTED ||
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
  if (h->kernel != SPMV_KERNEL_XPLAN && h->kernel != SPMV_KERNEL_SELL && h->kernel != SPMV_KERNEL_SELL_SORTED &&
      rk != SPMV_KERNEL_VECTOR && rk != SPMV_KERNEL_SCALAR && rk != SPMV_KERNEL_XSTAT && h->m_loc > 0 &&
      (rk == SPMV_KERNEL_MERGE || skewed)) {
    // skewed rows without a plan (a long row would pin one warp of the vector kernel): merge path
    spmv_status st = merge_setup(h);
    if (st != SPMV_OK) return fail(st);
    h->kernel = SPMV_KERNEL_MERGE;
    h->grid = h->vgrid;  // dot partials come from k_dot_partials
  }
  if (h->kernel == SPMV_KERNEL_XPLAN || h->kernel == SPMV_KERNEL_MERGE || h->kernel == SPMV_KERNEL_SELL ||
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
  for (size_t q = 0; q < h->peers.size(); ++q)
    if (h->peers[q] && h->peers[q] != h->fabric) cudaIpcCloseMemHandle(h->peers[q]);
  if (h->fabric) {
    cudaFree(h->fabric);
    if (h->xpad == h->fabric) h->xpad = nullptr;
  }
  void* bufs[] = {h->p2p_local, h->peer_table, h->mg.split_row, h->mg.split_nz, h->mg.head, h->mg.carry, h->mg.head_flag, h->xp.crow, h->xp.chunk_off, h->xp.tile0, h->xp.chunk_len, h->xp.seg, h->xp.row_slot,
                  h->xp.chunk_row, h->xp.plan, h->sl.pair_off, h->sl.vals, h->sl.cols, h->sl.perm, h->sl.seg, h->sl.seg_part, h->sl.seg_cnt,
                  h->seg, h->crow, h->ci_own, h->send_iv, h->xpad, h->z, h->r, h->q, h->p_single, h->part_pq, h->part_rr,
                  h->part_res, h->part_xz, h->part_zz, h->scal, h->out2, h->flags, h->s_vec, h->alpha2,
                  h->stage_x, h->stage_z};
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
static spmv_status exchange_x(spmv_csr_s* h, cudaStream_t s);

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

// ------------------------------------------------------------------ CG
static spmv_status cg_alloc(spmv_csr_s* h) {
  if (h->z) return SPMV_OK;
  const size_t nb = sizeof(double) * (size_t)std::max<int64_t>(h->m_loc, 1);
  const size_t pb = sizeof(double) * (size_t)std::max<int64_t>(std::max(std::max(h->grid, h->grid_vec), h->vgrid), 1);
  ST(ensure_buf((void**)&h->z, nb));
  ST(ensure_buf((void**)&h->r, nb));
  ST(ensure_buf((void**)&h->q, nb));
  if (!h->dist) ST(ensure_buf((void**)&h->p_single, nb));
  ST(ensure_buf((void**)&h->part_pq, pb));
  // [0],[1]: parity slots; [2]: ||b||^2 (init); [3..5]: rotating r.r of the single-reduction CG
  ST(ensure_buf((void**)&h->part_rr, 6 * pb));
  ST(ensure_buf((void**)&h->s_vec, nb));
  ST(ensure_buf((void**)&h->alpha2, sizeof(double) * 2));
  ST(ensure_buf((void**)&h->part_res, pb));
  ST(ensure_buf((void**)&h->part_xz, pb));
  ST(ensure_buf((void**)&h->part_zz, pb));
  ST(ensure_buf((void**)&h->scal, sizeof(double) * 16));
  ST(ensure_buf((void**)&h->out2, sizeof(double) * 2));
  ST(ensure_buf((void**)&h->flags, sizeof(int) * 4));
  CK(cudaMemset(h->flags, 0, sizeof(int) * 4));
  return SPMV_OK;
}

static P2PCtx p2p_ctx(spmv_csr_s* h) {
  P2PCtx c;
  c.peer = h->peer_table;
  c.off_exch = h->off_exch;
  c.off_flags = h->off_flags;
  c.epoch = h->p2p_local;
  c.slot_epoch = h->p2p_local + 1;
  c.ticket = reinterpret_cast<int*>(h->p2p_local + 2 + P2P_NSLOT);
  c.me = h->dist->rank;
  c.P = h->dist->nranks;
  c.send_iv = h->use_halo ? h->send_iv : nullptr;
  return c;
}

static bool use_p2p(const spmv_csr_s* h) { return h->dist && h->dist->p2p; }

// All-gather of this rank's slice (already at xpad + rank*maxlen) and wait.
static spmv_status exchange_x(spmv_csr_s* h, cudaStream_t s) {
  if (use_p2p(h)) {
    if (!h->p2p_connected) return arg_fail("p2p handle not connected (spmv_csr_p2p_connect)");
    const P2PCtx c = p2p_ctx(h);
    const int g = (int)std::max<int64_t>(1, std::min<int64_t>(cdiv(h->m_loc, 256), 2LL * num_sms(h->device)));
    if (h->dt == SPMV_F64) k_p2p_push_x<double><<<g, 256, 0, s>>>(h->m_loc, h->maxlen, c);
    else k_p2p_push_x<float><<<g, 256, 0, s>>>(h->m_loc, h->maxlen, c);
    LAUNCHED();
    k_p2p_wait_x<<<1, 1, 0, s>>>(c);
    LAUNCHED();
    return SPMV_OK;
  }
  const ncclDataType_t nt = h->dt == SPMV_F64 ? ncclDouble : ncclFloat;
  if (h->use_halo) {
    // halo exchange: send rank q the interval of my slice it reads, receive mine from every owner
    const int P = h->dist->nranks, me = h->dist->rank;
    char* xp = (char*)h->xpad;
    NK(ncclGroupStart());
    for (int q = 0; q < P; ++q) {
      if (q == me) continue;
      const long long* so = &h->halo[2 * ((size_t)q * P + me)];
      const long long* ro = &h->halo[2 * ((size_t)me * P + q)];
      if (so[1] > so[0])
        NK(ncclSend(xp + h->ts * (size_t)(me * h->maxlen + so[0]), (size_t)(so[1] - so[0]), nt, q, h->dist->comm, s));
      if (ro[1] > ro[0])
        NK(ncclRecv(xp + h->ts * (size_t)(q * h->maxlen + ro[0]), (size_t)(ro[1] - ro[0]), nt, q, h->dist->comm, s));
    }
    NK(ncclGroupEnd());
    return SPMV_OK;
  }
  NK(ncclAllGather((char*)h->xpad + h->ts * (size_t)(h->dist->rank * h->maxlen), h->xpad, (size_t)h->maxlen, nt,
                   h->dist->comm, s));
  return SPMV_OK;
}

static double* cg_p(spmv_csr_s* h) {
  if (!h->dist) return h->p_single;
  return (double*)h->xpad + h->dist->rank * h->maxlen;
}

// In distributed mode a SumSrc of per-CTA partials is finalized into scal[slot]
// and all-reduced over the ranks; single GPU returns the partials unchanged.
// The exchange-mode scalar source of `slot` (values pushed by every rank).
static SumSrc p2p_src(spmv_csr_s* h, int slot) {
  const P2PCtx c = p2p_ctx(h);
  SumSrc o;
  o.p = reinterpret_cast<const double*>(h->fabric + h->off_exch) + slot * c.P;
  o.count = -c.P;
  o.flags = reinterpret_cast<const unsigned long long*>(h->fabric + h->off_flags);
  o.epoch = c.slot_epoch + slot;
  o.me = c.me;
  return o;
}

static spmv_status reduce_src(spmv_csr_s* h, cudaStream_t s, SumSrc in, int slot, SumSrc* out) {
  if (!h->dist) { *out = in; return SPMV_OK; }
  if (use_p2p(h)) {
    if (!h->p2p_connected) return arg_fail("p2p handle not connected (spmv_csr_p2p_connect)");
    const P2PCtx c = p2p_ctx(h);
    k_p2p_push_sum<<<1, 32, 0, s>>>(in, slot, c);
    LAUNCHED();
    *out = p2p_src(h, slot);
    return SPMV_OK;
  }
  double* dst = h->scal + slot;
  k_finalize<<<1, 32, 0, s>>>(in, dst);
  LAUNCHED();
  NK(ncclAllReduce(dst, dst, 1, ncclDouble, ncclSum, h->dist->comm, s));
  *out = SumSrc{dst, 1};
  return SPMV_OK;
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
  if (h->cg_variant == 1) k_cg_init<<<vg, 256, 0, s>>>(h->m_loc, b, z, cg_p(h), h->r, prb);
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
  if (h->cg_variant == 1) {
    // single-reduction CG (cg_kernels.cuh k_cgcg): SpMV w = A r with w.r fused, then one update
    double* rv = p;  // the SpMV input slice holds r
    static const int kGamSlot[3] = {2, 3, 7};
    for (int c = 0; c < iters; ++c) {
      const int k = run->it++;
      SumSrc del;
      if (p2p) {
        P2PHook hs = base;
        hs.wait_x = 1;
        hs.push_slot = 1;
        ST(run_spmv(h, s, h->vals, xg, h->q, 1.0, 0.0, rv, h->part_pq, &hs));
        del = p2p_src(h, 1);
      } else {
        ST(gather_p(h, s));
        ST(run_spmv(h, s, h->vals, xg, h->q, 1.0, 0.0, rv, h->part_pq));
        ST(reduce_src(h, s, SumSrc{h->part_pq, sg}, 1, &del));
      }
      double* gnew = h->part_rr + (3 + (k + 1) % 3) * pstride;
      const int gslot = kGamSlot[(k + 1) % 3];
      P2PHook hz = base;
      hz.push_slot = p2p ? gslot : -1;
      const int64_t xoff = h->dist ? (int64_t)h->dist->rank * h->maxlen : 0;
      k_cgcg<<<vg, 256, 0, s>>>(n, k, run->rr_old, run->rr_prev, del, h->alpha2, h->r, h->s_vec, h->q, z, rv,
                                gnew, h->flags, tol, run->rr_b, hz, xoff);
      LAUNCHED();
      SumSrc g1;
      if (p2p) g1 = p2p_src(h, gslot);
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
      ST(run_spmv(h, s, h->vals, xg, h->q, 1.0, 0.0, p, h->part_pq, &hs));
      pq = p2p_src(h, 1);
    } else {
      ST(gather_p(h, s));
      ST(run_spmv(h, s, h->vals, xg, h->q, 1.0, 0.0, p, h->part_pq));
      ST(reduce_src(h, s, SumSrc{h->part_pq, sg}, 1, &pq));
    }
    double* pnew = h->part_rr + ((it + 1) & 1) * pstride;
    const int rslot = 2 + ((it + 1) & 1);
    P2PHook hz = base;
    hz.push_slot = p2p ? rslot : -1;
    k_cg_zr<<<vg, 256, 0, s>>>(n, pq, run->rr_old, p, h->q, z, h->r, pnew, h->flags, hz);
    LAUNCHED();
    SumSrc rr_new;
    if (p2p) rr_new = p2p_src(h, rslot);
    else ST(reduce_src(h, s, SumSrc{pnew, vg}, rslot, &rr_new));
    // p2p: the p update stores its slice into every peer's x buffer and publishes it
    const int64_t xoff = h->dist ? (int64_t)h->dist->rank * h->maxlen : 0;
    k_cg_p<<<vg, 256, 0, s>>>(n, rr_new, run->rr_old, h->r, p, h->flags, tol, run->rr_b, it, base, xoff);
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
  // z is final here: an external event lets the host copy of z overlap the residual
  cudaStreamCaptureStatus cst = cudaStreamCaptureStatusNone;
  CK(cudaStreamIsCapturing(s, &cst));
  if (cst == cudaStreamCaptureStatusActive) CK(cudaEventRecordWithFlags(h->ev_a, s, cudaEventRecordExternal));
  else CK(cudaEventRecord(h->ev_a, s));
  ST(cg_resid<true>(h, s, x, z));
  SumSrc res, xz, zz;
  const int vg = (int)h->vgrid;
  ST(reduce_src(h, s, SumSrc{h->part_res, vg}, 4, &res));
  ST(reduce_src(h, s, SumSrc{h->part_xz, vg}, 5, &xz));
  ST(reduce_src(h, s, SumSrc{h->part_zz, vg}, 6, &zz));
  k_npb_finish<<<vg, 256, 0, s>>>(h->m_loc, res, xz, zz, z, x, shift, out2);
  LAUNCHED();
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
  if (xd != x && h->m_loc > 0) {
    CK(cudaMemcpyAsync(x, xd, sizeof(double) * h->m_loc, cudaMemcpyDeviceToHost, s));
    sync = true;
  }
  bool copy_used = false;
  if (zd != z && h->m_loc > 0) {
    // z (host) is copied on a side stream as soon as the CG loop wrote it,
    // overlapping the residual SpMV and the finishing kernel
    if (!h->copy) CK(cudaStreamCreateWithFlags(&h->copy, cudaStreamNonBlocking));
    CK(cudaStreamWaitEvent(h->copy, h->ev_a, 0));
    CK(cudaMemcpyAsync(z, zd, sizeof(double) * h->m_loc, cudaMemcpyDeviceToHost, h->copy));
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

extern "C" spmv_status spmv_csr_update_values(spmv_csr_t h, const void* vals) {
  if (!h) return arg_fail("handle is NULL");
  CK(cudaSetDevice(h->device));
  ST(need_device(vals, h->device, "vals must be a device pointer", h->nnz == 0));
  h->vals = vals;
  if (h->xp.built) ST(xplan_pack(h, vals, 1));
  if (h->sl.built) ST(sell_pack(h, vals, 1));
  h->g_npb.reset();
  return SPMV_OK;
}

extern "C" spmv_status spmv_csr_set_cg_variant(spmv_csr_t h, int32_t variant) {
  if (!h) return arg_fail("handle is NULL");
  if (variant != 0 && variant != 1) return arg_fail("variant must be 0 (textbook) or 1 (single reduction)");
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

// ------------------------------------------------------ matrix-free stencil
// Tensor map of the stencil grid x (3-D: nx fastest, then ny, nz) for the TMA
// plane tiles of k_stencil27_box2: box (SBL::PX, 18, 1), no swizzle, zero fill
// outside the grid.  The driver entry point is fetched through the runtime
// (no link against libcuda).  false = not encodable (the caller keeps cp.async).
#ifndef ST_TMA_L2PROMO
#define ST_TMA_L2PROMO CU_TENSOR_MAP_L2_PROMOTION_L2_128B
#endif
static bool encode_stencil_map(CUtensorMap* tm, spmv_dtype dt, const void* x, int64_t nx, int64_t ny, int64_t nz) {
  using encode_fn = CUresult (*)(CUtensorMap*, CUtensorMapDataType, cuuint32_t, void*, const cuuint64_t*,
                                 const cuuint64_t*, const cuuint32_t*, const cuuint32_t*, CUtensorMapInterleave,
                                 CUtensorMapSwizzle, CUtensorMapL2promotion, CUtensorMapFloatOOBfill);
  static encode_fn fn = nullptr;
  static bool tried = false;
  if (!tried) {
    tried = true;
    void* p = nullptr;
    cudaDriverEntryPointQueryResult q;
    if (cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &p, cudaEnableDefault, &q) == cudaSuccess &&
        q == cudaDriverEntryPointSuccess)
      fn = reinterpret_cast<encode_fn>(p);
    else
      cudaGetLastError();
  }
  if (!fn) return false;
  const int64_t ts = dt == SPMV_F64 ? 8 : 4;
  if ((reinterpret_cast<uintptr_t>(x) & 15) || (nx * ts) % 16 || nx >= (1LL << 31) || ny >= (1LL << 31) ||
      nz >= (1LL << 31) || nx * ny * ts >= (1LL << 40))
    return false;
  const cuuint64_t dims[3] = {(cuuint64_t)nx, (cuuint64_t)ny, (cuuint64_t)nz};
  const cuuint64_t strides[2] = {(cuuint64_t)(nx * ts), (cuuint64_t)(nx * ny * ts)};
  const cuuint32_t box[3] = {(cuuint32_t)(dt == SPMV_F64 ? SBL<double, true>::PX : SBL<float, true>::PX),
                             (cuuint32_t)SB_PY, 1u};
  const cuuint32_t es[3] = {1u, 1u, 1u};
  const CUresult r = fn(tm, dt == SPMV_F64 ? CU_TENSOR_MAP_DATA_TYPE_FLOAT64 : CU_TENSOR_MAP_DATA_TYPE_FLOAT32, 3,
                        const_cast<void*>(x), dims, strides, box, es, CU_TENSOR_MAP_INTERLEAVE_NONE,
                        CU_TENSOR_MAP_SWIZZLE_NONE, ST_TMA_L2PROMO,
                        CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  return r == CUDA_SUCCESS;
}

extern "C" spmv_status stencil27_apply(spmv_dtype dt, int64_t nx, int64_t ny, int64_t nz, const double* w27,
                                       const void* x, void* y, double alpha, double beta, void* stream) {
  if (dt != SPMV_F64 && dt != SPMV_F32) return arg_fail("dtype must be SPMV_F64 or SPMV_F32");
  if (nx < 0 || ny < 0 || nz < 0) return arg_fail("grid dimensions must be >= 0");
  if (nx > 0 && ny > 0 && nz > 0 && (nx > INT64_MAX / ny || nx * ny > INT64_MAX / nz))
    return arg_fail("grid too large");
  const int64_t n = nx * ny * nz;
  if (n == 0) return SPMV_OK;
  if (nx > 2147483647LL / ST_TX || ny > 2147483647LL) return arg_fail("grid too large");
  int dev = 0;
  CK(cudaGetDevice(&dev));
  const size_t ts = dt == SPMV_F64 ? 8 : 4;
  ST(need_device(y, dev, "y must be a device pointer on the current device", false));
  if (alpha != 0.0) ST(need_device(x, dev, "x must be a device pointer on the current device", false));
  if (alpha != 0.0 && overlap(y, ts * (size_t)n, x, ts * (size_t)n)) {
    g_err = "y overlaps x";
    return SPMV_ERR_ALIAS;
  }
  cudaStream_t s = (cudaStream_t)stream;
  const int sms = num_sms(dev);
  if (alpha == 0.0) {  // A and x are not read (R6)
    const int64_t g = std::min<int64_t>(cdiv(n, 256), 4LL * sms);
    if (dt == SPMV_F64) k_scale<double><<<g, 256, 0, s>>>(n, (double*)y, beta);
    else k_scale<float><<<g, 256, 0, s>>>(n, (float*)y, (double)(float)beta);
    LAUNCHED();
    return SPMV_OK;
  }
  StencilArgs a;
  a.nx = nx; a.ny = ny; a.nz = nz;
  for (int i = 0; i < 27; ++i) a.w[i] = w27 ? w27[i] : (i == 13 ? 26.0 : -1.0);  // R19 Laplacian by default
  a.x = x; a.y = y;
  a.alpha = alpha; a.beta = beta;
  if (dt == SPMV_F32) {
    a.alpha = (double)(float)alpha;
    a.beta = (double)(float)beta;
    for (int i = 0; i < 27; ++i) a.w[i] = (double)(float)a.w[i];
  }
  // BOX form when the 26 neighbour weights are equal (R19's default among them);
  // SPMV_STENCIL_BOX=0 forces the general 27-weight form
  bool box = true;
  for (int i = 0; i < 27; ++i)
    if (i != 13 && a.w[i] != a.w[0]) box = false;
  int benv = 1;
  if (env_int("SPMV_STENCIL_BOX", &benv) && benv == 0) box = false;
  a.wn = a.w[0];
  a.wd = a.w[13] - a.w[0];
  void (*kfn)(StencilArgs) = dt == SPMV_F64 ? (box ? k_stencil27<double, true> : k_stencil27<double, false>)
                                            : (box ? k_stencil27<float, true> : k_stencil27<float, false>);
  // z ranges: ~8 CTAs per SM, each marching >= 16 planes (2 halo planes per range).
  // 256^3 with the cp.async ring (5 CTAs of 256 resident per SM, register-limited):
  // 52 planes per CTA 70.7 us, 26 (this rule) 66.6 us, 24 70.7 us, 13 70.7 us, 7 76.8 us
  // BOX with two columns per thread (k_stencil27_box2) unless SPMV_STENCIL_BOX2=0
  int b2env = 1;
  env_int("SPMV_STENCIL_BOX2", &b2env);
  const bool box2 = box && b2env != 0 && nx * ny < 2147483647LL;  // 32-bit in-plane offsets
  // TMA plane tiles (k_stencil27_box2<T, true>) unless SPMV_STENCIL_TMA=0 or the tensor map cannot be
  // encoded (row stride not a multiple of 16 B, x not 16-B aligned, sizes beyond the TMA limits)
  CUtensorMap tm;
  std::memset(&tm, 0, sizeof(tm));
  bool tma = false;
  if (box2) {
    int tenv = 1;
    env_int("SPMV_STENCIL_TMA", &tenv);
    tma = tenv != 0 && encode_stencil_map(&tm, dt, x, nx, ny, nz);
    // SPMV_STENCIL_TMA=2 (tests): the TMA form is required, no silent cp.async fallback
    if (tenv == 2 && !tma) return arg_fail("SPMV_STENCIL_TMA=2 but the grid's tensor map cannot be encoded");
  }
  void (*kfn2)(StencilArgs, const CUtensorMap) = nullptr;
  if (box2)
    kfn2 = dt == SPMV_F64 ? (tma ? k_stencil27_box2<double, true> : k_stencil27_box2<double, false>)
                          : (tma ? k_stencil27_box2<float, true> : k_stencil27_box2<float, false>);
  // TMA tiles start SHIFT columns left of a multiple of 64 (one more tile column when nx % 64 == 0;
  // handing that column to lane 31 of the last tile column instead measured 73.7 vs 61.4 us on 256^3:
  // the serial extra work makes those CTAs the tail)
  const int shift = !tma ? 0 : dt == SPMV_F64 ? SBL<double, true>::SHIFT : SBL<float, true>::SHIFT;
  const int64_t bx = cdiv(nx + shift, box2 ? SB_TX : ST_TX), by = cdiv(ny, box2 ? SB_TY : ST_TY);
  int64_t zs = std::max<int64_t>(1, std::min<int64_t>(cdiv(8LL * sms, bx * by), cdiv(nz, 16)));
  int zc = (int)cdiv(nz, zs);
  int env = 0;
  if (env_int("SPMV_STENCIL_ZCHUNK", &env) && env > 0) zc = env;
  zs = cdiv(nz, zc);
  a.zchunk = zc;
  if (by > 65535 || zs > 65535) return arg_fail("grid too large for the stencil launch");
  const dim3 grid((unsigned)bx, (unsigned)by, (unsigned)zs);
  if (box2) kfn2<<<grid, SB_NT, 0, s>>>(a, tm);
  else kfn<<<grid, ST_NT, 0, s>>>(a);
  LAUNCHED();
  return SPMV_OK;
}

extern "C" spmv_status spmv_dist_halo_host(const int32_t* rowptr, const int32_t* colidx, int64_t m,
                                           int32_t nranks, int64_t* halo) {
  if (!rowptr || !halo || nranks < 1) return arg_fail("bad halo arguments");
  const int P = nranks;
  std::vector<int64_t> b(P + 1);
  ST(spmv_csr_partition(rowptr, m, P, b.data()));
  std::vector<int64_t> lo((size_t)P * P, INT64_MAX), hi((size_t)P * P, -1);
  for (int r = 0; r < P; ++r)
    for (int64_t i = b[r]; i < b[r + 1]; ++i)
      for (int64_t k = rowptr[i]; k < rowptr[i + 1]; ++k) {
        const int64_t c = colidx[k];
        const int64_t sidx = (std::upper_bound(b.begin(), b.begin() + P, c) - b.begin()) - 1;
        if (sidx == r) continue;
        const size_t e = (size_t)r * P + sidx;
        lo[e] = std::min(lo[e], c - b[sidx]);
        hi[e] = std::max(hi[e], c - b[sidx]);
      }
  for (size_t e = 0; e < (size_t)P * P; ++e) {
    halo[2 * e] = hi[e] >= 0 ? lo[e] : 0;
    halo[2 * e + 1] = hi[e] >= 0 ? hi[e] + 1 : 0;
  }
  return SPMV_OK;
}

extern "C" spmv_status spmv_dist_halo(spmv_csr_t h, int64_t* halo, int32_t* used) {
  if (!h || !halo) return arg_fail("NULL argument");
  if (!h->dist) return arg_fail("not a distributed handle");
  for (size_t i = 0; i < h->halo.size(); ++i) halo[i] = h->halo[i];
  if (used) *used = h->use_halo ? 1 : 0;
  return SPMV_OK;
}

extern "C" spmv_status spmv_dist_colidx(spmv_csr_t h, int32_t* colidx_local_host) {
  if (!h || !colidx_local_host) return arg_fail("NULL argument");
  if (!h->dist) return arg_fail("not a distributed handle");
  CK(cudaSetDevice(h->device));
  CK(cudaMemcpy(colidx_local_host, h->ci_own, sizeof(int32_t) * (size_t)(h->k1 - h->k0),
                cudaMemcpyDeviceToHost));
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
  info->transport = h->dist ? (h->dist->p2p ? 2 : 1) : 0;
  info->nranks = h->dist ? h->dist->nranks : 1;
  info->sorted_cols = h->sorted;
  info->grid = h->grid;
  info->cluster = h->kernel == SPMV_KERNEL_XPLAN ? h->xp.B : h->kernel == SPMV_KERNEL_XSTAT ? h->xB : 0;
  info->plan_bytes = h->xp.built ? (int64_t)h->xp.bytes
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

// ------------------------------------------------------------------ dist
extern "C" spmv_status spmv_dist_get_unique_id(void* id128) {
  if (!id128) return arg_fail("id128 is NULL");
  static_assert(sizeof(ncclUniqueId) == 128, "ncclUniqueId is 128 bytes");
  NK(ncclGetUniqueId((ncclUniqueId*)id128));
  return SPMV_OK;
}

extern "C" spmv_status spmv_dist_init(spmv_dist_t* out, int32_t rank, int32_t nranks,
                                      const void* id128, int32_t device) {
  if (!out || !id128 || nranks < 1 || rank < 0 || rank >= nranks) return arg_fail("bad dist arguments");
  *out = nullptr;
  CK(cudaSetDevice(device));
  spmv_dist_s* d = new spmv_dist_s();
  d->rank = rank;
  d->nranks = nranks;
  d->device = device;
  ncclUniqueId id;
  memcpy(&id, id128, sizeof id);
  ncclResult_t r = ncclCommInitRank(&d->comm, nranks, id, rank);
  if (r != ncclSuccess) {
    g_err = std::string("ncclCommInitRank: ") + ncclGetErrorString(r);
    delete d;
    return SPMV_ERR_NCCL;
  }
  *out = d;
  return SPMV_OK;
}

extern "C" spmv_status spmv_dist_init_p2p(spmv_dist_t* out, int32_t rank, int32_t nranks, int32_t device) {
  if (!out || nranks < 1 || rank < 0 || rank >= nranks) return arg_fail("bad dist arguments");
  *out = nullptr;
  CK(cudaSetDevice(device));
  spmv_dist_s* d = new spmv_dist_s();
  d->rank = rank;
  d->nranks = nranks;
  d->device = device;
  d->p2p = 1;
  *out = d;
  return SPMV_OK;
}

extern "C" spmv_status spmv_csr_p2p_handle(spmv_csr_t h, void* handle64) {
  if (!h || !handle64) return arg_fail("NULL argument");
  if (!use_p2p(h)) return arg_fail("not a p2p distributed handle");
  static_assert(sizeof(cudaIpcMemHandle_t) == 64, "cudaIpcMemHandle_t is 64 bytes");
  CK(cudaSetDevice(h->device));
  cudaIpcMemHandle_t m;
  CK(cudaIpcGetMemHandle(&m, h->fabric));
  memcpy(handle64, &m, 64);
  return SPMV_OK;
}

extern "C" spmv_status spmv_csr_p2p_connect(spmv_csr_t h, const void* handles) {
  if (!h || !handles) return arg_fail("NULL argument");
  if (!use_p2p(h)) return arg_fail("not a p2p distributed handle");
  CK(cudaSetDevice(h->device));
  const int P = h->dist->nranks, me = h->dist->rank;
  for (int q = 0; q < P; ++q) {
    if (q == me || h->peers[q]) continue;
    cudaIpcMemHandle_t m;
    memcpy(&m, (const char*)handles + 64 * q, 64);
    void* ptr = nullptr;
    CK(cudaIpcOpenMemHandle(&ptr, m, cudaIpcMemLazyEnablePeerAccess));
    h->peers[q] = (unsigned char*)ptr;
  }
  CK(cudaMemcpy(h->peer_table, h->peers.data(), sizeof(unsigned char*) * P, cudaMemcpyHostToDevice));
  CK(cudaDeviceSynchronize());
  h->p2p_connected = true;
  return SPMV_OK;
}

extern "C" spmv_status spmv_dist_destroy(spmv_dist_t d) {
  if (!d) return SPMV_OK;
  spmv_status st = SPMV_OK;
  if (d->comm) {
    ncclResult_t r = ncclCommDestroy(d->comm);
    if (r != ncclSuccess) { g_err = ncclGetErrorString(r); st = SPMV_ERR_NCCL; }
  }
  delete d;
  return st;
}

// ------------------------------------------------------------------ idioms (NEXT-4)
#include "idioms_abi.cuh"
// ------------------------------------------------------------------ JDS-32 (NEXT-4, Parboil format)
#include "jds_abi.cuh"
