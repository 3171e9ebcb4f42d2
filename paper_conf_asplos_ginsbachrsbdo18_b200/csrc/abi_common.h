// abi_common.h -- host-side internals shared by the translation units of the
// C ABI (include/spmv.h): the handle type, error helpers and the functions one
// unit calls in another.  No arithmetic of the hot path lives here: every step
// runs in the kernels of the *.cuh headers.  P:a-b = /root/reference/PAPER.md
// lines; Rn = DESIGN.md reading n.
//
//   spmv_abi.cu     create / destroy / spmv_csr / introspection (8(a) a1, a2)
//   plans.cu        kernel plans (XPLAN, SELL, merge, XSTAT) and run_spmv
//   cg_driver.cu    CG and the NAS outer iteration (a3, a4; NEXT-1)
//   dist.cu         row-sharded mode: NCCL and peer-memory transports (a5)
//   stencil_abi.cu  matrix-free 27-point stencil (NEXT-3)
//   idioms_abi.cu, jds_abi.cu   NEXT-4
#pragma once
#include <algorithm>
#include <atomic>
#include <cmath>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <functional>
#include <string>
#include <vector>

#include <cuda_runtime.h>
#include <nccl.h>

#include "../../include/spmv.h"
#include "common.cuh"
#include "merge_kernel.cuh"
#include "sell_kernel.cuh"
#include "spmv_kernels.cuh"
#include "xplan_kernel.cuh"
#include "xstat_kernel.cuh"
#include "xt_kernel.cuh"

using namespace spmv;

// ------------------------------------------------------------------ errors
extern thread_local std::string g_err;      // spmv_last_error_string
extern std::atomic<uint64_t> g_launches;    // spmv_launch_count

inline spmv_status cuda_fail(cudaError_t e, const char* what, int line) {
  char buf[512];
  snprintf(buf, sizeof buf, "%s (line %d): %s", what, line, cudaGetErrorString(e));
  g_err = buf;
  return e == cudaErrorMemoryAllocation ? SPMV_ERR_NOMEM : SPMV_ERR_CUDA;
}
inline spmv_status arg_fail(const char* why) {
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
  int proxy = 0;              // 1: measurement proxy: rank r's share on one GPU, exchanges skipped
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
  // opts.l2_window: the persisting L2 window over x (0 = off)
  size_t l2win_bytes = 0, l2persist_bytes = 0;
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
    int dyn = 0, ncl_plan = 0;   // dyn: tiles popped from tq at run time; the plan has ncl_plan row ranges
    int* tq = nullptr;           // dyn: [0] next tile, [1] finished CTAs (reset by the last CTA)
    long long* cta_range = nullptr;  // small plans: [grid][2] chunk byte range per CTA (whole-range L2 prefetch)
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
    int bankperm = 1;  // k_xplan_bankperm after every pack (SPMV_XPLAN_PERM=0: CSR order within each row)
    // persisting-L2 access window over the plan (SPMV_XPLAN_PLANWIN=1; small plans that stay L2-resident)
    size_t win_bytes = 0;
    float win_ratio = 0.f;
  } xp;
  cudaStream_t side = nullptr;
  cudaEvent_t ev_fork = nullptr, ev_join = nullptr;
  // XT (TMA-streamed column-parted plan, xt_kernel.cuh)
  struct XtPlan {
    bool built = false;
    int B = 0, Q = 0, NB = 0, NS = 0, ncl = 0, ntiles = 0, xcap = 0;
    size_t smem = 0;
    int64_t bytes = 0, nchunks = 0, nstages = 0;
    unsigned char* plan = nullptr;
    int *cl_part = nullptr, *cl_tile0 = nullptr, *cta_w = nullptr, *cta_st0 = nullptr, *part_cl0 = nullptr;
    long long *cl_rows = nullptr, *cta_col0 = nullptr, *st_off = nullptr, *bcol = nullptr, *ck_off = nullptr;
    uint32_t* st_info = nullptr;
    uint2* ck_meta = nullptr;
    int *bseg = nullptr, *ck_len = nullptr, *row_slot = nullptr, *gcnt = nullptr;
    double* ypart = nullptr;
    void (*k)(XtArgs) = nullptr;
    void (*kdot)(XtArgs) = nullptr;
    void release() {
      void* bufs[] = {plan, cl_part, cl_tile0, cta_w, cta_st0, part_cl0, cl_rows, cta_col0, st_off, bcol, ck_off,
                      st_info, ck_meta, bseg, ck_len, row_slot, gcnt, ypart};
      for (void* q : bufs)
        if (q) cudaFree(q);
      *this = XtPlan();
    }
  } xt;
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
  // z, r, q, p_single, s_vec live in ONE allocation (cg_alloc), so one persisting-L2 window can keep
  // the CG vectors resident while the plan streams through L2 (SPMV_CG_L2WIN)
  unsigned char* cgws = nullptr;
  size_t cgws_bytes = 0;
  size_t cgwin_bytes = 0;
  float cgwin_ratio = 0.f;
  int cg_variant = 0;                          // 0 textbook (NPB conj_grad), 1 Chronopoulos-Gear, 2 persistent C-G
  int pdl = 1;                                 // programmatic dependent launch of the SpMV / k_cgcg chain (SPMV_PDL=0: off)
  unsigned int* gbar = nullptr;                // persistent CG: grid barrier counter
  double *part_pq = nullptr, *part_rr = nullptr, *part_res = nullptr, *part_xz = nullptr,
         *part_zz = nullptr, *scal = nullptr, *out2 = nullptr;
  int* flags = nullptr;
  double *stage_x = nullptr, *stage_z = nullptr;
  Graph g_npb;
};

// --------------------------------------------------------------- helpers
inline bool env_int(const char* name, int* v) {
  const char* s = getenv(name);
  if (!s || !*s) return false;
  *v = atoi(s);
  return true;
}

// Sweep-only knobs (loads in flight, prefetch, per-CTA timestamps, ...): read
// from the environment only in variant builds (-DSPMV_TUNING, tools/
// build_variants.sh); the product library ignores them.  The variant
// selectors the parity tests use (SPMV_KERNEL, SPMV_XPLAN_B, SPMV_STENCIL_*,
// SPMV_HIST, ...) stay runtime env_int reads, documented in DESIGN.md 7b.
inline bool tuning_env(const char* name, int* v) {
#ifdef SPMV_TUNING
  return env_int(name, v);
#else
  (void)name;
  (void)v;
  return false;
#endif
}

// Launch with programmatic stream serialization (PDL) when `pdl`: the kernel may
// start while its stream predecessor runs and synchronises with pdl_wait()
// (common.cuh).  Without it, an ordinary launch.
// `win` (nullable): a persisting access window carried by the launch.
template <typename... KArgs, typename... Args>
inline cudaError_t launch_maybe_pdl(void (*k)(KArgs...), dim3 grid, dim3 block, size_t smem, cudaStream_t s, bool pdl,
                                    const cudaAccessPolicyWindow* win, Args&&... args) {
  cudaLaunchConfig_t cfg = {};
  cfg.gridDim = grid;
  cfg.blockDim = block;
  cfg.dynamicSmemBytes = smem;
  cfg.stream = s;
  cudaLaunchAttribute at[2];
  cfg.attrs = at;
  cfg.numAttrs = 0;
  if (pdl) {
    at[cfg.numAttrs].id = cudaLaunchAttributeProgrammaticStreamSerialization;
    at[cfg.numAttrs].val.programmaticStreamSerializationAllowed = 1;
    ++cfg.numAttrs;
  }
  if (win) {
    at[cfg.numAttrs].id = cudaLaunchAttributeAccessPolicyWindow;
    at[cfg.numAttrs].val.accessPolicyWindow = *win;
    ++cfg.numAttrs;
  }
  return cudaLaunchKernelEx(&cfg, k, std::forward<Args>(args)...);
}

// The CG-vector window of a handle (nullptr when off).
inline const cudaAccessPolicyWindow* cg_window(const spmv_csr_s* h, cudaAccessPolicyWindow* w) {
  if (!h->cgwin_bytes) return nullptr;
  w->base_ptr = h->cgws;
  w->num_bytes = h->cgwin_bytes;
  w->hitRatio = h->cgwin_ratio;
  w->hitProp = cudaAccessPropertyPersisting;
  w->missProp = cudaAccessPropertyStreaming;
  return w;
}

inline int num_sms(int dev) {
  int v = kNumSMs;
  cudaDeviceGetAttribute(&v, cudaDevAttrMultiProcessorCount, dev);
  return v > 0 ? v : kNumSMs;
}

// 1 = device (or managed) memory of `dev`, 0 = host (pinned, pageable), -1 = error
inline int mem_kind(const void* p, int dev) {
  cudaPointerAttributes a;
  cudaError_t e = cudaPointerGetAttributes(&a, p);
  if (e != cudaSuccess) { cudaGetLastError(); return 0; }
  if (a.type == cudaMemoryTypeDevice || a.type == cudaMemoryTypeManaged)
    return a.device == dev ? 1 : -1;
  return 0;
}

inline spmv_status need_device(const void* p, int dev, const char* what, bool may_be_null) {
  if (!p) return may_be_null ? SPMV_OK : arg_fail(what);
  return mem_kind(p, dev) == 1 ? SPMV_OK : arg_fail(what);
}

inline bool overlap(const void* a, size_t na, const void* b, size_t nb) {
  if (!a || !b || na == 0 || nb == 0) return false;
  const uintptr_t a0 = (uintptr_t)a, b0 = (uintptr_t)b;
  return a0 < b0 + nb && b0 < a0 + na;
}

inline int64_t cdiv(int64_t a, int64_t b) { return (a + b - 1) / b; }

// SPMV_DEBUG=1: trace the create-time plan build on stderr (synchronising).
inline bool dbg() {
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

inline spmv_status ensure_buf(void** p, size_t bytes) {
  if (*p) return SPMV_OK;
  CK(cudaMalloc(p, bytes > 0 ? bytes : 8));
  return SPMV_OK;
}

// ------------------------------------------------------ across the units
// plans.cu
spmv_status xstat_setup(spmv_csr_s* h, bool* ok);
spmv_status xplan_build(spmv_csr_s* h, bool* ok);
spmv_status xplan_pack(spmv_csr_s* h, const void* vals, int values_only);
spmv_status sell_build(spmv_csr_s* h, double max_pad, int sorted, bool* ok);
spmv_status sell_pack(spmv_csr_s* h, const void* vals, int values_only);
spmv_status merge_setup(spmv_csr_s* h);
spmv_status xt_build(spmv_csr_s* h, bool* ok);
bool persist_eligible(const spmv_csr_s* h);
spmv_status launch_cg_persist(spmv_csr_s* h, cudaStream_t s, const void* x_input, double* r, double* p, double* sv,
                              double* w, double* z, double* part_d, double* part_g, int64_t pstride,
                              const double* gam0, int gam0_count, int iters);
spmv_status xt_pack(spmv_csr_s* h, const void* vals, int values_only);
spmv_status launch_xt(spmv_csr_s* h, cudaStream_t s, const void* x, void* y, double alpha, double beta,
                      const double* w, double* part, const P2PHook& hook);
// Local SpMV of the handle: y = alpha*A_loc*x + beta*y (+ partial w.y per CTA).
spmv_status run_spmv(spmv_csr_s* h, cudaStream_t s, const void* vals, const void* x, void* y, double alpha,
                     double beta, const double* w, double* part, const P2PHook* hk = nullptr);
// dist.cu
bool use_p2p(const spmv_csr_s* h);
P2PCtx p2p_ctx(spmv_csr_s* h);
SumSrc p2p_src(spmv_csr_s* h, int slot, int per);  // per: partials pushed per rank (1: one value)
int p2p_push_per(const spmv_csr_s* h, int64_t grid);  // per-CTA pushes for a producer of `grid` CTAs, else 0
int p2p_spmv_push_per(const spmv_csr_s* h);           // ... for the SpMV's fused dot
spmv_status exchange_x(spmv_csr_s* h, cudaStream_t s);
spmv_status reduce_src(spmv_csr_s* h, cudaStream_t s, SumSrc in, int slot, SumSrc* out);
