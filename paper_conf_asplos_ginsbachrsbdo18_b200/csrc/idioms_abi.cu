// idioms_abi.cu -- the C ABI of include/idioms.h (histogram, scalar
// reduction, NAS EP).  Shares the error/validation helpers of
// abi_common.h; the
// arithmetic is in idiom_kernels.cuh.  Rn = DESIGN.md reading n.
#include "abi_common.h"
#include "../../include/idioms.h"
#include "idiom_kernels.cuh"

static int cur_device(int* dev) { return cudaGetDevice(dev) == cudaSuccess ? 0 : -1; }

static bool aligned16(const void* p) { return ((uintptr_t)p & 15u) == 0; }

// ------------------------------------------------------------ scalar reduction
static int64_t red_grid(int64_t n, int sms) {
  // ~4 x 16-B loads in flight per thread, 2 CTAs of 512 per SM; small n: fewer CTAs
  return std::max<int64_t>(1, std::min<int64_t>({(int64_t)2 * sms, cdiv(n, 8LL * kRedThreads), kRedMaxGrid}));
}

extern "C" spmv_status idl_reduce_workspace(int64_t n, size_t* bytes) {
  if (!bytes) return arg_fail("bytes is NULL");
  if (n < 0) return arg_fail("n must be >= 0");
  *bytes = kWsHeader + sizeof(double) * kRedMaxGrid;
  return SPMV_OK;
}

extern "C" spmv_status idl_reduce(spmv_dtype dt, idl_red_op op, const void* a, const void* b, int64_t n,
                                  double* out, void* workspace, size_t workspace_bytes, void* stream) {
  if (dt != SPMV_F64 && dt != SPMV_F32) return arg_fail("dtype must be SPMV_F64 or SPMV_F32");
  if (op != IDL_RED_SUM && op != IDL_RED_DOT) return arg_fail("op must be IDL_RED_SUM or IDL_RED_DOT");
  if (n < 0) return arg_fail("n must be >= 0");
  if (op == IDL_RED_SUM && b) return arg_fail("b must be NULL for IDL_RED_SUM");
  size_t need = 0;
  ST(idl_reduce_workspace(n, &need));
  if (workspace_bytes < need) return arg_fail("workspace too small (idl_reduce_workspace)");
  int dev = 0;
  if (cur_device(&dev)) return arg_fail("no current CUDA device");
  ST(need_device(out, dev, "out must be a device pointer on the current device", false));
  ST(need_device(workspace, dev, "workspace must be a device pointer on the current device", false));
  if (n > 0) {
    ST(need_device(a, dev, "a must be a device pointer on the current device", false));
    if (op == IDL_RED_DOT) ST(need_device(b, dev, "b must be a device pointer on the current device", false));
  }
  const size_t ts = dt == SPMV_F64 ? 8 : 4;
  if (n > 0 && (overlap(out, 8, a, ts * (size_t)n) || (b && overlap(out, 8, b, ts * (size_t)n)))) {
    g_err = "out overlaps an input";
    return SPMV_ERR_ALIAS;
  }
  if (overlap(workspace, need, out, 8)) {
    g_err = "workspace overlaps out";
    return SPMV_ERR_ALIAS;
  }
  cudaStream_t s = (cudaStream_t)stream;
  const int64_t G = red_grid(n, num_sms(dev));
  const int W = dt == SPMV_F64 ? 2 : 4;
  const int64_t chunk = std::max<int64_t>(W, cdiv(cdiv(std::max<int64_t>(n, 1), G), W) * W);
  const int64_t grid = std::max<int64_t>(1, cdiv(std::max<int64_t>(n, 1), chunk));
  unsigned* ticket = (unsigned*)workspace;
  double* part = (double*)((char*)workspace + kWsHeader);
  const bool vec = aligned16(a) && (op == IDL_RED_SUM || aligned16(b));
  const bool dot = op == IDL_RED_DOT;
#define RED_LAUNCH(T)                                                                                     \
  do {                                                                                                    \
    const T* A_ = (const T*)a;                                                                            \
    const T* B_ = (const T*)b;                                                                            \
    if (dot) {                                                                                            \
      if (vec) k_reduce<T, true, true><<<(int)grid, kRedThreads, 0, s>>>(n, chunk, A_, B_, out, ticket, part);   \
      else k_reduce<T, true, false><<<(int)grid, kRedThreads, 0, s>>>(n, chunk, A_, B_, out, ticket, part);      \
    } else {                                                                                              \
      if (vec) k_reduce<T, false, true><<<(int)grid, kRedThreads, 0, s>>>(n, chunk, A_, B_, out, ticket, part);  \
      else k_reduce<T, false, false><<<(int)grid, kRedThreads, 0, s>>>(n, chunk, A_, B_, out, ticket, part);     \
    }                                                                                                     \
  } while (0)
  if (dt == SPMV_F64) RED_LAUNCH(double);
  else RED_LAUNCH(float);
#undef RED_LAUNCH
  LAUNCHED();
  return SPMV_OK;
}

// ------------------------------------------------------------------ histogram
static const int kHistSmemMax = 200 * 1024;  // dynamic shared memory of one 1024-thread CTA

static size_t hist_bin_bytes(idl_hist_kind kind) { return kind == IDL_HIST_SUM_F64 ? 8 : 4; }

// Bucketed counting (idiom_kernels.cuh K1-K4): eligible for the counting kinds
// when the bins exceed one CTA's shared memory, fit HB_MAXB buckets, and there
// are >= 2 keys per bin.  Workspace: [fixed part | cnt nb*G u32 | total nb u32 | keys n u16].
static int hb_grid(int sms) { return std::min(2 * sms, HB_THREADS); }
static bool hb_eligible(idl_hist_kind kind, int64_t n, int64_t nbins) {
  return kind != IDL_HIST_SUM_F64 && (size_t)4 * (size_t)nbins > (size_t)kHistSmemMax &&
         nbins <= (int64_t)HB_MAXB * HB_BW && n >= 2 * nbins && n < 4294967295LL;
}
static size_t hist_fixed_bytes(idl_hist_kind kind, int64_t nbins) {
  // saturating bins are counted in a uint32 workspace first (then min(255, old + count))
  return kind == IDL_HIST_SAT_U8 ? (((size_t)4 * (size_t)nbins + 255) & ~size_t(255)) : 256;
}
static size_t hb_bytes(int64_t n, int64_t nbins, int G) {
  const size_t nb = (size_t)cdiv(nbins, HB_BW);
  return ((4 * nb * (size_t)G + 4 * nb + 255) & ~size_t(255)) + 2 * (size_t)n + 256;
}

extern "C" spmv_status idl_histogram_workspace(idl_hist_kind kind, int64_t n, int64_t nbins, size_t* bytes) {
  if (!bytes) return arg_fail("bytes is NULL");
  if (kind < IDL_HIST_COUNT_U32 || kind > IDL_HIST_SUM_F64) return arg_fail("unknown histogram kind");
  if (n < 0 || nbins < 1 || nbins > 2147483647LL) return arg_fail("need n >= 0 and 1 <= nbins <= 2^31-1");
  size_t b = hist_fixed_bytes(kind, nbins);
  if (hb_eligible(kind, n, nbins)) b += hb_bytes(n, nbins, HB_THREADS);  // any grid up to HB_THREADS
  *bytes = b;
  return SPMV_OK;
}

static int hist_mode() {  // SPMV_HIST=smem|global|agg|bucket forces a variant (kernel sweeps), else auto
  const char* v = getenv("SPMV_HIST");
  if (!v) return 0;
  if (!strcmp(v, "smem")) return 1;
  if (!strcmp(v, "global")) return 2;
  if (!strcmp(v, "agg")) return 3;
  if (!strcmp(v, "bucket")) return 4;
  return 0;
}

extern "C" spmv_status idl_histogram(idl_hist_kind kind, const int32_t* keys, const double* w, int64_t n,
                                     int64_t nbins, void* bins, void* workspace, size_t workspace_bytes,
                                     void* stream) {
  size_t need = 0;
  ST(idl_histogram_workspace(kind, n, nbins, &need));  // validates kind, n, nbins
  (void)need;
  if (kind == IDL_HIST_SUM_F64 ? false : w != nullptr) return arg_fail("w must be NULL for the counting kinds");
  if (kind == IDL_HIST_SAT_U8 && n > 4294967295LL) return arg_fail("IDL_HIST_SAT_U8 needs n < 2^32");
  const size_t fixed = hist_fixed_bytes(kind, nbins);
  if (kind == IDL_HIST_SAT_U8 && workspace_bytes < fixed) return arg_fail("workspace too small (idl_histogram_workspace)");
  int dev = 0;
  if (cur_device(&dev)) return arg_fail("no current CUDA device");
  ST(need_device(bins, dev, "bins must be a device pointer on the current device", false));
  const int sms_ = num_sms(dev);
  const int hbG = hb_grid(sms_);
  const int mode0 = hist_mode();
  // bucketed counting when eligible and the caller's workspace holds it (older
  // callers that pass the fixed part only keep the atomic paths)
  // opt-in (SPMV_HIST=bucket): measured slower than the L2 atomics on NAS IS
  // class C (878 vs 748 us; its tile-staged scatter pass alone takes 566 us)
  const bool use_hb = hb_eligible(kind, n, nbins) && workspace && workspace_bytes >= fixed + hb_bytes(n, nbins, hbG) &&
                      mode0 == 4;
  if (kind == IDL_HIST_SAT_U8 || use_hb)
    ST(need_device(workspace, dev, "workspace must be a device pointer on the current device", false));
  if (n > 0) {
    ST(need_device(keys, dev, "keys must be a device pointer on the current device", false));
    if (kind == IDL_HIST_SUM_F64) ST(need_device(w, dev, "w must be a device pointer on the current device", false));
  }
  const size_t bb = kind == IDL_HIST_SAT_U8 ? 1 : hist_bin_bytes(kind);
  if (n > 0 && (overlap(bins, bb * (size_t)nbins, keys, 4 * (size_t)n) ||
                (w && overlap(bins, bb * (size_t)nbins, w, 8 * (size_t)n)))) {
    g_err = "bins overlap keys or w";
    return SPMV_ERR_ALIAS;
  }
  if (kind == IDL_HIST_SAT_U8 && overlap(workspace, need, bins, (size_t)nbins)) {
    g_err = "workspace overlaps bins";
    return SPMV_ERR_ALIAS;
  }
  if (n == 0) return SPMV_OK;
  cudaStream_t s = (cudaStream_t)stream;
  const int sms = num_sms(dev);
  if (use_hb) {
    if (overlap(workspace, fixed + hb_bytes(n, nbins, hbG), bins, (kind == IDL_HIST_SAT_U8 ? 1 : 4) * (size_t)nbins) ||
        overlap(workspace, fixed + hb_bytes(n, nbins, hbG), keys, 4 * (size_t)n)) {
      g_err = "workspace overlaps bins or keys";
      return SPMV_ERR_ALIAS;
    }
    const int nb = (int)cdiv(nbins, HB_BW);
    const int64_t chunk = cdiv(cdiv(n, hbG), 4) * 4;
    const int G = (int)cdiv(n, chunk);
    char* wb = (char*)workspace + fixed;
    unsigned* cnt = (unsigned*)wb;
    unsigned* total = cnt + (size_t)nb * G;
    uint16_t* sorted = (uint16_t*)(wb + ((4 * (size_t)nb * G + 4 * (size_t)nb + 255) & ~size_t(255)));
    k_hb_count<<<G, HB_THREADS, 0, s>>>(n, chunk, (int)nbins, nb, keys, cnt, aligned16(keys) ? 1 : 0);
    LAUNCHED();
    k_hb_scan<<<nb, HB_THREADS, 0, s>>>(G, cnt, total);
    LAUNCHED();
    CK(cudaFuncSetAttribute(k_hb_scatter, cudaFuncAttributeMaxDynamicSharedMemorySize, 4 * HB_TILE));
    k_hb_scatter<<<G, HB_THREADS, 4 * HB_TILE, s>>>(n, chunk, (int)nbins, nb, keys, cnt, total, sorted);
    LAUNCHED();
    const size_t sm4 = (size_t)4 * HB_BW;
    if (kind == IDL_HIST_COUNT_U32) {
      CK(cudaFuncSetAttribute(k_hb_bins<0>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)sm4));
      k_hb_bins<0><<<nb, HB_THREADS, sm4, s>>>((int)nbins, nb, total, sorted, bins);
    } else {
      CK(cudaFuncSetAttribute(k_hb_bins<1>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)sm4));
      k_hb_bins<1><<<nb, HB_THREADS, sm4, s>>>((int)nbins, nb, total, sorted, bins);
    }
    LAUNCHED();
    return SPMV_OK;
  }
  const int nb = (int)nbins;
  const int vec = aligned16(keys) ? 1 : 0;
  void* dst = kind == IDL_HIST_SAT_U8 ? workspace : bins;
  const size_t smem = hist_bin_bytes(kind) * (size_t)nbins;
  const int mode = hist_mode();
  // privatise in shared memory when the bins fit and each CTA has enough keys
  // to amortise zeroing and flushing its copy (>= 4 keys per bin)
  bool use_smem = smem <= (size_t)kHistSmemMax && n >= 4 * nbins;
  if (mode == 1) use_smem = smem <= (size_t)kHistSmemMax;
  if (mode >= 2) use_smem = false;
  if (use_smem) {
    const int64_t G = std::max<int64_t>(1, std::min<int64_t>(sms, cdiv(n, 4LL * nbins)));
    const int64_t chunk = cdiv(cdiv(n, G), 4) * 4;
    const int64_t grid = cdiv(n, chunk);
    switch (kind) {
      case IDL_HIST_COUNT_U32:
      case IDL_HIST_SAT_U8:
        CK(cudaFuncSetAttribute(k_hist_smem<0>, cudaFuncAttributeMaxDynamicSharedMemorySize, kHistSmemMax));
        k_hist_smem<0><<<(int)grid, kHistThreads, smem, s>>>(n, chunk, nb, keys, nullptr, (unsigned*)dst, vec);
        break;
      case IDL_HIST_SUM_F64:
        CK(cudaFuncSetAttribute(k_hist_smem<2>, cudaFuncAttributeMaxDynamicSharedMemorySize, kHistSmemMax));
        k_hist_smem<2><<<(int)grid, kHistThreads, smem, s>>>(n, chunk, nb, keys, w, (double*)dst, vec);
        break;
    }
  } else {
    const int64_t grid = std::max<int64_t>(1, std::min<int64_t>(8LL * sms, cdiv(n, 256LL * 4)));
    // warp aggregation pays for skewed keys (hot bins); the saturating kind is
    // Parboil histo's (hot spots), plain counting is IS's (spread keys)
    bool agg = kind == IDL_HIST_SAT_U8;
    if (mode == 2) agg = false;
    if (mode == 3) agg = kind != IDL_HIST_SUM_F64;
    if (kind == IDL_HIST_SUM_F64)
      k_hist_global<2, false><<<(int)grid, 256, 0, s>>>(n, nb, keys, w, (double*)dst, vec);
    else if (agg)
      k_hist_global<0, true><<<(int)grid, 256, 0, s>>>(n, nb, keys, nullptr, (unsigned*)dst, vec);
    else
      k_hist_global<0, false><<<(int)grid, 256, 0, s>>>(n, nb, keys, nullptr, (unsigned*)dst, vec);
  }
  LAUNCHED();
  if (kind == IDL_HIST_SAT_U8) {
    const int64_t g = std::max<int64_t>(1, std::min<int64_t>(cdiv(nbins, 256), 4LL * sms));
    k_hist_sat_fin<<<(int)g, 256, 0, s>>>(nbins, (unsigned*)workspace, (uint8_t*)bins);
    LAUNCHED();
  }
  return SPMV_OK;
}

// ----------------------------------------------------------------------- EP
static const int kEpMaxGrid = 4096;

extern "C" spmv_status ep_npb_workspace(size_t* bytes) {
  if (!bytes) return arg_fail("bytes is NULL");
  *bytes = kWsHeader + sizeof(double) * 12 * kEpMaxGrid;
  return SPMV_OK;
}

extern "C" spmv_status ep_npb(int32_t M, int64_t pair_begin, int64_t pair_count, double* out, void* workspace,
                              size_t workspace_bytes, void* stream) {
  if (M < 24 || M > 40) return arg_fail("M must be in [24, 40]");
  const int64_t total = (int64_t)1 << M;
  if (pair_begin < 0 || pair_count < 0 || pair_begin > total || pair_count > total - pair_begin)
    return arg_fail("pair range outside [0, 2^M)");
  size_t need = 0;
  ST(ep_npb_workspace(&need));
  if (workspace_bytes < need) return arg_fail("workspace too small (ep_npb_workspace)");
  int dev = 0;
  if (cur_device(&dev)) return arg_fail("no current CUDA device");
  ST(need_device(out, dev, "out must be a device pointer on the current device", false));
  ST(need_device(workspace, dev, "workspace must be a device pointer on the current device", false));
  if (overlap(workspace, need, out, 12 * sizeof(double))) {
    g_err = "workspace overlaps out";
    return SPMV_ERR_ALIAS;
  }
  cudaStream_t s = (cudaStream_t)stream;
  const int sms = num_sms(dev);
  // fixed thread count per SM count (deterministic sums): 8 CTAs of 256 per SM,
  // at least 64 pairs per thread (the LCG jump costs ~2*log2(p) multiplies)
  const int64_t T = std::max<int64_t>(1, std::min<int64_t>(8LL * sms * kEpThreads, cdiv(pair_count, 64)));
  const int64_t chunk = std::max<int64_t>(1, cdiv(pair_count, T));
  const int64_t grid = std::max<int64_t>(1, std::min<int64_t>(kEpMaxGrid, cdiv(cdiv(pair_count, chunk), kEpThreads)));
  int compact = 1;  // SPMV_EP_COMPACT=0: per-thread tally without the warp queue
  tuning_env("SPMV_EP_COMPACT", &compact);
  if (compact)
    k_ep<true><<<(int)grid, kEpThreads, 0, s>>>(pair_begin, pair_count, chunk, out, (unsigned*)workspace,
                                               (double*)((char*)workspace + kWsHeader));
  else
    k_ep<false><<<(int)grid, kEpThreads, 0, s>>>(pair_begin, pair_count, chunk, out, (unsigned*)workspace,
                                                (double*)((char*)workspace + kWsHeader));
  LAUNCHED();
  return SPMV_OK;
}
