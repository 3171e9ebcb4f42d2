// stencil_abi.cu -- stencil27_apply: the paper's Stencil
// idiom (Fig. 13) as a matrix-free 27-point operator; kernels in
// stencil_kernel.cuh.
#include "abi_common.h"
#include "stencil_kernel.cuh"

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
  // resolved once, thread-safe (function-local static initialisation)
  static const encode_fn fn = []() -> encode_fn {
    void* p = nullptr;
    cudaDriverEntryPointQueryResult q;
    if (cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &p, cudaEnableDefault, &q) == cudaSuccess &&
        q == cudaDriverEntryPointSuccess)
      return reinterpret_cast<encode_fn>(p);
    cudaGetLastError();
    return nullptr;
  }();
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
  int tenv = 1;
  env_int("SPMV_STENCIL_TMA", &tenv);
  // SPMV_STENCIL_TMA=2 (tests): the TMA form is required -- also when the weights or knobs rule out box2
  if (tenv == 2 && !box2) return arg_fail("SPMV_STENCIL_TMA=2 but the call does not take the box2 (TMA) form");
  if (box2) {
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
