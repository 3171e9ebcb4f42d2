// jds_abi.cu -- the JDS-32 entry points of include/spmv.h (spmv_jds_create,
// spmv_jds, spmv_jds_destroy; reading R34).  Shares the error/validation
// helpers of abi_common.h; kernels in
// jds_kernel.cuh.
#include "abi_common.h"
#include "jds_kernel.cuh"

struct spmv_jds_s {
  spmv_dtype dt = SPMV_F64;
  int64_t m = 0, n = 0, depth = 0, total = 0;
  const int32_t* perm = nullptr;
  const long long* jds_ptr = nullptr;
  const int32_t* idx = nullptr;
  const void* data = nullptr;
  int device = 0;
  cudaStream_t stream = nullptr;
  int4* units = nullptr;
  int nunits = 0;
  int4* fix = nullptr;
  int nfix = 0;
  double* parts = nullptr;
};

static void jds_free(spmv_jds_s* h) {
  if (!h) return;
  if (h->units) cudaFree(h->units);
  if (h->fix) cudaFree(h->fix);
  if (h->parts) cudaFree(h->parts);
  delete h;
}

extern "C" spmv_status spmv_jds_create(spmv_jds_t* out, spmv_dtype dt, int64_t m, int64_t n, int64_t depth,
                                       const int32_t* perm, const int64_t* jds_ptr, const int32_t* zcnt,
                                       const int32_t* indices, const void* data, void* stream) {
  if (!out) return arg_fail("out is NULL");
  *out = nullptr;
  if (dt != SPMV_F64 && dt != SPMV_F32) return arg_fail("dtype must be SPMV_F64 or SPMV_F32");
  if (m < 0 || n < 0 || depth < 0) return arg_fail("m, n, depth must be >= 0");
  if (m > 2147483647LL - 64) return arg_fail("m too large");
  int dev = 0;
  if (cudaGetDevice(&dev) != cudaSuccess) return arg_fail("no current CUDA device");
  const int64_t ns = cdiv(m, 32);
  if (m > 0) {
    ST(need_device(perm, dev, "perm must be a device pointer", false));
    ST(need_device(zcnt, dev, "zcnt must be a device pointer", false));
  }
  ST(need_device(jds_ptr, dev, "jds_ptr must be a device pointer", false));
  cudaStream_t s = (cudaStream_t)stream;
  // host copies of the small arrays: zcnt (m/32) and jds_ptr (depth+1)
  std::vector<int32_t> zc((size_t)ns);
  std::vector<long long> jp((size_t)depth + 1);
  if (ns) CK(cudaMemcpyAsync(zc.data(), zcnt, sizeof(int32_t) * ns, cudaMemcpyDeviceToHost, s));
  CK(cudaMemcpyAsync(jp.data(), jds_ptr, sizeof(long long) * (depth + 1), cudaMemcpyDeviceToHost, s));
  CK(cudaStreamSynchronize(s));
  // structure checks (O(m/32 + depth), always): zcnt non-increasing, depth = zcnt[0],
  // diagonal k spans exactly the 32-row slices with zcnt > k
  if (ns && (int64_t)zc[0] != depth) { g_err = "depth != zcnt[0]"; return SPMV_ERR_INDEX; }
  if (!ns && depth != 0) { g_err = "depth must be 0 when m == 0"; return SPMV_ERR_INDEX; }
  for (int64_t q = 0; q < ns; ++q)
    if (zc[q] < 0 || (q && zc[q] > zc[q - 1])) { g_err = "zcnt must be non-increasing and >= 0"; return SPMV_ERR_INDEX; }
  if (jp[0] != 0) { g_err = "jds_ptr[0] must be 0"; return SPMV_ERR_INDEX; }
  {
    int64_t q = ns;  // slices with zcnt > k (shrinks as k grows)
    for (int64_t k = 0; k < depth; ++k) {
      while (q > 0 && zc[q - 1] <= k) --q;
      if (jp[k + 1] - jp[k] != 32 * q) { g_err = "jds_ptr inconsistent with zcnt (R34)"; return SPMV_ERR_INDEX; }
    }
  }
  const int64_t total = jp[depth];
  if (total > 0) {
    ST(need_device(indices, dev, "indices must be a device pointer", false));
    ST(need_device(data, dev, "data must be a device pointer", false));
    if (n == 0) return arg_fail("entries need n >= 1");
  }
  // warp units: each slice in pieces of <= JDS_SEG steps (slices are already longest first)
  std::vector<int4> units, fix;
  int nparts = 0;
  for (int64_t q = 0; q < ns; ++q) {
    const int L = zc[q];
    const int pieces = L <= JDS_SEG ? 1 : (int)cdiv(L, JDS_SEG);
    if (pieces == 1) {
      units.push_back(make_int4((int)q, 0, L, -1));
    } else {
      fix.push_back(make_int4((int)q, nparts, pieces, 0));
      for (int p = 0; p < pieces; ++p)
        units.push_back(make_int4((int)q, p * JDS_SEG, std::min(L, (p + 1) * JDS_SEG), nparts + p));
      nparts += pieces;
    }
  }
  spmv_jds_s* h = new spmv_jds_s();
  h->dt = dt; h->m = m; h->n = n; h->depth = depth; h->total = total;
  h->perm = perm; h->jds_ptr = (const long long*)jds_ptr; h->idx = indices; h->data = data;
  h->device = dev; h->stream = s;
  h->nunits = (int)units.size();
  h->nfix = (int)fix.size();
  auto fail = [&](cudaError_t e) { jds_free(h); return cuda_fail(e, "spmv_jds_create", __LINE__); };
  cudaError_t e;
  if (h->nunits) {
    if ((e = cudaMalloc(&h->units, sizeof(int4) * units.size())) != cudaSuccess) return fail(e);
    if ((e = cudaMemcpyAsync(h->units, units.data(), sizeof(int4) * units.size(), cudaMemcpyHostToDevice, s)) != cudaSuccess) return fail(e);
  }
  if (h->nfix) {
    if ((e = cudaMalloc(&h->fix, sizeof(int4) * fix.size())) != cudaSuccess) return fail(e);
    if ((e = cudaMemcpyAsync(h->fix, fix.data(), sizeof(int4) * fix.size(), cudaMemcpyHostToDevice, s)) != cudaSuccess) return fail(e);
    if ((e = cudaMalloc(&h->parts, sizeof(double) * 32 * (size_t)nparts)) != cudaSuccess) return fail(e);
  }
  if ((e = cudaStreamSynchronize(s)) != cudaSuccess) return fail(e);
  *out = h;
  return SPMV_OK;
}

extern "C" spmv_status spmv_jds(spmv_jds_t h, const void* x, void* y, double alpha, double beta) {
  if (!h) return arg_fail("handle is NULL");
  if (h->m == 0) return SPMV_OK;
  CK(cudaSetDevice(h->device));
  const size_t ts = h->dt == SPMV_F64 ? 8 : 4;
  ST(need_device(y, h->device, "y must be a device pointer", false));
  if (alpha != 0.0 && h->total > 0) ST(need_device(x, h->device, "x must be a device pointer", false));
  if ((alpha != 0.0 && h->total > 0 && overlap(y, ts * (size_t)h->m, x, ts * (size_t)h->n)) ||
      overlap(y, ts * (size_t)h->m, h->data, ts * (size_t)h->total) ||
      overlap(y, ts * (size_t)h->m, h->idx, 4 * (size_t)h->total) ||
      overlap(y, ts * (size_t)h->m, h->perm, 4 * (size_t)h->m)) {
    g_err = "y overlaps an input";
    return SPMV_ERR_ALIAS;
  }
  cudaStream_t s = h->stream;
  const bool f32 = h->dt == SPMV_F32;
  const double a = f32 ? (double)(float)alpha : alpha, b = f32 ? (double)(float)beta : beta;
  if (a == 0.0) {  // A and x are not read (R6)
    const int64_t g = std::min<int64_t>(cdiv(h->m, 256), 4LL * num_sms(h->device));
    if (f32) k_scale<float><<<g, 256, 0, s>>>(h->m, (float*)y, b);
    else k_scale<double><<<g, 256, 0, s>>>(h->m, (double*)y, b);
    LAUNCHED();
    return SPMV_OK;
  }
  const unsigned g = (unsigned)cdiv((int64_t)h->nunits * 32, JDS_THREADS);
  if (f32)
    k_spmv_jds<float><<<g, JDS_THREADS, 0, s>>>(h->units, h->nunits, h->m, h->jds_ptr, h->idx, (const float*)h->data,
                                               (const float*)x, h->perm, (float*)y, a, b, h->parts);
  else
    k_spmv_jds<double><<<g, JDS_THREADS, 0, s>>>(h->units, h->nunits, h->m, h->jds_ptr, h->idx,
                                                (const double*)h->data, (const double*)x, h->perm, (double*)y, a, b,
                                                h->parts);
  LAUNCHED();
  if (h->nfix) {
    const unsigned gf = (unsigned)cdiv((int64_t)h->nfix * 32, JDS_THREADS);
    if (f32) k_jds_fixup<float><<<gf, JDS_THREADS, 0, s>>>(h->fix, h->nfix, h->m, h->parts, h->perm, (float*)y, a, b);
    else k_jds_fixup<double><<<gf, JDS_THREADS, 0, s>>>(h->fix, h->nfix, h->m, h->parts, h->perm, (double*)y, a, b);
    LAUNCHED();
  }
  return SPMV_OK;
}

extern "C" spmv_status spmv_jds_destroy(spmv_jds_t h) {
  if (!h) return SPMV_OK;
  cudaSetDevice(h->device);
  cudaError_t e = cudaStreamSynchronize(h->stream);
  jds_free(h);
  return e == cudaSuccess ? SPMV_OK : cuda_fail(e, "spmv_jds_destroy", __LINE__);
}
