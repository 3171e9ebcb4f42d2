// plan_xt.cu -- build and launch of the XT plan (xt_kernel.cuh):
// the column parts and blocks, the per-part nnz-balanced cluster row ranges,
// the SELL-32-sigma chunks per (cluster, tile, block), their packing into TMA
// stages of <= XT_SMAX bytes per CTA, and the kernel launch.  The paper's
// device-resident "lazy copy" of A (reading R26): built once at
// create, re-packed by spmv_csr_update_values.
#include "abi_common.h"

namespace {

struct XtShape {
  int B = 0, Q = 0, ncl = 0, sms = 0;
  std::vector<int> ncl_q;  // clusters per part
};

// Clusters of B: how many are co-resident with the kernel's shared memory.
spmv_status xt_clusters(void (*fn)(XtArgs), int B, size_t smem, int* out) {
  *out = 0;
  CK(cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem));
  if (B > 8) CK(cudaFuncSetAttribute(fn, cudaFuncAttributeNonPortableClusterSizeAllowed, 1));
  cudaLaunchConfig_t cfg = {};
  cfg.gridDim = dim3((unsigned)B, 1, 1);
  cfg.blockDim = dim3(XT_THREADS, 1, 1);
  cfg.dynamicSmemBytes = smem;
  cudaLaunchAttribute at[1];
  at[0].id = cudaLaunchAttributeClusterDimension;
  at[0].val.clusterDim.x = (unsigned)B;
  at[0].val.clusterDim.y = 1;
  at[0].val.clusterDim.z = 1;
  cfg.attrs = at;
  cfg.numAttrs = 1;
  int nc = 0;
  cudaError_t e = cudaOccupancyMaxActiveClusters(&nc, fn, &cfg);
  if (e != cudaSuccess) { cudaGetLastError(); nc = 0; }
  *out = nc;
  return SPMV_OK;
}

size_t xt_smem(int xcap, int ts, int NS) {
  return (((size_t)xcap * ts + 127) & ~size_t(127)) + (size_t)NS * XT_SMAX + (size_t)XT_K * XT_R * 8;
}

}  // namespace

spmv_status xt_pack(spmv_csr_s* h, const void* vals, int values_only) {
  auto& X = h->xt;
  cudaStream_t s = h->stream;
  const int64_t g = std::min<int64_t>(cdiv(h->m_loc * 32, 256), 16LL * num_sms(h->device));
  if (h->dt == SPMV_F64)
    k_xt_pack<double><<<g, 256, 0, s>>>(h->rp_loc, h->ci_loc, (const double*)vals, X.bseg, h->m_loc, X.NB, X.B, X.bcol,
                                        X.part_cl0, X.cl_rows, X.cl_tile0, X.ck_off, X.ck_len, X.row_slot, X.plan,
                                        values_only);
  else
    k_xt_pack<float><<<g, 256, 0, s>>>(h->rp_loc, h->ci_loc, (const float*)vals, X.bseg, h->m_loc, X.NB, X.B, X.bcol,
                                       X.part_cl0, X.cl_rows, X.cl_tile0, X.ck_off, X.ck_len, X.row_slot, X.plan,
                                       values_only);
  LAUNCHED();
  return SPMV_OK;
}

// Build the XT plan (create).  *ok = false if not eligible.
spmv_status xt_build(spmv_csr_s* h, bool* ok) {
  *ok = false;
  const int64_t m = h->m_loc, nx = h->nx, nnz = h->k1 - h->k0;
  if (!h->sorted || m == 0 || nx == 0 || nnz == 0 || m > 2147483647LL - XT_R) return SPMV_OK;
  const int ts = (int)h->ts;
  auto& X = h->xt;
  cudaStream_t s = h->stream;
  void (*fn)(XtArgs) = h->dt == SPMV_F64 ? k_spmv_xt<double, false> : k_spmv_xt<float, false>;
  void (*fnd)(XtArgs) = h->dt == SPMV_F64 ? k_spmv_xt<double, true> : nullptr;
  int NS = 7;
  env_int("SPMV_XT_NS", &NS);
  NS = std::max(3, std::min(NS, XT_NS_MAX));
  const size_t smem_cap = 227 * 1024 - 2048;  // dynamic smem of one CTA (static < 2 KB)
  const size_t fixed = (size_t)NS * XT_SMAX + (size_t)XT_K * XT_R * 8;
  if (smem_cap <= fixed + 1024) return SPMV_OK;
  const int64_t wmax = (int64_t)(((smem_cap - fixed) / ts - 1) & ~size_t(7));  // block width + pad <= x budget
  if (wmax < 64) return SPMV_OK;
  // cluster size: the one whose resident clusters (at most 16 parts) cover the most SMs; ties: fewer parts.
  int forcedB = 0, forcedQ = 0;
  env_int("SPMV_XT_B", &forcedB);
  env_int("SPMV_XT_Q", &forcedQ);
  XtShape best;
  for (int B : {2, 4, 8}) {  // >= 2: st.async / remote arrives need a real cluster
    if (forcedB && B != forcedB) continue;
    int nc = 0;
    ST(xt_clusters(fn, B, smem_cap, &nc));
    if (nc < 1) continue;
    int Q = (int)cdiv(nx, (int64_t)B * wmax);
    if (forcedQ >= Q) Q = forcedQ;
    if (Q > 16 || Q > nc) continue;
    XtShape sh;
    sh.B = B;
    sh.Q = Q;
    sh.ncl_q.assign(Q, nc / Q);
    for (int q = 0; q < nc % Q; ++q) sh.ncl_q[q] += 1;
    // rows: every cluster needs at least one 32-row group
    int tot = 0;
    for (int q = 0; q < Q; ++q) {
      sh.ncl_q[q] = (int)std::max<int64_t>(1, std::min<int64_t>(sh.ncl_q[q], cdiv(m, 32)));
      tot += sh.ncl_q[q];
    }
    sh.ncl = tot;
    sh.sms = tot * B;
    DBG("XT candidate B=%d Q=%d clusters=%d SMs=%d", B, Q, tot, sh.sms);
    if (best.B == 0 || sh.sms > best.sms || (sh.sms == best.sms && sh.Q < best.Q)) best = sh;
  }
  if (best.B == 0) return SPMV_OK;
  const int B = best.B, Q = best.Q, NB = Q * B, ncl = best.ncl;

  // ---- column blocks: parts with nnz in proportion to their clusters, blocks of equal nnz inside a part
  std::vector<int> hrp((size_t)m + 1);
  CK(cudaMemcpyAsync(hrp.data(), h->rp_loc, sizeof(int) * (m + 1), cudaMemcpyDeviceToHost, s));
  int* dcnt = nullptr;
  CK(cudaMalloc(&dcnt, sizeof(int) * (size_t)nx));
  CK(cudaMemsetAsync(dcnt, 0, sizeof(int) * (size_t)nx, s));
  k_col_count<<<(unsigned)std::min<int64_t>(cdiv(nnz, 256), 8LL * num_sms(h->device)), 256, 0, s>>>(
      h->k0, h->k1, h->ci_loc, dcnt);
  LAUNCHED();
  std::vector<int> ccnt((size_t)nx);
  CK(cudaMemcpyAsync(ccnt.data(), dcnt, sizeof(int) * (size_t)nx, cudaMemcpyDeviceToHost, s));
  CK(cudaStreamSynchronize(s));
  cudaFree(dcnt);
  std::vector<long long> cpre((size_t)nx + 1, 0);
  for (int64_t j = 0; j < nx; ++j) cpre[j + 1] = cpre[j] + ccnt[j];
  // target nnz at each block boundary: part q covers a share ncl_q/ncl, its B blocks equal shares of it
  std::vector<long long> bcol(NB + 1, 0);
  {
    long long cl_before = 0;
    for (int q = 0; q < Q; ++q) {
      for (int b = 0; b < B; ++b) {
        const int g = q * B + b;
        if (g == 0) continue;
        // share = (cl_before + ncl_q * b / B) / ncl
        const double share = ((double)cl_before + (double)best.ncl_q[q] * b / B) / ncl;
        const long long tgt = (long long)std::llround(share * (double)cpre[nx]);
        long long c0 = std::lower_bound(cpre.begin(), cpre.end(), tgt) - cpre.begin();
        c0 = std::min<long long>(std::max<long long>(c0 & ~7LL, bcol[g - 1]), nx);
        bcol[g] = c0;
      }
      cl_before += best.ncl_q[q];
    }
    bcol[NB] = nx;
  }
  int64_t wmx = 0;
  for (int g = 0; g < NB; ++g) wmx = std::max<int64_t>(wmx, bcol[g + 1] - bcol[g]);
  if (wmx > wmax || wmx > 65534) {
    // skewed column counts: equal widths (fit by construction of Q when parts are equal)
    for (int g = 0; g <= NB; ++g) bcol[g] = std::min<long long>(nx, ((nx * g / NB) + 7) & ~7LL);
    bcol[NB] = nx;
    wmx = 0;
    for (int g = 0; g < NB; ++g) wmx = std::max<int64_t>(wmx, bcol[g + 1] - bcol[g]);
    if (wmx > wmax || wmx > 65534) return SPMV_OK;
  }
  const int xcap = (int)((wmx + 1 + 7) & ~7LL);
  const size_t smem = xt_smem(xcap, ts, NS);
  DBG("XT B=%d Q=%d NB=%d ncl=%d wmax=%lld xcap=%d smem=%zu", B, Q, NB, ncl, (long long)wmx, xcap, smem);

  auto cleanup = [&]() { X.release(); };
  X.B = B; X.Q = Q; X.NB = NB; X.NS = NS; X.ncl = ncl; X.xcap = xcap; X.smem = smem; X.k = fn; X.kdot = fnd;
  CK(cudaMalloc(&X.bcol, sizeof(long long) * (NB + 1)));
  CK(cudaMemcpyAsync(X.bcol, bcol.data(), sizeof(long long) * (NB + 1), cudaMemcpyHostToDevice, s));
  CK(cudaMalloc(&X.bseg, sizeof(int) * (size_t)std::max(NB - 1, 1) * (size_t)m));
  if (NB > 1) {
    k_xt_splits<<<(unsigned)std::min<int64_t>(cdiv(m, 256), 8LL * num_sms(h->device)), 256, 0, s>>>(
        m, h->rp_loc, h->ci_loc, NB, X.bcol, X.bseg);
    LAUNCHED();
  }
  // ---- cluster row ranges: per part nnz-balanced over its clusters, at multiples of 32 rows
  std::vector<int> part_start(Q);  // block index of the first block of each part
  std::vector<int> hseg;
  if (Q > 1) {
    hseg.resize((size_t)(Q - 1) * m);
    for (int q = 1; q < Q; ++q)
      CK(cudaMemcpyAsync(hseg.data() + (size_t)(q - 1) * m, X.bseg + (size_t)(q * B - 1) * m, sizeof(int) * m,
                         cudaMemcpyDeviceToHost, s));
    CK(cudaStreamSynchronize(s));
  }
  auto pstart = [&](int q, int64_t i) -> long long { return q == 0 ? hrp[i] : hseg[(size_t)(q - 1) * m + i]; };
  auto pend = [&](int q, int64_t i) -> long long { return q == Q - 1 ? hrp[i + 1] : hseg[(size_t)q * m + i]; };
  std::vector<int> cl_part, cl_tile0, part_cl0(Q + 1, 0), tile_cl;
  std::vector<long long> cl_rows;
  std::vector<long long> pre((size_t)m + 1);
  int ntiles = 0;
  for (int q = 0; q < Q; ++q) {
    part_cl0[q] = (int)cl_part.size();
    pre[0] = 0;
    for (int64_t i = 0; i < m; ++i) pre[i + 1] = pre[i] + (pend(q, i) - pstart(q, i));
    const int nq = best.ncl_q[q];
    long long prev = 0;
    for (int r = 0; r < nq; ++r) {
      long long e;
      if (r == nq - 1) {
        e = m;
      } else {
        const long long tgt = (long long)((double)pre[m] * (r + 1) / nq);
        e = std::lower_bound(pre.begin(), pre.end(), tgt) - pre.begin();
        e = std::min<long long>(std::max<long long>((e + 16) & ~31LL, prev), m);
      }
      cl_part.push_back(q);
      cl_rows.push_back(prev);
      cl_rows.push_back(e);
      cl_tile0.push_back(ntiles);
      const int nt = (int)cdiv(e - prev, XT_R);
      for (int t = 0; t < nt; ++t) tile_cl.push_back((int)cl_part.size() - 1);
      ntiles += nt;
      prev = e;
    }
  }
  part_cl0[Q] = (int)cl_part.size();
  if ((int)cl_part.size() != ncl) return arg_fail("internal: XT cluster count");
  X.ntiles = ntiles;
  const int grid = ncl * B;
  // per-CTA column blocks
  std::vector<long long> cta_col0(grid);
  std::vector<int> cta_w(grid);
  for (int c = 0; c < ncl; ++c)
    for (int b = 0; b < B; ++b) {
      const int g = cl_part[c] * B + b;
      cta_col0[c * B + b] = bcol[g];
      cta_w[c * B + b] = (int)(bcol[g + 1] - bcol[g]);
    }
  auto up = [&](void** dst, const void* src, size_t bytes) -> spmv_status {
    CK(cudaMalloc(dst, std::max<size_t>(bytes, 16)));
    if (bytes) CK(cudaMemcpyAsync(*dst, src, bytes, cudaMemcpyHostToDevice, s));
    return SPMV_OK;
  };
  int* d_tile_cl = nullptr;
  ST(up((void**)&X.cl_part, cl_part.data(), sizeof(int) * ncl));
  ST(up((void**)&X.cl_rows, cl_rows.data(), sizeof(long long) * 2 * ncl));
  ST(up((void**)&X.cl_tile0, cl_tile0.data(), sizeof(int) * ncl));
  ST(up((void**)&X.part_cl0, part_cl0.data(), sizeof(int) * (Q + 1)));
  ST(up((void**)&X.cta_col0, cta_col0.data(), sizeof(long long) * grid));
  ST(up((void**)&X.cta_w, cta_w.data(), sizeof(int) * grid));
  ST(up((void**)&d_tile_cl, tile_cl.data(), sizeof(int) * tile_cl.size()));
  // ---- chunks: sort every (tile, block) by segment length
  const int64_t nch = (int64_t)ntiles * B * XT_NC;
  X.nchunks = nch;
  uint16_t* ck_row = nullptr;
  CK(cudaMalloc(&X.ck_len, sizeof(int) * std::max<int64_t>(nch, 1)));
  CK(cudaMalloc(&ck_row, sizeof(uint16_t) * 32 * std::max<int64_t>(nch, 1)));
  CK(cudaMalloc(&X.row_slot, sizeof(int) * (size_t)NB * (size_t)m));
  if (ntiles > 0) {
    k_xt_sell<<<(unsigned)(ntiles * B), XT_R, 0, s>>>(h->rp_loc, X.bseg, m, NB, B, d_tile_cl, X.cl_tile0, X.cl_part,
                                                   X.cl_rows, X.ck_len, ck_row, X.row_slot);
    LAUNCHED();
  }
  std::vector<int> len((size_t)std::max<int64_t>(nch, 1));
  CK(cudaMemcpyAsync(len.data(), X.ck_len, sizeof(int) * nch, cudaMemcpyDeviceToHost, s));
  CK(cudaStreamSynchronize(s));
  cudaFree(d_tile_cl);
  long long steps = 0;
  for (int64_t i = 0; i < nch; ++i) steps += len[i];
  if ((double)steps * 32.0 > 1.5 * (double)nnz + 64.0 * (double)nch) {  // SELL padding must stay moderate
    cudaFree(ck_row);
    cleanup();
    return SPMV_OK;
  }
  // ---- stream layout and TMA stages per CTA
  const int LMAX = ts == 8 ? xt_lmax<double>() : xt_lmax<float>();
  const long long step_bytes = 32LL * (ts + 2);
  std::vector<long long> ck_off((size_t)std::max<int64_t>(nch, 1)), st_off;
  std::vector<uint32_t> st_info;
  std::vector<uint2> ck_meta((size_t)std::max<int64_t>(nch, 1));
  std::vector<int> ck_pad((size_t)std::max<int64_t>(nch, 1)), cta_st0(grid + 1, 0);
  long long pos = 0;
  for (int c = 0; c < ncl; ++c) {
    const int nt = (int)cdiv(cl_rows[2 * c + 1] - cl_rows[2 * c], XT_R);
    for (int b = 0; b < B; ++b) {
      const int cta = c * B + b;
      cta_st0[cta] = (int)st_off.size();
      long long sbeg = pos, sbytes = 0;
      int snp = 0;
      auto close = [&]() {
        if (snp == 0) return;
        st_off.push_back(sbeg);
        st_info.push_back((uint32_t)sbytes | ((uint32_t)snp << 16));
        snp = 0;
        sbytes = 0;
      };
      for (int t = 0; t < nt; ++t)
        for (int j = 0; j < XT_NC; ++j) {
          const int64_t cid = ((int64_t)(cl_tile0[c] + t) * B + b) * XT_NC + j;
          const int L = len[cid];
          const int npc = std::max(1, (L + LMAX - 1) / LMAX);
          ck_off[cid] = pos;
          ck_pad[cid] = cta_w[cta];
          if (npc == 1) {
            const long long cb = XT_HDR + (long long)L * step_bytes;
            if (snp > 0 && (sbytes + cb > XT_SMAX || snp >= XT_EMPTY)) close();
            if (snp == 0) sbeg = pos;
            const int rel = (int)st_off.size() - cta_st0[cta];
            ck_meta[cid] = make_uint2((uint32_t)rel, (uint32_t)((pos - sbeg) / 16) | ((uint32_t)L << 16));
            sbytes += cb;
            snp += 1;
            pos += cb;
          } else {
            close();
            const int rel = (int)st_off.size() - cta_st0[cta];
            ck_meta[cid] = make_uint2((uint32_t)rel, (uint32_t)L << 16);
            for (int pc = 0; pc < npc; ++pc) {
              const int Lp = std::min(LMAX, L - pc * LMAX);
              const long long pb = (pc == 0 ? XT_HDR : 0) + (long long)Lp * step_bytes;
              sbeg = pos;
              sbytes = pb;
              snp = 1;
              pos += pb;
              close();
            }
          }
          if (L > 65535) { cudaFree(ck_row); cleanup(); return SPMV_OK; }
        }
      close();
    }
  }
  cta_st0[grid] = (int)st_off.size();
  X.nstages = (int64_t)st_off.size();
  X.bytes = pos;
  ST(up((void**)&X.ck_off, ck_off.data(), sizeof(long long) * nch));
  ST(up((void**)&X.ck_meta, ck_meta.data(), sizeof(uint2) * nch));
  ST(up((void**)&X.st_off, st_off.data(), sizeof(long long) * st_off.size()));
  ST(up((void**)&X.st_info, st_info.data(), sizeof(uint32_t) * st_info.size()));
  ST(up((void**)&X.cta_st0, cta_st0.data(), sizeof(int) * (grid + 1)));
  int* d_pad = nullptr;
  ST(up((void**)&d_pad, ck_pad.data(), sizeof(int) * nch));
  CK(cudaMalloc(&X.plan, (size_t)std::max<long long>(pos, 16)));
  if (nch > 0) {
    const unsigned g = (unsigned)std::min<int64_t>(nch, 16LL * num_sms(h->device));
    if (ts == 8) k_xt_fill<double><<<g, 256, 0, s>>>(X.plan, X.ck_off, X.ck_len, ck_row, d_pad, nch);
    else k_xt_fill<float><<<g, 256, 0, s>>>(X.plan, X.ck_off, X.ck_len, ck_row, d_pad, nch);
    LAUNCHED();
  }
  if (Q > 1) {
    CK(cudaMalloc(&X.ypart, sizeof(double) * (size_t)Q * (size_t)m));
    CK(cudaMalloc(&X.gcnt, sizeof(int) * (size_t)cdiv(m, 32)));
    CK(cudaMemsetAsync(X.gcnt, 0, sizeof(int) * (size_t)cdiv(m, 32), s));
  }
  ST(xt_pack(h, h->vals, 0));
  CK(cudaStreamSynchronize(s));
  cudaFree(d_pad);
  cudaFree(ck_row);
  CK(cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem));
  if (fnd) CK(cudaFuncSetAttribute(fnd, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem));
  if (B > 8) {
    CK(cudaFuncSetAttribute(fn, cudaFuncAttributeNonPortableClusterSizeAllowed, 1));
    if (fnd) CK(cudaFuncSetAttribute(fnd, cudaFuncAttributeNonPortableClusterSizeAllowed, 1));
  }
  DBG("XT built: %lld stages, %lld chunks, %lld plan bytes, %d tiles", (long long)X.nstages, (long long)nch,
      (long long)pos, ntiles);
  X.built = true;
  *ok = true;
  return SPMV_OK;
}

spmv_status launch_xt(spmv_csr_s* h, cudaStream_t s, const void* x, void* y, double alpha, double beta,
                      const double* w, double* part, const P2PHook& hook) {
  const auto& X = h->xt;
  if (part && X.Q > 1 && beta != 0.0) return arg_fail("internal: fused dot with beta != 0 over column parts");
  XtArgs a;
  a.m = h->m_loc;
  a.Q = X.Q;
  a.NS = X.NS;
  a.dyn = 1;
  env_int("SPMV_XT_DYN", &a.dyn);
  a.xcap = X.xcap;
  a.nx = h->nx;
  a.plan = X.plan;
  a.cl_part = X.cl_part;
  a.cl_rows = X.cl_rows;
  a.cl_tile0 = X.cl_tile0;
  a.cta_col0 = X.cta_col0;
  a.cta_w = X.cta_w;
  a.cta_st0 = X.cta_st0;
  a.st_off = X.st_off;
  a.st_info = X.st_info;
  a.ck_meta = X.ck_meta;
  a.x = x;
  a.y = y;
  a.alpha = alpha;
  a.beta = beta;
  if (h->dt == SPMV_F32) {
    a.alpha = (double)(float)alpha;
    a.beta = (double)(float)beta;
  }
  a.ypart = X.ypart;
  a.gcnt = X.gcnt;
  a.w = w;
  a.part = part;
  a.hk = hook;
  a.prof = nullptr;
#ifdef XT_PROF
  const size_t pn = (size_t)X.ncl * X.B * 32 * 8;
  CK(cudaMalloc(&a.prof, pn * 8));
  CK(cudaMemsetAsync(a.prof, 0, pn * 8, s));
#endif
  cudaLaunchConfig_t cfg = {};
  cfg.gridDim = dim3((unsigned)(X.ncl * X.B), 1, 1);
  cfg.blockDim = dim3(XT_THREADS, 1, 1);
  cfg.dynamicSmemBytes = X.smem;
  cfg.stream = s;
  cudaLaunchAttribute at[1];
  at[0].id = cudaLaunchAttributeClusterDimension;
  at[0].val.clusterDim.x = (unsigned)X.B;
  at[0].val.clusterDim.y = 1;
  at[0].val.clusterDim.z = 1;
  cfg.attrs = at;
  cfg.numAttrs = 1;
  CK(cudaLaunchKernelEx(&cfg, part ? X.kdot : X.k, a));
  LAUNCHED();
#ifdef XT_PROF
  {  // per-warp clock accounting, summarised on stderr (mean over CTAs of warps 1..31, and the producer)
    std::vector<unsigned long long> hp(pn);
    CK(cudaMemcpyAsync(hp.data(), a.prof, pn * 8, cudaMemcpyDeviceToHost, s));
    CK(cudaStreamSynchronize(s));
    cudaFree(a.prof);
    const char* nm[8] = {"tag", "full", "proc", "fbar", "fin", "rbar", "total", "chunks"};
    double cons[8] = {0}, fin[8] = {0}, prod[8] = {0};
    const int G = X.ncl * X.B;
    for (int c = 0; c < G; ++c)
      for (int w = 0; w < 32; ++w)
        for (int i = 0; i < 8; ++i)
          (w == 0 ? prod : w <= XT_NWC ? cons : fin)[i] += (double)hp[((size_t)c * 32 + w) * 8 + i];
    fprintf(stderr, "[xt prof] grid %d B %d Q %d NS %d; per consumer warp (mean, kclk):", G, X.B, X.Q, X.NS);
    for (int i : {0, 1, 2, 3, 6, 7}) fprintf(stderr, " %s %.1f", nm[i], cons[i] / (G * (double)XT_NWC) / (i == 7 ? 1.0 : 1e3));
    fprintf(stderr, "; finalizer: fin %.1f rbar %.1f total %.1f", fin[4] / (G * (double)XT_NFW) / 1e3,
            fin[5] / (G * (double)XT_NFW) / 1e3, fin[6] / (G * (double)XT_NFW) / 1e3);
    fprintf(stderr, "; producer total %.1f\n", prod[6] / G / 1e3);
  }
#endif
  return SPMV_OK;
}
