// dist.cu -- row-sharded mode: the x exchange and the
// scalar all-reduces of CG over NCCL or over the library's own peer-memory
// kernels (p2p_kernels.cuh), the halo tables (NEXT-2) and the transport
// set-up entry points.
#include "abi_common.h"
#include "cg_kernels.cuh"
#include "p2p_kernels.cuh"

P2PCtx p2p_ctx(spmv_csr_s* h) {
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

bool use_p2p(const spmv_csr_s* h) { return h->dist && h->dist->p2p; }

int p2p_push_per(const spmv_csr_s* h, int64_t grid) { return (grid >= 1 && grid <= P2P_PMAX) ? (int)grid : 0; }

// Partials per rank the SpMV's fused dot pushes: one per CTA for the static
// XPLAN grid (its partial count is its launch grid), else the last-CTA sum.
static int spmv_push_per(const spmv_csr_s* h) {
  const bool side = h->xp.mplan >= 0 && h->xp.mplan < h->m_loc;
  if (h->kernel != SPMV_KERNEL_XPLAN || !h->xp.built || h->xp.dyn || side) return 0;
  return p2p_push_per(h, (int64_t)h->xp.ncl * h->xp.B);
}
int p2p_spmv_push_per(const spmv_csr_s* h) { return spmv_push_per(h); }

// All-gather of this rank's slice (already at xpad + rank*maxlen) and wait.
spmv_status exchange_x(spmv_csr_s* h, cudaStream_t s) {
  if (h->dist->proxy) return SPMV_OK;  // measurement proxy: no communication
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

// In distributed mode a SumSrc of per-CTA partials is finalized into scal[slot]
// and all-reduced over the ranks; single GPU returns the partials unchanged.
// The exchange-mode scalar source of `slot` (values pushed by every rank).
SumSrc p2p_src(spmv_csr_s* h, int slot, int per) {
  const P2PCtx c = p2p_ctx(h);
  SumSrc o;
  o.p = reinterpret_cast<const double*>(h->fabric + h->off_exch) + (size_t)slot * c.P * P2P_PMAX;
  o.count = -c.P;
  o.per = per;
  o.flags = reinterpret_cast<const unsigned long long*>(h->fabric + h->off_flags);
  o.epoch = c.slot_epoch + slot;
  o.me = c.me;
  return o;
}

spmv_status reduce_src(spmv_csr_s* h, cudaStream_t s, SumSrc in, int slot, SumSrc* out) {
  if (!h->dist || h->dist->proxy) { *out = in; return SPMV_OK; }  // proxy: this rank's partials only
  if (use_p2p(h)) {
    if (!h->p2p_connected) return arg_fail("p2p handle not connected (spmv_csr_p2p_connect)");
    const P2PCtx c = p2p_ctx(h);
    k_p2p_push_sum<<<1, 32, 0, s>>>(in, slot, c);
    LAUNCHED();
    *out = p2p_src(h, slot, 1);
    return SPMV_OK;
  }
  double* dst = h->scal + slot;
  k_finalize<<<1, 32, 0, s>>>(in, dst);
  LAUNCHED();
  NK(ncclAllReduce(dst, dst, 1, ncclDouble, ncclSum, h->dist->comm, s));
  *out = SumSrc{dst, 1};
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

extern "C" spmv_status spmv_dist_init_proxy(spmv_dist_t* out, int32_t rank, int32_t nranks, int32_t device) {
  if (!out || nranks < 1 || rank < 0 || rank >= nranks) return arg_fail("bad dist arguments");
  *out = nullptr;
  CK(cudaSetDevice(device));
  spmv_dist_s* d = new spmv_dist_s();
  d->rank = rank;
  d->nranks = nranks;
  d->device = device;
  d->proxy = 1;
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
