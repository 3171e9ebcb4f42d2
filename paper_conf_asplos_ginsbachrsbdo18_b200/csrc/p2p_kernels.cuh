// p2p_kernels.cuh -- the distributed exchange of CG over peer memory
// (SURVEY 8(a) row a5, 8(e) "collective, stage 2"): CUDA-IPC-mapped buffers of
// every rank, reached over NVLink/NVSwitch by plain stores from our kernels.
// No NCCL on this path.
//
// Fabric of a rank (one cudaMalloc, IPC-exported):
//   xpad  [P * maxlen] T       gathered x / p (slice q written by rank q)
//   exch  [NSLOT][P][PMAX] double  pushed partials (slot s, rank q: one
//                                  value, or one per producing CTA)
//   flags [P]         u64      flags[q] = latest exchange epoch rank q completed
// plus local (never remote) counters: epoch (this rank's exchange count),
// slot_epoch[NSLOT+1] (epoch of the latest push of each slot / of x), ticket.
//
// A push writes the data into every peer (and itself); every CTA takes an
// acq_rel ticket at GPU scope and the last one fences at system scope,
// increments the local epoch e and stores flags[me] = e into every peer with
// st.release.sys.  A consumer waits until flags[q] >= e for all q != me with
// ld.acquire.sys, then reads.  All ranks run the same sequence of pushes, so
// epoch numbers agree.  Buffer reuse is safe by the CG data dependences: a
// peer can only push the next value of a slot after consuming something this
// rank pushes after it finished reading the slot.
#pragma once
#include "common.cuh"

namespace spmv {

// All-reduce, push half: sum `in` (fixed order) and push it into slot `slot`
// of every rank.  One CTA.
static __global__ void k_p2p_push_sum(SumSrc in, int slot, P2PCtx c) {
  __shared__ double s0;
  const double v = read_sum(in, &s0);
  if (threadIdx.x == 0) {
    for (int q = 0; q < c.P; ++q) {
      double* ex = reinterpret_cast<double*>(c.peer[q] + c.off_exch);
      ex[(size_t(slot) * c.P + c.me) * P2P_PMAX] = v;
    }
    p2p_signal(c, slot);
  }
}

// All-gather of x: this rank's slice (already at xpad + me*maxlen) is stored
// into every peer's xpad; the last CTA publishes.
template <typename T>
__global__ void __launch_bounds__(256)
k_p2p_push_x(int64_t n, int64_t maxlen, P2PCtx c) {
  const T* src = reinterpret_cast<const T*>(c.peer[c.me]) + int64_t(c.me) * maxlen;
  for (int64_t j = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; j < n; j += int64_t(gridDim.x) * blockDim.x) {
    const T v = src[j];
    for (int q = 0; q < c.P; ++q) {
      if (q == c.me || !p2p_sends(c, q, j)) continue;
      reinterpret_cast<T*>(c.peer[q])[int64_t(c.me) * maxlen + j] = v;
    }
  }
  __syncthreads();
  // acq_rel ticket at GPU scope; the last CTA fences at system scope and publishes
  if (threadIdx.x == 0 && ticket_acq_rel_gpu(c.ticket) == int(gridDim.x) - 1) {
    *c.ticket = 0;
    p2p_signal(c, P2P_XSLOT);
  }
}

// Block the stream until every peer's x slice of the latest x exchange landed.
static __global__ void k_p2p_wait_x(P2PCtx c) {
  const unsigned long long* flags = reinterpret_cast<const unsigned long long*>(c.peer[c.me] + c.off_flags);
  p2p_wait_flags(flags, c.me, c.P, c.slot_epoch[P2P_XSLOT]);
}

}  // namespace spmv
