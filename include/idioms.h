/*
 * idioms.h -- C ABI of the library's other data-parallel idioms (SURVEY 8(f)
 * NEXT-4): the generalised histogram (Fig. 11, described
 * at P:565-575) and the scalar reduction (Fig. 14, described at
 * P:591-595), plus NAS EP [ext:NPB-EP], the benchmark whose time is "about
 * 50% ... inside a detected histogram reduction" and which is
 * one of the paper's accelerated programs (Fig. 18, Table 3).
 *
 * Conventions (as include/spmv.h): extern "C", every call returns
 * spmv_status, nothing throws across the ABI.  Array arguments are
 * caller-owned DEVICE pointers on the current device (host pointers ->
 * SPMV_ERR_ARG); calls are asynchronous on `stream` (cudaStream_t, NULL =
 * legacy default stream); argument errors return synchronously with nothing
 * enqueued; kernel faults surface as SPMV_ERR_CUDA on a later call.
 *
 * Workspaces: every call takes a caller-owned device workspace of at least
 * the size its *_workspace query returns.  It must be ZERO-FILLED before its
 * first use (e.g. torch.zeros / cudaMemset); every call leaves it in a state
 * valid for the next call.  One workspace must not be used by two calls that
 * may run concurrently (different streams).
 *
 * Determinism: idl_reduce, ep_npb and the integer histograms return
 * bit-identical results run to run on the same GPU model (fixed grid, fixed
 * summation trees).  IDL_HIST_SUM_F64 uses floating-point atomics: its bins
 * vary run to run within reading R30's bound.
 */
#ifndef IDL_IDIOMS_B200_H
#define IDL_IDIOMS_B200_H
#include <stddef.h>
#include <stdint.h>

#include "spmv.h"

#ifdef __cplusplus
extern "C" {
#endif

/* ------------------------------------------------------ scalar reduction
 * Fig. 14: acc <- kernel(read_values[i], acc) over a For loop.
 *   op == IDL_RED_SUM: *out = sum_{i<n} a[i]          (b must be NULL)
 *   op == IDL_RED_DOT: *out = sum_{i<n} a[i] * b[i]   (the DotProductLoop
 *                       of P:560-564 without alpha/beta)
 * dt: SPMV_F64 or SPMV_F32 (fp32 inputs: terms formed and summed in double,
 * reading R5/R30); out is ONE device double.  n == 0 writes 0.
 * Accuracy (R30): |out - exact| <= (n + 64) * 2^-53 * sum|term|.
 * Any alignment is accepted (16-byte aligned inputs take the vector path). */
typedef enum { IDL_RED_SUM = 0, IDL_RED_DOT = 1 } idl_red_op;
spmv_status idl_reduce_workspace(int64_t n, size_t *bytes);
spmv_status idl_reduce(spmv_dtype dt, idl_red_op op, const void *a, const void *b, int64_t n,
                       double *out, void *workspace, size_t workspace_bytes, void *stream);

/* ------------------------------------------------- generalised histogram
 * Fig. 11: for i < n, a conditional read-modify-write of the bin
 * keys[i] (the index kernel is the identity on an int32 key array); the
 * condition is 0 <= keys[i] < nbins (reading R31: other keys are skipped).
 * The bins ACCUMULATE onto their current contents:
 *   IDL_HIST_COUNT_U32: uint32 bins, bins[k] += 1 (mod 2^32)   (NPB IS)
 *   IDL_HIST_SAT_U8   : uint8 bins,  if (bins[k] < 255) bins[k]++, i.e.
 *                       bins[k] = min(255, bins[k] + count_k)  (Parboil
 *                       histo, the "conditional" of P:566-569, R32)
 *   IDL_HIST_SUM_F64  : double bins, bins[k] += w[i]  (w: n doubles)
 * keys (int32[n]) and w are caller-owned device arrays; w must be NULL for
 * the two counting kinds.  bins must not overlap keys or w (SPMV_ERR_ALIAS).
 * nbins in [1, 2^31-1]; n in [0, 2^62]. */
typedef enum { IDL_HIST_COUNT_U32 = 0, IDL_HIST_SAT_U8 = 1, IDL_HIST_SUM_F64 = 2 } idl_hist_kind;
spmv_status idl_histogram_workspace(idl_hist_kind kind, int64_t n, int64_t nbins, size_t *bytes);
spmv_status idl_histogram(idl_hist_kind kind, const int32_t *keys, const double *w, int64_t n, int64_t nbins,
                          void *bins, void *workspace, size_t workspace_bytes, void *stream);

/* ------------------------------------------------------------------ NAS EP
 * [ext:NPB-EP]: for the Gaussian pairs with global index p in
 * [pair_begin, pair_begin + pair_count) of the class with 2^M pairs
 * (24 <= M <= 40): uniforms u_j = (271828183 * 5^(13 j) mod 2^46) * 2^-46,
 * pair p uses x1 = 2u_{2p+1} - 1, x2 = 2u_{2p+2} - 1; when
 * t = x1*x1 + x2*x2 <= 1 (products and sum rounded separately, no FMA, as
 * NPB's C), the deviates X = x1*s, Y = x2*s with s = sqrt(-2 ln t / t) are
 * tallied: q[(int)max(|X|,|Y|)] += 1 (the histogram idiom; l >= 10 skipped,
 * R31) and sx += X, sy += Y (the scalar-reduction idiom).
 * out: device double[12] = q[0..9], sx, sy (overwritten, not accumulated).
 * A rank of a sharded EP passes its own pair range (R33); the per-rank
 * results add up exactly in q and to rounding in sx, sy.
 * Accuracy: q exact unless a deviate lies within a few ulp of an integer;
 * sx, sy within 1e-8 relative of NPB's published values (NPB's own check). */
spmv_status ep_npb_workspace(size_t *bytes);
spmv_status ep_npb(int32_t M, int64_t pair_begin, int64_t pair_count, double *out, void *workspace,
                   size_t workspace_bytes, void *stream);

#ifdef __cplusplus
}
#endif
#endif /* IDL_IDIOMS_B200_H */
