"""B200-native CSR SpMV + CG: thin Python binding of libspmv_b200.so.

The library (include/spmv.h) implements the data-parallel hot path of the SPMV
idiom of Ginsbach et al., ASPLOS'18 (Fig. 4, Fig. 12, the
cuSPARSE call shape of Fig. 6) on hand-written sm_100a kernels.
This module only marshals arguments: torch tensors become raw device pointers
and every step of the path runs in the library's kernels.  There is no CPU
fallback: if the shared library is missing the import fails loudly.

Function names follow the C ABI: ``spmv_csr_create``, ``spmv_csr``,
``cg_solve``, ``cg_npb_outer``, ``spmv_csr_destroy`` (plus introspection and
the NCCL distributed-mode entry points).  ``CSRMatrix`` wraps a handle.
"""
from __future__ import annotations

import ctypes
import os

_HERE = os.path.dirname(os.path.abspath(__file__))
# SPMV_LIB_PATH: a variant build of tools/build_variants.sh (sweeps and diagnostics only)
LIB_PATH = os.environ.get("SPMV_LIB_PATH") or os.path.join(_HERE, "libspmv_b200.so")

if not os.path.exists(LIB_PATH):
    raise ImportError(
        f"{LIB_PATH} is missing: build it with `python -c 'import __graft_entry__ as g; g.build()'` "
        "(there is no CPU fallback)")

_lib = ctypes.CDLL(LIB_PATH)

_P, _I64, _I32, _D = ctypes.c_void_p, ctypes.c_int64, ctypes.c_int32, ctypes.c_double
_ST = ctypes.c_int

SPMV_OK, SPMV_ERR_ARG, SPMV_ERR_INDEX, SPMV_ERR_ALIAS, SPMV_ERR_CUDA = 0, 1, 2, 3, 4
SPMV_ERR_NCCL, SPMV_ERR_NOMEM, SPMV_ERR_BREAKDOWN, SPMV_ERR_UNSUPPORTED = 5, 6, 7, 8
SPMV_F64, SPMV_F32 = 0, 1
KERNELS = {"auto": 0, "scalar": 1, "vector": 2, "merge": 3, "xstat": 4, "xplan": 5, "sell": 6, "sellsort": 7, "xt": 8}
KERNEL_NAMES = {v: k for k, v in KERNELS.items()}


class SpmvOpts(ctypes.Structure):
    _fields_ = [("stream", _P), ("kernel", _I32), ("vec_lanes", _I32), ("validate", _I32),
                ("plan", _I32), ("dist", _P), ("l2_window", _I32)]


class SpmvInfo(ctypes.Structure):
    _fields_ = [("kernel", _I32), ("vec_lanes", _I32), ("row_min", _I64), ("row_max", _I64),
                ("row_mean", _D), ("row_cv", _D), ("m_local", _I64), ("row_begin", _I64),
                ("row_end", _I64), ("nnz_local", _I64), ("rank", _I32), ("nranks", _I32),
                ("sorted_cols", _I32), ("grid", _I64), ("cluster", _I32), ("plan_bytes", _I64),
                ("transport", _I32)]


def _decl(name, args, res=_ST):
    f = getattr(_lib, name)
    f.argtypes = args
    f.restype = res
    return f


spmv_csr_create_c = _decl("spmv_csr_create", [ctypes.POINTER(_P), _ST, _I64, _I64, _I64, _P, _P, _P,
                                               ctypes.POINTER(SpmvOpts)])
spmv_csr_c = _decl("spmv_csr", [_P, _I64, _I64, _I64, _P, _P, _P, _P, _P, _D, _D])
cg_solve_c = _decl("cg_solve", [_P, _P, _P, _I32, _D, ctypes.POINTER(_I32), ctypes.POINTER(_D)])
cg_npb_outer_c = _decl("cg_npb_outer", [_P, _P, _P, _I32, _D, _P])
spmv_cg_status_c = _decl("spmv_cg_status", [_P])
spmv_csr_set_cg_variant_c = _decl("spmv_csr_set_cg_variant", [_P, _I32])
spmv_csr_update_values_c = _decl("spmv_csr_update_values", [_P, _P])
spmv_csr_merge_splits_device_c = _decl("spmv_csr_merge_splits_device", [_P, _P, _P, _I64, ctypes.POINTER(_I64)])
spmv_csr_destroy_c = _decl("spmv_csr_destroy", [_P])
spmv_csr_partition_c = _decl("spmv_csr_partition", [_P, _I64, _I32, _P])
spmv_csr_merge_splits_c = _decl("spmv_csr_merge_splits", [_P, _I64, _I64, _P, _P])
spmv_csr_info_c = _decl("spmv_csr_info", [_P, ctypes.POINTER(SpmvInfo)])
spmv_launch_count = _decl("spmv_launch_count", [], ctypes.c_uint64)
spmv_status_string = _decl("spmv_status_string", [_ST], ctypes.c_char_p)
spmv_last_error_string = _decl("spmv_last_error_string", [], ctypes.c_char_p)
spmv_dist_get_unique_id_c = _decl("spmv_dist_get_unique_id", [_P])
spmv_dist_init_c = _decl("spmv_dist_init", [ctypes.POINTER(_P), _I32, _I32, _P, _I32])
spmv_dist_destroy_c = _decl("spmv_dist_destroy", [_P])
spmv_dist_init_p2p_c = _decl("spmv_dist_init_p2p", [ctypes.POINTER(_P), _I32, _I32, _I32])
spmv_dist_init_proxy_c = _decl("spmv_dist_init_proxy", [ctypes.POINTER(_P), _I32, _I32, _I32])
spmv_csr_p2p_handle_c = _decl("spmv_csr_p2p_handle", [_P, _P])
spmv_csr_p2p_connect_c = _decl("spmv_csr_p2p_connect", [_P, _P])
spmv_dist_plan_host_c = _decl("spmv_dist_plan_host", [_P, _P, _I64, _I32, _I32, _P, _P, _P])
spmv_dist_colidx_c = _decl("spmv_dist_colidx", [_P, _P])
spmv_dist_halo_host_c = _decl("spmv_dist_halo_host", [_P, _P, _I64, _I32, _P])
spmv_dist_halo_c = _decl("spmv_dist_halo", [_P, _P, _P])
stencil27_apply_c = _decl("stencil27_apply", [_ST, _I64, _I64, _I64, _P, _P, _P, _D, _D, _P])
spmv_jds_create_c = _decl("spmv_jds_create", [ctypes.POINTER(_P), _ST, _I64, _I64, _I64, _P, _P, _P, _P, _P, _P])
spmv_jds_c = _decl("spmv_jds", [_P, _P, _P, _D, _D])
spmv_jds_destroy_c = _decl("spmv_jds_destroy", [_P])
# include/idioms.h (histogram, scalar reduction, NAS EP)
_SZ = ctypes.c_size_t
idl_reduce_workspace_c = _decl("idl_reduce_workspace", [_I64, ctypes.POINTER(_SZ)])
idl_reduce_c = _decl("idl_reduce", [_ST, _ST, _P, _P, _I64, _P, _P, _SZ, _P])
idl_histogram_workspace_c = _decl("idl_histogram_workspace", [_ST, _I64, _I64, ctypes.POINTER(_SZ)])
idl_histogram_c = _decl("idl_histogram", [_ST, _P, _P, _I64, _I64, _P, _P, _SZ, _P])
ep_npb_workspace_c = _decl("ep_npb_workspace", [ctypes.POINTER(_SZ)])
ep_npb_c = _decl("ep_npb", [_I32, _I64, _I64, _P, _P, _SZ, _P])

# every symbol include/spmv.h declares (checked by tests/test_abi.py)
EXPORTS = ["spmv_csr_create", "spmv_csr", "cg_solve", "cg_npb_outer", "spmv_cg_status", "spmv_csr_set_cg_variant",
           "spmv_csr_update_values", "spmv_csr_merge_splits_device",
           "spmv_csr_destroy", "spmv_csr_partition", "spmv_csr_merge_splits", "spmv_csr_info",
           "spmv_launch_count", "spmv_status_string", "spmv_last_error_string",
           "spmv_dist_get_unique_id", "spmv_dist_init", "spmv_dist_destroy", "spmv_dist_plan_host",
           "spmv_dist_colidx", "spmv_dist_init_p2p", "spmv_dist_init_proxy", "spmv_csr_p2p_handle", "spmv_csr_p2p_connect",
           "spmv_dist_halo_host", "spmv_dist_halo", "stencil27_apply",
           "spmv_jds_create", "spmv_jds", "spmv_jds_destroy"]
# every symbol include/idioms.h declares
IDIOM_EXPORTS = ["idl_reduce_workspace", "idl_reduce", "idl_histogram_workspace", "idl_histogram",
                 "ep_npb_workspace", "ep_npb"]
IDL_RED_SUM, IDL_RED_DOT = 0, 1
IDL_HIST_COUNT_U32, IDL_HIST_SAT_U8, IDL_HIST_SUM_F64 = 0, 1, 2
HIST_KINDS = {"count": IDL_HIST_COUNT_U32, "sat_u8": IDL_HIST_SAT_U8, "sum_f64": IDL_HIST_SUM_F64}


class SpmvError(RuntimeError):
    def __init__(self, status, where):
        self.status = status
        msg = spmv_last_error_string().decode(errors="replace")
        super().__init__(f"{where}: {spmv_status_string(status).decode()} ({msg})")


def _check(st, where):
    if st != SPMV_OK:
        raise SpmvError(st, where)


def _ptr(t):
    """Raw data pointer of a torch tensor, numpy array, int or None."""
    if t is None:
        return None
    if isinstance(t, int):
        return t
    if hasattr(t, "data_ptr"):
        return t.data_ptr()
    if hasattr(t, "ctypes"):
        return t.ctypes.data
    raise TypeError(f"cannot take a pointer of {type(t)}")


# ----------------------------------------------------------------- host-side
def spmv_csr_partition(rowptr_host, nranks: int):
    """nnz-balanced row bounds (int64[nranks+1]) of a host rowptr (numpy int32)."""
    import numpy as np
    rp = np.ascontiguousarray(rowptr_host, dtype=np.int32)
    b = np.zeros(nranks + 1, dtype=np.int64)
    _check(spmv_csr_partition_c(rp.ctypes.data, rp.shape[0] - 1, nranks, b.ctypes.data),
           "spmv_csr_partition")
    return b


def spmv_csr_merge_splits(rowptr_host, pieces: int):
    import numpy as np
    rp = np.ascontiguousarray(rowptr_host, dtype=np.int32)
    sr = np.zeros(pieces + 1, dtype=np.int64)
    sn = np.zeros(pieces + 1, dtype=np.int64)
    _check(spmv_csr_merge_splits_c(rp.ctypes.data, rp.shape[0] - 1, pieces, sr.ctypes.data,
                                   sn.ctypes.data), "spmv_csr_merge_splits")
    return sr, sn


def spmv_dist_plan_host(rowptr_host, colidx_host, nranks: int, rank: int):
    """Host exchange plan of one rank: (bounds, maxlen, renumbered local colidx)."""
    import numpy as np
    rp = np.ascontiguousarray(rowptr_host, dtype=np.int32)
    ci = np.ascontiguousarray(colidx_host, dtype=np.int32)
    m = rp.shape[0] - 1
    b = np.zeros(nranks + 1, dtype=np.int64)
    ml = ctypes.c_int64(0)
    _check(spmv_dist_plan_host_c(rp.ctypes.data, ci.ctypes.data, m, nranks, rank, b.ctypes.data,
                                 ctypes.byref(ml), None), "spmv_dist_plan_host")
    loc = np.zeros(int(rp[b[rank + 1]]) - int(rp[b[rank]]), dtype=np.int32)
    _check(spmv_dist_plan_host_c(rp.ctypes.data, ci.ctypes.data, m, nranks, rank, b.ctypes.data,
                                 ctypes.byref(ml), loc.ctypes.data), "spmv_dist_plan_host")
    return b, ml.value, loc


def spmv_dist_halo_host(rowptr_host, colidx_host, nranks: int):
    """Halo intervals int64[nranks, nranks, 2]: [r, s] = [lo, hi) of rank s's
    slice that rank r reads (reading R27)."""
    import numpy as np
    rp = np.ascontiguousarray(rowptr_host, dtype=np.int32)
    ci = np.ascontiguousarray(colidx_host, dtype=np.int32)
    out = np.zeros((nranks, nranks, 2), dtype=np.int64)
    _check(spmv_dist_halo_host_c(rp.ctypes.data, ci.ctypes.data, rp.shape[0] - 1, nranks, out.ctypes.data),
           "spmv_dist_halo_host")
    return out


def stencil27_apply(nx: int, ny: int, nz: int, x, y, alpha: float = 1.0, beta: float = 0.0, w27=None,
                    stream=None):
    """Matrix-free 27-point stencil y <- alpha*A27 x + beta*y on an nx*ny*nz grid
    (the paper's Stencil idiom, Fig. 13; reading R19 weights unless w27 gives
    27 weights indexed (dz+1)*9+(dy+1)*3+(dx+1)).  Asynchronous."""
    import numpy as np
    import torch
    if y.dtype not in (torch.float64, torch.float32):
        raise ValueError("y must be float64 or float32")
    dt = SPMV_F64 if y.dtype == torch.float64 else SPMV_F32
    npts = int(nx) * int(ny) * int(nz)
    # the C ABI sees raw pointers only: dtype, layout and extent are checked here
    if not y.is_contiguous() or y.numel() < npts:
        raise ValueError(f"y must be contiguous with at least nx*ny*nz = {npts} elements")
    if alpha != 0.0:
        if x.dtype != y.dtype:
            raise ValueError(f"x.dtype {x.dtype} != y.dtype {y.dtype}")
        if not x.is_contiguous() or x.numel() < npts:
            raise ValueError(f"x must be contiguous with at least nx*ny*nz = {npts} elements")
    w = None if w27 is None else np.ascontiguousarray(w27, dtype=np.float64)
    if w is not None and w.shape != (27,):
        raise ValueError("w27 must hold 27 weights")
    if stream is None:
        stream = torch.cuda.current_stream(y.device).cuda_stream if y.is_cuda else 0
    _check(stencil27_apply_c(dt, nx, ny, nz, None if w is None else w.ctypes.data, _ptr(x), _ptr(y),
                             float(alpha), float(beta), stream), "stencil27_apply")
    return y


# ------------------------------------------------------------- distributed
class Dist:
    """Distributed context of the library.

    transport="nccl": an NCCL communicator bootstrapped through a torch process
    group (torch.distributed only broadcasts the 128-byte unique id).
    transport="p2p": no NCCL; exchanges run in the library's kernels over
    CUDA-IPC peer memory; IPC handles are all-gathered through the torch
    process group when a CSRMatrix is created.
    transport="proxy": single process, no communication: a handle does rank
    `rank`'s share of an nranks-way run on one GPU (measurement only,
    spmv_dist_init_proxy).
    """

    def __init__(self, rank: int, nranks: int, device: int, group=None, transport: str = "nccl"):
        self.group = group
        self.transport = transport
        self.rank, self.nranks, self.device = rank, nranks, device
        if transport == "proxy":
            h = _P()
            _check(spmv_dist_init_proxy_c(ctypes.byref(h), rank, nranks, device), "spmv_dist_init_proxy")
            self.handle = h
            return
        import torch.distributed as dist
        if transport == "p2p":
            h = _P()
            _check(spmv_dist_init_p2p_c(ctypes.byref(h), rank, nranks, device), "spmv_dist_init_p2p")
            self.handle = h
            return
        uid = (ctypes.c_char * 128)()
        if rank == 0:
            _check(spmv_dist_get_unique_id_c(ctypes.addressof(uid)), "spmv_dist_get_unique_id")
        buf = [bytes(uid)] if rank == 0 else [None]
        dist.broadcast_object_list(buf, src=0, group=group)
        ctypes.memmove(uid, buf[0], 128)
        h = _P()
        _check(spmv_dist_init_c(ctypes.byref(h), rank, nranks, ctypes.addressof(uid), device),
               "spmv_dist_init")
        self.handle = h
        self.rank, self.nranks, self.device = rank, nranks, device

    def close(self):
        if self.handle:
            _check(spmv_dist_destroy_c(self.handle), "spmv_dist_destroy")
            self.handle = None


# ------------------------------------------------------------------- handle
class CSRMatrix:
    """A device-resident CSR matrix handle (spmv_csr_create ... spmv_csr_destroy).

    rowptr/colidx/vals are torch CUDA tensors (int32, int32, float64|float32)
    that the caller keeps alive; the handle stores their pointers (the paper's
    lazy copying: A is uploaded once and stays resident).
    """

    def __init__(self, rowptr, colidx, vals, n: int | None = None, *, kernel: str = "auto",
                 vec_lanes: int = 0, validate: bool = False, stream=None, dist: Dist | None = None,
                 plan: bool = True, cg_variant: str = "textbook", l2_window: bool = False):
        import torch
        assert rowptr.dtype == torch.int32 and colidx.dtype == torch.int32
        assert vals.dtype in (torch.float64, torch.float32)
        self.rowptr, self.colidx, self.vals = rowptr, colidx, vals
        self.m = rowptr.numel() - 1
        self.n = self.m if n is None else int(n)
        self.dtype = vals.dtype
        self.dist = dist
        if stream is None:
            stream = torch.cuda.current_stream(rowptr.device)
        self.stream = stream
        o = SpmvOpts()
        o.stream = stream.cuda_stream
        o.kernel = KERNELS[kernel]
        o.vec_lanes = int(vec_lanes)
        o.validate = int(bool(validate))
        o.plan = int(bool(plan))
        o.dist = dist.handle if dist is not None else None
        o.l2_window = int(bool(l2_window))
        nnz = int(rowptr[-1].item()) - int(rowptr[0].item()) if self.m >= 0 else 0
        self.nnz = nnz
        h = _P()
        _check(spmv_csr_create_c(ctypes.byref(h), SPMV_F64 if vals.dtype == torch.float64 else SPMV_F32,
                                 self.m, self.n, nnz, _ptr(rowptr), _ptr(colidx), _ptr(vals),
                                 ctypes.byref(o)), "spmv_csr_create")
        self.handle = h
        if dist is not None and dist.transport == "p2p":
            import torch.distributed as tdist
            mine = (ctypes.c_char * 64)()
            _check(spmv_csr_p2p_handle_c(h, ctypes.addressof(mine)), "spmv_csr_p2p_handle")
            allh = [None] * dist.nranks
            tdist.all_gather_object(allh, bytes(mine), group=dist.group)
            buf = (ctypes.c_char * (64 * dist.nranks))()
            for q, hb in enumerate(allh):
                ctypes.memmove(ctypes.addressof(buf) + 64 * q, hb, 64)
            st = spmv_csr_p2p_connect_c(h, ctypes.addressof(buf))
            # every rank must agree before anyone uses the peer mappings
            oks = [None] * dist.nranks
            tdist.all_gather_object(oks, st == SPMV_OK, group=dist.group)
            if not all(oks):
                err = SpmvError(st if st != SPMV_OK else SPMV_ERR_CUDA, "spmv_csr_p2p_connect (some rank failed)")
                spmv_csr_destroy_c(h)
                self.handle = None
                raise err
            tdist.barrier(group=dist.group)
        self._info = self.info()
        if cg_variant != "textbook":
            self.set_cg_variant(cg_variant)

    CG_VARIANTS = {"textbook": 0, "cgcg": 1, "persist": 2}

    def set_cg_variant(self, variant: str):
        """'textbook' (NPB conj_grad), 'cgcg' (single-reduction Chronopoulos-Gear) or 'persist'
        (the single-reduction CG as one persistent kernel per solve, NEXT-1)."""
        _check(spmv_csr_set_cg_variant_c(self.handle, self.CG_VARIANTS[variant]), "spmv_csr_set_cg_variant")
        self.cg_variant = variant

    # -- calls ------------------------------------------------------------
    def spmv(self, x, y, alpha: float = 1.0, beta: float = 0.0, vals=None):
        """y <- alpha*A@x + beta*y (asynchronous on the handle's stream)."""
        v = self.vals if vals is None else vals
        _check(spmv_csr_c(self.handle, self.m, self.n, self.nnz, _ptr(self.rowptr), _ptr(self.colidx),
                          _ptr(v), _ptr(x), _ptr(y), float(alpha), float(beta)), "spmv_csr")
        return y

    def cg_solve(self, b, x, max_iter: int, tol: float = 0.0):
        """Textbook CG from x0=0 into x; returns (iterations, ||b - A x||).  Synchronous."""
        its = _I32(0)
        rn = _D(0.0)
        _check(cg_solve_c(self.handle, _ptr(b), _ptr(x), int(max_iter), float(tol), ctypes.byref(its),
                          ctypes.byref(rn)), "cg_solve")
        return its.value, rn.value

    def npb_outer(self, x, z, cgitmax: int, shift: float, out2):
        """One NAS CG outer iteration (x updated in place, z = CG(A, x)); out2 <- {zeta, rnorm}.
        Asynchronous when x, z, out2 are device tensors."""
        _check(cg_npb_outer_c(self.handle, _ptr(x), _ptr(z), int(cgitmax), float(shift), _ptr(out2)),
               "cg_npb_outer")
        return out2

    def dist_colidx(self):
        import numpy as np
        out = np.zeros(self._info["nnz_local"], dtype=np.int32)
        _check(spmv_dist_colidx_c(self.handle, out.ctypes.data), "spmv_dist_colidx")
        return out

    def dist_halo(self):
        """(device-computed halo table int64[P, P, 2], used-by-the-exchange flag)."""
        import numpy as np
        P = self._info["nranks"]
        out = np.zeros((P, P, 2), dtype=np.int64)
        used = _I32(0)
        _check(spmv_dist_halo_c(self.handle, out.ctypes.data, ctypes.byref(used)), "spmv_dist_halo")
        return out, bool(used.value)

    def merge_splits_device(self):
        """(split_row, split_nz) the MERGE kernel uses, or None."""
        import numpy as np
        cnt = _I64(0)
        _check(spmv_csr_merge_splits_device_c(self.handle, None, None, 0, ctypes.byref(cnt)), "merge_splits_device")
        if cnt.value == 0:
            return None
        sr = np.zeros(cnt.value, np.int64)
        sn = np.zeros(cnt.value, np.int64)
        _check(spmv_csr_merge_splits_device_c(self.handle, sr.ctypes.data, sn.ctypes.data, cnt.value,
                                              ctypes.byref(cnt)), "merge_splits_device")
        return sr, sn

    def update_values(self, vals):
        """Re-bind the values (same structure) and refresh the plan copy."""
        _check(spmv_csr_update_values_c(self.handle, _ptr(vals)), "spmv_csr_update_values")
        self.vals = vals

    def cg_status(self):
        _check(spmv_cg_status_c(self.handle), "spmv_cg_status")

    def info(self) -> dict:
        inf = SpmvInfo()
        _check(spmv_csr_info_c(self.handle, ctypes.byref(inf)), "spmv_csr_info")
        d = {f: getattr(inf, f) for f, _ in SpmvInfo._fields_}
        d["kernel_name"] = KERNEL_NAMES.get(d["kernel"], "?")
        return d

    @property
    def row_range(self):
        return self._info["row_begin"], self._info["row_end"]

    def destroy(self):
        if getattr(self, "handle", None):
            st = spmv_csr_destroy_c(self.handle)
            self.handle = None
            _check(st, "spmv_csr_destroy")

    def __del__(self):
        try:
            if getattr(self, "handle", None):
                spmv_csr_destroy_c(self.handle)
                self.handle = None
        except Exception:
            pass

    def __enter__(self):
        return self

    def __exit__(self, *a):
        self.destroy()


def launch_count() -> int:
    return int(spmv_launch_count())


# ------------------------------------------------------------------ idioms
# include/idioms.h: the histogram (Fig. 11), scalar reduction (Fig. 14) and
# NAS EP.  Workspaces are zero-filled device buffers (torch.zeros); pass one
# back in to avoid the allocation (bench loops do).

def _stream_of(t):
    import torch
    return torch.cuda.current_stream(t.device).cuda_stream


def _workspace(nbytes, device):
    import torch
    return torch.zeros(max(int(nbytes), 16), dtype=torch.uint8, device=device)


def idl_reduce_workspace(n: int) -> int:
    b = ctypes.c_size_t(0)
    _check(idl_reduce_workspace_c(int(n), ctypes.byref(b)), "idl_reduce_workspace")
    return b.value


def idl_reduce(a, b=None, out=None, workspace=None, stream=None):
    """Scalar reduction: sum(a) or dot(a, b) into a device float64 tensor of
    one element (returned).  fp32 inputs are summed in double.  Asynchronous."""
    import torch
    dt = SPMV_F64 if a.dtype == torch.float64 else SPMV_F32
    n = a.numel()
    if out is None:
        out = torch.empty(1, dtype=torch.float64, device=a.device)
    if workspace is None:
        workspace = _workspace(idl_reduce_workspace(n), a.device)
    op = IDL_RED_SUM if b is None else IDL_RED_DOT
    st = idl_reduce_c(dt, op, _ptr(a), _ptr(b), n, _ptr(out), _ptr(workspace), workspace.numel(),
                      _stream_of(out) if stream is None else stream)
    _check(st, "idl_reduce")
    return out


def idl_histogram_workspace(kind, n: int, nbins: int) -> int:
    k = HIST_KINDS[kind] if isinstance(kind, str) else int(kind)
    b = ctypes.c_size_t(0)
    _check(idl_histogram_workspace_c(k, int(n), int(nbins), ctypes.byref(b)), "idl_histogram_workspace")
    return b.value


def idl_histogram(kind, keys, bins, w=None, workspace=None, stream=None):
    """Generalised histogram accumulating into `bins` (uint32 / uint8 / float64
    device tensor for kind "count" / "sat_u8" / "sum_f64"); keys int32.
    Keys outside [0, len(bins)) are skipped.  Asynchronous; returns bins."""
    k = HIST_KINDS[kind] if isinstance(kind, str) else int(kind)
    n, nbins = keys.numel(), bins.numel()
    if workspace is None:
        workspace = _workspace(idl_histogram_workspace(k, n, nbins), bins.device)
    st = idl_histogram_c(k, _ptr(keys), _ptr(w), n, nbins, _ptr(bins), _ptr(workspace), workspace.numel(),
                         _stream_of(bins) if stream is None else stream)
    _check(st, "idl_histogram")
    return bins


def ep_shard_range(M: int, rank: int, nranks: int):
    """Reading R33: rank r of P owns pairs [floor(r*2^M/P), floor((r+1)*2^M/P)).
    Returns (pair_begin, pair_count); host-only."""
    total = 1 << M
    b0 = rank * total // nranks
    b1 = (rank + 1) * total // nranks
    return b0, b1 - b0


def ep_npb_workspace() -> int:
    b = ctypes.c_size_t(0)
    _check(ep_npb_workspace_c(ctypes.byref(b)), "ep_npb_workspace")
    return b.value


def ep_npb(M: int, pair_begin: int = 0, pair_count: int | None = None, out=None, workspace=None,
           device=None, stream=None):
    """NAS EP over pairs [pair_begin, pair_begin+pair_count) of class 2^M into a
    device float64[12] tensor: q[0..9], sx, sy (returned).  Asynchronous."""
    import torch
    if pair_count is None:
        pair_count = (1 << M) - pair_begin
    if out is None:
        out = torch.empty(12, dtype=torch.float64, device=device or torch.device("cuda", torch.cuda.current_device()))
    if workspace is None:
        workspace = _workspace(ep_npb_workspace(), out.device)
    st = ep_npb_c(int(M), int(pair_begin), int(pair_count), _ptr(out), _ptr(workspace), workspace.numel(),
                  _stream_of(out) if stream is None else stream)
    _check(st, "ep_npb")
    return out


# ------------------------------------------------------------------ JDS-32
class JDSMatrix:
    """Handle of spmv_jds_create (Parboil's jagged-diagonal layout, reading R34).

    perm/zcnt/indices int32, jds_ptr int64, data float64/float32: device tensors
    the caller keeps alive.  ``spmv(x, y)``: y (original row order) <- alpha*A x + beta*y.
    """

    def __init__(self, perm, jds_ptr, zcnt, indices, data, m: int, n: int, stream=None):
        import torch
        assert jds_ptr.dtype == torch.int64 and perm.dtype == torch.int32 and zcnt.dtype == torch.int32
        self._keep = (perm, jds_ptr, zcnt, indices, data)
        self.m, self.n = int(m), int(n)
        self.dtype = data.dtype
        if stream is None:
            stream = torch.cuda.current_stream(data.device)
        h = _P()
        _check(spmv_jds_create_c(ctypes.byref(h), SPMV_F64 if data.dtype == torch.float64 else SPMV_F32,
                                 self.m, self.n, jds_ptr.numel() - 1, _ptr(perm), _ptr(jds_ptr), _ptr(zcnt),
                                 _ptr(indices), _ptr(data), stream.cuda_stream), "spmv_jds_create")
        self.handle = h

    def spmv(self, x, y, alpha: float = 1.0, beta: float = 0.0):
        _check(spmv_jds_c(self.handle, _ptr(x), _ptr(y), float(alpha), float(beta)), "spmv_jds")
        return y

    def destroy(self):
        if getattr(self, "handle", None):
            st = spmv_jds_destroy_c(self.handle)
            self.handle = None
            _check(st, "spmv_jds_destroy")

    def __del__(self):
        try:
            self.destroy()
        except Exception:
            pass

    def __enter__(self):
        return self

    def __exit__(self, *a):
        self.destroy()
