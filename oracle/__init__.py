"""CPU oracle -- TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py`` (its
``cpu_baseline`` leg and ``--impl reference``) may import this package.  The
product package ``paper_conf_asplos_ginsbachrsbdo18_b200`` never imports it
and shares no code with it; the only shared module is the seeded input
generator ``gen`` (which holds none of the method's arithmetic).

The arithmetic lives in ``oracle_spmv.c`` (plain sequential fp64 C, each
function citing the PAPER.md passage it follows); this file only compiles it
with gcc (``-O3 -march=native -ffp-contract=off``) and marshals numpy arrays
through ctypes.
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "oracle_spmv.c")
_SRCS = [_SRC, os.path.join(_HERE, "oracle_idioms.c")]
_LIB = os.path.join(_HERE, "liboracle_spmv.so")
_lib = None

_P = ctypes.c_void_p
_I64 = ctypes.c_int64
_I32 = ctypes.c_int32
_D = ctypes.c_double


def build(force: bool = False) -> str:
    """Compile the oracle (gcc, no FMA contraction).  Returns the .so path."""
    if force or not os.path.exists(_LIB) or any(os.path.getmtime(_LIB) < os.path.getmtime(f) for f in _SRCS):
        tmp = _LIB + f".tmp{os.getpid()}"
        subprocess.check_call(
            ["gcc", "-O3", "-march=native", "-ffp-contract=off", "-std=c11", "-fPIC",
             "-shared", "-o", tmp, *_SRCS, "-lm"])
        os.replace(tmp, _LIB)
    return _LIB


def lib():
    global _lib
    if _lib is None:
        build()
        L = ctypes.CDLL(_LIB)
        L.oracle_spmv_f64.argtypes = [_I64, _P, _P, _P, _P, _P, _D, _D, _P, _P]
        L.oracle_spmv_f64.restype = None
        L.oracle_spmv_f32.argtypes = [_I64, _P, _P, _P, _P, _P, _D, _D, _P, _P]
        L.oracle_spmv_f32.restype = None
        L.oracle_cg.argtypes = [_I64, _P, _P, _P, _P, _P, _I32, _D, _P, _P]
        L.oracle_cg.restype = ctypes.c_int
        L.oracle_npb_outer.argtypes = [_I64, _P, _P, _P, _P, _P, _I32, _D, _P, _P]
        L.oracle_npb_outer.restype = ctypes.c_int
        L.oracle_spmv_jds.argtypes = [_I64, _P, _P, _P, _P, _P, _P, _P, _D, _D, _I32, _P, _P]
        L.oracle_spmv_jds.restype = None
        L.oracle_cg_cgcg.argtypes = [_I64, _P, _P, _P, _P, _P, _I32, _D, _P, _P]
        L.oracle_cg_cgcg.restype = ctypes.c_int
        L.oracle_npb_outer_v.argtypes = [_I64, _P, _P, _P, _P, _P, _I32, _D, _P, _P, _I32]
        L.oracle_npb_outer_v.restype = ctypes.c_int
        L.oracle_partition.argtypes = [_P, _I64, _I32, _P]
        L.oracle_partition.restype = None
        L.oracle_merge_path.argtypes = [_P, _I64, _I64, _P, _P]
        L.oracle_stencil27.argtypes = [_I64, _I64, _I64, _P, _P, _P, _D, _D, _P, _P]
        L.oracle_stencil27.restype = None
        L.oracle_merge_path.restype = None
        L.oracle_reduce_f64.argtypes = [_I64, _P, _P, _P, _P]
        L.oracle_reduce_f64.restype = None
        L.oracle_reduce_f32.argtypes = [_I64, _P, _P, _P, _P]
        L.oracle_reduce_f32.restype = None
        L.oracle_hist_count_u32.argtypes = [_I64, _P, _I64, _P]
        L.oracle_hist_count_u32.restype = None
        L.oracle_hist_sat_u8.argtypes = [_I64, _P, _I64, _P]
        L.oracle_hist_sat_u8.restype = None
        L.oracle_hist_sum_f64.argtypes = [_I64, _P, _P, _I64, _P, _P]
        L.oracle_hist_sum_f64.restype = None
        L.oracle_npb_randlc_stream.argtypes = [_D, _D, _I64, _P]
        L.oracle_npb_randlc_stream.restype = None
        L.oracle_ep.argtypes = [_I32, _I64, _I64, _P, _P, _P]
        L.oracle_ep.restype = ctypes.c_int
        _lib = L
    return _lib


def _ptr(a):
    return a.ctypes.data_as(ctypes.c_void_p) if a is not None else None


def _c(a, dt):
    return np.ascontiguousarray(a, dtype=dt)


def spmv(rowptr, colidx, vals, x, y_old=None, alpha=1.0, beta=0.0):
    """y_ref, bound = alpha*A@x + beta*y_old with fp64 accumulation.

    vals/x/y_old may be float64 or float32 (then products are formed in double
    from the fp32 inputs, alpha/beta rounded to float first).
    """
    rowptr = _c(rowptr, np.int32)
    colidx = _c(colidx, np.int32)
    m = rowptr.shape[0] - 1
    f32 = np.asarray(vals).dtype == np.float32
    dt = np.float32 if f32 else np.float64
    vals = _c(vals, dt)
    x = _c(x, dt)
    yo = _c(y_old, dt) if y_old is not None else np.zeros(max(m, 1), dtype=dt)
    y_ref = np.empty(max(m, 1), dtype=np.float64)
    bound = np.empty(max(m, 1), dtype=np.float64)
    fn = lib().oracle_spmv_f32 if f32 else lib().oracle_spmv_f64
    fn(m, _ptr(rowptr), _ptr(colidx), _ptr(vals), _ptr(x), _ptr(yo), float(alpha),
       float(beta), _ptr(y_ref), _ptr(bound))
    return y_ref[:m], bound[:m]


def cg(rowptr, colidx, vals, b, max_iter, tol=0.0, variant=0):
    """CG from x0=0: variant 0 textbook (NPB conj_grad), 1 Chronopoulos-Gear
    single reduction.  Returns (z, iters, rnorm, status)."""
    rowptr = _c(rowptr, np.int32)
    colidx = _c(colidx, np.int32)
    vals = _c(vals, np.float64)
    b = _c(b, np.float64)
    n = rowptr.shape[0] - 1
    z = np.zeros(max(n, 1))
    its = ctypes.c_int32(0)
    rn = ctypes.c_double(0.0)
    fn = lib().oracle_cg_cgcg if variant == 1 else lib().oracle_cg
    st = fn(n, _ptr(rowptr), _ptr(colidx), _ptr(vals), _ptr(b), _ptr(z),
            int(max_iter), float(tol), ctypes.byref(its), ctypes.byref(rn))
    return z[:n], its.value, rn.value, st


def npb_outer(rowptr, colidx, vals, x, cgitmax, shift, variant=0):
    """One NAS CG outer iteration; x (float64, contiguous) updated in place.
    variant: 0 textbook CG, 1 Chronopoulos-Gear.  Returns (z, zeta, rnorm).
    """
    assert x.dtype == np.float64 and x.flags.c_contiguous
    rowptr = _c(rowptr, np.int32)
    colidx = _c(colidx, np.int32)
    vals = _c(vals, np.float64)
    n = rowptr.shape[0] - 1
    z = np.zeros(n)
    zeta = ctypes.c_double(0.0)
    rn = ctypes.c_double(0.0)
    lib().oracle_npb_outer_v(n, _ptr(rowptr), _ptr(colidx), _ptr(vals), _ptr(x), _ptr(z),
                             int(cgitmax), float(shift), ctypes.byref(zeta), ctypes.byref(rn), int(variant))
    return z, zeta.value, rn.value


def npb_run(rowptr, colidx, vals, niter, shift, cgitmax=25, on_iter=None, variant=0):
    """NPB CG benchmark driver: x=1; NITER outer iterations; returns zetas, rnorms.

    (The untimed warm-up iteration of NPB resets x=1 afterwards and so does not
    change any zeta; it is not repeated here.)
    """
    n = len(rowptr) - 1
    x = np.ones(n)
    zetas, rnorms = [], []
    for it in range(niter):
        _, zeta, rn = npb_outer(rowptr, colidx, vals, x, cgitmax, shift, variant)
        zetas.append(zeta)
        rnorms.append(rn)
        if on_iter:
            on_iter(it, zeta, rn)
    return np.array(zetas), np.array(rnorms)


def partition(rowptr, nranks):
    rowptr = _c(rowptr, np.int32)
    m = rowptr.shape[0] - 1
    bounds = np.zeros(nranks + 1, dtype=np.int64)
    lib().oracle_partition(_ptr(rowptr), m, int(nranks), _ptr(bounds))
    return bounds


def merge_path(rowptr, pieces):
    rowptr = _c(rowptr, np.int32)
    m = rowptr.shape[0] - 1
    sr = np.zeros(pieces + 1, dtype=np.int64)
    sn = np.zeros(pieces + 1, dtype=np.int64)
    lib().oracle_merge_path(_ptr(rowptr), m, int(pieces), _ptr(sr), _ptr(sn))
    return sr, sn


LAPLACE27 = np.array([-1.0] * 13 + [26.0] + [-1.0] * 13)  # reading R19 weights, w[(dz+1)*9+(dy+1)*3+(dx+1)]


def stencil27(nx, ny, nz, x, w=None, y_old=None, alpha=1.0, beta=0.0):
    """Matrix-free 27-point stencil (Fig. 13 Stencil idiom, R19): (y_ref, bound)."""
    w = LAPLACE27 if w is None else np.ascontiguousarray(w, dtype=np.float64)
    assert w.shape == (27,)
    n = nx * ny * nz
    x = _c(x, np.float64)
    yo = _c(y_old if y_old is not None else np.zeros(n), np.float64)
    y = np.empty(n)
    b = np.empty(n)
    lib().oracle_stencil27(nx, ny, nz, _ptr(w), _ptr(x), _ptr(yo), alpha, beta, _ptr(y), _ptr(b))
    return y, b


# ---------------------------------------------------------------- idioms
# Scalar reduction (Fig. 14), generalised histogram (Fig. 11), NAS EP.

def reduce(a, b=None):
    """(sum, bound): sequential sum of a[i] (or a[i]*b[i]) in fp64 and sum|term|."""
    f32 = np.asarray(a).dtype == np.float32
    dt = np.float32 if f32 else np.float64
    a = _c(a, dt)
    b = _c(b, dt) if b is not None else None
    s = ctypes.c_double(0.0)
    bd = ctypes.c_double(0.0)
    fn = lib().oracle_reduce_f32 if f32 else lib().oracle_reduce_f64
    fn(a.shape[0], _ptr(a), _ptr(b), ctypes.byref(s), ctypes.byref(bd))
    return s.value, bd.value


def hist_count_u32(keys, nbins, bins=None):
    keys = _c(keys, np.int32)
    out = np.zeros(max(nbins, 1), np.uint32) if bins is None else _c(bins, np.uint32).copy()
    lib().oracle_hist_count_u32(keys.shape[0], _ptr(keys), int(nbins), _ptr(out))
    return out[:nbins]


def hist_sat_u8(keys, nbins, bins=None):
    keys = _c(keys, np.int32)
    out = np.zeros(max(nbins, 1), np.uint8) if bins is None else _c(bins, np.uint8).copy()
    lib().oracle_hist_sat_u8(keys.shape[0], _ptr(keys), int(nbins), _ptr(out))
    return out[:nbins]


def hist_sum_f64(keys, w, nbins, bins=None):
    """(bins, bound): weighted histogram and the per-bin sum of |w| (+|old|)."""
    keys = _c(keys, np.int32)
    w = _c(w, np.float64)
    out = np.zeros(max(nbins, 1)) if bins is None else _c(bins, np.float64).copy()
    bound = np.zeros(max(nbins, 1))
    lib().oracle_hist_sum_f64(keys.shape[0], _ptr(keys), _ptr(w), int(nbins), _ptr(out), _ptr(bound))
    return out[:nbins], bound[:nbins]


def npb_randlc_stream(count, seed=314159265.0, a=1220703125.0):
    out = np.empty(count)
    lib().oracle_npb_randlc_stream(float(seed), float(a), int(count), _ptr(out))
    return out


def ep(M, pair_begin=0, pair_count=None):
    """NAS EP over pairs [pair_begin, pair_begin+pair_count) of class 2^M.

    Returns (q[10], sx, sy)."""
    if pair_count is None:
        pair_count = (1 << M) - pair_begin
    q = np.zeros(10)
    sx = ctypes.c_double(0.0)
    sy = ctypes.c_double(0.0)
    st = lib().oracle_ep(int(M), int(pair_begin), int(pair_count), _ptr(q), ctypes.byref(sx), ctypes.byref(sy))
    if st != 0:
        raise ValueError(f"oracle_ep: bad arguments (status {st})")
    return q, sx.value, sy.value


def spmv_jds(J, x, y_old=None, alpha=1.0, beta=0.0):
    """y_ref, bound on the JDS-32 layout J (gen.JDS): y indexed by ORIGINAL row."""
    f32 = J.data.dtype == np.float32
    dt = np.float32 if f32 else np.float64
    x = _c(x, dt)
    yo = _c(y_old, dt) if y_old is not None else np.zeros(max(J.m, 1), dtype=dt)
    y_ref = np.empty(max(J.m, 1))
    bound = np.empty(max(J.m, 1))
    lib().oracle_spmv_jds(J.m, _ptr(_c(J.perm, np.int32)), _ptr(_c(J.jds_ptr, np.int64)), _ptr(_c(J.zcnt, np.int32)),
                          _ptr(_c(J.indices, np.int32)), _ptr(_c(J.data, dt)), _ptr(x), _ptr(yo),
                          float(alpha), float(beta), int(f32), _ptr(y_ref), _ptr(bound))
    return y_ref[:J.m], bound[:J.m]


# ---------------------------------------------------------------- CPU baseline
# oracle_omp.c: the textbook-CG loops of oracle_spmv.c with OpenMP
# schedule(static) row/element loops, for bench.py's all-core CPU baseline
# (BASELINE.md section 3).  Not pinned, never used for parity.
_OMP_SRC = os.path.join(_HERE, "oracle_omp.c")
_OMP_LIB = os.path.join(_HERE, "liboracle_omp.so")
_omp = None


def build_omp(force: bool = False) -> str:
    if force or not os.path.exists(_OMP_LIB) or os.path.getmtime(_OMP_LIB) < os.path.getmtime(_OMP_SRC):
        tmp = _OMP_LIB + f".tmp{os.getpid()}"
        subprocess.check_call(["gcc", "-O3", "-march=native", "-ffp-contract=off", "-std=c11", "-fPIC", "-fopenmp",
                               "-shared", "-o", tmp, _OMP_SRC, "-lm"])
        os.replace(tmp, _OMP_LIB)
    return _OMP_LIB


def npb_outer_omp(rowptr, colidx, vals, x, cgitmax, shift, nthreads=0):
    """oracle_omp.c's NAS outer iteration on nthreads OpenMP threads (0 = all);
    returns (z, zeta, rnorm, threads_used)."""
    global _omp
    if _omp is None:
        build_omp()
        _omp = ctypes.CDLL(_OMP_LIB)
        _omp.omp_npb_outer.argtypes = [_I64, _P, _P, _P, _P, _P, _I32, _D, _P, _P, _I32]
        _omp.omp_npb_outer.restype = ctypes.c_int
    assert x.dtype == np.float64 and x.flags.c_contiguous
    rowptr = _c(rowptr, np.int32)
    colidx = _c(colidx, np.int32)
    vals = _c(vals, np.float64)
    n = rowptr.shape[0] - 1
    z = np.zeros(n)
    zeta = ctypes.c_double(0.0)
    rn = ctypes.c_double(0.0)
    used = _omp.omp_npb_outer(n, _ptr(rowptr), _ptr(colidx), _ptr(vals), _ptr(x), _ptr(z), int(cgitmax),
                              float(shift), ctypes.byref(zeta), ctypes.byref(rn), int(nthreads))
    return z, zeta.value, rn.value, used

