"""Seeded synthetic inputs shared by the oracle tests and the CUDA path.

This module holds none of the method's arithmetic (no SpMV, no CG).  It builds
CSR matrices and vectors with the shapes of the paper's workloads (DESIGN.md
section 4): the NAS CG makea matrix [ext:NPB] (the matrix of the SpMV idiom of
Fig. 4), a Parboil-spmv-shaped power-law matrix (BJ.cfg[2]), the
27-point stencil (BJ.cfg[4]) and the 1-D Laplacian.  The heavy loops are in
``gen.c`` (compiled with gcc on first use); this file marshals numpy arrays.
"""
from __future__ import annotations

import ctypes
import os
import subprocess
from dataclasses import dataclass

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "gen.c")
_LIB = os.path.join(_HERE, "libgen.so")
_lib = None

# NPB CG class parameters [ext:NPB]: (NA, NONZER, NITER, SHIFT); RCOND = 0.1
NPB_CLASSES = {
    "S": (1400, 7, 15, 10.0),
    "W": (7000, 8, 15, 12.0),
    "A": (14000, 11, 15, 20.0),
    "B": (75000, 13, 75, 60.0),
    "C": (150000, 15, 75, 110.0),
}
NPB_RCOND = 0.1
NPB_CGITMAX = 25
# NPB published verification values of zeta [ext:NPB] (tolerance 1e-10)
NPB_ZETA = {
    "S": 8.5971775078648,
    "W": 10.362595087124,
    "A": 17.130235054029,
    "B": 22.712745482631,
    "C": 28.973605592845,
}

PARBOIL_SEED = 20180324
PARBOIL_M = 1 << 20
PARBOIL_LMAX = 10000.0
PARBOIL_BETA = 0.545


def build(force: bool = False) -> str:
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        tmp = _LIB + f".tmp{os.getpid()}"
        subprocess.check_call(["gcc", "-O2", "-std=c11", "-fPIC", "-shared", "-o", tmp, _SRC, "-lm"])
        os.replace(tmp, _LIB)
    return _LIB


def _L():
    global _lib
    if _lib is None:
        build()
        L = ctypes.CDLL(_LIB)
        P, I64, I32, D, U64 = ctypes.c_void_p, ctypes.c_int64, ctypes.c_int32, ctypes.c_double, ctypes.c_uint64
        L.gen_makea.argtypes = [I64, I32, D, D]
        L.gen_makea.restype = P
        L.gen_powerlaw.argtypes = [I64, I64, D, D, U64]
        L.gen_powerlaw.restype = P
        L.gen_stencil27.argtypes = [I64]
        L.gen_stencil27.restype = P
        L.gen_laplace1d.argtypes = [I64]
        L.gen_laplace1d.restype = P
        for f in (L.gen_m, L.gen_n, L.gen_nnz):
            f.argtypes = [P]
            f.restype = I64
        L.gen_copy.argtypes = [P, P, P, P, ctypes.c_int]
        L.gen_copy.restype = None
        L.gen_free.argtypes = [P]
        L.gen_free.restype = None
        L.gen_randlc_stream.argtypes = [U64, U64, I64, P]
        L.gen_randlc_stream.restype = None
        L.gen_uniform_f64.argtypes = [U64, U64, I64, P]
        L.gen_uniform_f64.restype = None
        L.gen_uniform_f32.argtypes = [U64, U64, I64, P]
        L.gen_uniform_f32.restype = None
        L.gen_is_keys.argtypes = [I64, I64, U64, U64, P]
        L.gen_is_keys.restype = None
        L.gen_histo_image.argtypes = [I64, I64, I32, U64, P]
        L.gen_histo_image.restype = None
        _lib = L
    return _lib


@dataclass
class CSR:
    """Host CSR matrix: rowptr int32[m+1], colidx int32[nnz], vals float64/32[nnz]."""
    m: int
    n: int
    rowptr: np.ndarray
    colidx: np.ndarray
    vals: np.ndarray
    name: str = ""

    @property
    def nnz(self) -> int:
        return int(self.rowptr[self.m]) - int(self.rowptr[0])

    def row_lengths(self) -> np.ndarray:
        return np.diff(self.rowptr.astype(np.int64))

    def astype(self, dt) -> "CSR":
        return CSR(self.m, self.n, self.rowptr, self.colidx, self.vals.astype(dt), self.name)

    def bytes_per_spmv(self, beta_nonzero: bool = False) -> int:
        """Algorithmic bytes of one SpMV: nnz*(sizeof(T)+4) + 4*(m+1)
        + sizeof(T)*n (x once) + sizeof(T)*m (y written) [+ sizeof(T)*m if beta != 0]."""
        t = self.vals.dtype.itemsize
        b = self.nnz * (t + 4) + 4 * (self.m + 1) + t * self.n + t * self.m
        return b + (t * self.m if beta_nonzero else 0)


def _take(ptr, f32: bool, name: str) -> CSR:
    L = _L()
    if not ptr:
        raise MemoryError("generator failed")
    try:
        m, n, nnz = L.gen_m(ptr), L.gen_n(ptr), L.gen_nnz(ptr)
        rowptr = np.empty(m + 1, np.int32)
        colidx = np.empty(nnz, np.int32)
        vals = np.empty(nnz, np.float32 if f32 else np.float64)
        L.gen_copy(ptr, rowptr.ctypes.data, colidx.ctypes.data, vals.ctypes.data, 1 if f32 else 0)
    finally:
        L.gen_free(ptr)
    return CSR(int(m), int(n), rowptr, colidx, vals, name)


def makea(cls: str | None = None, *, n: int | None = None, nonzer: int | None = None,
          shift: float | None = None, rcond: float = NPB_RCOND) -> CSR:
    """NAS CG makea matrix for an NPB class ('S','W','A','B','C') or explicit params."""
    if cls is not None:
        n, nonzer, _, shift = NPB_CLASSES[cls]
    return _take(_L().gen_makea(int(n), int(nonzer), float(rcond), float(shift)), False,
                 f"makea-{cls or n}")


def powerlaw(m: int = PARBOIL_M, n: int | None = None, lmax: float = PARBOIL_LMAX,
             beta: float = PARBOIL_BETA, seed: int = PARBOIL_SEED, f32: bool = True) -> CSR:
    n = m if n is None else n
    return _take(_L().gen_powerlaw(int(m), int(n), float(lmax), float(beta), int(seed)), f32,
                 f"powerlaw-{m}")


def stencil27(N: int) -> CSR:
    return _take(_L().gen_stencil27(int(N)), False, f"stencil27-{N}")


def laplace1d(n: int) -> CSR:
    return _take(_L().gen_laplace1d(int(n)), False, f"laplace1d-{n}")


def randlc_stream(count: int, seed: int = 314159265, a: int = 1220703125) -> np.ndarray:
    out = np.empty(count, np.float64)
    _L().gen_randlc_stream(seed, a, count, out.ctypes.data)
    return out


def uniform(count: int, seed: int, stream: int = 7, f32: bool = False) -> np.ndarray:
    """U[-1,1) vector from the counter-based splitmix64 (seed, stream, index)."""
    out = np.empty(count, np.float32 if f32 else np.float64)
    fn = _L().gen_uniform_f32 if f32 else _L().gen_uniform_f64
    fn(int(seed), int(stream), int(count), out.ctypes.data)
    return out


def from_dense(A: np.ndarray, dtype=np.float64) -> CSR:
    """CSR (row-major, ascending columns) of a small dense matrix; test helper."""
    A = np.asarray(A)
    m, n = A.shape
    rows, cols = np.nonzero(A)
    rowptr = np.zeros(m + 1, np.int32)
    np.add.at(rowptr, rows + 1, 1)
    rowptr = np.cumsum(rowptr).astype(np.int32)
    return CSR(m, n, rowptr, cols.astype(np.int32), A[rows, cols].astype(dtype), "dense")


def from_coo(m: int, n: int, rows, cols, vals, dtype=np.float64) -> CSR:
    """CSR keeping the given entry order within each row (duplicates kept); test helper."""
    rows = np.asarray(rows, np.int64)
    order = np.argsort(rows, kind="stable")
    rowptr = np.zeros(m + 1, np.int64)
    np.add.at(rowptr, rows + 1, 1)
    rowptr = np.cumsum(rowptr).astype(np.int32)
    return CSR(m, n, rowptr, np.asarray(cols, np.int32)[order],
               np.asarray(vals, dtype)[order], "coo")


# ------------------------------------------------------------- idiom inputs
# NPB IS class parameters [ext:NPB-IS]: (TOTAL_KEYS_LOG_2, MAX_KEY_LOG_2)
NPB_IS_CLASSES = {"S": (16, 11), "W": (20, 16), "A": (23, 19), "B": (25, 21), "C": (27, 23)}
# NPB EP classes [ext:NPB-EP]: M (2^M Gaussian pairs)
NPB_EP_CLASSES = {"S": 24, "W": 25, "A": 28, "B": 30, "C": 32}
# Parboil-histo-shaped image (reading R32): 996x1040 pixels, 4096x256 uint8 bins
HISTO_NPIX = 996 * 1040
HISTO_NBINS = 4096 * 256
HISTO_HOT = 64
HISTO_SEED = 20180324


def is_keys(cls: str | None = None, *, n: int | None = None, max_key: int | None = None,
            seed: int = 314159265, a: int = 1220703125) -> np.ndarray:
    """NPB IS create_seq keys (int32) of a class or of explicit (n, max_key)."""
    if cls is not None:
        lk, lm = NPB_IS_CLASSES[cls]
        n, max_key = 1 << lk, 1 << lm
    out = np.empty(n, np.int32)
    _L().gen_is_keys(int(n), int(max_key), int(seed), int(a), out.ctypes.data)
    return out


def histo_image(npix: int = HISTO_NPIX, nbins: int = HISTO_NBINS, hot: int = HISTO_HOT,
                seed: int = HISTO_SEED) -> np.ndarray:
    """Parboil-histo-shaped pixel values in [0, nbins) with hot spots (int32)."""
    out = np.empty(npix, np.int32)
    _L().gen_histo_image(int(npix), int(nbins), int(hot), int(seed), out.ctypes.data)
    return out


# --------------------------------------------------- JDS-32 layout (R34)
@dataclass
class JDS:
    """Jagged-diagonal layout of a CSR matrix (Parboil spmv's format, reading R34).

    perm[i]   original row at sorted position i (decreasing length, stable)
    zcnt[s]   diagonal steps of slice s = positions [32s, 32s+32) (its longest row)
    jds_ptr   int64[depth+1]: diagonal k occupies [jds_ptr[k], jds_ptr[k+1]) and holds
              positions 0 .. jds_ptr[k+1]-jds_ptr[k]-1 (whole slices with zcnt > k)
    indices, data: entry jds_ptr[k]+i = step k of position i (value 0, column 0 padding)
    """
    m: int
    n: int
    perm: np.ndarray
    zcnt: np.ndarray
    jds_ptr: np.ndarray
    indices: np.ndarray
    data: np.ndarray

    @property
    def depth(self) -> int:
        return len(self.jds_ptr) - 1


def csr_to_jds(A: CSR) -> JDS:
    """Pure layout transform (no arithmetic): CSR -> JDS-32, entries in CSR order per row."""
    m = A.m
    L = A.row_lengths().astype(np.int64)
    perm = np.argsort(-L, kind="stable").astype(np.int32)
    Ls = L[perm]
    ns = (m + 31) // 32
    zcnt = Ls[0::32].astype(np.int32) if m else np.zeros(0, np.int32)
    depth = int(zcnt[0]) if ns else 0
    # positions covered by diagonal k: 32 * #{slices with zcnt > k} (zcnt is non-increasing)
    cover = np.array([32 * int(np.searchsorted(-zcnt, -k, side="left")) for k in range(depth)], np.int64)
    jds_ptr = np.zeros(depth + 1, np.int64)
    jds_ptr[1:] = np.cumsum(cover)
    tot = int(jds_ptr[-1])
    indices = np.zeros(tot, np.int32)
    data = np.zeros(tot, A.vals.dtype)
    start = A.rowptr[:-1].astype(np.int64)[perm] if m else np.zeros(0, np.int64)
    for k in range(depth):
        c = int(cover[k])
        i = np.arange(min(c, m))
        ok = Ls[i] > k
        src = start[i[ok]] + k
        dst = jds_ptr[k] + i[ok]
        indices[dst] = A.colidx[src]
        data[dst] = A.vals[src]
    return JDS(m, A.n, perm, zcnt, jds_ptr, indices, data)
