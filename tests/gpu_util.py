"""Helpers for the -m gpu parity tests (not a test module)."""
import numpy as np

TOL = {np.float64: 1e-12, np.float32: 1e-5}  # BJ.ns per-row tolerance


def to_dev(A, dev, vals=None):
    import torch
    rp = torch.from_numpy(np.ascontiguousarray(A.rowptr)).to(dev)
    ci = torch.from_numpy(np.ascontiguousarray(A.colidx)).to(dev)
    va = torch.from_numpy(np.ascontiguousarray(A.vals if vals is None else vals)).to(dev)
    return rp, ci, va


def check_rows(y_gpu, y_ref, bound, dtype, what=""):
    """|y - y_ref| <= tol * bound per row (bound == 0 -> exact; +0 == -0)."""
    y = np.asarray(y_gpu, dtype=np.float64)
    tol = TOL[np.dtype(dtype).type]
    err = np.abs(y - y_ref)
    bad = ~(err <= tol * bound)
    # NaN/inf in the reference must be matched exactly
    both_nan = np.isnan(y) & np.isnan(y_ref)
    bad &= ~both_nan
    if bad.any():
        i = int(np.nonzero(bad)[0][0])
        raise AssertionError(f"{what}: {int(bad.sum())} rows out of tolerance; first row {i}: "
                             f"gpu {y[i]!r} ref {y_ref[i]!r} bound {bound[i]!r}")
    return float(np.max(err / np.where(bound > 0, bound, 1.0))) if len(err) else 0.0
