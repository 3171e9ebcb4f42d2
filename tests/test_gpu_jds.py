"""GPU parity of spmv_jds (the JDS-32 layout of Parboil spmv, reading R34,
SURVEY 8(f) NEXT-4) against the JDS oracle row by row (R11 tolerance), at the
full Parboil-shaped size (fp32, every row), with the BLAS alpha/beta
conventions, structure checks and determinism."""
import numpy as np
import pytest

import gen
import oracle
from gpu_util import check_rows

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def sp():
    import torch
    import paper_conf_asplos_ginsbachrsbdo18_b200 as sp
    torch.cuda.set_device(0)
    return sp


def _dev(a):
    import torch
    return torch.from_numpy(np.ascontiguousarray(a)).cuda()


def _handle(sp, J):
    return sp.JDSMatrix(_dev(J.perm), _dev(J.jds_ptr), _dev(J.zcnt), _dev(J.indices), _dev(J.data), J.m, J.n)


def _cases():
    rows = np.array([0, 0, 2, 5, 5, 5, 40]); cols = np.array([3, 1, 0, 2, 9, 4, 7])
    skew = gen.powerlaw(m=20_000, lmax=5000.0, seed=9, f32=False)     # slices split into many units
    return [gen.makea("S"), gen.laplace1d(1000), gen.from_coo(41, 10, rows, cols, np.arange(1.0, 8.0)),
            gen.from_dense(np.zeros((3, 4))), skew, gen.stencil27(12)]


@pytest.mark.parametrize("f32", [False, True])
def test_jds_zoo_alpha_beta(sp, f32):
    import torch
    for A in _cases():
        A = A.astype(np.float32) if f32 else A
        J = gen.csr_to_jds(A)
        dt = np.float32 if f32 else np.float64
        x = gen.uniform(A.n, seed=1, f32=f32)
        yo = gen.uniform(A.m, seed=2, f32=f32)
        with _handle(sp, J) as M:
            for al, be in ((1.0, 0.0), (-1.5, 0.25), (0.0, 2.0), (0.0, 0.0)):
                y = _dev(yo.copy())
                if be == 0.0:
                    y.fill_(float("nan"))                              # beta == 0: y is write-only (R6)
                M.spmv(_dev(x), y, al, be)
                ref, bound = oracle.spmv_jds(J, x, yo, al, be)
                check_rows(y.cpu().numpy().astype(np.float64), ref, bound, dt, f"{A.name} a={al} b={be}")


def test_jds_parboil_full_size_every_row(sp):
    """BJ.cfg[2] shape (2^20 rows, ~11.5M nnz, rows up to 10,000) in fp32."""
    A = gen.powerlaw()
    J = gen.csr_to_jds(A)
    x = gen.uniform(A.n, seed=5, f32=True)
    y = _dev(np.zeros(A.m, np.float32))
    with _handle(sp, J) as M:
        M.spmv(_dev(x), y)
        got = y.cpu().numpy()
        ref, bound = oracle.spmv_jds(J, x)
        check_rows(got.astype(np.float64), ref, bound, np.float32, "parboil jds")
        y2 = _dev(np.zeros(A.m, np.float32))
        M.spmv(_dev(x), y2)
        assert np.array_equal(got, y2.cpu().numpy())                    # deterministic (no atomics)
    # and equal to the CSR path's oracle: the layout does not change the per-row terms
    ref_csr, bound_csr = oracle.spmv(A.rowptr, A.colidx, A.vals, x)
    check_rows(got.astype(np.float64), ref_csr, bound_csr, np.float32, "parboil jds vs csr oracle")


def test_jds_structure_errors(sp):
    A = gen.makea("S")
    J = gen.csr_to_jds(A)
    bad = J.jds_ptr.copy()
    bad[3] += 32
    with pytest.raises(sp.SpmvError) as e:
        sp.JDSMatrix(_dev(J.perm), _dev(bad), _dev(J.zcnt), _dev(J.indices), _dev(J.data), J.m, J.n)
    assert e.value.status == sp.SPMV_ERR_INDEX
    z = J.zcnt.copy()
    z[-1] = z[0] + 1
    with pytest.raises(sp.SpmvError):
        sp.JDSMatrix(_dev(J.perm), _dev(J.jds_ptr), _dev(z), _dev(J.indices), _dev(J.data), J.m, J.n)
    with _handle(sp, J) as M:
        d = M._keep[4]
        with pytest.raises(sp.SpmvError) as e:
            M.spmv(_dev(gen.uniform(A.n, seed=1)), d[:A.m])             # y inside data
        assert e.value.status == sp.SPMV_ERR_ALIAS
