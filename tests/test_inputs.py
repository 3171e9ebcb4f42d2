"""Generator tests (CPU): shapes and structure of the synthetic workloads
(DESIGN.md section 4), and closed forms that pin the 27-point stencil."""
import numpy as np
import pytest

import gen
import oracle


@pytest.mark.parametrize("N", [1, 2, 3, 6])
def test_stencil27_structure_and_closed_form(N):
    A = gen.stencil27(N)
    assert A.m == N ** 3 and A.nnz == (3 * N - 2) ** 3
    L = A.row_lengths()
    # row-length multiset {27:(N-2)^3, 18:6(N-2)^2, 12:12(N-2), 8:8} (N >= 2)
    if N >= 2:
        k = N - 2
        want = {27: k ** 3, 18: 6 * k * k, 12: 12 * k, 8: 8}
        got = {v: int((L == v).sum()) for v in set(L.tolist())}
        assert {a: b for a, b in want.items() if b} == got
    # (A.1)_i = 27 - cnt_i  (centre 26, neighbours -1)
    y, _ = oracle.spmv(A.rowptr, A.colidx, A.vals, np.ones(A.n))
    assert np.array_equal(y, 27.0 - L)
    # interior rows of A.(affine function) vanish... up to the centre term:
    # A = 27 I - (box-sum) so for an affine f, (A f)_i = 27 f_i - 27 f_i = 0 inside
    if N >= 3:
        z, yy, x = np.meshgrid(np.arange(N), np.arange(N), np.arange(N), indexing="ij")
        f = (2.0 * x + 3.0 * yy - 5.0 * z + 1.0).ravel()
        y, _ = oracle.spmv(A.rowptr, A.colidx, A.vals, f)
        interior = ((x > 0) & (x < N - 1) & (yy > 0) & (yy < N - 1) & (z > 0) & (z < N - 1)).ravel()
        assert np.all(y[interior] == 0.0)


def test_stencil27_columns_sorted():
    A = gen.stencil27(5)
    for i in range(A.m):
        c = A.colidx[A.rowptr[i]:A.rowptr[i + 1]]
        assert np.all(np.diff(c) > 0)


def test_powerlaw_shape_small():
    m = 1 << 14
    A = gen.powerlaw(m=m, lmax=1000.0, beta=0.545, seed=7)
    L = A.row_lengths()
    ref = np.maximum(1, np.floor(1000.0 * np.arange(1, m + 1, dtype=np.float64) ** -0.545)).astype(np.int64)
    assert np.array_equal(np.sort(L), np.sort(ref))
    for i in np.nonzero(L > 1)[0][:500]:
        c = A.colidx[A.rowptr[i]:A.rowptr[i + 1]]
        assert np.all(np.diff(c) > 0) and c.min() >= 0 and c.max() < m
    assert A.vals.dtype == np.float32 and np.all(np.abs(A.vals) <= 1)
    # deterministic
    B = gen.powerlaw(m=m, lmax=1000.0, beta=0.545, seed=7)
    assert np.array_equal(A.colidx, B.colidx) and np.array_equal(A.vals, B.vals)


@pytest.mark.slow
def test_powerlaw_parboil_size():
    A = gen.powerlaw()
    L = A.row_lengths()
    assert A.m == 1 << 20 and A.nnz == 11518867
    assert L.min() == 5 and L.max() == 10000 and int((L >= 1024).sum()) == 65


def test_uniform_range_and_determinism():
    a = gen.uniform(10000, seed=3)
    b = gen.uniform(10000, seed=3)
    c = gen.uniform(10000, seed=4)
    assert np.array_equal(a, b) and not np.array_equal(a, c)
    assert a.min() >= -1 and a.max() < 1 and abs(a.mean()) < 0.05
