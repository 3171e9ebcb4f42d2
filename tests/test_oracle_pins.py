"""Pins for the CPU oracle (oracle/oracle_spmv.c) against facts that do not come
from the oracle itself: closed forms, exact integer brute force, published NPB
verification values, and characterising properties of the partition and
merge-path splits.  All CPU (-m "not gpu").

Each pin is chosen so a plausible oracle bug fails it: a dropped term (dense
brute force, Laplacian closed forms), a wrong sign/index (permutation, j and j^2
Laplacian forms), transposed operands (non-square and non-symmetric brute
force), beta/alpha mix-ups (alpha/beta tests), a wrong CG update (Laplacian CG
closed form, NPB zeta).
"""
import os

import numpy as np
import pytest

import gen
import oracle

GOLD = os.path.join(os.path.dirname(__file__), "golden")


def _read_golden(name):
    rows = []
    with open(os.path.join(GOLD, name)) as f:
        for line in f:
            if line.startswith("#") or not line.strip():
                continue
            rows.append(line.split())
    return rows


# ---------------------------------------------------------------- SpMV pins
def test_identity_exact():
    n = 257
    A = gen.from_dense(np.eye(n))
    x = gen.uniform(n, seed=1)
    y, b = oracle.spmv(A.rowptr, A.colidx, A.vals, x)
    assert np.array_equal(y, x)
    assert np.array_equal(b, np.abs(x))


def test_permutation_exact():
    n = 300
    rng = np.random.default_rng(3)
    pi = rng.permutation(n)
    A = gen.from_coo(n, n, np.arange(n), pi, np.ones(n))
    x = gen.uniform(n, seed=2)
    y, _ = oracle.spmv(A.rowptr, A.colidx, A.vals, x)
    assert np.array_equal(y, x[pi])


def test_diagonal_exact():
    n = 123
    d = gen.uniform(n, seed=5)
    x = gen.uniform(n, seed=6)
    A = gen.from_coo(n, n, np.arange(n), np.arange(n), d)
    y, _ = oracle.spmv(A.rowptr, A.colidx, A.vals, x)
    assert np.array_equal(y, d * x)  # one correctly rounded product per row


@pytest.mark.parametrize("density", [0.0, 0.05, 0.3, 1.0])
@pytest.mark.parametrize("shape", [(1, 1), (7, 13), (64, 64), (40, 3)])
def test_dense_bruteforce_exact(density, shape):
    """Small-integer A, x: every partial sum is an exact integer in fp64."""
    m, n = shape
    rng = np.random.default_rng(int(density * 100) + m * 7 + n)
    A = rng.integers(-9, 10, size=(m, n)) * (rng.random((m, n)) < density)
    x = rng.integers(-9, 10, size=n)
    ref = A.astype(np.int64) @ x.astype(np.int64)
    C = gen.from_dense(A.astype(np.float64))
    y, b = oracle.spmv(C.rowptr, C.colidx, C.vals, x.astype(np.float64))
    assert np.array_equal(y, ref.astype(np.float64))
    assert np.array_equal(b, (np.abs(A) @ np.abs(x)).astype(np.float64))
    # fp32 variant: same exact integers
    y32, _ = oracle.spmv(C.rowptr, C.colidx, C.vals.astype(np.float32), x.astype(np.float32))
    assert np.array_equal(y32, ref.astype(np.float64))


def test_duplicates_unsorted_offset_rowptr_empty_rows():
    """Reading R10 (duplicates/unsorted summed), R2 (rowptr[0] != 0), R7 (empty rows written)."""
    m, n = 6, 5
    rows = [0, 0, 0, 2, 2, 2, 2, 5]
    cols = [4, 1, 4, 0, 3, 0, 3, 2]
    vals = [1, 2, 3, 4, 5, 6, 7, 8]
    C = gen.from_coo(m, n, rows, cols, vals)
    dense = np.zeros((m, n), np.int64)
    for r, c, v in zip(rows, cols, vals):
        dense[r, c] += v
    x = np.array([1.0, -2.0, 3.0, 5.0, 7.0])
    ref = dense @ x.astype(np.int64)
    # shift the arrays: rowptr[0] = 11, arrays carry 11 junk leading entries
    off = 11
    colidx = np.concatenate([np.full(off, 10**6, np.int32), C.colidx])
    v = np.concatenate([np.full(off, np.nan), C.vals])
    y, _ = oracle.spmv(C.rowptr + off, colidx, v, x)
    assert np.array_equal(y, ref.astype(np.float64))
    assert y[1] == 0.0 and y[3] == 0.0 and y[4] == 0.0


def test_alpha_beta_conventions():
    rng = np.random.default_rng(11)
    m, n = 17, 9
    A = rng.integers(-5, 6, size=(m, n)) * (rng.random((m, n)) < 0.5)
    x = rng.integers(-5, 6, size=n).astype(np.float64)
    yo = rng.integers(-5, 6, size=m).astype(np.float64)
    C = gen.from_dense(A.astype(np.float64))
    y, _ = oracle.spmv(C.rowptr, C.colidx, C.vals, x, yo, alpha=2.0, beta=-3.0)
    assert np.array_equal(y, 2.0 * (A @ x) - 3.0 * yo)
    # beta == 0: y_old is not read (NaN must not propagate)
    y, _ = oracle.spmv(C.rowptr, C.colidx, C.vals, x, np.full(m, np.nan), alpha=1.0, beta=0.0)
    assert np.array_equal(y, A @ x)
    # alpha == 0: A and x are not read
    xn = np.full(n, np.nan)
    y, _ = oracle.spmv(C.rowptr, C.colidx, C.vals, xn, yo, alpha=0.0, beta=2.0)
    assert np.array_equal(y, 2.0 * yo)


@pytest.mark.parametrize("n", [2, 3, 10, 1000, 65537])
def test_laplace1d_closed_forms(n):
    A = gen.laplace1d(n)
    j = np.arange(n, dtype=np.float64)
    y, _ = oracle.spmv(A.rowptr, A.colidx, A.vals, np.ones(n))
    e = np.zeros(n); e[0] += 1; e[-1] += 1
    assert np.array_equal(y, e)
    y, _ = oracle.spmv(A.rowptr, A.colidx, A.vals, j)
    ref = np.zeros(n); ref[0] = -1; ref[-1] = n
    assert np.array_equal(y, ref)
    y, _ = oracle.spmv(A.rowptr, A.colidx, A.vals, j * j)
    ref = np.full(n, -2.0); ref[0] = -1; ref[-1] = float(n) * n - 2
    assert np.array_equal(y, ref)


def test_nonsymmetric_orientation():
    """Transposed operand check: a strictly upper-triangular shift matrix."""
    n = 50
    A = gen.from_coo(n, n, np.arange(n - 1), np.arange(1, n), np.ones(n - 1))
    x = np.arange(n, dtype=np.float64)
    y, _ = oracle.spmv(A.rowptr, A.colidx, A.vals, x)
    assert np.array_equal(y[:-1], x[1:]) and y[-1] == 0.0


# ------------------------------------------------------------------ CG pins
@pytest.mark.parametrize("n", [1, 2, 5, 16, 64])
def test_cg_laplace1d_closed_form(n):
    """A=tridiag(-1,2,-1), b=1: z_j=(j+1)(n-j)/2; CG terminates in <= n steps."""
    A = gen.laplace1d(n)
    z, its, rn, st = oracle.cg(A.rowptr, A.colidx, A.vals, np.ones(n), max_iter=n, tol=1e-14)
    j = np.arange(n)
    ref = (j + 1) * (n - j) / 2.0
    assert st == 0
    assert np.allclose(z, ref, rtol=1e-10, atol=0)
    assert rn <= 1e-10 * np.sqrt(n) * ref.max()


def test_cg_diagonal_one_step():
    """Diagonal c*I: CG reaches b/c after one iteration exactly (up to one rounding)."""
    n = 40
    A = gen.from_coo(n, n, np.arange(n), np.arange(n), np.full(n, 4.0))
    b = gen.uniform(n, seed=9)
    z, its, rn, st = oracle.cg(A.rowptr, A.colidx, A.vals, b, max_iter=1)
    assert st == 0 and its == 1
    assert np.allclose(z, b / 4.0, rtol=1e-15, atol=0)


def test_cg_breakdown_zero_rhs():
    A = gen.laplace1d(8)
    z, its, rn, st = oracle.cg(A.rowptr, A.colidx, A.vals, np.zeros(8), max_iter=5)
    assert st == 7 and its == 0


# Single-reduction (Chronopoulos-Gear) CG oracle, NEXT-1: pinned to the same
# closed forms, to exact termination, and to the textbook oracle's iterates.
@pytest.mark.parametrize("n", [1, 2, 5, 16, 64])
def test_cgcg_laplace1d_closed_form(n):
    A = gen.laplace1d(n)
    z, its, rn, st = oracle.cg(A.rowptr, A.colidx, A.vals, np.ones(n), max_iter=n, tol=1e-14, variant=1)
    j = np.arange(n)
    ref = (j + 1) * (n - j) / 2.0
    assert st == 0
    assert np.allclose(z, ref, rtol=1e-10, atol=0)


def test_cgcg_small_integer_spd_exact_solution():
    """A = B^T B + n I with small integers, x* integer: n steps reach x* (rounding only)."""
    rng = np.random.default_rng(3)
    n = 12
    B = rng.integers(-3, 4, size=(n, n)).astype(np.float64)
    Ad = B.T @ B + n * np.eye(n)
    xs = rng.integers(-5, 6, size=n).astype(np.float64)
    b = Ad @ xs
    A = gen.from_dense(Ad)
    z, its, rn, st = oracle.cg(A.rowptr, A.colidx, A.vals, b, max_iter=n, variant=1)
    assert st == 0 and its == n
    assert np.allclose(z, xs, rtol=0, atol=1e-9)


@pytest.mark.parametrize("k", [1, 2, 3, 10, 25])
def test_cgcg_iterates_equal_textbook(k):
    """Mathematically identical iterates: z_k of both oracles agree to rounding on makea S."""
    A = gen.makea("S")
    b = np.ones(A.n)
    z0, _, _, _ = oracle.cg(A.rowptr, A.colidx, A.vals, b, max_iter=k)
    z1, its, _, st = oracle.cg(A.rowptr, A.colidx, A.vals, b, max_iter=k, variant=1)
    assert st == 0 and its == k
    assert np.max(np.abs(z1 - z0)) <= 1e-12 * np.max(np.abs(z0))


def test_cgcg_one_step_and_breakdown():
    n = 40
    A = gen.from_coo(n, n, np.arange(n), np.arange(n), np.full(n, 4.0))
    b = gen.uniform(n, seed=9)
    z, its, rn, st = oracle.cg(A.rowptr, A.colidx, A.vals, b, max_iter=1, variant=1)
    assert st == 0 and its == 1 and np.allclose(z, b / 4.0, rtol=1e-15, atol=0)
    L = gen.laplace1d(8)
    z, its, rn, st = oracle.cg(L.rowptr, L.colidx, L.vals, np.zeros(8), max_iter=5, variant=1)
    assert st == 7 and its == 0


@pytest.mark.parametrize("cls", ["S", "W"])
def test_cgcg_npb_zeta_published(cls):
    g = {r[0]: r[1:] for r in _read_golden("npb_zeta.txt")}[cls]
    niter, shift, zeta_ref = int(g[2]), float(g[3]), float(g[4])
    A = gen.makea(cls)
    zetas, rnorms = oracle.npb_run(A.rowptr, A.colidx, A.vals, niter, shift, variant=1)
    assert abs(zetas[-1] - zeta_ref) / zeta_ref <= 1e-10
    assert rnorms.max() <= 1e-11


def test_randlc_against_bigint():
    """NPB randlc: x <- 5^13 x mod 2^46 (exact integer recurrence)."""
    vals = gen.randlc_stream(2000)
    x, a = 314159265, 1220703125
    for i in range(2000):
        x = (a * x) % (1 << 46)
        assert vals[i] == x / float(1 << 46)


@pytest.mark.parametrize("cls", ["S", "W", "A"])
def test_makea_nnz_golden(cls):
    g = {r[0]: r[1:] for r in _read_golden("npb_nnz.txt")}[cls]
    A = gen.makea(cls)
    L = A.row_lengths()
    assert A.nnz == int(g[0]) and L.min() == int(g[1]) and L.max() == int(g[2])
    # pattern symmetric, columns ascending, diagonal present (reading R16)
    assert np.all(np.diff(A.colidx.astype(np.int64))[np.diff(np.repeat(np.arange(A.m), L)) == 0] > 0)


@pytest.mark.parametrize("cls", ["S", "W", "A"])
def test_npb_zeta_published(cls):
    """The oracle's NAS CG run reproduces the published zeta within 1e-10 and
    keeps rnorm <= 1e-11 at every outer iteration."""
    g = {r[0]: r[1:] for r in _read_golden("npb_zeta.txt")}[cls]
    na, nonzer, niter, shift, zeta_ref = int(g[0]), int(g[1]), int(g[2]), float(g[3]), float(g[4])
    A = gen.makea(cls)
    assert A.m == na
    zetas, rnorms = oracle.npb_run(A.rowptr, A.colidx, A.vals, niter, shift)
    assert abs(zetas[-1] - zeta_ref) / zeta_ref <= 1e-10
    assert rnorms.max() <= 1e-11


# ------------------------------------------------------- partition / merge
def _rowptr_cases():
    rng = np.random.default_rng(5)
    cases = [np.array([0], np.int32), np.array([0, 0, 0], np.int32), np.array([0, 5], np.int32),
             np.array([3, 3, 10, 10, 11], np.int32)]
    for m in [1, 2, 7, 33]:
        L = rng.integers(0, 9, size=m)
        L[rng.random(m) < 0.2] = 0
        cases.append((np.concatenate([[0], np.cumsum(L)]) + rng.integers(0, 4)).astype(np.int32))
    skew = np.zeros(20, np.int64); skew[3] = 100
    cases.append(np.concatenate([[0], np.cumsum(skew)]).astype(np.int32))
    return cases


@pytest.mark.parametrize("P", [1, 2, 3, 4, 8])
def test_partition_characterisation(P):
    """b_r is the unique i with prefix(i) >= t_r and (i == 0 or prefix(i-1) < t_r)."""
    for rp in _rowptr_cases():
        m = len(rp) - 1
        b = oracle.partition(rp, P)
        pre = rp.astype(np.int64) - rp[0]
        nnz = int(pre[-1])
        assert b[0] == 0 and b[P] == m and np.all(np.diff(b) >= 0)
        for r in range(1, P):
            t = (r * nnz) // P
            cands = [i for i in range(m + 1) if pre[i] >= t and (i == 0 or pre[i - 1] < t)]
            assert cands == [b[r]]


@pytest.mark.parametrize("C", [1, 2, 5, 16])
def test_merge_path_characterisation(C):
    for rp in _rowptr_cases():
        m = len(rp) - 1
        A = rp[1:].astype(np.int64) - rp[0]
        nnz = int(rp[-1]) - int(rp[0])
        sr, sn = oracle.merge_path(rp, C)
        for c in range(C + 1):
            d = (c * (m + nnz)) // C
            cands = [(i, d - i) for i in range(0, min(d, m) + 1)
                     if 0 <= d - i <= nnz
                     and (i == 0 or A[i - 1] <= d - i)
                     and (i == m or d - i == 0 or A[i] > d - i - 1)]
            assert cands == [(sr[c], sn[c])], (rp, c, cands, sr[c], sn[c])


# ---------------------------------------------------------------- stencil27
# oracle_stencil27 (Fig. 13 Stencil idiom, reading R19), pinned to closed
# forms, exact shifts, and the CSR oracle on the generator's matrix.

@pytest.mark.parametrize("dims", [(1, 1, 1), (2, 3, 5), (7, 4, 3), (9, 9, 9)])
def test_stencil27_laplace_closed_forms(dims):
    nx, ny, nz = dims
    n = nx * ny * nz
    i = np.arange(n)
    xx, yy, zz = i % nx, (i // nx) % ny, i // (nx * ny)
    cnt = np.ones(n, dtype=np.int64)
    for c, N in ((xx, nx), (yy, ny), (zz, nz)):
        cnt *= (np.minimum(c + 1, N - 1) - np.maximum(c - 1, 0) + 1)
    y, b = oracle.stencil27(nx, ny, nz, np.ones(n))
    assert np.array_equal(y, (27 - cnt).astype(np.float64))  # A*1 = 26 - (cnt - 1)
    # affine fields vanish on interior points (weights sum to 0, symmetric offsets)
    f = 3.0 + 2.0 * xx - 5.0 * yy + 7.0 * zz
    y, _ = oracle.stencil27(nx, ny, nz, f)
    inner = (xx > 0) & (xx < nx - 1) & (yy > 0) & (yy < ny - 1) & (zz > 0) & (zz < nz - 1)
    assert np.all(y[inner] == 0.0)


@pytest.mark.parametrize("d", [(0, 0, 0), (1, 0, 0), (-1, 1, 0), (1, -1, -1), (0, 0, 1)])
def test_stencil27_one_hot_weight_is_a_shift(d):
    """w = e_d: y[p] = x[p + d] when p + d is inside the grid, else 0 (exact)."""
    nx, ny, nz = 6, 5, 4
    dx, dy, dz = d
    w = np.zeros(27)
    w[(dz + 1) * 9 + (dy + 1) * 3 + (dx + 1)] = 1.0
    x = gen.uniform(nx * ny * nz, seed=3)
    y, _ = oracle.stencil27(nx, ny, nz, x, w=w)
    for z in range(nz):
        for yy in range(ny):
            for xx in range(nx):
                p = xx + nx * (yy + ny * z)
                q = (xx + dx, yy + dy, z + dz)
                inside = 0 <= q[0] < nx and 0 <= q[1] < ny and 0 <= q[2] < nz
                assert y[p] == (x[q[0] + nx * (q[1] + ny * q[2])] if inside else 0.0)


@pytest.mark.parametrize("N", [2, 5, 12])
def test_stencil27_equals_csr_oracle_bitwise(N):
    """R19 weights on an N^3 grid == oracle_spmv_f64 on gen.stencil27(N): same
    terms in the same (ascending column) order, so bit for bit; alpha/beta too."""
    A = gen.stencil27(N)
    x = gen.uniform(A.n, seed=4)
    y0 = gen.uniform(A.m, seed=5)
    for a, b in [(1.0, 0.0), (-2.5, 0.5), (0.0, 3.0)]:
        ys, bs = oracle.stencil27(N, N, N, x, y_old=y0, alpha=a, beta=b)
        yc, bc = oracle.spmv(A.rowptr, A.colidx, A.vals, x, y0, a, b)
        assert np.array_equal(ys, yc) and np.array_equal(bs, bc)


# ------------------------------------------------- JDS-32 (Parboil format, R34)
def _jds_cases():
    cases = [gen.makea("S"), gen.powerlaw(m=5000, lmax=700.0, seed=4), gen.laplace1d(33),
             gen.from_dense(np.zeros((3, 4))), gen.from_dense(np.eye(1))]
    rows = np.array([0, 0, 2, 5, 5, 5, 40]); cols = np.array([3, 1, 0, 2, 9, 4, 7])
    cases.append(gen.from_coo(41, 10, rows, cols, np.arange(1.0, 8.0)))   # empty rows, m % 32 != 0
    return cases


@pytest.mark.parametrize("f32", [False, True])
def test_jds_oracle_equals_csr_oracle(f32):
    """The JDS layout changes only the storage order: per row the same terms in
    the same order (padding adds exact zeros), so the results are bit-identical."""
    for A in _jds_cases():
        A = A.astype(np.float32) if f32 else A
        J = gen.csr_to_jds(A)
        assert np.all(np.diff(J.zcnt) <= 0) and sorted(J.perm.tolist()) == list(range(A.m))
        x = gen.uniform(A.n, seed=2, f32=f32)
        yo = gen.uniform(A.m, seed=3, f32=f32)
        for al, be in ((1.0, 0.0), (-2.5, 0.5), (0.0, 3.0)):
            y1, b1 = oracle.spmv(A.rowptr, A.colidx, A.vals, x, yo, al, be)
            y2, b2 = oracle.spmv_jds(J, x, yo, al, be)
            assert np.array_equal(y1, y2) and np.array_equal(b1, b2), (A.name, al, be)


def test_jds_tiny_by_hand():
    """3x3 [[1,0,2],[0,0,0],[3,4,5]] x=(1,10,100): rows sorted (2,0,1); y = (201, 0, 543)."""
    A = gen.from_dense(np.array([[1.0, 0, 2], [0, 0, 0], [3, 4, 5]]))
    J = gen.csr_to_jds(A)
    assert J.perm.tolist() == [2, 0, 1] and J.zcnt.tolist() == [3] and J.jds_ptr.tolist() == [0, 32, 64, 96]
    y, _ = oracle.spmv_jds(J, np.array([1.0, 10.0, 100.0]))
    assert y.tolist() == [201.0, 0.0, 543.0]
