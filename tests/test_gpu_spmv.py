"""GPU parity of spmv_csr against the CPU oracle (element by element, per-row
tolerance of BJ.ns: 1e-12 (fp64) / 1e-5 (fp32) of sum_k |a_ik x_k|), through
the C ABI.  Covers every kernel variant, the adversarial zoo of SURVEY 4.3,
the alpha/beta conventions, the error paths, and the full-size NAS B/C and
Parboil-shaped matrices of BASELINE.json."""
import numpy as np
import pytest

import gen
import oracle
from gpu_util import check_rows, to_dev

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def torch_dev():
    import torch
    return torch, torch.device("cuda:0")


@pytest.fixture(scope="module")
def sp():
    import paper_conf_asplos_ginsbachrsbdo18_b200 as sp
    return sp


def run_case(sp, torch, dev, A, x_h, *, alpha=1.0, beta=0.0, y0=None, kernel="auto", lanes=0,
             validate=True, what=""):
    f32 = A.vals.dtype == np.float32
    tdt = torch.float32 if f32 else torch.float64
    rp, ci, va = to_dev(A, dev)
    x = torch.from_numpy(np.ascontiguousarray(x_h)).to(dev)
    y_old = y0 if y0 is not None else np.full(A.m, np.nan, dtype=A.vals.dtype)
    y = torch.from_numpy(y_old.copy()).to(dev)
    if lanes and kernel == "auto":
        kernel = "vector"
    with sp.CSRMatrix(rp, ci, va, A.n, kernel=kernel, vec_lanes=lanes, validate=validate) as M:
        M.spmv(x, y, alpha, beta)
        torch.cuda.synchronize()
        info = M.info()
    y_ref, bound = oracle.spmv(A.rowptr, A.colidx, A.vals, x_h, y_old, alpha, beta)
    check_rows(y.cpu().numpy(), y_ref, bound, A.vals.dtype, what)
    return info


def zoo():
    """(name, CSR) adversarial cases; the paper's silent corners."""
    r = np.random.default_rng(42)
    cases = []
    cases.append(("m0", gen.CSR(0, 5, np.zeros(1, np.int32), np.zeros(0, np.int32), np.zeros(0))))
    cases.append(("nnz0", gen.CSR(7, 3, np.zeros(8, np.int32), np.zeros(0, np.int32), np.zeros(0))))
    cases.append(("n1", gen.from_dense(r.standard_normal((9, 1)))))
    rp = np.array([0, 0, 0, 3, 3, 5, 5, 5, 5], np.int32)
    cases.append(("trailing_empty", gen.CSR(8, 4, rp, r.integers(0, 4, 5).astype(np.int32), r.standard_normal(5))))
    L = r.integers(0, 6, 3000)
    L[1234] = 100000
    rp = np.concatenate([[0], np.cumsum(L)]).astype(np.int32)
    nnz = int(rp[-1])
    cases.append(("one_long_row", gen.CSR(3000, 5000, rp, r.integers(0, 5000, nnz).astype(np.int32), r.standard_normal(nnz))))
    rows = r.integers(0, 50, 2000)
    cases.append(("dups_unsorted", gen.from_coo(50, 20, rows, r.integers(0, 20, 2000), r.standard_normal(2000))))
    A = gen.powerlaw(m=20000, lmax=3000.0, beta=0.6, seed=5, f32=False)
    cases.append(("powerlaw_small", A))
    cases.append(("laplace1d", gen.laplace1d(100001)))
    cases.append(("stencil27_9", gen.stencil27(9)))
    cases.append(("makea_S", gen.makea("S")))
    return cases


ZOO = zoo()


@pytest.mark.parametrize("lanes", [0, 1, 2, 4, 8, 16, 32])
@pytest.mark.parametrize("name,A", ZOO, ids=[c[0] for c in ZOO])
def test_zoo_fp64(sp, torch_dev, name, A, lanes):
    torch, dev = torch_dev
    x = gen.uniform(A.n, seed=11)
    run_case(sp, torch, dev, A, x, lanes=lanes, what=f"{name} lanes={lanes}")


@pytest.mark.parametrize("name,A", ZOO, ids=[c[0] for c in ZOO])
def test_zoo_fp32(sp, torch_dev, name, A):
    torch, dev = torch_dev
    A32 = A.astype(np.float32)
    x = gen.uniform(A.n, seed=12, f32=True)
    run_case(sp, torch, dev, A32, x, what=f"{name} fp32")


@pytest.mark.parametrize("unroll", ["2", "4", "8"])
def test_unroll_variants(sp, torch_dev, unroll, monkeypatch):
    torch, dev = torch_dev
    monkeypatch.setenv("SPMV_UNROLL", unroll)
    A = gen.makea("W")
    for lanes in (4, 32):
        run_case(sp, torch, dev, A, gen.uniform(A.n, seed=3), lanes=lanes, what=f"unroll {unroll}")


@pytest.mark.parametrize("alpha,beta", [(1.0, 0.0), (2.5, 0.0), (1.0, 1.0), (-0.5, 3.0), (0.0, 2.0),
                                        (0.0, 0.0)])
@pytest.mark.parametrize("f32", [False, True])
def test_alpha_beta(sp, torch_dev, alpha, beta, f32):
    torch, dev = torch_dev
    A = gen.makea("S")
    if f32:
        A = A.astype(np.float32)
    x = gen.uniform(A.n, seed=4, f32=f32)
    if alpha == 0.0:
        x = np.full(A.n, np.nan, dtype=x.dtype)  # A and x must not be read
    y0 = gen.uniform(A.m, seed=5, f32=f32)
    if beta == 0.0:
        y0 = np.full(A.m, np.nan, dtype=y0.dtype)  # y must not be read
    run_case(sp, torch, dev, A, x, alpha=alpha, beta=beta, y0=y0, what=f"a={alpha} b={beta}")


def test_rowptr_offset_and_misaligned_views(sp, torch_dev):
    """rowptr[0] != 0 (R2) and base pointers misaligned to 16 B (views at offset 1)."""
    torch, dev = torch_dev
    A = gen.makea("S")
    off = 3
    rp = torch.from_numpy(A.rowptr + off).to(dev)
    ci_full = torch.from_numpy(np.concatenate([np.full(off, 0, np.int32), A.colidx])).to(dev)
    va_full = torch.from_numpy(np.concatenate([np.full(off, np.nan), A.vals])).to(dev)
    # misalign: shift the whole structure by one element inside a bigger buffer
    ci_buf = torch.zeros(ci_full.numel() + 1, dtype=torch.int32, device=dev)
    va_buf = torch.zeros(va_full.numel() + 1, dtype=torch.float64, device=dev)
    ci_buf[1:] = ci_full
    va_buf[1:] = va_full
    ci, va = ci_buf[1:], va_buf[1:]
    x_h = gen.uniform(A.n, seed=8)
    xb = torch.zeros(A.n + 1, dtype=torch.float64, device=dev)
    xb[1:] = torch.from_numpy(x_h).to(dev)
    x = xb[1:]
    y = torch.full((A.m,), float("nan"), dtype=torch.float64, device=dev)
    with sp.CSRMatrix(rp, ci, va, A.n, validate=True) as M:
        M.spmv(x, y)
        torch.cuda.synchronize()
    y_ref, bound = oracle.spmv(A.rowptr, A.colidx, A.vals, x_h)
    check_rows(y.cpu().numpy(), y_ref, bound, np.float64, "offset/misaligned")


def test_vals_may_change_per_call(sp, torch_dev):
    torch, dev = torch_dev
    A = gen.makea("S")
    rp, ci, va = to_dev(A, dev)
    v2_h = gen.uniform(A.nnz, seed=21)
    v2 = torch.from_numpy(v2_h).to(dev)
    x_h = gen.uniform(A.n, seed=22)
    x = torch.from_numpy(x_h).to(dev)
    y = torch.empty(A.m, dtype=torch.float64, device=dev)
    with sp.CSRMatrix(rp, ci, va, A.n) as M:
        M.spmv(x, y, vals=v2)
        torch.cuda.synchronize()
    y_ref, bound = oracle.spmv(A.rowptr, A.colidx, v2_h, x_h)
    check_rows(y.cpu().numpy(), y_ref, bound, np.float64, "vals per call")


def test_errors(sp, torch_dev):
    torch, dev = torch_dev
    A = gen.makea("S")
    rp, ci, va = to_dev(A, dev)
    x = torch.zeros(A.n, dtype=torch.float64, device=dev)
    y = torch.zeros(A.m, dtype=torch.float64, device=dev)
    M = sp.CSRMatrix(rp, ci, va, A.n)
    # aliasing: y == x (R13)
    with pytest.raises(sp.SpmvError) as e:
        M.spmv(y[: A.n], y)
    assert e.value.status == sp.SPMV_ERR_ALIAS
    with pytest.raises(sp.SpmvError) as e:
        M.spmv(x, va[: A.m])
    assert e.value.status == sp.SPMV_ERR_ALIAS
    # host pointer where a device pointer is needed
    xh = torch.zeros(A.n, dtype=torch.float64)
    with pytest.raises(sp.SpmvError) as e:
        M.spmv(xh, y)
    assert e.value.status == sp.SPMV_ERR_ARG
    # structure binding mismatch
    import ctypes
    st = sp.spmv_csr_c(M.handle, A.m + 1, A.n, A.nnz, rp.data_ptr(), ci.data_ptr(), va.data_ptr(),
                       x.data_ptr(), y.data_ptr(), 1.0, 0.0)
    assert st == sp.SPMV_ERR_ARG
    M.destroy()
    # nnz mismatch at create (R1)
    h = ctypes.c_void_p()
    st = sp.spmv_csr_create_c(ctypes.byref(h), 0, A.m, A.n, A.nnz + 1, rp.data_ptr(), ci.data_ptr(),
                              va.data_ptr(), None)
    assert st == sp.SPMV_ERR_ARG
    # validate: column out of range, decreasing rowptr
    bad = ci.clone()
    bad[5] = A.n
    with pytest.raises(sp.SpmvError) as e:
        sp.CSRMatrix(rp, bad, va, A.n, validate=True)
    assert e.value.status == sp.SPMV_ERR_INDEX
    rp2 = rp.clone()
    rp2[10] = rp2[12] + 1
    rp2[11] = rp2[12] + 1  # keeps rowptr[m] - rowptr[0] == nnz
    with pytest.raises(sp.SpmvError) as e:
        sp.CSRMatrix(rp2, ci, va, A.n, validate=True)
    assert e.value.status == sp.SPMV_ERR_INDEX


def test_launch_count_increases(sp, torch_dev):
    torch, dev = torch_dev
    A = gen.makea("S")
    rp, ci, va = to_dev(A, dev)
    x = torch.ones(A.n, dtype=torch.float64, device=dev)
    y = torch.empty(A.m, dtype=torch.float64, device=dev)
    with sp.CSRMatrix(rp, ci, va, A.n) as M:
        c0 = sp.launch_count()
        for _ in range(5):
            M.spmv(x, y)
        assert sp.launch_count() - c0 == 5


@pytest.mark.parametrize("cls", ["B", "C"])
def test_nas_full_size(sp, torch_dev, cls):
    """BJ.cfg[1], BJ.cfg[3]: every row of the full-size matrix, in the launch
    configuration bench.py times (auto kernel)."""
    torch, dev = torch_dev
    A = gen.makea(cls)
    x = gen.uniform(A.n, seed=31)
    info = run_case(sp, torch, dev, A, x, what=f"NAS {cls}")
    assert info["kernel_name"] == "xplan", info  # the auto choice for NAS-shaped matrices


def test_parboil_full_size_fp32(sp, torch_dev):
    """BJ.cfg[2]: 1M rows, power-law row lengths, fp32."""
    torch, dev = torch_dev
    A = gen.powerlaw()
    x = gen.uniform(A.n, seed=41, f32=True)
    run_case(sp, torch, dev, A, x, what="parboil fp32")
    # sanity of the tolerance: the plain fp32 sequential loop also passes
    rp, ci, v = A.rowptr, A.colidx, A.vals
    rows = np.arange(0, A.m, 997)
    y_ref, bound = oracle.spmv(rp, ci, v, x)
    for i in rows:
        s = np.float32(0)
        for k in range(rp[i], rp[i + 1]):
            s = np.float32(s + np.float32(v[k] * x[ci[k]]))
        assert abs(float(s) - y_ref[i]) <= 1e-5 * bound[i]


def _sample_rows(A, rows):
    """Sub-CSR of the given rows (same columns) for per-row oracle checks."""
    lens = (A.rowptr[rows + 1] - A.rowptr[rows]).astype(np.int64)
    rp = np.concatenate([[0], np.cumsum(lens)]).astype(np.int32)
    idx = np.concatenate([np.arange(A.rowptr[i], A.rowptr[i + 1]) for i in rows])
    return gen.CSR(len(rows), A.n, rp, A.colidx[idx], A.vals[idx])


@pytest.fixture(scope="module")
def stencil256():
    return gen.stencil27(256)


@pytest.mark.parametrize("kernel", ["auto", "vector"])
def test_stencil256_full_size(sp, torch_dev, stencil256, kernel):  # auto = the SELL plan
    """BJ.cfg[4] at full size (16.8M rows, 449,455,096 nnz, fp64), in the launch
    configuration bench/sweep time: (1) A*1 = 27 - cnt_i on EVERY row, exact
    (R19: centre 26, neighbours -1; all partial sums are small integers);
    (2) a random x on 4096 sampled rows (every boundary class included) vs the
    oracle, per-row tolerance."""
    torch, dev = torch_dev
    A = stencil256
    N = 256
    assert A.nnz == (3 * N - 2) ** 3
    rp, ci, va = to_dev(A, dev)
    y = torch.empty(A.m, dtype=torch.float64, device=dev)
    ones = torch.ones(A.n, dtype=torch.float64, device=dev)
    with sp.CSRMatrix(rp, ci, va, A.n, kernel=kernel) as M:
        if kernel == "auto":
            assert M.info()["kernel_name"] == "sell"
        M.spmv(ones, y)
        torch.cuda.synchronize()
        yo = y.cpu().numpy()
        i = np.arange(A.m)
        xx, yy, zz = i % N, (i // N) % N, i // (N * N)
        cnt = 1
        for c in (xx, yy, zz):
            cnt = cnt * (3 - (c == 0) - (c == N - 1))
        assert np.array_equal(yo, (27 - cnt).astype(np.float64)), "A*1 closed form"
        x_h = gen.uniform(A.n, seed=77)
        M.spmv(torch.from_numpy(x_h).to(dev), y)
        torch.cuda.synchronize()
        rng = np.random.default_rng(5)
        rows = np.unique(np.concatenate([rng.integers(0, A.m, 4000), [0, N - 1, N * N - 1, A.m - 1,
                                                                       N * N * (N // 2) + N * (N // 2) + N // 2]]))
        S = _sample_rows(A, rows)
        y_ref, bound = oracle.spmv(S.rowptr, S.colidx, S.vals, x_h)
        check_rows(y[torch.from_numpy(rows).to(dev)].cpu().numpy(), y_ref, bound, np.float64, f"stencil256 {kernel}")


@pytest.mark.parametrize("cfg", [{}, {"SPMV_XSTAT_B": "2"}, {"SPMV_XSTAT_B": "8"},
                                 {"SPMV_XSTAT_G": "4"}, {"SPMV_XSTAT_G": "32", "SPMV_XSTAT_B": "3"},
                                 {"SPMV_XSTAT_CLUSTERS": "1"}])
@pytest.mark.parametrize("name,A", ZOO, ids=[c[0] for c in ZOO])
def test_zoo_xstat(sp, torch_dev, name, A, cfg, monkeypatch):
    """x-stationary cluster kernel (thread-block clusters + DSMEM reduction):
    every zoo case with sorted columns, several cluster sizes / lane groups /
    cluster counts (1 cluster = many row tiles, exercises the triple buffer)."""
    torch, dev = torch_dev
    for k, v in cfg.items():
        monkeypatch.setenv(k, v)
    x = gen.uniform(A.n, seed=13)
    info = run_case(sp, torch, dev, A, x, kernel="xstat", what=f"{name} xstat {cfg}")
    k = np.arange(A.rowptr[0] + 1, A.rowptr[-1])
    starts = np.zeros(A.colidx.shape[0] + 1, bool)
    starts[A.rowptr[:-1]] = True
    inner = ~starts[k]
    sorted_cols = bool(np.all(A.colidx[k][inner] > A.colidx[k - 1][inner]))
    if sorted_cols and A.m > 0:
        assert info["kernel_name"] == "xstat", info
    A32 = A.astype(np.float32)
    run_case(sp, torch, dev, A32, gen.uniform(A.n, seed=14, f32=True), kernel="xstat",
             what=f"{name} xstat fp32 {cfg}")


def test_xstat_alpha_beta_and_offset(sp, torch_dev):
    torch, dev = torch_dev
    A = gen.makea("W")
    x = gen.uniform(A.n, seed=15)
    y0 = gen.uniform(A.m, seed=16)
    for a, b in [(2.0, -1.0), (0.0, 3.0), (1.0, 0.0)]:
        run_case(sp, torch, dev, A, x, alpha=a, beta=b, y0=y0, kernel="xstat", what=f"xstat a={a} b={b}")


@pytest.mark.parametrize("cfg", [{}, {"SPMV_XPLAN_B": "2"}, {"SPMV_XPLAN_B": "4"}, {"SPMV_XPLAN_B": "8"},
                                 {"SPMV_XPLAN_CLUSTERS": "1"}, {"SPMV_XPLAN_CLUSTERS": "3", "SPMV_XPLAN_B": "2"},
                                 {"SPMV_XPLAN_DYN": "1"}, {"SPMV_XPLAN_DYN": "1", "SPMV_XPLAN_CLUSTERS": "2"}])
@pytest.mark.parametrize("name,A", ZOO, ids=[c[0] for c in ZOO])
def test_zoo_xplan(sp, torch_dev, name, A, cfg, monkeypatch):
    """x-stationary kernel over the column-blocked SELL-32 plan (clusters,
    st.async partials to the owning CTA, mbarrier transaction counts):
    cluster sizes and few clusters (many tiles per cluster: exercises the
    triple-buffered receive arrays and the split barrier).  Skewed matrices
    whose SELL padding would exceed 1.5x fall back to the zero-copy kernel."""
    torch, dev = torch_dev
    for k, v in cfg.items():
        monkeypatch.setenv(k, v)
    x = gen.uniform(A.n, seed=17)
    info = run_case(sp, torch, dev, A, x, kernel="xplan", what=f"{name} xplan {cfg}")
    if name in ("laplace1d", "stencil27_9", "makea_S", "n1"):
        assert info["kernel_name"] == "xplan", info
        assert info["plan_bytes"] >= A.nnz * 10
    A32 = A.astype(np.float32)
    run_case(sp, torch, dev, A32, gen.uniform(A.n, seed=18, f32=True), kernel="xplan",
             what=f"{name} xplan fp32 {cfg}")


def test_xplan_alpha_beta_update_values(sp, torch_dev):
    torch, dev = torch_dev
    A = gen.makea("A")
    x_h = gen.uniform(A.n, seed=19)
    y0 = gen.uniform(A.m, seed=20)
    for a, b in [(2.0, -1.0), (0.0, 3.0), (1.0, 0.0), (-1.5, 1.0)]:
        info = run_case(sp, torch, dev, A, x_h, alpha=a, beta=b, y0=y0, kernel="xplan", what=f"xplan a={a} b={b}")
        assert info["kernel_name"] == "xplan"
    # in-place value change + update_values (the paper's lazy-copy flag)
    rp, ci, va = to_dev(A, dev)
    x = torch.from_numpy(x_h).to(dev)
    y = torch.empty(A.m, dtype=torch.float64, device=dev)
    with sp.CSRMatrix(rp, ci, va, A.n, kernel="xplan") as M:
        assert M.info()["kernel_name"] == "xplan"
        v2_h = gen.uniform(A.nnz, seed=23)
        va.copy_(torch.from_numpy(v2_h))
        M.update_values(va)
        M.spmv(x, y)
        torch.cuda.synchronize()
    y_ref, bound = oracle.spmv(A.rowptr, A.colidx, v2_h, x_h)
    check_rows(y.cpu().numpy(), y_ref, bound, np.float64, "xplan update_values")


def test_plan_off_uses_zero_copy(sp, torch_dev):
    torch, dev = torch_dev
    A = gen.makea("S")
    rp, ci, va = to_dev(A, dev)
    with sp.CSRMatrix(rp, ci, va, A.n, plan=False) as M:
        inf = M.info()
        assert inf["kernel_name"] == "vector" and inf["plan_bytes"] == 0


@pytest.mark.parametrize("name,A", ZOO, ids=[c[0] for c in ZOO])
def test_zoo_merge(sp, torch_dev, name, A):
    """Merge-path kernel (equal rows+nnz tiles, segmented-scan carries,
    tile-order fix-up of rows spanning tiles) on every zoo case, fp64 and fp32,
    and its device splits equal the host/oracle splits bit for bit (R21)."""
    torch, dev = torch_dev
    x = gen.uniform(A.n, seed=19)
    info = run_case(sp, torch, dev, A, x, kernel="merge", what=f"{name} merge")
    if A.m > 0:
        assert info["kernel_name"] == "merge"
        rp, ci, va = to_dev(A, dev)
        with sp.CSRMatrix(rp, ci, va, A.n, kernel="merge") as M:
            sr, sn = M.merge_splits_device()
        C = len(sr) - 1
        orr, onz = oracle.merge_path(A.rowptr, C)
        assert np.array_equal(sr, orr) and np.array_equal(sn, onz)
    A32 = A.astype(np.float32)
    run_case(sp, torch, dev, A32, gen.uniform(A.n, seed=20, f32=True), kernel="merge", what=f"{name} merge fp32")
    y0 = gen.uniform(A.m, seed=21)
    run_case(sp, torch, dev, A, x, alpha=-2.0, beta=0.5, y0=y0, kernel="merge", what=f"{name} merge a/b")


@pytest.mark.parametrize("name,A", ZOO, ids=[c[0] for c in ZOO])
def test_zoo_sell(sp, torch_dev, name, A):
    """SELL-32 plan with global x gathers (forced: any padding), fp64 and fp32,
    alpha/beta with NaN in y_old, and the zero-copy fallback for a per-call
    vals pointer."""
    torch, dev = torch_dev
    x = gen.uniform(A.n, seed=25)
    info = run_case(sp, torch, dev, A, x, kernel="sell", what=f"{name} sell")
    if A.m > 0 and A.nnz > 0:
        assert info["kernel_name"] == "sell" and info["plan_bytes"] >= A.nnz * 12
    A32 = A.astype(np.float32)
    run_case(sp, torch, dev, A32, gen.uniform(A.n, seed=26, f32=True), kernel="sell", what=f"{name} sell fp32")
    y0 = gen.uniform(A.m, seed=27)
    run_case(sp, torch, dev, A, x, alpha=-2.0, beta=0.5, y0=y0, kernel="sell", what=f"{name} sell a/b")
    run_case(sp, torch, dev, A, x, alpha=0.0, beta=2.0, y0=y0, kernel="sell", what=f"{name} sell a=0")


def test_sell_auto_update_values_and_vals_override(sp, torch_dev):
    """auto + plan picks SELL for the 27-point stencil at N=96 (x = 7 MB,
    beyond the shared memory of a 16-CTA cluster); then in-place values +
    update_values, and a different vals pointer (zero-copy path)."""
    torch, dev = torch_dev
    A = gen.stencil27(96)
    x_h = gen.uniform(A.n, seed=28)
    info = run_case(sp, torch, dev, A, x_h, what="stencil64 auto")
    assert info["kernel_name"] == "sell", info
    rp, ci, va = to_dev(A, dev)
    x = torch.from_numpy(x_h).to(dev)
    y = torch.empty(A.m, dtype=torch.float64, device=dev)
    v2_h = gen.uniform(A.nnz, seed=29)
    with sp.CSRMatrix(rp, ci, va, A.n) as M:
        va.copy_(torch.from_numpy(v2_h))
        M.update_values(va)
        M.spmv(x, y)
        torch.cuda.synchronize()
        y_ref, bound = oracle.spmv(A.rowptr, A.colidx, v2_h, x_h)
        check_rows(y.cpu().numpy(), y_ref, bound, np.float64, "sell update_values")
        v3 = torch.from_numpy(gen.uniform(A.nnz, seed=30)).to(dev)
        M.spmv(x, y, vals=v3)
        torch.cuda.synchronize()
        y_ref, bound = oracle.spmv(A.rowptr, A.colidx, v3.cpu().numpy(), x_h)
        check_rows(y.cpu().numpy(), y_ref, bound, np.float64, "sell vals override")


def test_parboil_auto_kernels(sp, torch_dev):
    """BJ.cfg[2] (power law, fp32): auto picks the length-sorted SELL plan, and
    the merge path without a plan; both every row against the oracle."""
    torch, dev = torch_dev
    A = gen.powerlaw()
    x = gen.uniform(A.n, seed=42, f32=True)
    info = run_case(sp, torch, dev, A, x, what="parboil auto")
    assert info["kernel_name"] == "sellsort"
    rp, ci, va = to_dev(A, dev)
    with sp.CSRMatrix(rp, ci, va, A.n, plan=False) as M:
        assert M.info()["kernel_name"] == "merge"


@pytest.mark.parametrize("name,A", ZOO, ids=[c[0] for c in ZOO])
def test_zoo_sellsort(sp, torch_dev, name, A):
    """Length-sorted SELL (forced: any padding), long rows (> 64) warp-per-row
    from the CSR, y through the permutation: fp64, fp32, alpha/beta."""
    torch, dev = torch_dev
    x = gen.uniform(A.n, seed=31)
    info = run_case(sp, torch, dev, A, x, kernel="sellsort", what=f"{name} sellsort")
    if A.m > 0 and A.nnz > 0:
        assert info["kernel_name"] == "sellsort"
    A32 = A.astype(np.float32)
    run_case(sp, torch, dev, A32, gen.uniform(A.n, seed=32, f32=True), kernel="sellsort",
             what=f"{name} sellsort fp32")
    y0 = gen.uniform(A.m, seed=33)
    run_case(sp, torch, dev, A, x, alpha=1.5, beta=-0.5, y0=y0, kernel="sellsort", what=f"{name} sellsort a/b")


def test_sellsort_update_values(sp, torch_dev):
    torch, dev = torch_dev
    A = gen.powerlaw(m=50000, lmax=5000.0, seed=9, f32=False)
    x_h = gen.uniform(A.n, seed=34)
    rp, ci, va = to_dev(A, dev)
    y = torch.empty(A.m, dtype=torch.float64, device=dev)
    v2_h = gen.uniform(A.nnz, seed=35)
    with sp.CSRMatrix(rp, ci, va, A.n, kernel="sellsort") as M:
        assert M.info()["kernel_name"] == "sellsort"
        va.copy_(torch.from_numpy(v2_h))
        M.update_values(va)
        M.spmv(torch.from_numpy(x_h).to(dev), y)
        torch.cuda.synchronize()
    y_ref, bound = oracle.spmv(A.rowptr, A.colidx, v2_h, x_h)
    check_rows(y.cpu().numpy(), y_ref, bound, np.float64, "sellsort update_values")


@pytest.mark.parametrize("kernel", ["vector", "merge", "sell", "sellsort", "auto"])
@pytest.mark.parametrize("name", ["powerlaw_small", "makea_S", "stencil27_9"])
def test_l2_window_parity(sp, torch_dev, kernel, name):
    """opts.l2_window (the persisting L2 window over x, BJ.ns) changes caching
    only: results stay within the per-row bound (and equal the no-window run
    bit for bit -- same kernel, same summation order), fp64 and fp32."""
    torch, dev = torch_dev
    A = dict(ZOO)[name]
    for f32 in (False, True):
        B = A.astype(np.float32) if f32 else A
        tdt = torch.float32 if f32 else torch.float64
        x_h = gen.uniform(A.n, seed=61, f32=f32)
        rp, ci, va = to_dev(B, dev)
        x = torch.from_numpy(x_h).to(dev)
        ys = []
        for win in (False, True):
            y = torch.full((A.m,), float("nan"), dtype=tdt, device=dev)
            with sp.CSRMatrix(rp, ci, va, A.n, kernel=kernel, l2_window=win) as M:
                M.spmv(x, y)
                torch.cuda.synchronize()
            ys.append(y.cpu().numpy())
        y_ref, bound = oracle.spmv(B.rowptr, B.colidx, B.vals, x_h)
        check_rows(ys[1], y_ref, bound, B.vals.dtype, f"{name} {kernel} l2_window f32={f32}")
        assert np.array_equal(ys[0].view(np.uint8), ys[1].view(np.uint8))


@pytest.mark.parametrize("perm", ["0", "1"])
@pytest.mark.parametrize("f32", [False, True])
def test_xplan_bankperm(sp, torch_dev, perm, f32, monkeypatch):
    """k_xplan_bankperm: the per-row step order of the plan is
    re-arranged for shared-memory banks.  Parity with and without it, bit-identical
    results from two independent creates (the permutation is deterministic), and
    update_values twice in a row (each re-pack restores the pads, then re-permutes)."""
    torch, dev = torch_dev
    monkeypatch.setenv("SPMV_XPLAN_PERM", perm)
    A = gen.makea("W")
    if f32:
        A = A.astype(np.float32)
    x_h = gen.uniform(A.n, seed=41, f32=f32)
    rp, ci, va = to_dev(A, dev)
    x = torch.from_numpy(x_h).to(dev)
    ys = []
    for _ in range(2):
        y = torch.empty(A.m, dtype=va.dtype, device=dev)
        with sp.CSRMatrix(rp, ci, va, A.n, kernel="xplan") as M:
            assert M.info()["kernel_name"] == "xplan"
            M.spmv(x, y)
            torch.cuda.synchronize()
        ys.append(y.cpu().numpy())
    assert np.array_equal(ys[0].view(np.uint8), ys[1].view(np.uint8))
    y_ref, bound = oracle.spmv(A.rowptr, A.colidx, A.vals, x_h)
    check_rows(ys[0], y_ref, bound, A.vals.dtype, f"bankperm={perm}")
    y = torch.empty(A.m, dtype=va.dtype, device=dev)
    with sp.CSRMatrix(rp, ci, va, A.n, kernel="xplan") as M:
        for seed in (42, 43):
            v_h = gen.uniform(A.nnz, seed=seed, f32=f32)
            va.copy_(torch.from_numpy(v_h))
            M.update_values(va)
            M.spmv(x, y)
            torch.cuda.synchronize()
            y_ref, bound = oracle.spmv(A.rowptr, A.colidx, v_h, x_h)
            check_rows(y.cpu().numpy(), y_ref, bound, A.vals.dtype, f"bankperm={perm} update_values {seed}")
        # the re-packed plan equals a fresh one: same bits as a new handle on the same values
        y2 = torch.empty_like(y)
        with sp.CSRMatrix(rp, ci, va, A.n, kernel="xplan") as M2:
            M2.spmv(x, y2)
            torch.cuda.synchronize()
        assert torch.equal(y, y2)
