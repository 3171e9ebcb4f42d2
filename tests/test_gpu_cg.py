"""GPU CG parity (cg_solve, cg_npb_outer) through the C ABI: the 1-D Laplacian
closed form, the oracle's iterates, and the published NPB zeta values for
classes S..C within 1e-10 (BJ.cfg[0], BJ.cfg[3])."""
import numpy as np
import pytest

import gen
import oracle
from gpu_util import to_dev

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def torch_dev():
    import torch
    return torch, torch.device("cuda:0")


@pytest.fixture(scope="module")
def sp():
    import paper_conf_asplos_ginsbachrsbdo18_b200 as sp
    return sp


@pytest.mark.parametrize("n", [1, 5, 16, 64])
def test_cg_laplace1d_closed_form(sp, torch_dev, n):
    torch, dev = torch_dev
    A = gen.laplace1d(n)
    rp, ci, va = to_dev(A, dev)
    b = torch.ones(n, dtype=torch.float64, device=dev)
    x = torch.empty(n, dtype=torch.float64, device=dev)
    with sp.CSRMatrix(rp, ci, va, n) as M:
        its, rn = M.cg_solve(b, x, max_iter=n, tol=1e-14)
    j = np.arange(n)
    ref = (j + 1) * (n - j) / 2.0
    assert np.allclose(x.cpu().numpy(), ref, rtol=1e-10, atol=0)
    assert 1 <= its <= n


def test_cg_matches_oracle_iterates(sp, torch_dev):
    torch, dev = torch_dev
    A = gen.makea("S")
    rp, ci, va = to_dev(A, dev)
    b_h = gen.uniform(A.n, seed=3)
    b = torch.from_numpy(b_h).to(dev)
    x = torch.empty_like(b)
    with sp.CSRMatrix(rp, ci, va, A.n) as M:
        for k in (1, 2, 7, 25):
            its, rn = M.cg_solve(b, x, max_iter=k)
            z_ref, its_ref, rn_ref, st = oracle.cg(A.rowptr, A.colidx, A.vals, b_h, k)
            assert its == its_ref == k
            assert np.allclose(x.cpu().numpy(), z_ref, rtol=1e-10, atol=1e-13)
            assert abs(rn - rn_ref) <= 1e-9 * max(rn_ref, 1e-300) + 1e-14


def test_cg_host_buffers_equal_device(sp, torch_dev):
    """The staged host-pointer path computes exactly the device path."""
    torch, dev = torch_dev
    A = gen.makea("S")
    rp, ci, va = to_dev(A, dev)
    b_h = gen.uniform(A.n, seed=4)
    with sp.CSRMatrix(rp, ci, va, A.n) as M:
        xd = torch.empty(A.n, dtype=torch.float64, device=dev)
        M.cg_solve(torch.from_numpy(b_h).to(dev), xd, 10)
        xh = torch.empty(A.n, dtype=torch.float64).pin_memory()
        M.cg_solve(torch.from_numpy(b_h).pin_memory(), xh, 10)
        xp = np.empty(A.n)
        M.cg_solve(b_h, xp, 10)  # pageable numpy
    assert np.array_equal(xd.cpu().numpy(), xh.numpy())
    assert np.array_equal(xd.cpu().numpy(), xp)


def test_cg_tol_early_stop(sp, torch_dev):
    torch, dev = torch_dev
    A = gen.laplace1d(200)
    rp, ci, va = to_dev(A, dev)
    b = torch.ones(200, dtype=torch.float64, device=dev)
    x = torch.empty_like(b)
    with sp.CSRMatrix(rp, ci, va, 200) as M:
        its, rn = M.cg_solve(b, x, max_iter=1000, tol=1e-10)
    z, its_ref, rn_ref, st = oracle.cg(A.rowptr, A.colidx, A.vals, np.ones(200), 1000, 1e-10)
    assert abs(its - its_ref) <= 1 and its < 1000
    assert rn <= 1e-8 * np.sqrt(200) * 5050


def test_cg_breakdown(sp, torch_dev):
    torch, dev = torch_dev
    A = gen.laplace1d(8)
    rp, ci, va = to_dev(A, dev)
    b = torch.zeros(8, dtype=torch.float64, device=dev)
    x = torch.empty_like(b)
    with sp.CSRMatrix(rp, ci, va, 8) as M:
        with pytest.raises(sp.SpmvError) as e:
            M.cg_solve(b, x, 3)
        assert e.value.status == sp.SPMV_ERR_BREAKDOWN


def test_npb_host_z_equals_device_z(sp, torch_dev):
    """The host copy of z (made on a side stream after an event inside the NPB
    graph, overlapping the residual) equals the device-path z bit for bit."""
    torch, dev = torch_dev
    A = gen.makea("S")
    rp, ci, va = to_dev(A, dev)
    with sp.CSRMatrix(rp, ci, va, A.n) as M:
        xd = torch.ones(A.n, dtype=torch.float64, device=dev)
        zd = torch.empty_like(xd)
        od = torch.zeros(2, dtype=torch.float64, device=dev)
        xh = torch.ones(A.n, dtype=torch.float64).pin_memory()
        zh = torch.empty(A.n, dtype=torch.float64).pin_memory()
        oh = torch.zeros(2, dtype=torch.float64).pin_memory()
        for it in range(4):
            M.npb_outer(xd, zd, 25, 10.0, od)
            M.npb_outer(xh, zh, 25, 10.0, oh)
            torch.cuda.synchronize()
            assert torch.equal(zd.cpu(), zh) and torch.equal(xd.cpu(), xh), it
            assert torch.equal(od.cpu(), oh)


def test_npb_host_graph_replay(sp, torch_dev):
    """Several host-buffer calls in a row on ONE handle replay the same captured
    graph (the side-stream z copy waits on the external event of the earlier
    capture): every call's host z, x and {zeta, rnorm} equal a device-buffer run
    on a second handle bit for bit."""
    torch, dev = torch_dev
    A = gen.makea("S")
    rp, ci, va = to_dev(A, dev)
    with sp.CSRMatrix(rp, ci, va, A.n) as Mh, sp.CSRMatrix(rp, ci, va, A.n) as Md:
        xd = torch.ones(A.n, dtype=torch.float64, device=dev)
        zd = torch.empty_like(xd)
        od = torch.zeros(2, dtype=torch.float64, device=dev)
        xh = torch.ones(A.n, dtype=torch.float64).pin_memory()
        zh = torch.empty(A.n, dtype=torch.float64).pin_memory()
        oh = torch.zeros(2, dtype=torch.float64).pin_memory()
        for it in range(5):
            zh.fill_(float("nan"))  # a stale or missing copy shows
            Mh.npb_outer(xh, zh, 25, 10.0, oh)  # synchronous (host buffers)
            Md.npb_outer(xd, zd, 25, 10.0, od)
            torch.cuda.synchronize()
            assert torch.equal(zd.cpu(), zh) and torch.equal(xd.cpu(), xh), it
            assert torch.equal(od.cpu(), oh), it


def _npb(sp, torch, dev, cls, niter=None, host=False):
    na, nonzer, NITER, shift = gen.NPB_CLASSES[cls]
    A = gen.makea(cls)
    rp, ci, va = to_dev(A, dev)
    niter = NITER if niter is None else niter
    zetas, rnorms = [], []
    with sp.CSRMatrix(rp, ci, va, A.n) as M:
        if host:
            x = np.ones(A.n)
            z = np.empty(A.n)
            out2 = np.zeros(2)
            for _ in range(niter):
                M.npb_outer(x, z, gen.NPB_CGITMAX, shift, out2)
                zetas.append(out2[0]); rnorms.append(out2[1])
        else:
            x = torch.ones(A.n, dtype=torch.float64, device=dev)
            z = torch.empty_like(x)
            out = torch.zeros((niter, 2), dtype=torch.float64, device=dev)
            for it in range(niter):
                M.npb_outer(x, z, gen.NPB_CGITMAX, shift, out[it])
            M.cg_status()
            o = out.cpu().numpy()
            zetas, rnorms = list(o[:, 0]), list(o[:, 1])
    return A, np.array(zetas), np.array(rnorms)


@pytest.mark.parametrize("cls", ["S", "W", "A", "B", "C"])
def test_npb_zeta_published(sp, torch_dev, cls):
    torch, dev = torch_dev
    A, zetas, rnorms = _npb(sp, torch, dev, cls)
    ref = gen.NPB_ZETA[cls]
    assert abs(zetas[-1] - ref) / ref <= 1e-10, (zetas[-1], ref)
    assert rnorms.max() <= 1e-11


@pytest.mark.parametrize("cls", ["S", "W", "A"])
def test_npb_matches_oracle_each_iteration(sp, torch_dev, cls):
    torch, dev = torch_dev
    A, zetas, rnorms = _npb(sp, torch, dev, cls)
    zr, rr = oracle.npb_run(A.rowptr, A.colidx, A.vals, gen.NPB_CLASSES[cls][2], gen.NPB_CLASSES[cls][3])
    assert np.allclose(zetas, zr, rtol=1e-11, atol=0)


def test_npb_host_path_bitexact(sp, torch_dev):
    torch, dev = torch_dev
    _, zd, rd = _npb(sp, torch, dev, "S", niter=4)
    _, zh, rh = _npb(sp, torch, dev, "S", niter=4, host=True)
    assert np.array_equal(zd, zh) and np.array_equal(rd, rh)


def test_npb_graph_vs_eager_bitexact(sp, torch_dev, monkeypatch):
    torch, dev = torch_dev
    _, z1, r1 = _npb(sp, torch, dev, "S", niter=3)
    monkeypatch.setenv("SPMV_GRAPH", "0")
    _, z2, r2 = _npb(sp, torch, dev, "S", niter=3)
    assert np.array_equal(z1, z2) and np.array_equal(r1, r2)


@pytest.mark.parametrize("kernel", ["merge", "vector", "xstat", "xplan", "sell", "sellsort", "xt", "xplan_dyn"])
def test_npb_s_every_kernel(sp, torch_dev, kernel, monkeypatch):
    """NPB class S zeta with every SpMV kernel inside CG (fused or separate dot)."""
    torch, dev = torch_dev
    na, nonzer, niter, shift = gen.NPB_CLASSES["S"]
    A = gen.makea("S")
    rp, ci, va = to_dev(A, dev)
    if kernel == "xplan_dyn":  # XPLAN with dynamic tile scheduling (per-tile dot partials)
        monkeypatch.setenv("SPMV_XPLAN_DYN", "1")
        kernel = "xplan"
    with sp.CSRMatrix(rp, ci, va, A.n, kernel=kernel) as M:
        assert M.info()["kernel_name"] == kernel
        x = torch.ones(A.n, dtype=torch.float64, device=dev)
        z = torch.empty_like(x)
        out = torch.zeros(2, dtype=torch.float64, device=dev)
        for _ in range(niter):
            M.npb_outer(x, z, 25, shift, out)
        zeta = float(out[0].item())
    assert abs(zeta - gen.NPB_ZETA["S"]) / gen.NPB_ZETA["S"] <= 1e-10


def test_cg_sellsort_multisegment_rows(sp, torch_dev):
    """Length-sorted SELL with rows split into several warp segments (arrowhead
    matrix: dense first row/column of 3000 entries): CG iterates match the
    oracle, and two identical solves are bit-identical (the separate dot pass
    keeps the scalars deterministic although segment completion order varies)."""
    torch, dev = torch_dev
    n = 3000
    rows = np.concatenate([np.zeros(n, np.int64), np.arange(1, n), np.arange(1, n)])
    cols = np.concatenate([np.arange(n), np.zeros(n - 1, np.int64), np.arange(1, n)])
    vals = np.concatenate([np.full(n, 0.5), np.full(n - 1, 0.5), np.full(n - 1, 4.0)])
    vals[0] = float(n)  # A[0,0]: diagonally dominant -> SPD
    A = gen.from_coo(n, n, rows, cols, vals)
    rp, ci, va = to_dev(A, dev)
    b_h = gen.uniform(n, seed=12)
    b = torch.from_numpy(b_h).to(dev)
    xs = []
    with sp.CSRMatrix(rp, ci, va, n, kernel="sellsort") as M:
        assert M.info()["kernel_name"] == "sellsort"
        for _ in range(2):
            x = torch.empty_like(b)
            its, rn = M.cg_solve(b, x, max_iter=20)
            xs.append(x.cpu().numpy())
    z_ref, its_ref, rn_ref, st = oracle.cg(A.rowptr, A.colidx, A.vals, b_h, 20)
    assert np.allclose(xs[0], z_ref, rtol=1e-10, atol=1e-13)
    assert np.array_equal(xs[0], xs[1])
