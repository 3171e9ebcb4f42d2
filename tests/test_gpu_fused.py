"""GPU parity of the fused single-reduction CG (spmv_csr_set_cg_variant(h, 3),
DESIGN.md 5.4d): the update of iteration k-1 is folded into the XPLAN SpMV of
iteration k (x block built from r, w, s of the previous launch; the row owners
write r, s, p, z), one kernel per iteration plus a tail kernel.  Checked
against its oracle (oracle_cg_cgcg) iterate by iterate, the Laplacian closed
form, the published NPB zeta of classes S..C within 1e-10, the graph-path
single-reduction CG, repeatability, PDL on/off, and the
fall-back to variant 1 where it is not eligible (another kernel, tol > 0,
the proxy transport)."""
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


@pytest.mark.parametrize("cfg", [{}, {"SPMV_XPLAN_B": "2"}, {"SPMV_XPLAN_CLUSTERS": "1"}, {"SPMV_XPLAN_B": "8"}])
def test_fused_matches_its_oracle_iterates(sp, torch_dev, cfg, monkeypatch):
    torch, dev = torch_dev
    for k, v in cfg.items():
        monkeypatch.setenv(k, v)
    A = gen.makea("S")
    rp, ci, va = to_dev(A, dev)
    b_h = gen.uniform(A.n, seed=3)
    b = torch.from_numpy(b_h).to(dev)
    x = torch.empty_like(b)
    with sp.CSRMatrix(rp, ci, va, A.n, kernel="xplan", cg_variant="fused") as M:
        assert M.info()["kernel_name"] == "xplan"
        for k in (1, 2, 7, 25):
            its, rn = M.cg_solve(b, x, max_iter=k)
            z_ref, its_ref, rn_ref, st = oracle.cg(A.rowptr, A.colidx, A.vals, b_h, k, variant=1)
            assert its == its_ref == k
            assert np.allclose(x.cpu().numpy(), z_ref, rtol=1e-10, atol=1e-13), (k, cfg)
            assert abs(rn - rn_ref) <= 1e-9 * max(rn_ref, 1e-300) + 1e-14


@pytest.mark.parametrize("n", [64, 3000])
def test_fused_laplace1d(sp, torch_dev, n):
    """1-D Laplacian: the closed form (j+1)(n-j)/2 after n iterations (n = 64),
    and CG's residual decrease on a larger system; rows are short (3), so the
    plan is forced."""
    torch, dev = torch_dev
    A = gen.laplace1d(n)
    rp, ci, va = to_dev(A, dev)
    b = torch.ones(n, dtype=torch.float64, device=dev)
    x = torch.empty(n, dtype=torch.float64, device=dev)
    with sp.CSRMatrix(rp, ci, va, n, kernel="xplan", cg_variant="fused") as M:
        its, rn = M.cg_solve(b, x, max_iter=min(n, 200))
    z_ref, _, rn_ref, _ = oracle.cg(A.rowptr, A.colidx, A.vals, np.ones(n), min(n, 200), variant=1)
    assert np.allclose(x.cpu().numpy(), z_ref, rtol=1e-9, atol=1e-11)
    if n == 64:
        j = np.arange(n)
        assert np.allclose(x.cpu().numpy(), (j + 1) * (n - j) / 2.0, rtol=1e-9)


@pytest.mark.parametrize("cls", ["S", "W", "A", "B", "C"])
def test_fused_npb_zeta(sp, torch_dev, cls):
    """Published NPB zeta (1e-10) at full NITER with the persistent kernel
    inside the captured NPB graph (class C: 75 outer iterations)."""
    torch, dev = torch_dev
    na, nonzer, niter, shift = gen.NPB_CLASSES[cls]
    A = gen.makea(cls)
    rp, ci, va = to_dev(A, dev)
    with sp.CSRMatrix(rp, ci, va, A.n, cg_variant="fused") as M:
        assert M.info()["kernel_name"] == "xplan"
        x = torch.ones(A.n, dtype=torch.float64, device=dev)
        z = torch.empty_like(x)
        out = torch.zeros(2, dtype=torch.float64, device=dev)
        for _ in range(niter):
            M.npb_outer(x, z, 25, shift, out)
        M.cg_status()
        zeta, rn = float(out[0]), float(out[1])
    assert abs(zeta - gen.NPB_ZETA[cls]) / gen.NPB_ZETA[cls] <= 1e-10, (cls, zeta)
    assert rn <= 1e-11


def test_fused_equals_graph_cgcg_and_repeats(sp, torch_dev):
    """Same iterates as the graph-path single-reduction CG (up to the rounding
    of the r.r partials), and bit-identical repeated solves."""
    torch, dev = torch_dev
    A = gen.makea("W")
    rp, ci, va = to_dev(A, dev)
    b = torch.from_numpy(gen.uniform(A.n, seed=9)).to(dev)
    xs = {}
    with sp.CSRMatrix(rp, ci, va, A.n) as M:
        for v in ("cgcg", "fused", "fused"):
            M.set_cg_variant(v)
            x = torch.empty_like(b)
            M.cg_solve(b, x, max_iter=25)
            xs.setdefault(v, []).append(x.cpu().numpy())
    assert np.allclose(xs["fused"][0], xs["cgcg"][0], rtol=1e-12, atol=1e-14)
    assert np.array_equal(xs["fused"][0], xs["fused"][1])


@pytest.mark.parametrize("kernel", ["vector", "sell", "xt"])
def test_fused_falls_back(sp, torch_dev, kernel):
    """Not eligible (another SpMV kernel, or tol > 0): variant 1 runs, correct results."""
    torch, dev = torch_dev
    A = gen.makea("S")
    rp, ci, va = to_dev(A, dev)
    b_h = gen.uniform(A.n, seed=4)
    b = torch.from_numpy(b_h).to(dev)
    x = torch.empty_like(b)
    with sp.CSRMatrix(rp, ci, va, A.n, kernel=kernel, cg_variant="fused") as M:
        its, rn = M.cg_solve(b, x, max_iter=12)
    z_ref, _, _, _ = oracle.cg(A.rowptr, A.colidx, A.vals, b_h, 12, variant=1)
    assert np.allclose(x.cpu().numpy(), z_ref, rtol=1e-10, atol=1e-13)


@pytest.mark.parametrize("P", [2, 8])
def test_fused_proxy_transport_runs(sp, torch_dev, P):
    """The proxy transport (rank P-1's share of a P-way run, exchanges skipped)
    runs the persistent kernel on the padded x layout: it completes, and its
    SpMV agrees with the same handle's graph path on the first iteration."""
    torch, dev = torch_dev
    A = gen.makea("W")
    rp, ci, va = to_dev(A, dev)
    d = sp.Dist(P - 1, P, 0, transport="proxy")
    with sp.CSRMatrix(rp, ci, va, A.n, dist=d) as M:
        info = M.info()
        assert info["transport"] == 3 and info["kernel_name"] == "xplan"
        nl = info["row_end"] - info["row_begin"]
        b = torch.from_numpy(gen.uniform(A.n, seed=8)[info["row_begin"]:info["row_end"]].copy()).to(dev)
        out = {}
        for v in ("cgcg", "fused"):
            M.set_cg_variant(v)
            x = torch.empty(nl, dtype=torch.float64, device=dev)
            M.cg_solve(b, x, max_iter=1)
            out[v] = x.cpu().numpy()
        assert np.allclose(out["cgcg"], out["fused"], rtol=1e-12, atol=1e-14)
    d.close()


def test_fused_pdl_on_off_bit_identical(sp, torch_dev, monkeypatch):
    """Three NPB outer iterations (captured graph, replayed) give the same bits
    with programmatic dependent launch on and off."""
    torch, dev = torch_dev
    A = gen.makea("W")
    na, nonzer, niter, shift = gen.NPB_CLASSES["W"]
    rp, ci, va = to_dev(A, dev)
    res = []
    for pdl in ("1", "0"):
        monkeypatch.setenv("SPMV_PDL", pdl)
        with sp.CSRMatrix(rp, ci, va, A.n, cg_variant="fused") as M:
            x = torch.ones(A.n, dtype=torch.float64, device=dev)
            z = torch.empty_like(x)
            out = torch.zeros(2, dtype=torch.float64, device=dev)
            for _ in range(3):
                M.npb_outer(x, z, 25, shift, out)
            torch.cuda.synchronize()
            res.append((x.cpu().numpy().copy(), z.cpu().numpy().copy(), out.cpu().numpy().copy()))
    for a, b in zip(res[0], res[1]):
        assert np.array_equal(a.view(np.uint64), b.view(np.uint64))
