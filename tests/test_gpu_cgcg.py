"""GPU parity of the single-reduction CG (Chronopoulos & Gear, SURVEY 8(f)
NEXT-1; spmv_csr_set_cg_variant(h, 1)) through the C ABI: its own oracle
(oracle_cg_cgcg) iterate by iterate, the Laplacian closed form, the published
NPB zeta of classes S..C within 1e-10, bit-exactness of graph vs eager and of
the distributed 1-rank transports, and switching variants on one handle."""
import os
import socket

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
def test_cgcg_laplace1d_closed_form(sp, torch_dev, n):
    torch, dev = torch_dev
    A = gen.laplace1d(n)
    rp, ci, va = to_dev(A, dev)
    b = torch.ones(n, dtype=torch.float64, device=dev)
    x = torch.empty(n, dtype=torch.float64, device=dev)
    with sp.CSRMatrix(rp, ci, va, n, cg_variant="cgcg") as M:
        its, rn = M.cg_solve(b, x, max_iter=n, tol=1e-14)
    j = np.arange(n)
    assert np.allclose(x.cpu().numpy(), (j + 1) * (n - j) / 2.0, rtol=1e-10, atol=0)
    assert 1 <= its <= n


@pytest.mark.parametrize("kernel", ["auto", "vector", "sellsort"])
def test_cgcg_matches_its_oracle_iterates(sp, torch_dev, kernel):
    torch, dev = torch_dev
    A = gen.makea("S")
    rp, ci, va = to_dev(A, dev)
    b_h = gen.uniform(A.n, seed=3)
    b = torch.from_numpy(b_h).to(dev)
    x = torch.empty_like(b)
    with sp.CSRMatrix(rp, ci, va, A.n, kernel=kernel, cg_variant="cgcg") as M:
        for k in (1, 2, 7, 25):
            its, rn = M.cg_solve(b, x, max_iter=k)
            z_ref, its_ref, rn_ref, st = oracle.cg(A.rowptr, A.colidx, A.vals, b_h, k, variant=1)
            assert its == its_ref == k
            assert np.allclose(x.cpu().numpy(), z_ref, rtol=1e-10, atol=1e-13)
            assert abs(rn - rn_ref) <= 1e-9 * max(rn_ref, 1e-300) + 1e-14


def test_cgcg_tol_early_stop_and_breakdown(sp, torch_dev):
    torch, dev = torch_dev
    A = gen.laplace1d(200)
    rp, ci, va = to_dev(A, dev)
    b = torch.ones(200, dtype=torch.float64, device=dev)
    x = torch.empty_like(b)
    with sp.CSRMatrix(rp, ci, va, 200, cg_variant="cgcg") as M:
        its, rn = M.cg_solve(b, x, max_iter=1000, tol=1e-10)
        z, its_ref, rn_ref, st = oracle.cg(A.rowptr, A.colidx, A.vals, np.ones(200), 1000, 1e-10, variant=1)
        assert abs(its - its_ref) <= 1 and its < 1000
        assert rn <= 1e-8 * np.sqrt(200) * 5050
        with pytest.raises(sp.SpmvError) as e:
            M.cg_solve(torch.zeros_like(b), x, 3)
        assert e.value.status == sp.SPMV_ERR_BREAKDOWN


def _npb(sp, torch, dev, cls, niter=None, variant="cgcg", dist=None):
    na, nonzer, NITER, shift = gen.NPB_CLASSES[cls]
    A = gen.makea(cls)
    rp, ci, va = to_dev(A, dev)
    niter = NITER if niter is None else niter
    with sp.CSRMatrix(rp, ci, va, A.n, cg_variant=variant, dist=dist) as M:
        x = torch.ones(A.n, dtype=torch.float64, device=dev)
        z = torch.empty_like(x)
        out = torch.zeros((niter, 2), dtype=torch.float64, device=dev)
        for it in range(niter):
            M.npb_outer(x, z, gen.NPB_CGITMAX, shift, out[it])
        M.cg_status()
        o = out.cpu().numpy()
    return A, o[:, 0], o[:, 1]


@pytest.mark.parametrize("cls", ["S", "W", "A", "B", "C"])
def test_cgcg_npb_zeta_published(sp, torch_dev, cls):
    torch, dev = torch_dev
    A, zetas, rnorms = _npb(sp, torch, dev, cls)
    ref = gen.NPB_ZETA[cls]
    assert abs(zetas[-1] - ref) / ref <= 1e-10, (zetas[-1], ref)
    assert rnorms.max() <= 1e-11


@pytest.mark.parametrize("cls", ["S", "W"])
def test_cgcg_npb_matches_oracle_each_iteration(sp, torch_dev, cls):
    torch, dev = torch_dev
    A, zetas, rnorms = _npb(sp, torch, dev, cls)
    zr, rr = oracle.npb_run(A.rowptr, A.colidx, A.vals, gen.NPB_CLASSES[cls][2], gen.NPB_CLASSES[cls][3],
                            variant=1)
    assert np.allclose(zetas, zr, rtol=1e-11, atol=0)


def test_cgcg_graph_vs_eager_bitexact(sp, torch_dev, monkeypatch):
    torch, dev = torch_dev
    _, z1, r1 = _npb(sp, torch, dev, "S", niter=3)
    monkeypatch.setenv("SPMV_GRAPH", "0")
    _, z2, r2 = _npb(sp, torch, dev, "S", niter=3)
    assert np.array_equal(z1, z2) and np.array_equal(r1, r2)


def test_variant_switch_on_one_handle(sp, torch_dev):
    """textbook -> cgcg -> textbook on one handle equals fresh handles bit for bit."""
    torch, dev = torch_dev
    A = gen.makea("S")
    rp, ci, va = to_dev(A, dev)
    b = torch.from_numpy(gen.uniform(A.n, seed=8)).to(dev)

    def solve(M):
        x = torch.empty_like(b)
        M.cg_solve(b, x, 25)
        return x.cpu().numpy()

    fresh = {}
    for v in ("textbook", "cgcg"):
        with sp.CSRMatrix(rp, ci, va, A.n, cg_variant=v) as M:
            fresh[v] = solve(M)
    assert not np.array_equal(fresh["textbook"], fresh["cgcg"])   # different rounding ...
    assert np.allclose(fresh["textbook"], fresh["cgcg"], rtol=1e-10, atol=1e-13)   # ... same mathematics
    with sp.CSRMatrix(rp, ci, va, A.n) as M:
        for v in ("textbook", "cgcg", "textbook"):
            M.set_cg_variant(v)
            assert np.array_equal(solve(M), fresh[v])


@pytest.fixture(scope="module")
def dists():
    import torch
    import torch.distributed as tdist

    import paper_conf_asplos_ginsbachrsbdo18_b200 as sp
    if not tdist.is_initialized():
        s = socket.socket()
        s.bind(("127.0.0.1", 0))
        port = s.getsockname()[1]
        s.close()
        tdist.init_process_group("gloo", init_method=f"tcp://127.0.0.1:{port}", rank=0, world_size=1)
    dn = sp.Dist(0, 1, 0)
    dp = sp.Dist(0, 1, 0, transport="p2p")
    yield dn, dp
    dp.close()
    dn.close()


def test_cgcg_dist1_transports_bitexact(sp, torch_dev, dists):
    """NCCL and p2p 1-rank transports (scalar exchange slots, fused x push of r)
    reproduce the single-GPU single-reduction CG bit for bit."""
    torch, dev = torch_dev
    _, z0, r0 = _npb(sp, torch, dev, "S", niter=3)
    for d in dists:
        _, z1, r1 = _npb(sp, torch, dev, "S", niter=3, dist=d)
        assert np.array_equal(z0, z1) and np.array_equal(r0, r1)
