"""GPU parity of the XT kernel (TMA-streamed, column-parted x-stationary plan,
DESIGN.md 5.2b) against the CPU oracle, per row with the BJ.ns tolerance.

Covers: the adversarial zoo with forced cluster sizes B and part counts Q
(Q > 1 exercises the cross-part group tickets), ring depths, multi-piece
chunks (rows longer than one TMA stage), alpha/beta with NaN probes,
update_values, determinism, the NAS CG zeta with Q > 1 (the per-part fused
dot), and the full-size class-C matrix in the bench's launch configuration."""
import numpy as np
import pytest

import gen
import oracle
from gpu_util import check_rows, to_dev
from test_gpu_spmv import ZOO, run_case

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def torch_dev():
    import torch
    return torch, torch.device("cuda:0")


@pytest.fixture(scope="module")
def sp():
    import paper_conf_asplos_ginsbachrsbdo18_b200 as sp
    return sp


def _sorted_cols(A):
    if A.m == 0 or A.nnz == 0:
        return False
    k = np.arange(A.rowptr[0] + 1, A.rowptr[-1])
    starts = np.zeros(A.colidx.shape[0] + 1, bool)
    starts[A.rowptr[:-1]] = True
    inner = ~starts[k]
    return bool(np.all(A.colidx[k][inner] > A.colidx[k - 1][inner]))


CFGS = [{}, {"SPMV_XT_B": "2", "SPMV_XT_Q": "3"}, {"SPMV_XT_B": "4", "SPMV_XT_Q": "2"},
        {"SPMV_XT_B": "8"}, {"SPMV_XT_B": "2", "SPMV_XT_Q": "5"}, {"SPMV_XT_NS": "3", "SPMV_XT_Q": "2"},
        {"SPMV_XT_B": "2", "SPMV_XT_Q": "16"}]


@pytest.mark.parametrize("cfg", CFGS, ids=[str(c) for c in CFGS])
@pytest.mark.parametrize("name,A", ZOO, ids=[c[0] for c in ZOO])
def test_zoo_xt(sp, torch_dev, name, A, cfg, monkeypatch):
    torch, dev = torch_dev
    for k, v in cfg.items():
        monkeypatch.setenv(k, v)
    x = gen.uniform(A.n, seed=51)
    info = run_case(sp, torch, dev, A, x, kernel="xt", what=f"{name} xt {cfg}")
    if name in ("laplace1d", "stencil27_9", "makea_S", "n1"):
        assert info["kernel_name"] == "xt", info
    A32 = A.astype(np.float32)
    run_case(sp, torch, dev, A32, gen.uniform(A.n, seed=52, f32=True), kernel="xt", what=f"{name} xt fp32 {cfg}")
    y0 = gen.uniform(A.m, seed=53)
    run_case(sp, torch, dev, A, x, alpha=-1.5, beta=0.5, y0=y0, kernel="xt", what=f"{name} xt a/b {cfg}")


def _long_rows_matrix(seed=3):
    """3000 x 4000, 40 sorted random columns per row, plus 64 rows of 3000
    entries: their chunk segments are far longer than one TMA stage (51 fp64
    steps), so their chunks are split into pieces across several stages."""
    r = np.random.default_rng(seed)
    m, n = 3000, 4000
    L = np.full(m, 40)
    L[1024 + 128:1024 + 192] = 3000  # two whole chunks of one tile (little SELL padding)
    rp = np.concatenate([[0], np.cumsum(L)]).astype(np.int32)
    cols = np.concatenate([np.sort(r.choice(n, l, replace=False)) for l in L]).astype(np.int32)
    return gen.CSR(m, n, rp, cols, r.standard_normal(int(rp[-1])))


@pytest.mark.parametrize("cfg", [{}, {"SPMV_XT_Q": "2"}, {"SPMV_XT_B": "4"}])
def test_xt_multipiece_chunks(sp, torch_dev, cfg, monkeypatch):
    torch, dev = torch_dev
    for k, v in cfg.items():
        monkeypatch.setenv(k, v)
    A = _long_rows_matrix()
    x = gen.uniform(A.n, seed=54)
    info = run_case(sp, torch, dev, A, x, kernel="xt", what=f"long rows {cfg}")
    assert info["kernel_name"] == "xt", info
    run_case(sp, torch, dev, A.astype(np.float32), gen.uniform(A.n, seed=55, f32=True), kernel="xt",
             what=f"long rows fp32 {cfg}")


@pytest.mark.parametrize("q", ["1", "3"])
def test_xt_alpha_beta_update_values_deterministic(sp, torch_dev, q, monkeypatch):
    torch, dev = torch_dev
    monkeypatch.setenv("SPMV_XT_Q", q)
    A = gen.makea("A")
    x_h = gen.uniform(A.n, seed=56)
    y0 = gen.uniform(A.m, seed=57)
    for a, b in [(2.0, -1.0), (0.0, 3.0), (1.0, 0.0), (-1.5, 1.0)]:
        xin = x_h if a != 0.0 else np.full(A.n, np.nan)
        info = run_case(sp, torch, dev, A, xin, alpha=a, beta=b, y0=y0, kernel="xt", what=f"xt a={a} b={b} Q={q}")
        assert info["kernel_name"] == "xt"
    rp, ci, va = to_dev(A, dev)
    x = torch.from_numpy(x_h).to(dev)
    y = torch.empty(A.m, dtype=torch.float64, device=dev)
    y2 = torch.empty_like(y)
    with sp.CSRMatrix(rp, ci, va, A.n, kernel="xt") as M:
        assert M.info()["kernel_name"] == "xt"
        # determinism: repeated launches are bit-identical (fixed summation orders)
        M.spmv(x, y)
        for _ in range(3):
            M.spmv(x, y2)
            torch.cuda.synchronize()
            assert torch.equal(y, y2)
        # in-place value change + update_values (the paper's lazy-copy flag)
        v2_h = gen.uniform(A.nnz, seed=58)
        va.copy_(torch.from_numpy(v2_h))
        M.update_values(va)
        M.spmv(x, y)
        torch.cuda.synchronize()
    y_ref, bound = oracle.spmv(A.rowptr, A.colidx, v2_h, x_h)
    check_rows(y.cpu().numpy(), y_ref, bound, np.float64, "xt update_values")


@pytest.mark.parametrize("cfg", [{"SPMV_XT_Q": "3"}, {"SPMV_XT_B": "4", "SPMV_XT_Q": "2"}, {"SPMV_XT_B": "8"}])
@pytest.mark.parametrize("variant", ["textbook", "cgcg"])
def test_xt_npb_zeta_parts(sp, torch_dev, cfg, variant, monkeypatch):
    """NPB class S and W zeta (published, 1e-10) with the fused CG dot taken
    per column part (Q > 1: w.y = sum_q w.y_q)."""
    torch, dev = torch_dev
    for k, v in cfg.items():
        monkeypatch.setenv(k, v)
    for cls in ("S", "W"):
        na, nonzer, niter, shift = gen.NPB_CLASSES[cls]
        A = gen.makea(cls)
        rp, ci, va = to_dev(A, dev)
        with sp.CSRMatrix(rp, ci, va, A.n, kernel="xt") as M:
            assert M.info()["kernel_name"] == "xt"
            M.set_cg_variant(variant)
            x = torch.ones(A.n, dtype=torch.float64, device=dev)
            z = torch.empty_like(x)
            out = torch.zeros(2, dtype=torch.float64, device=dev)
            for _ in range(niter):
                M.npb_outer(x, z, 25, shift, out)
            zeta = float(out[0].item())
        assert abs(zeta - gen.NPB_ZETA[cls]) / gen.NPB_ZETA[cls] <= 1e-10, (cls, zeta)


def test_xt_class_c_every_row(sp, torch_dev):
    """BJ.cfg[3] at full size through the XT plan: every row vs the oracle."""
    torch, dev = torch_dev
    A = gen.makea("C")
    x = gen.uniform(A.n, seed=59)
    info = run_case(sp, torch, dev, A, x, kernel="xt", what="NAS C xt")
    assert info["kernel_name"] == "xt" and info["cluster"] in (1, 2, 4, 8), info
