"""Distributed mode on one GPU (NCCL communicator of size 1; the driver's GPU
tier has one GPU): the rank-local path (partition kernel, renumbered colidx,
padded all-gather, all-reduced CG scalars) must reproduce the single-GPU
results bit for bit, and the device exchange plan must equal the host plan.
Multi-rank orchestration is covered on CPU by test_dist_gloo.py."""
import os
import socket

import numpy as np
import pytest

import gen
from gpu_util import to_dev

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def env():
    import torch
    import torch.distributed as dist

    import paper_conf_asplos_ginsbachrsbdo18_b200 as sp
    if not dist.is_initialized():
        s = socket.socket()
        s.bind(("127.0.0.1", 0))
        port = s.getsockname()[1]
        s.close()
        dist.init_process_group("gloo", init_method=f"tcp://127.0.0.1:{port}", rank=0, world_size=1)
    d = sp.Dist(0, 1, 0)
    yield torch, torch.device("cuda:0"), sp, d
    d.close()


@pytest.mark.parametrize("cls", ["S", "W"])
def test_dist1_spmv_bitexact(env, cls):
    torch, dev, sp, d = env
    A = gen.makea(cls)
    rp, ci, va = to_dev(A, dev)
    x = torch.from_numpy(gen.uniform(A.n, seed=5)).to(dev)
    y1 = torch.empty(A.m, dtype=torch.float64, device=dev)
    y2 = torch.empty_like(y1)
    with sp.CSRMatrix(rp, ci, va, A.n) as M1, sp.CSRMatrix(rp, ci, va, A.n, dist=d) as M2:
        M1.spmv(x, y1)
        M2.spmv(x, y2)
        torch.cuda.synchronize()
        b, ml, loc = sp.spmv_dist_plan_host(A.rowptr, A.colidx, 1, 0)
        assert np.array_equal(M2.dist_colidx(), loc)
        assert M2.info()["row_begin"] == 0 and M2.info()["row_end"] == A.m
    assert torch.equal(y1, y2)


def test_dist1_npb_bitexact(env):
    torch, dev, sp, d = env
    A = gen.makea("S")
    rp, ci, va = to_dev(A, dev)
    res = []
    for dd in (None, d):
        with sp.CSRMatrix(rp, ci, va, A.n, dist=dd) as M:
            x = torch.ones(A.n, dtype=torch.float64, device=dev)
            z = torch.empty_like(x)
            out = torch.zeros((3, 2), dtype=torch.float64, device=dev)
            for it in range(3):
                M.npb_outer(x, z, 25, 10.0, out[it])
            torch.cuda.synchronize()
            res.append(out.cpu().numpy())
    assert np.array_equal(res[0], res[1])


def test_dist1_cg_solve(env):
    torch, dev, sp, d = env
    A = gen.laplace1d(50)
    rp, ci, va = to_dev(A, dev)
    b = torch.ones(50, dtype=torch.float64, device=dev)
    x = torch.empty_like(b)
    with sp.CSRMatrix(rp, ci, va, 50, dist=d) as M:
        its, rn = M.cg_solve(b, x, 50, tol=1e-13)
    j = np.arange(50)
    assert np.allclose(x.cpu().numpy(), (j + 1) * (50 - j) / 2.0, rtol=1e-10)


@pytest.fixture(scope="module")
def p2p1(env):
    torch, dev, sp, d = env
    dp = sp.Dist(0, 1, 0, transport="p2p")
    yield dp
    dp.close()


def test_p2p1_spmv_and_npb_bitexact(env, p2p1):
    """1-rank p2p transport (push/wait kernels, exchange-mode scalar sources)
    reproduces the single-GPU results bit for bit."""
    torch, dev, sp, d = env
    A = gen.makea("S")
    rp, ci, va = to_dev(A, dev)
    x = torch.from_numpy(gen.uniform(A.n, seed=5)).to(dev)
    y1 = torch.empty(A.m, dtype=torch.float64, device=dev)
    y2 = torch.empty_like(y1)
    res = []
    for dd in (None, p2p1):
        with sp.CSRMatrix(rp, ci, va, A.n, dist=dd) as M:
            M.spmv(x, y1 if dd is None else y2)
            xs = torch.ones(A.n, dtype=torch.float64, device=dev)
            z = torch.empty_like(xs)
            out = torch.zeros((3, 2), dtype=torch.float64, device=dev)
            for it in range(3):
                M.npb_outer(xs, z, 25, 10.0, out[it])
            torch.cuda.synchronize()
            res.append(out.cpu().numpy())
            if dd is not None:
                assert M.info()["transport"] == 2
    assert torch.equal(y1, y2)
    assert np.array_equal(res[0], res[1])
