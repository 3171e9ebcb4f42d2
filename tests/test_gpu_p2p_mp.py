"""Two ranks of the p2p transport as two processes sharing the one GPU of the
development box (CUDA IPC works across processes on one device; NCCL would
refuse duplicate GPUs).  Exercises the multi-rank exchange protocol of
p2p_kernels.cuh -- peer stores, epoch flags with release/acquire at system
scope, last-CTA publication, rank-order scalar sums -- end to end: row-sharded
SpMV against the oracle and NAS class-S CG against the published zeta."""
import os
import socket

import numpy as np
import pytest
import torch.multiprocessing as mp

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
pytestmark = pytest.mark.gpu


def _worker(rank, world, port, q):
    import sys
    sys.path.insert(0, ROOT)
    import torch
    import torch.distributed as dist

    import gen
    import oracle
    import paper_conf_asplos_ginsbachrsbdo18_b200 as sp
    try:
        dist.init_process_group("gloo", init_method=f"tcp://127.0.0.1:{port}", rank=rank, world_size=world)
        dev = torch.device("cuda:0")
        torch.cuda.set_device(dev)
        d = sp.Dist(rank, world, 0, transport="p2p")
        out = {}
        for cls in ("S", "W"):
            A = gen.makea(cls)
            rp = torch.from_numpy(A.rowptr).to(dev)
            ci = torch.from_numpy(A.colidx).to(dev)
            va = torch.from_numpy(A.vals).to(dev)
            for kernel in ("auto", "vector"):
                with sp.CSRMatrix(rp, ci, va, A.n, dist=d, kernel=kernel) as M:
                    b0, b1 = M.row_range
                    x_h = gen.uniform(A.n, seed=9)
                    x = torch.from_numpy(x_h[b0:b1].copy()).to(dev)
                    y = torch.empty(b1 - b0, dtype=torch.float64, device=dev)
                    M.spmv(x, y)
                    torch.cuda.synchronize()
                    y_ref, bound = oracle.spmv(A.rowptr, A.colidx, A.vals, x_h)
                    err = np.abs(y.cpu().numpy() - y_ref[b0:b1])
                    assert np.all(err <= 1e-12 * bound[b0:b1]), f"{cls} {kernel} spmv rank {rank}"
                    if cls == "S":
                        na, nonzer, niter, shift = gen.NPB_CLASSES[cls]
                        xs = torch.ones(b1 - b0, dtype=torch.float64, device=dev)
                        z = torch.empty_like(xs)
                        o2 = torch.zeros(2, dtype=torch.float64, device=dev)
                        for _ in range(niter):
                            M.npb_outer(xs, z, 25, shift, o2)
                        torch.cuda.synchronize()
                        out[kernel] = float(o2[0].item())
                        if kernel == "auto":  # NEXT-1: single-reduction CG over the p2p transport
                            M.set_cg_variant("cgcg")
                            xs.fill_(1.0)
                            for _ in range(niter):
                                M.npb_outer(xs, z, 25, shift, o2)
                            torch.cuda.synchronize()
                            out["cgcg"] = float(o2[0].item())
                            M.set_cg_variant("textbook")
        # halo exchange (NEXT-2): the stencil's ranks only exchange boundary planes
        A = gen.stencil27(20)
        rp = torch.from_numpy(A.rowptr).to(dev)
        ci = torch.from_numpy(A.colidx).to(dev)
        va = torch.from_numpy(A.vals).to(dev)
        for kernel in ("auto", "sell", "vector"):
            with sp.CSRMatrix(rp, ci, va, A.n, dist=d, kernel=kernel) as M:
                halo, used = M.dist_halo()
                assert used, "stencil halo should be used"
                assert np.array_equal(halo, sp.spmv_dist_halo_host(A.rowptr, A.colidx, world))
                b0, b1 = M.row_range
                x_h = gen.uniform(A.n, seed=10)
                x = torch.from_numpy(x_h[b0:b1].copy()).to(dev)
                y = torch.empty(b1 - b0, dtype=torch.float64, device=dev)
                for rep in range(3):  # repeated exchanges reuse the epochs
                    M.spmv(x, y)
                torch.cuda.synchronize()
                y_ref, bound = oracle.spmv(A.rowptr, A.colidx, A.vals, x_h)
                err = np.abs(y.cpu().numpy() - y_ref[b0:b1])
                assert np.all(err <= 1e-12 * bound[b0:b1]), f"stencil {kernel} halo spmv rank {rank}"
                bvec = torch.ones(b1 - b0, dtype=torch.float64, device=dev)
                xs = torch.empty_like(bvec)
                its, rn = M.cg_solve(bvec, xs, 200, tol=1e-10)
                assert rn <= 1e-9 * np.sqrt(A.n), (kernel, its, rn)
                out[f"stencil_{kernel}_its"] = its
                if kernel == "auto":  # single-reduction CG with early stop over the p2p transport
                    M.set_cg_variant("cgcg")
                    its2, rn2 = M.cg_solve(bvec, xs, 200, tol=1e-10)
                    M.set_cg_variant("textbook")
                    assert rn2 <= 1e-9 * np.sqrt(A.n) and abs(its2 - its) <= 1, (its, its2, rn2)
                    out["stencil_cgcg_its"] = its2
        dist.barrier()
        d.close()
        dist.destroy_process_group()
        q.put((rank, "ok", out))
    except Exception as e:  # pragma: no cover
        import traceback
        q.put((rank, "".join(traceback.format_exception(e)), None))


def test_p2p_two_processes_one_gpu():
    import gen
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    port = s.getsockname()[1]
    s.close()
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    ps = [ctx.Process(target=_worker, args=(r, 2, port, q)) for r in range(2)]
    for p in ps:
        p.start()
    res = [q.get(timeout=600) for _ in ps]
    for p in ps:
        p.join(timeout=60)
    for r, msg, out in res:
        assert msg == "ok", f"rank {r}: {msg}"
        for kernel, zeta in out.items():
            if kernel.startswith("stencil"):
                continue
            assert abs(zeta - gen.NPB_ZETA["S"]) / gen.NPB_ZETA["S"] <= 1e-10, (r, kernel, zeta)
    # both ranks computed identical scalars (rank-order sums of pushed values)
    assert res[0][2] == res[1][2]
