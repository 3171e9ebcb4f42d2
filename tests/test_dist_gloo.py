"""Distributed orchestration without GPUs (world_size 2 and 3, gloo on CPU).

Each rank computes the library's host exchange plan (nnz-balanced partition +
columns renumbered into the padded gather layout, spmv_dist_plan_host), the
ranks exchange their x slices with an all-gather (gloo here, NCCL on the GPU
path), each rank runs the oracle SpMV on its row block against the padded x,
and the gathered y must equal the global oracle SpMV bit for bit (row-local
computation: each row's summation order does not depend on the partition).
The plan's partition is also checked against the oracle's on every rank."""
import os
import socket

import numpy as np
import pytest
import torch.multiprocessing as mp

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _halo_brute(A, bounds, world):
    """Reading R27 written out: per (reader r, owner s != r), min and max of
    c - b_s over the columns c of r's rows owned by s; [0, 0) if none."""
    import numpy as np
    out = np.zeros((world, world, 2), dtype=np.int64)
    rows = np.repeat(np.arange(A.m), np.diff(A.rowptr))
    reader = np.searchsorted(bounds, rows, side="right") - 1
    owner = np.searchsorted(bounds, A.colidx, side="right") - 1
    for r in range(world):
        for s_ in range(world):
            sel = (reader == r) & (owner == s_)
            if r != s_ and sel.any():
                li = A.colidx[sel].astype(np.int64) - bounds[s_]
                out[r, s_] = (li.min(), li.max() + 1)
    return out


def _worker(rank, world, port, cls, q):
    import sys
    sys.path.insert(0, ROOT)
    import torch
    import torch.distributed as dist

    import gen
    import oracle
    import paper_conf_asplos_ginsbachrsbdo18_b200 as sp
    try:
        dist.init_process_group("gloo", init_method=f"tcp://127.0.0.1:{port}", rank=rank,
                                world_size=world)
        if cls == "powerlaw":
            A = gen.powerlaw(m=5000, lmax=800.0, seed=2, f32=False)
        elif cls == "stencil":
            A = gen.stencil27(12)
        else:
            A = gen.makea(cls)
        bounds, maxlen, ci_loc = sp.spmv_dist_plan_host(A.rowptr, A.colidx, world, rank)
        assert np.array_equal(bounds, oracle.partition(A.rowptr, world))
        x = gen.uniform(A.n, seed=77)
        b0, b1 = int(bounds[rank]), int(bounds[rank + 1])
        # exchange: padded all-gather of the rank slices
        mine = torch.zeros(maxlen, dtype=torch.float64)
        mine[: b1 - b0] = torch.from_numpy(x[b0:b1])
        parts = [torch.zeros(maxlen, dtype=torch.float64) for _ in range(world)]
        dist.all_gather(parts, mine)
        xpad = torch.cat(parts).numpy()
        # halo intervals (NEXT-2, R27): keep only what each owner would send
        # this rank; everything else becomes NaN, so a missed column shows
        halo = sp.spmv_dist_halo_host(A.rowptr, A.colidx, world)
        assert np.array_equal(halo, _halo_brute(A, bounds, world))
        for s_ in range(world):
            if s_ == rank:
                continue
            lo, hi = halo[rank, s_]
            seg = xpad[s_ * maxlen:(s_ + 1) * maxlen]
            seg[:lo] = np.nan
            seg[hi:] = np.nan
        if cls == "stencil":  # at most one plane + one line + 1 from a neighbour, nothing from others
            for s_ in range(world):
                ln = halo[rank, s_, 1] - halo[rank, s_, 0]
                if s_ != rank and abs(s_ - rank) == 1:
                    assert 12 * 12 <= ln <= 12 * 12 + 12 + 1, ln
                elif s_ != rank:
                    assert ln == 0
        # local block, rebased rowptr, renumbered columns
        rp_loc = (A.rowptr[b0:b1 + 1] - A.rowptr[b0]).astype(np.int32)
        v_loc = A.vals[A.rowptr[b0]:A.rowptr[b1]]
        y_loc, _ = oracle.spmv(rp_loc, ci_loc, v_loc, xpad)
        # gather y slices (variable length: pad) and compare on rank 0
        ypad = torch.zeros(maxlen, dtype=torch.float64)
        ypad[: b1 - b0] = torch.from_numpy(y_loc)
        ys = [torch.zeros(maxlen, dtype=torch.float64) for _ in range(world)]
        dist.all_gather(ys, ypad)
        if rank == 0:
            y = np.concatenate([ys[r].numpy()[: int(bounds[r + 1] - bounds[r])] for r in range(world)])
            y_ref, _ = oracle.spmv(A.rowptr, A.colidx, A.vals, x)
            assert np.array_equal(y, y_ref), "distributed result differs from global oracle"
        dist.barrier()
        dist.destroy_process_group()
        q.put((rank, "ok"))
    except Exception as e:  # pragma: no cover
        import traceback
        q.put((rank, "".join(traceback.format_exception(e))))


@pytest.mark.parametrize("world", [2, 3])
@pytest.mark.parametrize("cls", ["S", "powerlaw", "stencil"])
def test_dist_plan_gloo(world, cls):
    from paper_conf_asplos_ginsbachrsbdo18_b200 import build
    build.build()
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    ps = [ctx.Process(target=_worker, args=(r, world, port, cls, q)) for r in range(world)]
    for p in ps:
        p.start()
    res = [q.get(timeout=300) for _ in ps]
    for p in ps:
        p.join(timeout=60)
    for r, msg in res:
        assert msg == "ok", f"rank {r}: {msg}"


def _ep_worker(rank, world, port, q):
    import sys
    sys.path.insert(0, ROOT)
    import numpy as np
    import torch
    import torch.distributed as dist

    import oracle
    from paper_conf_asplos_ginsbachrsbdo18_b200 import ep_shard_range
    try:
        dist.init_process_group("gloo", init_method=f"tcp://127.0.0.1:{port}", rank=rank, world_size=world)
        M = 24
        b0, cnt = ep_shard_range(M, rank, world)
        qq, sx, sy = oracle.ep(M, b0, cnt)
        mine = torch.tensor(np.concatenate([qq, [sx, sy]]), dtype=torch.float64)
        parts = [torch.zeros(12, dtype=torch.float64) for _ in range(world)]
        dist.all_gather(parts, mine)
        tot = torch.zeros(12, dtype=torch.float64)
        for p in parts:           # rank order: every rank gets the same sums
            tot += p
        dist.destroy_process_group()
        q.put((rank, "ok", tot.numpy().tolist(), (b0, cnt)))
    except Exception as e:  # pragma: no cover
        import traceback
        q.put((rank, "".join(traceback.format_exception(e)), None, None))


@pytest.mark.parametrize("world", [2, 3])
def test_ep_sharded_gloo(world):
    """NAS EP sharded by pair ranges (R33) over gloo ranks: the rank-order sum of
    the per-rank tallies equals the single-process oracle (q exactly)."""
    import oracle
    port = _free_port()
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    ps = [ctx.Process(target=_ep_worker, args=(r, world, port, q)) for r in range(world)]
    for p in ps:
        p.start()
    res = [q.get(timeout=300) for _ in ps]
    for p in ps:
        p.join(timeout=60)
    ranges = sorted(r[3] for r in res)
    assert ranges[0][0] == 0 and sum(c for _, c in ranges) == 1 << 24
    assert all(ranges[i][0] + ranges[i][1] == ranges[i + 1][0] for i in range(world - 1))
    qf, sxf, syf = oracle.ep(24)
    for rank, msg, tot, _ in res:
        assert msg == "ok", msg
        tot = np.array(tot)
        assert np.array_equal(tot[:10], qf)
        assert abs(tot[10] - sxf) <= 1e-10 * abs(sxf) and abs(tot[11] - syf) <= 1e-10 * abs(syf)
    assert res[0][2] == res[-1][2]
