#!/usr/bin/env python3
"""Small invocations of every kernel family of the library, for the
compute-sanitizer tier (memcheck / racecheck / synccheck; VERDICT r1 item 5,
SURVEY T6).  Each case runs once on tiny inputs and is checked against the
oracle, so a sanitizer run also exercises correct executions.

usage: compute-sanitizer --tool memcheck --error-exitcode 9 python tools/sanitize_cases.py [case ...]
"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402
import torch  # noqa: E402

import gen  # noqa: E402
import oracle  # noqa: E402
import paper_conf_asplos_ginsbachrsbdo18_b200 as sp  # noqa: E402

dev = torch.device("cuda:0")


def spmv_case(A, kernel, env=None, f32=False):
    env = env or {}
    old = {k: os.environ.get(k) for k in env}
    os.environ.update(env)
    try:
        B = A.astype(np.float32) if f32 else A
        rp, ci, va = (torch.from_numpy(np.ascontiguousarray(a)).to(dev) for a in (B.rowptr, B.colidx, B.vals))
        x_h = gen.uniform(A.n, seed=3, f32=f32)
        x = torch.from_numpy(x_h).to(dev)
        y = torch.empty(A.m, dtype=va.dtype, device=dev)
        with sp.CSRMatrix(rp, ci, va, A.n, kernel=kernel) as M:
            M.spmv(x, y)
            torch.cuda.synchronize()
            name = M.info()["kernel_name"]
        y_ref, bound = oracle.spmv(B.rowptr, B.colidx, B.vals, x_h)
        tol = 1e-5 if f32 else 1e-12
        assert np.all(np.abs(y.cpu().numpy() - y_ref) <= tol * bound), (kernel, env)
        return name
    finally:
        for k, v in old.items():
            if v is None:
                os.environ.pop(k, None)
            else:
                os.environ[k] = v


def cg_case(kernel, variant, env=None):
    env = env or {}
    os.environ.update(env)
    A = gen.makea("S")
    rp, ci, va = (torch.from_numpy(a).to(dev) for a in (A.rowptr, A.colidx, A.vals))
    with sp.CSRMatrix(rp, ci, va, A.n, kernel=kernel) as M:
        M.set_cg_variant(variant)
        x = torch.ones(A.n, dtype=torch.float64, device=dev)
        z = torch.empty_like(x)
        out = torch.zeros(2, dtype=torch.float64, device=dev)
        M.npb_outer(x, z, 25, 10.0, out)
        torch.cuda.synchronize()
    for k in env:
        os.environ.pop(k, None)
    _, zeta, _ = oracle.npb_outer(A.rowptr, A.colidx, A.vals, np.ones(A.n), 25, 10.0,
                                  variant=0 if variant == "textbook" else 1)
    assert abs(float(out[0]) - zeta) <= 1e-10 * abs(zeta)


def _p2p_worker(rank, world, port, q):
    import torch.distributed as dist
    try:
        dist.init_process_group("gloo", init_method=f"tcp://127.0.0.1:{port}", rank=rank, world_size=world)
        torch.cuda.set_device(dev)
        d = sp.Dist(rank, world, 0, transport="p2p")
        A = gen.makea("S")
        t = lambda v: torch.from_numpy(np.ascontiguousarray(v)).to(dev)  # noqa: E731
        with sp.CSRMatrix(t(A.rowptr), t(A.colidx), t(A.vals), A.n, dist=d) as M:
            b0, b1 = M.row_range
            x_h = gen.uniform(A.n, seed=9)
            y = torch.empty(b1 - b0, dtype=torch.float64, device=dev)
            M.spmv(t(x_h[b0:b1]), y)
            torch.cuda.synchronize()
            y_ref, bound = oracle.spmv(A.rowptr, A.colidx, A.vals, x_h)
            assert np.all(np.abs(y.cpu().numpy() - y_ref[b0:b1]) <= 1e-12 * bound[b0:b1])
            zeta = {}
            for variant in ("textbook", "cgcg"):
                M.set_cg_variant(variant)
                xs = torch.ones(b1 - b0, dtype=torch.float64, device=dev)
                z = torch.empty_like(xs)
                o2 = torch.zeros(2, dtype=torch.float64, device=dev)
                M.npb_outer(xs, z, 25, 10.0, o2)
                torch.cuda.synchronize()
                zeta[variant] = float(o2[0])
            _, zr, _ = oracle.npb_outer(A.rowptr, A.colidx, A.vals, np.ones(A.n), 25, 10.0, variant=0)
            assert abs(zeta["textbook"] - zr) <= 1e-10 * abs(zr), zeta
        S = gen.stencil27(12)
        with sp.CSRMatrix(t(S.rowptr), t(S.colidx), t(S.vals), S.n, dist=d) as M:
            b0, b1 = M.row_range
            x_h = gen.uniform(S.n, seed=10)
            y = torch.empty(b1 - b0, dtype=torch.float64, device=dev)
            for _ in range(2):
                M.spmv(t(x_h[b0:b1]), y)
            torch.cuda.synchronize()
            y_ref, bound = oracle.spmv(S.rowptr, S.colidx, S.vals, x_h)
            assert np.all(np.abs(y.cpu().numpy() - y_ref[b0:b1]) <= 1e-12 * bound[b0:b1])
        dist.barrier()
        d.close()
        dist.destroy_process_group()
        # under compute-sanitizer --target-processes all the tool is injected into this child too
        q.put((rank, "ok", os.environ.get("CUDA_INJECTION64_PATH", "")))
    except Exception as e:  # pragma: no cover
        import traceback
        q.put((rank, "".join(traceback.format_exception(e)), ""))


def p2p_case():
    """Two ranks of the p2p transport as two processes on the one GPU (CUDA IPC
    peer stores, epoch flags, last-CTA publication), as tests/test_gpu_p2p_mp.py."""
    import socket
    import torch.multiprocessing as mp
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    port = s.getsockname()[1]
    s.close()
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    ps = [ctx.Process(target=_p2p_worker, args=(r, 2, port, q)) for r in range(2)]
    for p in ps:
        p.start()
    res = [q.get(timeout=900) for _ in ps]
    for p in ps:
        p.join(timeout=60)
    for r, msg, inj in res:
        assert msg == "ok", f"rank {r}: {msg}"
        print(f"p2p rank {r} ok; sanitizer injection: {inj or 'none'}", flush=True)


def stencil_case(env=None):
    env = env or {}
    os.environ.update(env)
    dims = (64, 20, 9)
    n = dims[0] * dims[1] * dims[2]
    x_h = gen.uniform(n, seed=4)
    y = torch.empty(n, dtype=torch.float64, device=dev)
    sp.stencil27_apply(*dims, torch.from_numpy(x_h).to(dev), y)
    torch.cuda.synchronize()
    for k in env:
        os.environ.pop(k, None)
    y_ref, bound = oracle.stencil27(*dims, x_h)
    assert np.all(np.abs(y.cpu().numpy() - y_ref) <= 1e-12 * bound)


def idioms_case():
    keys = gen.is_keys("S")
    bins = torch.zeros(1 << 11, dtype=torch.uint32, device=dev)
    sp.idl_histogram("count", torch.from_numpy(keys).to(dev), bins)
    assert np.array_equal(bins.cpu().numpy(), oracle.hist_count_u32(keys, 1 << 11))
    a_h = gen.uniform(20001, seed=5)
    r = sp.idl_reduce(torch.from_numpy(a_h).to(dev)).item()
    r_ref, bnd = oracle.reduce(a_h)
    assert abs(r - r_ref) <= 2 * (20001 + 64) * 2.0 ** -53 * bnd
    ep = sp.ep_npb(24, 0, 1 << 14, device=dev).cpu().numpy()
    q, sx, sy = oracle.ep(24, 0, 1 << 14)
    assert np.array_equal(ep[:10], q)


def jds_case():
    A = gen.makea("S")
    J = gen.csr_to_jds(A)
    t = lambda v: torch.from_numpy(np.ascontiguousarray(v)).to(dev)  # noqa: E731
    x_h = gen.uniform(A.n, seed=6)
    with sp.JDSMatrix(t(J.perm), t(J.jds_ptr), t(J.zcnt), t(J.indices), t(J.data), J.m, J.n) as M:
        y = torch.empty(A.m, dtype=torch.float64, device=dev)
        M.spmv(t(x_h), y)
        torch.cuda.synchronize()
    y_ref, b = oracle.spmv_jds(J, x_h)
    assert np.all(np.abs(y.cpu().numpy() - y_ref) <= 1e-12 * b)


CASES = {
    "xplan": lambda: [spmv_case(gen.makea("S"), "xplan", {"SPMV_XPLAN_B": b}) for b in ("2", "4", "8")]
    + [spmv_case(gen.makea("S"), "xplan", {"SPMV_XPLAN_CLUSTERS": "1"}),
       spmv_case(gen.makea("S"), "xplan", {"SPMV_XPLAN_DYN": "1"})],
    "xt": lambda: [spmv_case(gen.makea("S"), "xt", {"SPMV_XT_Q": q}) for q in ("1", "3")],
    "sell": lambda: [spmv_case(gen.stencil27(9), "sell"), spmv_case(gen.stencil27(9), "sell", f32=True)],
    "sellsort": lambda: spmv_case(gen.powerlaw(m=4000, lmax=1500.0, beta=0.6, seed=5, f32=False), "sellsort"),
    "merge": lambda: spmv_case(gen.powerlaw(m=4000, lmax=1500.0, beta=0.6, seed=5, f32=False), "merge"),
    "vector": lambda: spmv_case(gen.makea("S"), "vector"),
    "xstat": lambda: spmv_case(gen.makea("S"), "xstat"),
    "cg": lambda: [cg_case("xplan", "cgcg"), cg_case("xplan", "textbook"), cg_case("sell", "cgcg")],
    "persist": lambda: cg_case("xplan", "persist"),
    "p2p": p2p_case,
    "stencil": lambda: [stencil_case(), stencil_case({"SPMV_STENCIL_TMA": "0"}), stencil_case({"SPMV_STENCIL_BOX": "0"})],
    "jds": jds_case,
    "idioms": idioms_case,
}

def p2p_rank_main(rank, port):
    """One rank of the p2p case as its own top-level process, so that a
    compute-sanitizer wrapping this command certainly instruments it:
    tests/test_gpu_sanitizer.py starts two of these, each under the tool."""
    import queue
    q = queue.Queue()
    _p2p_worker(rank, 2, port, q)
    r, msg, _ = q.get()
    assert msg == "ok", f"rank {r}: {msg}"
    print(f"p2p rank {r} OK", flush=True)


if __name__ == "__main__":
    if sys.argv[1:2] == ["p2prank"]:
        p2p_rank_main(int(sys.argv[2]), int(sys.argv[3]))
        print("sanitize cases OK")
        sys.exit(0)
    names = sys.argv[1:] or list(CASES)
    for nm in names:
        CASES[nm]()
        print(f"case {nm} OK", flush=True)
    print("sanitize cases OK")
