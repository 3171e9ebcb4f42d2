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
    "stencil": lambda: [stencil_case(), stencil_case({"SPMV_STENCIL_TMA": "0"}), stencil_case({"SPMV_STENCIL_BOX": "0"})],
    "jds": jds_case,
    "idioms": idioms_case,
}

if __name__ == "__main__":
    names = sys.argv[1:] or list(CASES)
    for nm in names:
        CASES[nm]()
        print(f"case {nm} OK", flush=True)
    print("sanitize cases OK")
