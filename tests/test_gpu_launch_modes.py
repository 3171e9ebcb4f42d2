"""Launch-mode switches that must not change a single bit:
programmatic dependent launch of the CG chain (SPMV_PDL) and the persisting-L2
window over the XPLAN plan (SPMV_XPLAN_PLANWIN) only change how the kernels are
scheduled and cached, not what they compute.  Each is compared on and off, on
the NPB outer iteration (captured graph, zeta/rnorm/z) and on cg_solve, with the
published zeta as the anchor (the SpMV inside the CG loop)."""
import numpy as np
import pytest

import gen
from gpu_util import to_dev

pytestmark = pytest.mark.gpu


def _run(monkeypatch, env, value, cls, variant):
    import torch

    import paper_conf_asplos_ginsbachrsbdo18_b200 as sp
    monkeypatch.setenv(env, value)
    dev = torch.device("cuda:0")
    A = gen.makea(cls)
    na, nonzer, niter, shift = gen.NPB_CLASSES[cls]
    rp, ci, va = to_dev(A, dev)
    s = torch.cuda.Stream(dev)
    with torch.cuda.stream(s):
        with sp.CSRMatrix(rp, ci, va, A.n, cg_variant=variant) as M:
            x = torch.ones(A.n, dtype=torch.float64, device=dev)
            z = torch.empty_like(x)
            out2 = torch.zeros(2, dtype=torch.float64, device=dev)
            zetas = []
            for _ in range(niter):
                M.npb_outer(x, z, gen.NPB_CGITMAX, shift, out2)
                zetas.append(out2.cpu().numpy().copy())
            torch.cuda.synchronize()
            b = torch.from_numpy(gen.uniform(A.n, seed=9)).to(dev)
            xs = torch.empty_like(b)
            its, rn = M.cg_solve(b, xs, max_iter=17)
            torch.cuda.synchronize()
    return np.array(zetas), z.cpu().numpy(), xs.cpu().numpy(), rn


@pytest.mark.parametrize("variant", ["cgcg", "textbook"])
@pytest.mark.parametrize("cls", ["S", "W"])
def test_pdl_on_off_bit_identical(monkeypatch, cls, variant):
    on = _run(monkeypatch, "SPMV_PDL", "1", cls, variant)
    off = _run(monkeypatch, "SPMV_PDL", "0", cls, variant)
    for a, b in zip(on[:3], off[:3]):
        assert np.array_equal(a.view(np.uint64), b.view(np.uint64))
    assert on[3] == off[3]
    assert abs(on[0][-1][0] - gen.NPB_ZETA[cls]) / gen.NPB_ZETA[cls] <= 1e-10


@pytest.mark.parametrize("variant", ["cgcg", "persist"])
def test_plan_window_on_off_bit_identical(monkeypatch, variant):
    on = _run(monkeypatch, "SPMV_XPLAN_PLANWIN", "1", "W", variant)
    off = _run(monkeypatch, "SPMV_XPLAN_PLANWIN", "0", "W", variant)
    for a, b in zip(on[:3], off[:3]):
        assert np.array_equal(a.view(np.uint64), b.view(np.uint64))
    assert abs(on[0][-1][0] - gen.NPB_ZETA["W"]) / gen.NPB_ZETA["W"] <= 1e-10
