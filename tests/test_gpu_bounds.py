"""Out-of-range accesses without compute-sanitizer (closed on this pool, see
test_gpu_sanitizer.py): every operand of spmv_csr is a view into a larger
device buffer whose guard regions on both sides hold NaN (inputs) or a
sentinel bit pattern (the output).  A kernel that reads x, vals or y outside
its extent turns a row into NaN; one that writes y outside [0, m) changes a
guard word.  Run over every kernel family on the ragged / skewed shapes of
the adversarial zoo, compared row by row with the oracle (the
Fig. 4 loop, and P:878-888, section 6.3: soundness of sparse accesses)."""
import numpy as np
import pytest

import gen
import oracle
from gpu_util import check_rows

pytestmark = pytest.mark.gpu

G = 4099  # guard elements on each side (odd: shifts the views off 16-B alignment too)
SENT = -1.2345678e300


def _guarded(torch, dev, h, fill):
    buf = torch.full((h.size + 2 * G,), fill, dtype=torch.from_numpy(h[:0]).dtype, device=dev)
    buf[G:G + h.size] = torch.from_numpy(np.ascontiguousarray(h)).to(dev)
    return buf, buf[G:G + h.size]


def _cases():
    r = np.random.default_rng(7)
    L = r.integers(0, 9, 5000)
    L[17] = 4000
    rp = np.concatenate([[0], np.cumsum(L)]).astype(np.int32)
    skew = gen.CSR(5000, 7001, rp, r.integers(0, 7001, int(rp[-1])).astype(np.int32), r.standard_normal(int(rp[-1])))
    return [("makea_S", gen.makea("S")), ("makea_W", gen.makea("W")), ("skew_ragged", skew),
            ("stencil27_11", gen.stencil27(11)), ("laplace1d", gen.laplace1d(33333))]


CASES = _cases()


@pytest.mark.parametrize("kernel", ["auto", "vector", "merge", "xstat", "xplan", "sell", "sellsort", "xt"])
@pytest.mark.parametrize("name,A", CASES, ids=[c[0] for c in CASES])
@pytest.mark.parametrize("beta", [0.0, 1.5])
def test_guard_regions(name, A, kernel, beta):
    import torch

    import paper_conf_asplos_ginsbachrsbdo18_b200 as sp
    dev = torch.device("cuda:0")
    rpb, rp = _guarded(torch, dev, A.rowptr, 0)
    cib, ci = _guarded(torch, dev, A.colidx, 0)
    vab, va = _guarded(torch, dev, A.vals, float("nan"))
    x_h = gen.uniform(A.n, seed=31)
    xb, x = _guarded(torch, dev, x_h, float("nan"))
    y0 = gen.uniform(A.m, seed=32)
    yb, y = _guarded(torch, dev, y0, SENT)
    try:
        M = sp.CSRMatrix(rp, ci, va, A.n, kernel=kernel)
    except RuntimeError as e:  # a plan kernel that does not apply to this shape is refused at create
        pytest.skip(f"{kernel} not applicable to {name}: {e}")
    with M:
        for _ in range(2):  # twice: the second call runs on warmed plan buffers
            y.copy_(torch.from_numpy(y0).to(dev))
            M.spmv(x, y, 1.0, beta)
        torch.cuda.synchronize()
    yh = yb.cpu().numpy()
    assert np.all(yh[:G] == SENT) and np.all(yh[G + A.m:] == SENT), f"{name}/{kernel}: y written out of range"
    y_ref, bound = oracle.spmv(A.rowptr, A.colidx, A.vals, x_h, y0, 1.0, beta)
    check_rows(yh[G:G + A.m], y_ref, bound, np.float64, f"{name}/{kernel} beta={beta}")


@pytest.mark.parametrize("variant", ["textbook", "cgcg", "persist"])
def test_guard_regions_cg(variant):
    """cg_solve with b and x as guarded views (NaN around b, sentinel around x):
    no read outside b (the solution would turn NaN), no write outside x."""
    import torch

    import paper_conf_asplos_ginsbachrsbdo18_b200 as sp
    dev = torch.device("cuda:0")
    A = gen.makea("S")
    rp = torch.from_numpy(A.rowptr).to(dev)
    ci = torch.from_numpy(A.colidx).to(dev)
    va = torch.from_numpy(A.vals).to(dev)
    b_h = gen.uniform(A.n, seed=33)
    bb, b = _guarded(torch, dev, b_h, float("nan"))
    xb, x = _guarded(torch, dev, np.zeros(A.n), SENT)
    with sp.CSRMatrix(rp, ci, va, A.n, cg_variant=variant) as M:
        its, rn = M.cg_solve(b, x, max_iter=10)
        torch.cuda.synchronize()
    xh = xb.cpu().numpy()
    assert np.all(xh[:G] == SENT) and np.all(xh[G + A.n:] == SENT), f"{variant}: x written out of range"
    z_ref, _, _, _ = oracle.cg(A.rowptr, A.colidx, A.vals, b_h, 10, variant=0 if variant == "textbook" else 1)
    assert np.allclose(xh[G:G + A.n], z_ref, rtol=1e-10, atol=1e-13)


@pytest.mark.parametrize("dims", [(16, 16, 16), (17, 9, 5), (64, 3, 7)])
def test_guard_regions_stencil(dims):
    """stencil27_apply on guarded views: the zero boundary must come from the kernel,
    not from reading past the grid (NaN guards around x, sentinels around y)."""
    import torch

    import paper_conf_asplos_ginsbachrsbdo18_b200 as sp
    dev = torch.device("cuda:0")
    nx, ny, nz = dims
    n = nx * ny * nz
    x_h = gen.uniform(n, seed=34)
    xb, x = _guarded(torch, dev, x_h, float("nan"))
    y0 = gen.uniform(n, seed=35)
    yb, y = _guarded(torch, dev, y0, SENT)
    sp.stencil27_apply(nx, ny, nz, x, y, 1.0, 0.5)
    torch.cuda.synchronize()
    yh = yb.cpu().numpy()
    assert np.all(yh[:G] == SENT) and np.all(yh[G + n:] == SENT), f"{dims}: y written out of range"
    y_ref, bound = oracle.stencil27(nx, ny, nz, x_h, y_old=y0, alpha=1.0, beta=0.5)
    check_rows(yh[G:G + n], y_ref, bound, np.float64, f"stencil {dims}")


@pytest.mark.parametrize("kind", ["count", "sat_u8"])
def test_guard_regions_histogram(kind):
    """idl_histogram with guarded bins: keys outside [0, nbins) are skipped, and no
    bin outside the view is touched (sentinel guards around the bins)."""
    import torch

    import paper_conf_asplos_ginsbachrsbdo18_b200 as sp
    dev = torch.device("cuda:0")
    nbins = 5000
    r = np.random.default_rng(36)
    keys_h = r.integers(-50, nbins + 50, 200003).astype(np.int32)  # includes out-of-range keys
    keys = torch.from_numpy(keys_h).to(dev)
    ndt = np.uint32 if kind == "count" else np.uint8
    sent = 0xA5A5A5A5 if kind == "count" else 0xA5
    init = np.full(nbins + 2 * G, sent, dtype=ndt)
    init[G:G + nbins] = 0
    binsb = torch.from_numpy(init).to(dev)
    sp.idl_histogram(kind, keys, binsb[G:G + nbins])
    torch.cuda.synchronize()
    hb = binsb.cpu().numpy()
    assert np.all(hb[:G] == sent) and np.all(hb[G + nbins:] == sent), f"{kind}: bins written out of range"
    ref = oracle.hist_count_u32(keys_h, nbins) if kind == "count" else oracle.hist_sat_u8(keys_h, nbins)
    assert np.array_equal(hb[G:G + nbins], ref)
