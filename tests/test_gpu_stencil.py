"""GPU parity of the matrix-free 27-point stencil (stencil27_apply, NEXT-3:
the paper's Stencil idiom, Fig. 13) against oracle_stencil27, point by point
within BJ.ns's bound (1e-12 fp64 / 1e-5 fp32 of sum |w x|: the kernel uses
FMA like the CSR kernels, reading R11); integer-valued inputs are compared
exactly (every partial sum is an exact integer).  Ragged tiles in every
dimension, several z-range splits, random weights, alpha/beta with NaN
probes, the full 256^3 grid of BJ.cfg[4], and agreement with the CSR SpMV of
the same operator."""
import numpy as np
import pytest

import gen
import oracle
from gpu_util import check_rows, to_dev

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def env():
    import torch

    import paper_conf_asplos_ginsbachrsbdo18_b200 as sp
    return torch, torch.device("cuda:0"), sp


def _run(env, dims, x_h, w=None, y0=None, alpha=1.0, beta=0.0, f32=False):
    torch, dev, sp = env
    nx, ny, nz = dims
    n = nx * ny * nz
    dt = np.float32 if f32 else np.float64
    x = torch.from_numpy(np.ascontiguousarray(x_h, dtype=dt)).to(dev)
    yo = np.full(n, np.nan, dtype=dt) if y0 is None else np.ascontiguousarray(y0, dtype=dt)
    y = torch.from_numpy(yo.copy()).to(dev)
    sp.stencil27_apply(nx, ny, nz, x, y, alpha, beta, w27=w)
    torch.cuda.synchronize()
    wref = None if w is None else (np.asarray(w, np.float32).astype(np.float64) if f32 else w)
    y_ref, bound = oracle.stencil27(nx, ny, nz, np.asarray(x_h, dt).astype(np.float64), w=wref,
                                    y_old=yo.astype(np.float64), alpha=alpha, beta=beta)
    return y.cpu().numpy(), y_ref, bound


DIMS = [(1, 1, 1), (2, 3, 5), (33, 9, 17), (31, 70, 40), (64, 64, 64), (5, 1, 130)]


@pytest.mark.parametrize("dims", DIMS)
@pytest.mark.parametrize("weights", ["laplace", "random"])
def test_stencil_bitexact_fp64(env, dims, weights):
    n = dims[0] * dims[1] * dims[2]
    w = None if weights == "laplace" else gen.uniform(27, seed=7)
    y, y_ref, bound = _run(env, dims, gen.uniform(n, seed=1), w=w)
    check_rows(y, y_ref, bound, np.float64, f"stencil {dims} {weights}")
    # small-integer x and weights: every partial sum is exact -> exact equality
    r = np.random.default_rng(dims[0] + 7 * dims[1])
    wi = None if w is None else r.integers(-3, 4, 27).astype(np.float64)
    y, y_ref, _ = _run(env, dims, r.integers(-5, 6, n).astype(np.float64), w=wi)
    assert np.array_equal(y, y_ref)


@pytest.mark.parametrize("zchunk", ["1", "3", "7"])
def test_stencil_z_ranges(env, zchunk, monkeypatch):
    monkeypatch.setenv("SPMV_STENCIL_ZCHUNK", zchunk)
    dims = (40, 12, 23)
    y, y_ref, bound = _run(env, dims, gen.uniform(40 * 12 * 23, seed=2), w=gen.uniform(27, seed=8))
    check_rows(y, y_ref, bound, np.float64, f"stencil zchunk {zchunk}")


@pytest.mark.parametrize("alpha,beta", [(2.5, 0.0), (-1.0, 0.5), (0.0, 3.0), (0.0, 0.0), (1.0, 1.0)])
@pytest.mark.parametrize("f32", [False, True])
@pytest.mark.parametrize("wkind", ["random", "laplace"])
def test_stencil_alpha_beta(env, alpha, beta, f32, wkind):
    dims = (17, 9, 11)
    n = 17 * 9 * 11
    x = gen.uniform(n, seed=3, f32=f32)
    if alpha == 0.0:
        x = np.full(n, np.nan, dtype=x.dtype)  # must not be read
    y0 = gen.uniform(n, seed=4, f32=f32)
    if beta == 0.0:
        y0 = np.full(n, np.nan, dtype=y0.dtype)  # must not be read
    w = gen.uniform(27, seed=9) if wkind == "random" else None   # laplace: the BOX form
    y, y_ref, bound = _run(env, dims, x, w=w, y0=y0, alpha=alpha, beta=beta, f32=f32)
    check_rows(y, y_ref, bound, np.float32 if f32 else np.float64, f"stencil f32={f32} a={alpha} b={beta}")


def test_stencil_equals_csr_spmv(env):
    """R19 weights: the matrix-free operator and spmv_csr on gen.stencil27 agree
    (auto kernel; per-row tolerance), and both agree with the CSR oracle."""
    torch, dev, sp = env
    N = 48
    A = gen.stencil27(N)
    x_h = gen.uniform(A.n, seed=5)
    y_mf, y_ref, bound = _run(env, (N, N, N), x_h)
    rp, ci, va = to_dev(A, dev)
    y = torch.empty(A.m, dtype=torch.float64, device=dev)
    with sp.CSRMatrix(rp, ci, va, A.n) as M:
        M.spmv(torch.from_numpy(x_h).to(dev), y)
        torch.cuda.synchronize()
    yc_ref, bc = oracle.spmv(A.rowptr, A.colidx, A.vals, x_h)
    assert np.array_equal(y_ref, yc_ref)
    check_rows(y.cpu().numpy(), y_mf, bound, np.float64, "csr vs matrix-free")


def test_stencil_errors(env):
    torch, dev, sp = env
    x = torch.zeros(1000, dtype=torch.float64, device=dev)
    with pytest.raises(sp.SpmvError) as e:
        sp.stencil27_apply(10, 10, 10, x, x)
    assert e.value.status == sp.SPMV_ERR_ALIAS
    with pytest.raises(sp.SpmvError) as e:
        sp.stencil27_apply(10, 10, 10, x, torch.zeros(1000, dtype=torch.float64))  # host y
    assert e.value.status == sp.SPMV_ERR_ARG
    with pytest.raises(ValueError):
        sp.stencil27_apply(10, 10, 10, x, torch.zeros_like(x), w27=np.ones(5))


def test_stencil256_full_size(env):
    """BJ.cfg[4]'s grid (256^3 = 16,777,216 points) matrix-free, fp64: every
    point against the oracle within the bound; A*1 = 27 - cnt exactly."""
    torch, dev, sp = env
    N = 256
    n = N ** 3
    x_h = gen.uniform(n, seed=6)
    y, y_ref, bound = _run(env, (N, N, N), x_h)
    check_rows(y, y_ref, bound, np.float64, "stencil 256^3")
    ones = torch.ones(n, dtype=torch.float64, device=dev)
    yy = torch.empty_like(ones)
    sp.stencil27_apply(N, N, N, ones, yy)
    torch.cuda.synchronize()
    i = np.arange(n)
    cnt = 1
    for c in (i % N, (i // N) % N, i // (N * N)):
        cnt = cnt * (3 - (c == 0) - (c == N - 1))
    assert np.array_equal(yy.cpu().numpy(), (27 - cnt).astype(np.float64))


@pytest.mark.parametrize("dims", [(33, 9, 17), (64, 64, 64), (5, 1, 130), (65, 17, 3), (2, 2, 2)])
def test_stencil_box_form(env, dims, monkeypatch):
    """Equal neighbour weights select the separable box-sum form: R19's Laplacian,
    all 27 weights equal, and an arbitrary (centre, neighbour) pair; each within
    the R11 bound of the oracle, and close to the general 27-FMA form."""
    n = dims[0] * dims[1] * dims[2]
    x = gen.uniform(n, seed=11)
    for w in (None, np.full(27, 0.37), np.where(np.arange(27) == 13, 5.5, -0.25)):
        y, y_ref, bound = _run(env, dims, x, w=w)
        check_rows(y, y_ref, bound, np.float64, f"box {dims}")
        monkeypatch.setenv("SPMV_STENCIL_BOX2", "0")                    # one column per thread
        y1, _, _ = _run(env, dims, x, w=w)
        monkeypatch.delenv("SPMV_STENCIL_BOX2")
        check_rows(y1, y_ref, bound, np.float64, f"box1 {dims}")
        monkeypatch.setenv("SPMV_STENCIL_BOX", "0")
        y2, _, _ = _run(env, dims, x, w=w)
        monkeypatch.delenv("SPMV_STENCIL_BOX")
        check_rows(y2, y_ref, bound, np.float64, f"general {dims}")


@pytest.mark.parametrize("dims", [(2, 2, 2), (64, 64, 64), (66, 17, 9), (128, 33, 40), (200, 3, 70), (192, 5, 7)])
@pytest.mark.parametrize("f32", [False, True])
@pytest.mark.parametrize("zchunk", [None, "5"])
def test_stencil_box2_tma_equals_cpasync(env, dims, f32, zchunk, monkeypatch):
    """The TMA plane tiles of k_stencil27_box2 (default when nx*sizeof(T) is a
    multiple of 16 B; the tensor map's out-of-bound fill supplies the halo,
    planes outside the grid are zero-filled by the CTA) stage the same values
    as the cp.async ring (SPMV_STENCIL_TMA=0): the outputs are bit-identical,
    and both are within the bound of the oracle.  Ragged x/y tiles, 1-plane
    grids' neighbours, several z ranges per column."""
    n = dims[0] * dims[1] * dims[2]
    x = gen.uniform(n, seed=12)
    if zchunk:
        monkeypatch.setenv("SPMV_STENCIL_ZCHUNK", zchunk)
    y0 = gen.uniform(n, seed=13)
    y_t, y_ref, bound = _run(env, dims, x, y0=y0, alpha=1.5, beta=-0.5, f32=f32)
    monkeypatch.setenv("SPMV_STENCIL_TMA", "0")
    y_c, _, _ = _run(env, dims, x, y0=y0, alpha=1.5, beta=-0.5, f32=f32)
    monkeypatch.delenv("SPMV_STENCIL_TMA")
    assert np.array_equal(y_t.view(np.uint64 if not f32 else np.uint32), y_c.view(np.uint64 if not f32 else np.uint32))
    check_rows(y_t, y_ref, bound, np.float32 if f32 else np.float64, f"tma {dims}")


def test_stencil_tma_path_is_taken(env, monkeypatch):
    """SPMV_STENCIL_TMA=2 makes the TMA form mandatory (argument error instead of the
    cp.async fallback): the 256^3 grid and even fp64 rows take it (so the TMA parity
    tests above exercise the tensor-map path), odd rows (nx*8 not a multiple of 16 B)
    cannot."""
    torch, dev, sp = env
    monkeypatch.setenv("SPMV_STENCIL_TMA", "2")
    for dims in [(256, 256, 256), (64, 64, 64), (66, 17, 9), (2, 3, 5)]:
        n = dims[0] * dims[1] * dims[2]
        x = torch.rand(n, dtype=torch.float64, device=dev)
        sp.stencil27_apply(*dims, x, torch.empty_like(x))
    torch.cuda.synchronize()
    x = torch.rand(33 * 9 * 17, dtype=torch.float64, device=dev)
    with pytest.raises(sp.SpmvError) as e:
        sp.stencil27_apply(33, 9, 17, x, torch.empty_like(x))
    assert e.value.status == sp.SPMV_ERR_ARG


def test_stencil_binding_checks(env):
    """The binding checks what the raw-pointer ABI cannot: x and y dtypes agree,
    both are contiguous and hold nx*ny*nz elements."""
    torch, dev, sp = env
    n = 8 * 8 * 8
    x = torch.rand(n, dtype=torch.float64, device=dev)
    with pytest.raises(ValueError):
        sp.stencil27_apply(8, 8, 8, x.float(), torch.empty_like(x))
    with pytest.raises(ValueError):
        sp.stencil27_apply(8, 8, 8, x, torch.empty(n - 1, dtype=torch.float64, device=dev))
    with pytest.raises(ValueError):
        sp.stencil27_apply(8, 8, 8, x[: n - 1], torch.empty_like(x))
    with pytest.raises(ValueError):
        sp.stencil27_apply(8, 8, 8, torch.rand(2 * n, dtype=torch.float64, device=dev)[::2], torch.empty_like(x))


def test_stencil_tma_mandatory_rejects_general_weights(env, monkeypatch):
    """SPMV_STENCIL_TMA=2 with general weights (no box2 form) is an argument
    error, not a silent cp.async run."""
    torch, dev, sp = env
    monkeypatch.setenv("SPMV_STENCIL_TMA", "2")
    x = torch.rand(64 ** 3, dtype=torch.float64, device=dev)
    w = np.arange(27, dtype=np.float64)
    with pytest.raises(sp.SpmvError) as e:
        sp.stencil27_apply(64, 64, 64, x, torch.empty_like(x), w27=w)
    assert e.value.status == sp.SPMV_ERR_ARG
