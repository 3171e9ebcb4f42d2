"""GPU parity of the idiom kernels (include/idioms.h) against
the CPU oracle (oracle/oracle_idioms.c), element by element on the same seeded
inputs; integer results bit-exact, floating-point results within reading R30's
bound; plus the published NPB EP values at the full class sizes (BJ-scale
inputs the oracle cannot finish quickly) and run-to-run determinism.
"""
import math
import os

import numpy as np
import pytest

import gen
import oracle

pytestmark = pytest.mark.gpu
U = 2.0 ** -53
GOLD = os.path.join(os.path.dirname(__file__), "golden")


@pytest.fixture(scope="module")
def sp():
    import torch
    import paper_conf_asplos_ginsbachrsbdo18_b200 as sp
    torch.cuda.set_device(0)
    return sp


def _dev(a):
    import torch
    return torch.from_numpy(np.ascontiguousarray(a)).cuda()


def _sync():
    import torch
    torch.cuda.synchronize()


# ------------------------------------------------------------ scalar reduction
def _red_bound(n, bound):
    # both sides' rounding (oracle sequential, GPU chunked trees): R30
    return 2.0 * (n + 64) * U * bound


@pytest.mark.parametrize("dt", [np.float64, np.float32])
@pytest.mark.parametrize("n", [0, 1, 3, 7, 1000, 4097, 1_000_003, 12_345_679])
def test_reduce_sum_dot_vs_oracle(sp, dt, n):
    a = gen.uniform(n, seed=n + 1, f32=dt == np.float32)
    b = gen.uniform(n, seed=n + 2, f32=dt == np.float32)
    da, db = _dev(a), _dev(b)
    for bb, db_ in ((None, None), (b, db)):
        ref, bound = oracle.reduce(a, bb)
        got = float(sp.idl_reduce(da, db_).item())
        assert abs(got - ref) <= _red_bound(n, bound), (n, got, ref, bound)


def test_reduce_exact_integers_and_misaligned_views(sp):
    n = 1_000_001
    a = np.arange(1, n + 1, dtype=np.float64)
    da = _dev(a)
    assert sp.idl_reduce(da).item() == n * (n + 1) // 2
    for off in (1, 2, 3):                                        # 8-B and 4-B offsets: scalar path
        assert sp.idl_reduce(da[off:]).item() == n * (n + 1) // 2 - off * (off + 1) // 2
    f = np.arange(0, 4099, dtype=np.float32)
    df = _dev(f)
    assert sp.idl_reduce(df[1:], df[:-1]).item() == float(sum(i * (i - 1) for i in range(1, 4099)))


def test_reduce_deterministic_and_workspace_reuse(sp):
    import torch
    a = _dev(gen.uniform(3_000_017, seed=5))
    b = _dev(gen.uniform(3_000_017, seed=6))
    ws = torch.zeros(sp.idl_reduce_workspace(a.numel()), dtype=torch.uint8, device="cuda")
    outs = [sp.idl_reduce(a, b, workspace=ws).item() for _ in range(5)]
    assert len(set(outs)) == 1
    assert sp.idl_reduce(a, workspace=ws).item() == sp.idl_reduce(a).item()


def test_reduce_full_size_2pow27(sp):
    n = 1 << 27                                                  # 1 GiB of fp64 (NPB IS/EP scale)
    a = gen.uniform(n, seed=77)
    ref, bound = oracle.reduce(a)
    got = sp.idl_reduce(_dev(a)).item()
    assert abs(got - ref) <= _red_bound(n, bound)


def test_reduce_errors(sp):
    import torch
    a = torch.ones(10, dtype=torch.float64, device="cuda")
    with pytest.raises(sp.SpmvError):
        sp.idl_reduce(a.cpu(), out=torch.empty(1, dtype=torch.float64, device="cuda"))   # host input
    with pytest.raises(sp.SpmvError):
        sp.idl_reduce(a, out=a[3:4])                              # out inside a -> alias
    ws = torch.zeros(8, dtype=torch.uint8, device="cuda")
    with pytest.raises(sp.SpmvError):
        sp.idl_reduce(a, workspace=ws)                            # too small


# ------------------------------------------------------------------ histogram
def _keys(n, nbins, seed):
    r = np.random.default_rng(seed)
    return r.integers(-3, nbins + 3, size=n).astype(np.int32)


@pytest.mark.parametrize("mode", ["auto", "smem", "global", "agg"])
@pytest.mark.parametrize("n,nbins", [(1, 1), (1000, 7), (300_001, 2048), (2_000_003, 50_000),
                                     (1_000_000, 1 << 20)])
def test_hist_count_exact(sp, monkeypatch, mode, n, nbins):
    import torch
    if mode != "auto":
        monkeypatch.setenv("SPMV_HIST", mode)
    k = _keys(n, nbins, seed=n ^ nbins)
    old = (np.arange(nbins) * 7).astype(np.uint32)
    ref = oracle.hist_count_u32(k, nbins, old)
    bins = _dev(old)
    sp.idl_histogram("count", _dev(k), bins)
    assert np.array_equal(bins.cpu().numpy(), ref)
    dk = _dev(k)
    bins2 = torch.zeros(nbins, dtype=torch.uint32, device="cuda")
    sp.idl_histogram("count", dk[1:], bins2)                        # unaligned keys view
    assert np.array_equal(bins2.cpu().numpy(), oracle.hist_count_u32(k[1:], nbins))


@pytest.mark.parametrize("cls", ["S", "A", "B", "C"])
def test_hist_count_npb_is_keys(sp, cls):
    """NPB IS key counting (key_buff1[key]++) at every class size up to C (2^27 keys)."""
    import torch
    lk, lm = gen.NPB_IS_CLASSES[cls]
    keys = gen.is_keys(cls)
    ref = oracle.hist_count_u32(keys, 1 << lm)
    bins = torch.zeros(1 << lm, dtype=torch.uint32, device="cuda")
    sp.idl_histogram("count", _dev(keys), bins)
    got = bins.cpu().numpy()
    assert np.array_equal(got, ref) and int(got.sum(dtype=np.int64)) == 1 << lk


@pytest.mark.parametrize("mode", ["auto", "smem", "global", "agg"])
def test_hist_sat_u8_parboil_image(sp, monkeypatch, mode):
    import torch
    if mode != "auto":
        monkeypatch.setenv("SPMV_HIST", mode)
    img = gen.histo_image()
    for nbins in (gen.HISTO_NBINS, 40_000):                       # global and (forced) smem shapes
        k = img % nbins
        old = (np.arange(nbins) % 256).astype(np.uint8)
        ref = oracle.hist_sat_u8(k, nbins, old)
        bins = _dev(old)
        ws = torch.zeros(sp.idl_histogram_workspace("sat_u8", k.size, nbins), dtype=torch.uint8, device="cuda")
        sp.idl_histogram("sat_u8", _dev(k), bins, workspace=ws)
        assert np.array_equal(bins.cpu().numpy(), ref)
        bins.zero_()                                               # workspace left zeroed: reuse
        sp.idl_histogram("sat_u8", _dev(k), bins, workspace=ws)
        assert np.array_equal(bins.cpu().numpy(), oracle.hist_sat_u8(k, nbins))


def test_hist_sat_u8_single_hot_key(sp):
    import torch
    k = np.full(5_000_000, 3, np.int32)
    bins = torch.zeros(8, dtype=torch.uint8, device="cuda")
    sp.idl_histogram("sat_u8", _dev(k), bins)
    assert bins.cpu().numpy().tolist() == [0, 0, 0, 255, 0, 0, 0, 0]


@pytest.mark.parametrize("n,nbins", [(10, 3), (1_000_003, 1000), (2_000_000, 300_000)])
def test_hist_sum_f64_within_bound(sp, n, nbins):
    k = _keys(n, nbins, seed=n + 3)
    w = gen.uniform(n, seed=n + 4)
    old = gen.uniform(nbins, seed=9)
    ref, bound = oracle.hist_sum_f64(k, w, nbins, old)
    bins = _dev(old)
    sp.idl_histogram("sum_f64", _dev(k), bins, w=_dev(w))
    got = bins.cpu().numpy()
    cnt = np.bincount(k[(k >= 0) & (k < nbins)], minlength=nbins)
    assert np.all(np.abs(got - ref) <= 2.0 * (cnt + 2) * U * bound)
    wi = np.random.default_rng(2).integers(-100, 100, size=n).astype(np.float64)   # exact
    bins = _dev(np.zeros(nbins))
    sp.idl_histogram("sum_f64", _dev(k), bins, w=_dev(wi))
    assert np.array_equal(bins.cpu().numpy(), oracle.hist_sum_f64(k, wi, nbins)[0])


def test_hist_errors(sp):
    import torch
    k = torch.zeros(10, dtype=torch.int32, device="cuda")
    bins = torch.zeros(4, dtype=torch.uint32, device="cuda")
    with pytest.raises(sp.SpmvError):
        sp.idl_histogram("count", k, bins, w=torch.zeros(10, dtype=torch.float64, device="cuda"))
    with pytest.raises(sp.SpmvError):
        sp.idl_histogram("count", k, k.view(torch.uint32)[:4])    # bins overlap keys
    sp.idl_histogram("count", k[:0], bins)                         # n = 0: no-op
    assert not bins.cpu().numpy().any()


# ------------------------------------------------------------------------ EP
def _golden_ep():
    with open(os.path.join(GOLD, "npb_ep.txt")) as f:
        return {r[0]: (int(r[1]), float(r[2]), float(r[3]))
                for r in (ln.split() for ln in f if ln.strip() and not ln.startswith("#"))}


@pytest.mark.parametrize("cls", ["S", "W"])
def test_ep_vs_oracle(sp, cls):
    M, sxv, syv = _golden_ep()[cls]
    q, sx, sy = oracle.ep(M)
    out = sp.ep_npb(M).cpu().numpy()
    assert np.array_equal(out[:10], q)                             # integer tallies: exact
    assert abs(out[10] - sx) <= 1e-10 * abs(sxv) and abs(out[11] - sy) <= 1e-10 * abs(syv)


@pytest.mark.parametrize("cls", ["S", "W", "A", "B", "C"])
def test_ep_published_values_full_classes(sp, cls):
    """Full class sizes (C: 2^32 pairs) against NPB's published sx, sy (NPB's 1e-8)."""
    M, sxv, syv = _golden_ep()[cls]
    out = sp.ep_npb(M).cpu().numpy()
    assert abs(out[10] - sxv) <= 1e-8 * abs(sxv) and abs(out[11] - syv) <= 1e-8 * abs(syv)
    assert out[:10].sum() == pytest.approx(math.pi / 4 * 2.0 ** M, rel=1e-3)


def test_ep_ranges_shards_and_determinism(sp):
    import torch
    M = 24
    cuts = [0, 1, 65_535, 65_537, 3_000_000, 1 << 24]               # ragged shards across batches
    parts = [sp.ep_npb(M, a, b - a).cpu().numpy() for a, b in zip(cuts[:-1], cuts[1:])]
    full = sp.ep_npb(M).cpu().numpy()
    tot = np.sum(parts, axis=0)
    assert np.array_equal(tot[:10], full[:10])
    assert abs(tot[10] - full[10]) <= 1e-10 * abs(full[10]) and abs(tot[11] - full[11]) <= 1e-10 * abs(full[11])
    for (a, b), p in zip(zip(cuts[:-1], cuts[1:]), parts):
        if b - a <= 3_000_000:
            q, sx, sy = oracle.ep(M, a, b - a)
            assert np.array_equal(p[:10], q)
            assert abs(p[10] - sx) <= 1e-9 * max(1.0, abs(sx)) and abs(p[11] - sy) <= 1e-9 * max(1.0, abs(sy))
    ws = torch.zeros(sp.ep_npb_workspace(), dtype=torch.uint8, device="cuda")
    runs = [sp.ep_npb(25, workspace=ws).cpu().numpy().tobytes() for _ in range(3)]
    assert len(set(runs)) == 1
    z = sp.ep_npb(M, 5, 0).cpu().numpy()
    assert not z.any()


@pytest.mark.parametrize("kind", ["count", "sat_u8"])
@pytest.mark.parametrize("n,nbins", [(3_000_001, 1_000_003), (600_000, 65_537), (5_000_000, 2_000_000)])
def test_hist_bucketed_exact(sp, monkeypatch, kind, n, nbins):
    """Bucketed counting (partition by key >> 15, shared-memory counts per bucket;
    opt-in via SPMV_HIST=bucket): out-of-range keys skipped, accumulation onto
    old bins, unaligned key views."""
    import torch
    monkeypatch.setenv("SPMV_HIST", "bucket")
    r = np.random.default_rng(n)
    hot = r.integers(0, nbins, size=16)
    k = np.where(r.random(n) < 0.3, hot[r.integers(0, 16, size=n)], r.integers(-7, nbins + 7, size=n)).astype(np.int32)
    dt = np.uint32 if kind == "count" else np.uint8
    old = (np.arange(nbins) % (7 if kind == "count" else 200)).astype(dt)
    for view in (slice(None), slice(1, None)):
        kk = k[view]
        ref = (oracle.hist_count_u32(kk, nbins, old) if kind == "count" else oracle.hist_sat_u8(kk, nbins, old))
        bins = _dev(old)
        wsb = sp.idl_histogram_workspace(kind, kk.size, nbins)
        assert wsb > 2 * kk.size                                   # the bucketed path's scratch is offered
        ws = torch.zeros(wsb, dtype=torch.uint8, device="cuda")
        sp.idl_histogram(kind, _dev(k)[view], bins, workspace=ws)
        assert np.array_equal(bins.cpu().numpy(), ref), (kind, n, nbins, view)
