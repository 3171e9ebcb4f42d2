"""Pins for the idiom oracle (oracle/oracle_idioms.c: scalar reduction, Fig. 14;
generalised histogram, Fig. 11; NAS EP) against facts that do not come from the
oracle: exact integer closed forms, numpy/math library routines on the same
data (bincount, fsum), published NPB EP and IS verification values, and the
range-additivity of EP.  All CPU (-m "not gpu").

Plausible bugs each pin catches: a dropped or doubled term (closed-form sums,
bincount), a wrong operand in the dot (one-hot dot), a lost condition
(out-of-range keys, saturation at 255), a wrong acceptance test, deviate or
annulus index in EP (published sx, sy; sum q), a wrong batch seed (published
values at M > MK, range additivity across batches), a wrong key generator or
off-by-one in the count (published IS ranks).
"""
import math
import os

import numpy as np
import pytest

import gen
import oracle

GOLD = os.path.join(os.path.dirname(__file__), "golden")
U = 2.0 ** -53


def _golden(name):
    with open(os.path.join(GOLD, name)) as f:
        return [ln.split() for ln in f if ln.strip() and not ln.startswith("#")]


# ------------------------------------------------------------ scalar reduction
def test_reduce_empty_is_zero():
    s, b = oracle.reduce(np.zeros(0))
    assert s == 0.0 and b == 0.0


@pytest.mark.parametrize("n", [1, 2, 1000, 100_003])
def test_reduce_integer_closed_forms(n):
    a = np.arange(1, n + 1, dtype=np.float64)
    s, b = oracle.reduce(a)
    assert s == n * (n + 1) // 2 and b == s                       # exact: every partial < 2^53
    alt = a * np.where(np.arange(n) % 2 == 0, 1.0, -1.0)         # 1 - 2 + 3 - ...
    s2, b2 = oracle.reduce(alt)
    assert s2 == ((n + 1) // 2 if n % 2 else -(n // 2))
    assert b2 == n * (n + 1) // 2
    s3, _ = oracle.reduce(a, a)                                    # sum of squares
    assert s3 == n * (n + 1) * (2 * n + 1) // 6


def test_reduce_dot_one_hot_picks_operands():
    v = gen.uniform(777, seed=3)
    w = gen.uniform(777, seed=4)
    for j in (0, 5, 776):
        e = np.zeros(777)
        e[j] = 1.0
        assert oracle.reduce(e, v)[0] == v[j]
        assert oracle.reduce(v, e)[0] == v[j]
        e[j] = 2.0
        assert oracle.reduce(e, w)[0] == 2.0 * w[j]


@pytest.mark.parametrize("n", [10, 4096, 1_000_001])
def test_reduce_against_fsum(n):
    a = gen.uniform(n, seed=11)
    b = gen.uniform(n, seed=12)
    s, bound = oracle.reduce(a)
    assert abs(s - math.fsum(a)) <= n * U * bound
    assert bound == pytest.approx(math.fsum(np.abs(a)), rel=n * U)
    sd, bd = oracle.reduce(a, b)
    assert abs(sd - math.fsum(a * b)) <= (n + 1) * U * bd


def test_reduce_f32_terms_in_double():
    a = gen.uniform(5000, seed=5, f32=True)
    b = gen.uniform(5000, seed=6, f32=True)
    s, bound = oracle.reduce(a, b)
    exact = math.fsum(a.astype(np.float64) * b.astype(np.float64))   # float*float is exact in double
    assert abs(s - exact) <= 5000 * U * bound
    ints = np.arange(1000, dtype=np.float32)
    assert oracle.reduce(ints)[0] == 999 * 1000 // 2


# ------------------------------------------------------------------ histogram
def _keys(n, nbins, seed, lo=-5, hi_extra=5):
    r = np.random.default_rng(seed)
    return r.integers(lo, nbins + hi_extra, size=n).astype(np.int32)


@pytest.mark.parametrize("n,nbins", [(0, 10), (1, 1), (10_000, 7), (200_000, 65_536), (50_000, 1_000_003)])
def test_hist_count_matches_bincount(n, nbins):
    k = _keys(n, nbins, seed=n + nbins)
    inr = k[(k >= 0) & (k < nbins)]
    ref = np.bincount(inr, minlength=nbins).astype(np.uint32)
    got = oracle.hist_count_u32(k, nbins)
    assert np.array_equal(got, ref)
    old = np.arange(nbins, dtype=np.uint32)                      # accumulates onto existing bins
    assert np.array_equal(oracle.hist_count_u32(k, nbins, old), old + ref)


def test_hist_count_npb_is_class_s_a_b_ranks():
    """Published NPB IS partial verification (tests/golden/npb_is.txt): 10 iterations x 5 ranks."""
    rows = _golden("npb_is.txt")
    for cls in ("S", "A", "B"):
        lk, lm = gen.NPB_IS_CLASSES[cls]
        nkeys, max_key = 1 << lk, 1 << lm
        keys = gen.is_keys(cls)
        assert keys.min() >= 0 and keys.max() < max_key
        tests = [(int(r[2]), int(r[3]), int(r[4]), int(r[5])) for r in rows if r[0] == cls]
        assert len(tests) == 5
        for it in range(1, 11):
            keys[it] = it
            keys[it + 10] = max_key - it
            cum = np.cumsum(oracle.hist_count_u32(keys, max_key).astype(np.int64))
            assert cum[-1] == nkeys
            for idx, rank, sign, off in tests:
                k = int(keys[idx])
                assert 0 < k <= nkeys - 1
                assert cum[k - 1] == rank + sign * (it - off), (cls, it, idx)


@pytest.mark.parametrize("n,nbins", [(0, 5), (30_000, 100), (300_000, 1 << 20)])
def test_hist_sat_u8_is_min_255(n, nbins):
    k = _keys(n, nbins, seed=7 * n + 1)
    inr = k[(k >= 0) & (k < nbins)]
    cnt = np.bincount(inr, minlength=nbins).astype(np.int64)
    got = oracle.hist_sat_u8(k, nbins)
    assert np.array_equal(got, np.minimum(cnt, 255).astype(np.uint8))
    old = (np.arange(nbins) % 256).astype(np.uint8)
    got2 = oracle.hist_sat_u8(k, nbins, old)
    assert np.array_equal(got2, np.minimum(old.astype(np.int64) + cnt, 255).astype(np.uint8))


def test_hist_sat_u8_single_hot_key():
    k = np.full(100_000, 3, np.int32)
    got = oracle.hist_sat_u8(k, 8)
    assert got[3] == 255 and got.sum() == 255
    assert oracle.hist_sat_u8(k[:254], 8)[3] == 254


def test_hist_parboil_image_shape():
    img = gen.histo_image()
    assert img.shape == (gen.HISTO_NPIX,) and img.min() >= 0 and img.max() < gen.HISTO_NBINS
    h = oracle.hist_sat_u8(img, gen.HISTO_NBINS)
    cnt = np.bincount(img, minlength=gen.HISTO_NBINS)
    assert np.array_equal(h, np.minimum(cnt, 255))
    assert (h == 255).sum() > 100                                  # hot spots saturate (R32)


def test_hist_sum_f64_integer_weights_exact_and_fsum():
    n, nbins = 100_000, 1000
    k = _keys(n, nbins, seed=99)
    inr = (k >= 0) & (k < nbins)
    wi = np.random.default_rng(1).integers(-1000, 1000, size=n).astype(np.float64)
    got, bound = oracle.hist_sum_f64(k, wi, nbins)
    assert np.array_equal(got, np.bincount(k[inr], weights=wi[inr], minlength=nbins))
    assert np.array_equal(bound, np.bincount(k[inr], weights=np.abs(wi[inr]), minlength=nbins))
    w = gen.uniform(n, seed=2)
    got, bound = oracle.hist_sum_f64(k, w, nbins)
    for b in (0, 17, 999):
        sel = w[inr & (k == b)]
        assert abs(got[b] - math.fsum(sel)) <= len(sel) * U * bound[b]


# ------------------------------------------------------------------------ EP
def test_npb_randlc_double_arithmetic_equals_bigint():
    """NPB's 23-bit-split double randlc is the exact LCG x <- 5^13 x mod 2^46."""
    for seed in (271828183, 314159265):
        got = oracle.npb_randlc_stream(3000, seed=float(seed))
        x = seed
        for i in range(3000):
            x = (1220703125 * x) % (1 << 46)
            assert got[i] == x / float(1 << 46)


@pytest.mark.parametrize("cls", ["S", "W"])
def test_ep_published_sums(cls):
    rows = {r[0]: r for r in _golden("npb_ep.txt")}
    M, sxv, syv = int(rows[cls][1]), float(rows[cls][2]), float(rows[cls][3])
    q, sx, sy = oracle.ep(M)
    assert abs(sx - sxv) <= 1e-8 * abs(sxv) and abs(sy - syv) <= 1e-8 * abs(syv)
    npairs = 1 << M
    assert q.sum() == pytest.approx(np.pi / 4 * npairs, rel=1e-3)   # acceptance rate pi/4
    assert np.all(np.diff(q[:6]) < 0) and q[0] > 0


def test_ep_range_additivity_across_batches():
    """Tallies over [0,a) + [a,b) equal [0,b): batch seeds (kk > 0) and pair ranges agree."""
    M = 24
    a, b = 70_000, 200_000                                        # crosses the 65536-pair batches
    q1, sx1, sy1 = oracle.ep(M, 0, a)
    q2, sx2, sy2 = oracle.ep(M, a, b - a)
    q, sx, sy = oracle.ep(M, 0, b)
    assert np.array_equal(q1 + q2, q)
    assert sx1 + sx2 == pytest.approx(sx, rel=1e-12, abs=1e-9)
    assert sy1 + sy2 == pytest.approx(sy, rel=1e-12, abs=1e-9)
    q0, sx0, sy0 = oracle.ep(M, 5, 0)
    assert q0.sum() == 0 and sx0 == 0.0 and sy0 == 0.0
    with pytest.raises(ValueError):
        oracle.ep(M, (1 << M) - 1, 2)


def test_ep_first_pairs_by_hand():
    """The first pairs recomputed from the published LCG definition (big integers)."""
    x, vals = 271828183, []
    for _ in range(40):
        x = (1220703125 * x) % (1 << 46)
        vals.append(x / float(1 << 46))
    acc, sx = 0, 0.0
    for i in range(20):
        x1, x2 = 2.0 * vals[2 * i] - 1.0, 2.0 * vals[2 * i + 1] - 1.0
        t = x1 * x1 + x2 * x2
        if t <= 1.0:
            acc += 1
            sx += x1 * math.sqrt(-2.0 * math.log(t) / t)
    q, osx, _ = oracle.ep(24, 0, 20)
    assert q.sum() == acc
    assert osx == pytest.approx(sx, rel=1e-13)
