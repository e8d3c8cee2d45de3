"""Pins for oracle/stats.py (readings R10, R11) against numpy's own estimators.

mean = numpy mean, var = numpy var(ddof=1), histogram = numpy.histogram with explicit
edges plus under/overflow counts, quantile = numpy.quantile(method='inverted_cdf')
(Hyndman-Fan type 1) for width-1 bins.  Missing samples (-1, reading R9) are excluded.
"""
import math

import numpy as np

from oracle.stats import ensemble_stats, hist_bin


def _raw(seed, T=7, S=3, N=301, lo=0, hi=60, miss=0.1):
    rng = np.random.default_rng(seed)
    raw = rng.integers(lo, hi, size=(T, S, N)).astype(np.int32)
    # missing = an instance frozen from some k on (all species together)
    for i in range(N):
        if rng.random() < miss:
            k0 = int(rng.integers(1, T))
            raw[k0:, :, i] = -1
    return raw


def test_moments_match_numpy():
    raw = _raw(1)
    st = ensemble_stats(raw, [0, 0, 0], [1, 1, 1], 64, (0.05, 0.5, 0.95))
    for k in range(raw.shape[0]):
        pres = raw[k, 0] >= 0
        assert st.n[k] == pres.sum()
        for s in range(raw.shape[1]):
            x = raw[k, s, pres].astype(np.int64)
            assert st.sum[k, s] == int(x.sum()) and st.sumsq[k, s] == int((x * x).sum())
            assert math.isclose(st.mean[k, s], x.mean(), rel_tol=1e-15)
            assert math.isclose(st.var[k, s], x.var(ddof=1), rel_tol=1e-12)


def test_quantiles_inverted_cdf():
    raw = _raw(2, hi=40)
    qs = (0.0, 0.05, 0.25, 0.5, 0.75, 0.95, 1.0, 0.333)
    st = ensemble_stats(raw, [0, 0, 0], [1, 1, 1], 64, qs)
    for k in range(raw.shape[0]):
        pres = raw[k, 0] >= 0
        for s in range(raw.shape[1]):
            x = raw[k, s, pres]
            for qi, q in enumerate(qs):
                assert st.quantile[k, s, qi] == np.quantile(x, q, method="inverted_cdf"), (k, s, q)


def test_histogram_edges():
    raw = _raw(3, lo=-5, hi=300)
    lo, width, B = [0, 10, -3], [4, 16, 1], 16
    st = ensemble_stats(raw, lo, width, B, (0.5,))
    for k in range(raw.shape[0]):
        pres = raw[k, 0] >= 0
        for s in range(raw.shape[1]):
            x = raw[k, s, pres]
            edges = lo[s] + width[s] * np.arange(B + 1)
            inner, _ = np.histogram(x, bins=edges)
            # numpy's last bin is closed on the right; ours is half-open -> count separately
            inner[-1] -= int((x == edges[-1]).sum())
            assert st.hist[k, s, 0] == (x < lo[s]).sum()
            assert np.array_equal(st.hist[k, s, 1:B + 1], inner)
            assert st.hist[k, s, B + 1] == (x >= edges[-1]).sum()
    assert hist_bin(-1, 0, 1, 4) == 0 and hist_bin(0, 0, 1, 4) == 1 and hist_bin(3, 0, 1, 4) == 4
    assert hist_bin(4, 0, 1, 4) == 5


def test_small_n_edge_cases():
    raw = np.full((2, 1, 3), -1, dtype=np.int32)
    raw[0, 0, 0] = 5
    st = ensemble_stats(raw, [0], [1], 8, (0.5,))
    assert st.n.tolist() == [1, 0]
    assert st.mean[0, 0] == 5.0 and math.isnan(st.var[0, 0])
    assert math.isnan(st.mean[1, 0]) and math.isnan(st.quantile[1, 0, 0])
    assert st.quantile[0, 0, 0] == 5.0
