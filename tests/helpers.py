"""Test helpers: run the product path on the GPU and compare it with the oracle."""
import math

import numpy as np

import oracle
from oracle.stats import ensemble_stats


def gpu_run(model_def, n_total, first, count, t_end, dt, seed, *, hist_bins=256, hist_width=1, hist_lo=0,
            quantiles=(0.05, 0.25, 0.5, 0.75, 0.95), raw=True, copy_raw=True, **opts):
    """Product path: load, simulate [first, first+count), return (result, raw, flags, reactions, model)
    (raw = None when raw samples are off or copy_raw is False; read them with model.samples)."""
    import paper_conf_icdcsw_aldinuccidpmtt14_b200 as cwc
    m = cwc.Model.from_def(model_def, hist_bins=hist_bins, hist_width=hist_width, hist_lo=hist_lo,
                           quantiles=quantiles, raw_samples=raw, **opts)
    m.simulate_range(n_total, first, count, t_end, dt, seed)
    res = m.finalize()
    samples = m.samples(0, count) if raw and copy_raw else None
    flags, reactions, _ = m.records(0, count)
    return res, samples, flags, reactions, m


def numpy_stats(raw, lo, width, B):
    """Exact integer stats of raw [T][S][N] samples (-1 missing), numpy-vectorised."""
    T, S, N = raw.shape
    present = raw[:, 0, :] >= 0
    n = present.sum(axis=1).astype(np.int64)
    x = np.where(present[:, None, :], raw, 0).astype(np.int64)
    ssum = x.sum(axis=2)
    sq = x * x
    sqlo = (sq & 0xFFFFFFFF).sum(axis=2)
    sqhi = (sq >> 32).sum(axis=2)
    hist = np.zeros((T, S, B + 2), dtype=np.int64)
    for s in range(S):
        d = raw[:, s, :].astype(np.int64) - lo[s]
        b = np.where(d < 0, 0, np.minimum(d // width[s], B) + 1)
        b = np.where(d >= B * width[s], B + 1, b)
        for k in range(T):
            hist[k, s] = np.bincount(b[k][present[k]], minlength=B + 2)
    return n, ssum, sqlo, sqhi, hist


def assert_stats_match_raw(res, raw):
    B = res.hist.shape[2] - 2
    n, ssum, sqlo, sqhi, hist = numpy_stats(raw, res.hist_lo, res.hist_width, B)
    assert np.array_equal(res.n, n)
    assert np.array_equal(res.sum, ssum)
    assert np.array_equal(res.sqlo, sqlo)
    assert np.array_equal(res.sqhi, sqhi)
    assert np.array_equal(res.hist, hist)


def assert_matches_oracle_stats(res, oraw, quantiles):
    """GPU finalised stats == oracle stats computed from the oracle's own raw samples."""
    B = res.hist.shape[2] - 2
    st = ensemble_stats(oraw, list(res.hist_lo), list(res.hist_width), B, quantiles)
    assert np.array_equal(res.n, st.n)
    T, S = res.sum.shape
    exact = res.sumsq_exact()
    for k in range(T):
        for s in range(S):
            assert int(res.sum[k, s]) == st.sum[k, s]
            assert exact[k, s] == st.sumsq[k, s]
    assert np.array_equal(res.hist, st.hist)
    same = lambda a, b: np.array_equal(a, b, equal_nan=True)  # noqa: E731
    assert same(res.mean, st.mean)
    assert same(res.var, st.var)
    assert same(res.quantile, st.quantile)
