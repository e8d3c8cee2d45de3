"""ORACLE (test infrastructure only) — ensemble statistics of trajectory cuts.

PAPER.md: a cut is "an array containing the results of all simulations at a given
simulation time" (§IV.A.2); cuts feed statistical engines computing mean and
variance (Fig. 2 label P:L407, on-line estimators P:L689-691).  Histograms/quantiles come
from north_star (cf. StochSimGPU).  Readings R10 (unbiased variance) and R11
(fixed-width histogram with under/overflow bins, inverted-CDF quantiles) in DESIGN.md §3.

Everything is computed from the raw integer samples by its plain definition, with Python
integers for exactness.  Pins: numpy's mean/var/quantile(method='inverted_cdf') on the
same samples (tests/test_oracle_stats.py).
"""
from __future__ import annotations

import math
from dataclasses import dataclass
from typing import Sequence

import numpy as np


@dataclass
class EnsembleStats:
    n: np.ndarray          # [T] int64: instances present at cut k
    sum: np.ndarray        # [T,S] object (Python int)
    sumsq: np.ndarray      # [T,S] object (Python int)
    mean: np.ndarray       # [T,S] float64
    var: np.ndarray        # [T,S] float64, NaN if n < 2
    hist: np.ndarray       # [T,S,B+2] int64: underflow, B bins, overflow
    quantile: np.ndarray   # [T,S,Q] float64
    quantiles: tuple


def hist_bin(x: int, lo: int, width: int, B: int) -> int:
    """0 = underflow (x < lo); 1..B = [lo+(b-1)w, lo+bw); B+1 = overflow."""
    if x < lo:
        return 0
    b = (x - lo) // width
    return B + 1 if b >= B else b + 1


def quantile_from_hist(counts: Sequence[int], n: int, q: float, lo: int, width: int) -> float:
    """Inverted CDF (Hyndman-Fan type 1): smallest bin whose cumulative count reaches
    ceil(q*n) (at least 1); the value is the bin's left edge (exact when width = 1)."""
    if n == 0:
        return math.nan
    need = max(1, math.ceil(q * n))
    c = 0
    for b, cnt in enumerate(counts):
        c += int(cnt)
        if c >= need:
            if b == 0:
                return -math.inf
            if b == len(counts) - 1:
                return math.inf
            return float(lo + width * (b - 1))
    return math.inf


def ensemble_stats(raw: np.ndarray, lo: Sequence[int], width: Sequence[int], B: int,
                   quantiles: Sequence[float]) -> EnsembleStats:
    """raw: [T][S][count] int32 with -1 marking a missing sample (reading R9)."""
    T, S, _ = raw.shape
    n = np.zeros(T, dtype=np.int64)
    ssum = np.empty((T, S), dtype=object)
    ssq = np.empty((T, S), dtype=object)
    mean = np.full((T, S), math.nan)
    var = np.full((T, S), math.nan)
    hist = np.zeros((T, S, B + 2), dtype=np.int64)
    Q = len(quantiles)
    qv = np.full((T, S, Q), math.nan)
    for k in range(T):
        present = raw[k, 0, :] >= 0
        nk = int(present.sum())
        n[k] = nk
        for s in range(S):
            xs = [int(v) for v in raw[k, s, present]]
            sm = sum(xs)
            sq = sum(v * v for v in xs)
            ssum[k, s] = sm
            ssq[k, s] = sq
            if nk > 0:
                mean[k, s] = float(sm) / float(nk)
            if nk > 1:
                var[k, s] = float(nk * sq - sm * sm) / float(nk * (nk - 1))
            for v in xs:
                hist[k, s, hist_bin(v, lo[s], width[s], B)] += 1
            for qi, q in enumerate(quantiles):
                qv[k, s, qi] = quantile_from_hist(hist[k, s], nk, q, lo[s], width[s])
    return EnsembleStats(n, ssum, ssq, mean, var, hist, qv, tuple(quantiles))
