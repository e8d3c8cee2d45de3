"""ORACLE (test infrastructure only) — on-line oscillation-period analysis of trajectory cuts.

PAPER.md P:L541-545 (§V.B): "We compute the period of each oscillation and plot the moving
average of more than 200 simulations of the local period"; the analysis runs on sliding
windows over the stream of cuts (§IV.A.2).  The paper defines neither the period
detector nor the window; reading R19 fixes them:

* observable: one flat species s*, sampled on the cut grid (x_k = x_{s*}(t_k), present cuts);
* events: a Schmitt trigger with integer thresholds lo < hi — the detector is armed by a cut
  with x_k <= lo and fires (an "oscillation peak event", disarming it) at the first later cut
  with x_k >= hi;
* the m-th period of an instance is p_m = e_m - e_{m-1} cuts between consecutive events;
* per cut k (exact integers): ev[k] = events at k; pc_n/pc_sum/pc_sq[k] = periods completing
  at k; lp_n/lp_sum/lp_sq[k] = "local period" — the last completed period of every instance
  present at cut k that has one;
* finalize: mean local period per cut and the sliding-window ("moving") average of the periods
  completed in the W cuts ending at k, both in time units (x dt).

Pins: tests/test_oracle_period.py (hand-built series with hand-counted events).
"""
from __future__ import annotations

from dataclasses import dataclass

import numpy as np


@dataclass
class PeriodStats:
    ev: np.ndarray        # [T] int
    pc_n: np.ndarray      # [T]
    pc_sum: np.ndarray    # [T]
    pc_sq: np.ndarray     # [T] object (Python int)
    lp_n: np.ndarray
    lp_sum: np.ndarray
    lp_sq: np.ndarray     # object


def detect(series, lo: int, hi: int):
    """Events and (completion cut, period) pairs of one instance's cut series (-1 = missing)."""
    armed = False
    last = None
    events, periods = [], []
    for k, x in enumerate(series):
        if x < 0:
            break                      # frozen after an overflow: no further cuts (R9)
        if x <= lo:
            armed = True
        if armed and x >= hi:
            events.append(k)
            armed = False
            if last is not None:
                periods.append((k, k - last))
            last = k
    return events, periods


def period_stats(raw: np.ndarray, species: int, lo: int, hi: int) -> PeriodStats:
    """raw: [T][S][count] int32 cuts (-1 missing)."""
    T = raw.shape[0]
    ev = np.zeros(T, dtype=np.int64)
    pc_n = np.zeros(T, dtype=np.int64)
    pc_sum = np.zeros(T, dtype=np.int64)
    pc_sq = np.array([0] * T, dtype=object)
    lp_n = np.zeros(T, dtype=np.int64)
    lp_sum = np.zeros(T, dtype=np.int64)
    lp_sq = np.array([0] * T, dtype=object)
    for i in range(raw.shape[2]):
        series = [int(v) for v in raw[:, species, i]]
        events, periods = detect(series, lo, hi)
        for k in events:
            ev[k] += 1
        done = {k: p for k, p in periods}
        local = None
        for k, x in enumerate(series):
            if x < 0:
                break
            if k in done:
                local = done[k]
                pc_n[k] += 1
                pc_sum[k] += local
                pc_sq[k] += local * local
            if local is not None:
                lp_n[k] += 1
                lp_sum[k] += local
                lp_sq[k] += local * local
    return PeriodStats(ev, pc_n, pc_sum, pc_sq, lp_n, lp_sum, lp_sq)


def finalize(ps: PeriodStats, dt: float, window: int):
    """Mean local period per cut, the W-cut moving average of completed periods (time units) and
    the unbiased variance of the local period (time^2): (mean, moving average, variance)."""
    T = len(ps.ev)
    lp_mean = np.array([float(int(ps.lp_sum[k])) / float(int(ps.lp_n[k])) * dt if ps.lp_n[k] else np.nan
                        for k in range(T)])
    lp_var = np.full(T, np.nan)
    for k in range(T):
        n = int(ps.lp_n[k])
        if n > 1:
            s, q = int(ps.lp_sum[k]), int(ps.lp_sq[k])
            lp_var[k] = float(n * q - s * s) / float(n * (n - 1)) * dt * dt
    ma = np.full(T, np.nan)
    for k in range(T):
        a = max(0, k - window + 1)
        n = int(ps.pc_n[a:k + 1].sum())
        s = int(ps.pc_sum[a:k + 1].sum())
        if n:
            ma[k] = float(s) / float(n) * dt
    return lp_mean, ma, lp_var
