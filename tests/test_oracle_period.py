"""Pins for oracle/period.py (reading R19) on hand-built cut series with hand-counted events."""
import numpy as np

from oracle.period import detect, finalize, period_stats


def test_schmitt_trigger_events():
    lo, hi = 2, 8
    #         0  1  2  3  4  5  6  7  8  9 10 11 12 13
    series = [5, 9, 1, 4, 8, 9, 3, 2, 5, 9, 0, 10, 1, 7]
    # armed at k=2 (1 <= 2) -> fires at k=4 (8 >= 8); k=1 is not an event (never armed);
    # re-armed at k=7 (2 <= 2) -> fires at k=9; armed at k=10 -> fires at k=11; k=12 arms only
    events, periods = detect(series, lo, hi)
    assert events == [4, 9, 11]
    assert periods == [(9, 5), (11, 2)]


def test_no_rearm_without_dip_and_missing_cuts():
    assert detect([0, 9, 9, 5, 9, 9], 2, 8) == ([1], [])
    # a frozen (overflowed) instance contributes nothing after its last present cut
    assert detect([0, 9, 0, -1, -1], 2, 8) == ([1], [])


def test_period_stats_and_moving_average():
    lo, hi = 2, 8
    a = [0, 9, 0, 0, 9, 1, 9, 1, 1, 1]      # events 1, 4, 6 -> periods 3 (at 4), 2 (at 6)
    b = [9, 0, 1, 9, 1, 1, 1, 1, 9, 9]      # events 3, 8 -> period 5 (at 8)
    raw = np.array([a, b], dtype=np.int32).T[:, None, :]   # [T=10][S=1][2]
    ps = period_stats(raw, 0, lo, hi)
    assert ps.ev.tolist() == [0, 1, 0, 1, 1, 0, 1, 0, 1, 0]
    assert ps.pc_n.tolist() == [0, 0, 0, 0, 1, 0, 1, 0, 1, 0]
    assert ps.pc_sum.tolist() == [0, 0, 0, 0, 3, 0, 2, 0, 5, 0]
    # local period: a has 3 from k=4, 2 from k=6; b has 5 from k=8
    assert ps.lp_n.tolist() == [0, 0, 0, 0, 1, 1, 1, 1, 2, 2]
    assert ps.lp_sum.tolist() == [0, 0, 0, 0, 3, 3, 2, 2, 7, 7]
    assert list(ps.lp_sq) == [0, 0, 0, 0, 9, 9, 4, 4, 29, 29]
    lp_mean, ma, lp_var = finalize(ps, 0.5, window=3)
    assert lp_var[8] == (2 * 29 - 49) / 2 * 0.25 and np.isnan(lp_var[7])
    assert lp_mean[4] == 1.5 and lp_mean[9] == 3.5 * 0.5 and np.isnan(lp_mean[3])
    # window of 3 cuts ending at k: periods completing in [k-2, k]
    assert np.isnan(ma[3]) and ma[4] == 1.5 and ma[6] == (3 + 2) / 2 * 0.5 and ma[8] == (2 + 5) / 2 * 0.5
    assert ma[9] == 5 * 0.5
