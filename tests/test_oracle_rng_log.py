"""Pins for the oracle's RNG stream (reading R3) and CWC-log (reading R4).

Philox4x32-10 is pinned to the Random123 known-answer vectors (tests/golden); the uniform
mapping is pinned by its exact bit pattern; CWC-log is pinned to the mathematical log
computed by mpmath at 60 significant digits (error <= 1 ulp on the whole input range the
SSA uses, u in [2^-53, 1)).
"""
import math
import os
import struct

import numpy as np
import pytest

GOLDEN = os.path.join(os.path.dirname(__file__), "golden")


def _kat():
    rows = []
    with open(os.path.join(GOLDEN, "philox4x32_10_kat.txt")) as f:
        for line in f:
            if line.startswith("#") or not line.strip():
                continue
            v = [int(t, 16) for t in line.split()]
            rows.append((v[0:4], v[4:6], v[6:10]))
    return rows


def test_philox_known_answers(oracle_lib):
    rows = _kat()
    assert len(rows) == 3
    for ctr, key, out in rows:
        assert list(oracle_lib.philox4x32_10(ctr, key)) == out


def test_u01_bit_pattern(oracle_lib):
    # u = (2m+1) 2^-53, m = top 52 bits of (hi:lo)
    assert oracle_lib.u01(0, 0) == 2.0 ** -53
    assert oracle_lib.u01(0xFFFFFFFF, 0xFFFFFFFF) == 1.0 - 2.0 ** -53
    assert oracle_lib.u01(0xFFF, 0) == 2.0 ** -53            # low 12 bits dropped
    assert oracle_lib.u01(0x1000, 0) == 3 * 2.0 ** -53
    assert oracle_lib.u01(0, 0x80000000) == 0.5 + 2.0 ** -53
    rng = np.random.default_rng(1)
    for lo, hi in rng.integers(0, 2 ** 32, size=(2000, 2), dtype=np.uint64):
        u = oracle_lib.u01(int(lo), int(hi))
        m = ((int(hi) << 32) | int(lo)) >> 12
        assert 0.0 < u < 1.0
        assert u == (2 * m + 1) / 2.0 ** 53


def _ulp(x):
    return math.ulp(x)


def test_cwclog_within_one_ulp(oracle_lib):
    mpmath = pytest.importorskip("mpmath")
    mpmath.mp.dps = 60
    rng = np.random.default_rng(12345)
    us = list(rng.random(6000))
    # log-uniform over the full SSA range [2^-53, 1)
    us += list(np.exp2(-rng.random(4000) * 53.0))
    # table-boundary and special neighbourhoods
    for e in range(-53, 1):
        for z in (0.6875, 0.6875 + 1e-12, 0.75, 0.999, 1.0 - 2 ** -53, 1.0, 1.0 + 2 ** -52, 1.0078125,
                  1.2, 1.375 - 2 ** -52):
            v = math.ldexp(z, e)
            if 2 ** -53 <= v < 1.0:
                us.append(v)
    us += [2 ** -53, 1 - 2 ** -53, 0.5, 0.25, 1 - 2 ** -20]
    worst = 0.0
    for u in us:
        got = oracle_lib.cwclog(float(u))
        ref = mpmath.log(mpmath.mpf(float(u)))
        err = abs(mpmath.mpf(got) - ref) / mpmath.mpf(_ulp(float(ref)))
        worst = max(worst, float(err))
        assert err <= 1.0, (u, got, float(ref))
    assert worst < 1.0


def test_cwclog_table_shape(oracle_lib):
    invc, logc, logclo = oracle_lib.cwclog_table()
    assert invc[79] == 1.0 and invc[80] == 1.0 and logc[79] == 0.0 and logc[80] == 0.0
    # |log(c_i)| grows away from the entries around 1
    assert np.all(np.abs(logc[:79]) > 0) and np.all(np.abs(logc[81:]) > 0)
    # invc_i * c_i ~ 1 within an ulp for the midpoints
    for i in list(range(0, 79)) + list(range(81, 128)):
        zlo = struct.unpack("<d", struct.pack("<Q", 0x3FE6000000000000 + (i << 45)))[0]
        zhi = struct.unpack("<d", struct.pack("<Q", 0x3FE6000000000000 + ((i + 1) << 45)))[0]
        c = (zlo + zhi) / 2
        assert abs(invc[i] * c - 1.0) < 2e-16
        assert abs(logc[i] - math.log(c)) < 2e-16
        assert abs(logclo[i]) <= math.ulp(logc[i]) / 2
