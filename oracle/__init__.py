"""ORACLE — test infrastructure only.

Plain, slow, obviously-correct CPU reference of the CWC ensemble-SSA hot path
(readings R1-R15 in DESIGN.md §3).

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s ``cpu_baseline`` /
``--impl reference`` legs may import this package.  It shares no code with the product
package ``paper_conf_icdcsw_aldinuccidpmtt14_b200`` and never imports it; the one module
both sides import is ``workloads`` (inputs only).

Parts:
  * ``ssa.c``        — Philox4x32-10, CWC-log, direct-method SSA, sampler (C, -ffp-contract=off)
  * ``cwc_terms.py`` — CWC parser + tree matching -> flat reactions (Python)
  * ``stats.py``     — ensemble statistics from raw samples (exact integers, numpy)
"""
from __future__ import annotations

import ctypes
import os
import subprocess
from dataclasses import dataclass
from typing import Optional, Sequence

import numpy as np

from .cwc_terms import CWCError, FlatModel, flatten, flatten_def  # noqa: F401

_HERE = os.path.dirname(os.path.abspath(__file__))
_SO = os.path.join(_HERE, "liboracle.so")
_SRC = os.path.join(_HERE, "ssa.c")

FLAG_ABSORBED = 1
FLAG_OVERFLOWED = 2


def build(force: bool = False) -> str:
    """Compile oracle/ssa.c -> oracle/liboracle.so (gcc, -O2 -ffp-contract=off)."""
    if force or not os.path.exists(_SO) or os.path.getmtime(_SO) < os.path.getmtime(_SRC):
        cmd = ["gcc", "-O2", "-ffp-contract=off", "-fno-fast-math", "-std=c11", "-fPIC", "-shared",
               "-pthread", "-o", _SO + ".tmp", _SRC, "-lm"]
        subprocess.check_call(cmd)
        os.replace(_SO + ".tmp", _SO)
    return _SO


class _Model(ctypes.Structure):
    _fields_ = [
        ("S", ctypes.c_int32), ("M", ctypes.c_int32),
        ("x0", ctypes.POINTER(ctypes.c_int32)),
        ("k", ctypes.POINTER(ctypes.c_double)),
        ("n_react", ctypes.POINTER(ctypes.c_int32)),
        ("react_s", ctypes.POINTER(ctypes.c_int32)),
        ("react_r", ctypes.POINTER(ctypes.c_int32)),
        ("delta", ctypes.POINTER(ctypes.c_int32)),
        ("x_cap", ctypes.c_int64),
        ("law", ctypes.POINTER(ctypes.c_int32)),
        ("law_s", ctypes.POINTER(ctypes.c_int32)),
        ("law_K", ctypes.POINTER(ctypes.c_double)),
        ("law_n", ctypes.POINTER(ctypes.c_int32)),
    ]


_lib = None


def lib():
    global _lib
    if _lib is None:
        _lib = ctypes.CDLL(build())
        _lib.oracle_philox4x32_10.argtypes = [ctypes.POINTER(ctypes.c_uint32)] * 3
        _lib.oracle_u01.argtypes = [ctypes.c_uint32, ctypes.c_uint32]
        _lib.oracle_u01.restype = ctypes.c_double
        _lib.oracle_cwclog.argtypes = [ctypes.c_double]
        _lib.oracle_cwclog.restype = ctypes.c_double
        _lib.oracle_cwclog_table.argtypes = [ctypes.POINTER(ctypes.c_double)] * 3
        _lib.oracle_simulate.argtypes = [
            ctypes.POINTER(_Model), ctypes.c_int64, ctypes.c_int64, ctypes.c_int64, ctypes.c_double,
            ctypes.c_uint64, ctypes.c_int32, ctypes.c_void_p, ctypes.c_void_p, ctypes.c_void_p]
        _lib.oracle_simulate.restype = ctypes.c_int
        _lib.oracle_propensities.argtypes = [ctypes.POINTER(_Model), ctypes.c_void_p,
                                             ctypes.c_void_p, ctypes.c_void_p]
    return _lib


def philox4x32_10(ctr: Sequence[int], key: Sequence[int]):
    c = (ctypes.c_uint32 * 4)(*ctr)
    k = (ctypes.c_uint32 * 2)(*key)
    o = (ctypes.c_uint32 * 4)()
    lib().oracle_philox4x32_10(c, k, o)
    return tuple(o)


def u01(lo: int, hi: int) -> float:
    return lib().oracle_u01(lo, hi)


def cwclog(x: float) -> float:
    return lib().oracle_cwclog(x)


def cwclog_table():
    a = (ctypes.c_double * 128)()
    b = (ctypes.c_double * 128)()
    c = (ctypes.c_double * 128)()
    lib().oracle_cwclog_table(a, b, c)
    return np.array(a), np.array(b), np.array(c)


class CModel:
    """Flat model marshalled for ssa.c (keeps the numpy buffers alive)."""

    def __init__(self, fm: FlatModel):
        S, M = len(fm.names), len(fm.rates)
        self.fm = fm
        self.S, self.M = S, M
        self.x0 = np.array(fm.x0, dtype=np.int32)
        self.k = np.array(fm.rates, dtype=np.float64) if M else np.zeros(1)
        self.n_react = np.array([len(r) for r in fm.reactants] or [0], dtype=np.int32)
        self.react_s = np.zeros(max(M, 1) * 4, dtype=np.int32)
        self.react_r = np.zeros(max(M, 1) * 4, dtype=np.int32)
        for j, rl in enumerate(fm.reactants):
            for e, (s, r) in enumerate(rl):
                self.react_s[j * 4 + e] = s
                self.react_r[j * 4 + e] = r
        self.delta = np.array(fm.delta, dtype=np.int32).reshape(-1) if M else np.zeros(1, np.int32)
        nz = max(M, 1)
        self.law = np.array(fm.law or [0] * nz, dtype=np.int32)
        self.law_s = np.array(fm.law_species or [-1] * nz, dtype=np.int32)
        self.law_K = np.array(fm.law_K or [0.0] * nz, dtype=np.float64)
        self.law_n = np.array(fm.law_n or [1] * nz, dtype=np.int32)
        P = lambda a, t: a.ctypes.data_as(ctypes.POINTER(t))  # noqa: E731
        self.c = _Model(S, M, P(self.x0, ctypes.c_int32), P(self.k, ctypes.c_double),
                        P(self.n_react, ctypes.c_int32), P(self.react_s, ctypes.c_int32),
                        P(self.react_r, ctypes.c_int32), P(self.delta, ctypes.c_int32), fm.x_cap,
                        P(self.law, ctypes.c_int32), P(self.law_s, ctypes.c_int32),
                        P(self.law_K, ctypes.c_double), P(self.law_n, ctypes.c_int32))

    def propensities(self, x):
        x = np.ascontiguousarray(x, dtype=np.int32)
        a = np.zeros(max(self.M, 1))
        cum = np.zeros(max(self.M, 1))
        lib().oracle_propensities(ctypes.byref(self.c), x.ctypes.data, a.ctypes.data, cum.ctypes.data)
        return a[: self.M], cum[: self.M]


def grid_K(t_end: float, dt: float) -> int:
    """K = llround(t_end/dt); |K*dt - t_end| <= 1e-9*max(1, t_end) (reading R13)."""
    if not (dt > 0) or not (t_end >= 0):
        raise CWCError("invalid", "need dt > 0 and t_end >= 0")
    K = int(round(t_end / dt))
    if abs(K * dt - t_end) > 1e-9 * max(1.0, t_end):
        raise CWCError("invalid", "t_end is not a multiple of sample_dt")
    return K


@dataclass
class OracleRun:
    raw: Optional[np.ndarray]    # [T][S][count] int32, -1 = missing
    flags: np.ndarray            # [count] uint8
    reactions: np.ndarray        # [count] int64
    first: int
    K: int


def simulate(model, first: int, count: int, t_end: float, dt: float, seed: int,
             nthreads: int = 1, raw: bool = True) -> OracleRun:
    """Simulate global instances [first, first+count). ``model`` is a ModelDef, FlatModel or CModel."""
    if isinstance(model, CModel):
        cm = model
    else:
        fm = model if isinstance(model, FlatModel) else flatten_def(model)
        cm = CModel(fm)
    K = grid_K(t_end, dt)
    rawbuf = np.empty((K + 1, cm.S, count), dtype=np.int32) if raw else None
    flags = np.zeros(count, dtype=np.uint8)
    reactions = np.zeros(count, dtype=np.int64)
    rc = lib().oracle_simulate(ctypes.byref(cm.c), first, count, K, dt, seed, nthreads,
                               rawbuf.ctypes.data if raw else None, flags.ctypes.data,
                               reactions.ctypes.data)
    if rc != 0:
        raise CWCError("invalid", "oracle_simulate rejected its arguments")
    return OracleRun(rawbuf, flags, reactions, first, K)
