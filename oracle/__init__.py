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
        ("gate_s", ctypes.POINTER(ctypes.c_int32)),
        ("gate_k", ctypes.POINTER(ctypes.c_int32)),
        ("place_off", ctypes.POINTER(ctypes.c_int32)),
        ("place_alive", ctypes.POINTER(ctypes.c_int32)),
        ("add_off", ctypes.POINTER(ctypes.c_int32)),
        ("add_s", ctypes.POINTER(ctypes.c_int32)),
        ("add_n", ctypes.POINTER(ctypes.c_int32)),
        ("xfer_off", ctypes.POINTER(ctypes.c_int32)),
        ("xfer_src", ctypes.POINTER(ctypes.c_int32)),
        ("xfer_dst", ctypes.POINTER(ctypes.c_int32)),
        ("sentinel", ctypes.c_int32),
    ]

RMAX = 8  # reactant entries per flat reaction (ORACLE_RMAX in ssa.c)


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
        _lib.oracle_step_with_draws.argtypes = [
            ctypes.POINTER(_Model), ctypes.c_void_p, ctypes.POINTER(ctypes.c_double), ctypes.POINTER(ctypes.c_int64),
            ctypes.c_int64, ctypes.c_double, ctypes.c_int32, ctypes.c_void_p, ctypes.c_void_p, ctypes.c_void_p,
            ctypes.c_void_p, ctypes.POINTER(ctypes.c_int32)]
        _lib.oracle_step_with_draws.restype = ctypes.c_int
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
        self.react_s = np.zeros(max(M, 1) * RMAX, dtype=np.int32)
        self.react_r = np.zeros(max(M, 1) * RMAX, dtype=np.int32)
        for j, rl in enumerate(fm.reactants):
            if len(rl) > RMAX:
                raise CWCError("unsupported", f"flat reaction {j} has more than {RMAX} reactant species")
            for e, (s, r) in enumerate(rl):
                self.react_s[j * RMAX + e] = s
                self.react_r[j * RMAX + e] = r
        self.delta = np.array(fm.delta, dtype=np.int32).reshape(-1) if M else np.zeros(1, np.int32)
        nz = max(M, 1)
        self.law = np.array(fm.law or [0] * nz, dtype=np.int32)
        self.law_s = np.array(fm.law_species or [-1] * nz, dtype=np.int32)
        self.law_K = np.array(fm.law_K or [0.0] * nz, dtype=np.float64)
        self.law_n = np.array(fm.law_n or [1] * nz, dtype=np.int32)
        # reading R20: gates, creations (place), destructions (transfer), the "#full" sentinel
        self.gate_s = np.array(fm.gate_species or [-1] * nz, dtype=np.int32)
        self.gate_k = np.array(fm.gate_kind or [0] * nz, dtype=np.int32)
        place = fm.place or [[] for _ in range(M)]
        xfer = fm.transfer or [[] for _ in range(M)]
        self.place_off = np.cumsum([0] + [len(p) for p in place]).astype(np.int32)
        self.place_alive = np.array([al for p in place for al, _ in p] or [0], dtype=np.int32)
        self.add_off = np.cumsum([0] + [len(ad) for p in place for _, ad in p]).astype(np.int32)
        self.add_s = np.array([sp for p in place for _, ad in p for sp, _ in ad] or [0], dtype=np.int32)
        self.add_n = np.array([n for p in place for _, ad in p for _, n in ad] or [0], dtype=np.int32)
        self.xfer_off = np.cumsum([0] + [len(x) for x in xfer]).astype(np.int32)
        self.xfer_src = np.array([a for x in xfer for a, _ in x] or [0], dtype=np.int32)
        self.xfer_dst = np.array([b for x in xfer for _, b in x] or [0], dtype=np.int32)
        P = lambda a, t: a.ctypes.data_as(ctypes.POINTER(t))  # noqa: E731
        I = lambda a: P(a, ctypes.c_int32)  # noqa: E731
        self.c = _Model(S, M, I(self.x0), P(self.k, ctypes.c_double),
                        I(self.n_react), I(self.react_s), I(self.react_r), I(self.delta), fm.x_cap,
                        I(self.law), I(self.law_s), P(self.law_K, ctypes.c_double), I(self.law_n),
                        I(self.gate_s), I(self.gate_k), I(self.place_off), I(self.place_alive),
                        I(self.add_off), I(self.add_s), I(self.add_n), I(self.xfer_off), I(self.xfer_src),
                        I(self.xfer_dst), int(fm.sentinel))

    def propensities(self, x):
        x = np.ascontiguousarray(x, dtype=np.int32)
        a = np.zeros(max(self.M, 1))
        cum = np.zeros(max(self.M, 1))
        lib().oracle_propensities(ctypes.byref(self.c), x.ctypes.data, a.ctypes.data, cum.ctypes.data)
        return a[: self.M], cum[: self.M]


# status of an injected-draw step (ssa.c ssa_step)
STEP_JUMP, STEP_ABSORBED, STEP_OVERFLOWED, STEP_HORIZON = 0, 1, 2, 3


@dataclass
class StepRun:
    x: np.ndarray          # [S] state after the steps
    t: float               # time of the last applied jump
    k: int                 # next cut index
    status: int            # STEP_* of the last step taken
    n_done: int            # steps taken (the last one may be a non-jump)
    js: np.ndarray         # [n_done] selected reaction of each step (-1: no jump)
    cuts: np.ndarray       # [K+1][S] cuts emitted (-2 = not emitted by these steps, -1 = missing)


def step_with_draws(model, x, t: float, k: int, K: int, dt: float, u_tau, u_sel) -> StepRun:
    """Injected-draw trajectory: from state (x, t, next cut k), the direct-method steps of ssa.c
    with the given uniforms instead of Philox draws (R6/R7 pins with crafted draws; the
    device counterpart is cwc_selftest_step)."""
    cm = model if isinstance(model, CModel) else CModel(model if isinstance(model, FlatModel) else flatten_def(model))
    xs = np.ascontiguousarray(x, dtype=np.int32).copy()
    ut = np.ascontiguousarray(u_tau, dtype=np.float64)
    us = np.ascontiguousarray(u_sel, dtype=np.float64)
    n = len(ut)
    cuts = np.full((K + 1, cm.S), -2, dtype=np.int32)
    js = np.full(max(n, 1), -1, dtype=np.int32)
    tt = ctypes.c_double(t)
    kk = ctypes.c_int64(k)
    nd = ctypes.c_int32(0)
    st = lib().oracle_step_with_draws(ctypes.byref(cm.c), xs.ctypes.data, ctypes.byref(tt), ctypes.byref(kk), K, dt,
                                      n, ut.ctypes.data, us.ctypes.data, cuts.ctypes.data, js.ctypes.data,
                                      ctypes.byref(nd))
    if st < 0:
        raise CWCError("invalid", "oracle_step_with_draws rejected its arguments")
    return StepRun(xs, tt.value, kk.value, st, nd.value, js[: nd.value], cuts)


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
