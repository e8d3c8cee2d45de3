"""Python API over the C ABI (include/cwc.h).  Marshalling only — every step of the hot path
runs in the NVRTC-compiled sm_100a kernel behind ``cwc_simulate_range``.

    m = Model(species, rules, rates, initial_term, x_cap=..., hist_bins=..., hist_width=...)
    res = m.simulate(n_instances, t_end, sample_dt, seed)      # synchronous, host results
    res.mean[k, s], res.var[k, s], res.quantile[k, s, q], res.hist[k, s, b]

PyTorch only provides device memory and streams: ``DeviceBuffers`` allocates the stats / raw /
scratch buffers as torch tensors and binds them, and ``simulate_range`` enqueues on a torch
stream so the caller can time it with CUDA events and all-reduce the stats with NCCL.
"""
from __future__ import annotations

import ctypes
import weakref
from dataclasses import dataclass
from typing import List, Optional, Sequence

import numpy as np

from . import _lib
from ._lib import CWCError, check, lib  # noqa: F401


def _stream_handle(stream):
    """cudaStream_t of a torch.cuda.Stream / raw handle; None = torch's current stream (the legacy
    default stream, 0, when CUDA is unavailable — the library then reports CWC_E_CUDA)."""
    if stream is None:
        import torch
        stream = torch.cuda.current_stream() if torch.cuda.is_available() else 0
    if hasattr(stream, "cuda_stream"):
        stream = stream.cuda_stream
    return int(stream) if stream else 0


def _ptr(a: np.ndarray):
    return ctypes.c_void_p(a.ctypes.data)


@dataclass
class EnsembleResult:
    """Finalised ensemble statistics of one simulation (cwc_stats_t as numpy arrays)."""

    times: np.ndarray       # [T]
    n: np.ndarray           # [T] int64
    sum: np.ndarray         # [T,S] int64
    sqlo: np.ndarray        # [T,S] int64
    sqhi: np.ndarray        # [T,S] int64
    sumsq: np.ndarray       # [T,S] float64 (rounded)
    mean: np.ndarray        # [T,S]
    var: np.ndarray         # [T,S]
    hist: np.ndarray        # [T,S,B+2] int64
    hist_lo: np.ndarray     # [S]
    hist_width: np.ndarray  # [S]
    q: np.ndarray           # [Q]
    quantile: np.ndarray    # [T,S,Q]
    reactions: int
    absorbed: int
    overflowed: int
    finished: int
    kernel_ms: float
    species: List[str]
    cuts_final: int = -1    # cuts [0, cuts_final) are final (T after finalize; a snapshot may be less)
    pool_full: int = 0      # overflowed instances frozen by a full compartment pool (R20)
    launches: int = 1       # kernels the simulation launched (SSA + compaction)
    raw_staged: int = 0     # raw cuts staged per lane in shared memory (option raw_stage)

    @property
    def frozen_fraction(self) -> float:
        """Fraction of the finished instances frozen before t_end (X_cap overflow or a full pool)."""
        return self.overflowed / self.finished if self.finished else 0.0

    def sumsq_exact(self) -> np.ndarray:
        out = np.empty(self.sqlo.shape, dtype=object)
        for idx in np.ndindex(self.sqlo.shape):
            out[idx] = (int(self.sqhi[idx]) << 32) + int(self.sqlo[idx])
        return out


class Model:
    """A loaded CWC model (cwc_model_load) with its options."""

    def __init__(self, species: Sequence[str], rules: Sequence[str], rates: Sequence[float], initial_term: str,
                 *, x_cap: Optional[int] = None, hist_bins: Optional[int] = None, hist_width=None, hist_lo=None,
                 quantiles: Optional[Sequence[float]] = None, raw_samples: bool = True,
                 quantum_samples: int = 0, block_threads: Optional[int] = None, refill: bool = True,
                 blocks_per_sm: int = 0, device: Optional[int] = None, period_species=None,
                 period_lo: int = 0, period_hi: int = 1, period_window: int = 1, capacity=None,
                 pool_auto: bool = True, **options):
        sp = (ctypes.c_char_p * len(species))(*[s.encode() for s in species])
        rl = (ctypes.c_char_p * max(len(rules), 1))(*[r.encode() for r in rules])
        rt = (ctypes.c_double * max(len(rates), 1))(*[float(k) for k in rates])
        h = ctypes.c_void_p()
        check(lib.cwc_model_load(ctypes.byref(h), len(species), sp, len(rules), rl, rt, initial_term.encode()))
        self._h = h
        self._info_cache = None
        self._bound_buffers = None   # DeviceBuffers bound to the handle (kept alive while bound)
        self._capacity = {k: int(v) for k, v in dict(capacity or {}).items()}
        # reading R20': a simulation in which some instance found a compartment pool full is repeated
        # with every pool capacity doubled (simulate / dist.simulate_sharded), until none is full
        self.pool_auto = bool(pool_auto)
        self._opts = dict(x_cap=x_cap, hist_bins=hist_bins, hist_width=hist_width, hist_lo=hist_lo,
                          quantiles=quantiles, raw_samples=raw_samples, quantum_samples=quantum_samples,
                          block_threads=block_threads, refill=refill, blocks_per_sm=blocks_per_sm, device=device,
                          period_species=period_species, period_lo=period_lo, period_hi=period_hi,
                          period_window=period_window, options=options)
        for label, c in self._capacity.items():   # re-flattens: before species options (R20)
            self.set_option(f"capacity.{label}", int(c))
        self._apply_options(**self._opts)

    def _apply_options(self, *, x_cap, hist_bins, hist_width, hist_lo, quantiles, raw_samples, quantum_samples,
                       block_threads, refill, blocks_per_sm, device, period_species, period_lo, period_hi,
                       period_window, options):
        if x_cap is not None:
            self.set_option("x_cap", int(x_cap))
        if hist_bins is not None:
            self.set_option("hist_bins", int(hist_bins))
        for key, val in (("hist_width", hist_width), ("hist_lo", hist_lo)):
            if val is None:
                continue
            if isinstance(val, dict):
                for name, v in val.items():
                    self.set_option(f"{key}.{name}", int(v))
            else:
                self.set_option(key, int(val))
        if quantiles is not None:
            self.set_quantiles(quantiles)
        self.set_option("raw_samples", 1 if raw_samples else 0)
        self.set_option("quantum_samples", int(quantum_samples))
        if block_threads is not None:
            self.set_option("block_threads", int(block_threads))
        self.set_option("refill", 1 if refill else 0)
        self.set_option("blocks_per_sm", int(blocks_per_sm))
        for key, val in options.items():
            self.set_option(key, int(val))
        if period_species is not None:   # on-line oscillation-period analysis (R19)
            if isinstance(period_species, str):
                self.set_option(f"period_species.{period_species}", 1)
            else:
                self.set_option("period_species", int(period_species))
            self.set_option("period_lo", int(period_lo))
            self.set_option("period_hi", int(period_hi))
            self.set_option("period_window", int(period_window))
        if device is not None:
            self.set_option("device", int(device))

    # ------------------------------------------------------------ compartment pools (R20, R20')
    def pool_capacities(self) -> dict:
        """Slots per pool of every dynamic compartment label ({} for static models)."""
        labels = sorted({n.split(":", 1)[1].split("@", 1)[0] for n in self.info()["names"] if n.startswith("#free:")})
        return {lab: self._capacity.get(lab, 8) for lab in labels}

    def grow_pools(self) -> bool:
        """Double every pool capacity (max 4096), re-flatten and re-apply this model's options.
        Returns False when no pool can grow (static model, or every pool at 4096 slots)."""
        caps = self.pool_capacities()
        grown = {lab: min(4096, 2 * c) for lab, c in caps.items()}
        if not caps or grown == caps:
            return False
        for lab, c in grown.items():
            self._capacity[lab] = c
            self.set_option(f"capacity.{lab}", c)
        self._info_cache = None
        self._apply_options(**self._opts)
        return True

    @classmethod
    def from_def(cls, mdef, **kw) -> "Model":
        """Load a workloads.ModelDef-like object (species, rules, rates, initial_term, x_cap)."""
        if getattr(mdef, "x_cap", None) is not None and "x_cap" not in kw:
            kw["x_cap"] = mdef.x_cap
        if getattr(mdef, "capacity", None) and "capacity" not in kw:
            kw["capacity"] = dict(mdef.capacity)
        return cls(mdef.species, mdef.rules, mdef.rates, mdef.initial_term, **kw)

    def close(self):
        if getattr(self, "_h", None):
            lib.cwc_model_free(self._h)
            self._h = None
        self._bound_buffers = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass

    @property
    def handle(self):
        return self._h

    # ---------------------------------------------------------------- options / info
    def set_option(self, key: str, value: int) -> None:
        check(lib.cwc_set_option_i64(self._h, key.encode(), int(value)))
        self._info_cache = None

    def set_quantiles(self, qs: Sequence[float]) -> None:
        arr = (ctypes.c_double * max(len(qs), 1))(*[float(q) for q in qs])
        check(lib.cwc_set_quantiles(self._h, len(qs), arr))

    def info(self) -> dict:
        if self._info_cache is None:
            mi = _lib.ModelInfo()
            check(lib.cwc_model_info(self._h, ctypes.byref(mi)))
            S, M = mi.n_species, mi.n_reactions
            R = _lib.MAX_REACTANTS
            nre = [mi.n_reactants[j] for j in range(M)]
            self._info_cache = dict(
                names=[mi.species_names[s].decode() for s in range(S)],
                x0=[mi.x0[s] for s in range(S)],
                rates=[mi.rates[j] for j in range(M)],
                reactants=[[(mi.reactant_species[j * R + e], mi.reactant_order[j * R + e]) for e in range(nre[j])]
                           for j in range(M)],
                delta=[[mi.delta[j * S + s] for s in range(S)] for j in range(M)],
                rule_of=[mi.rule_of[j] for j in range(M)],
                x_cap=mi.x_cap, x_cap_max=mi.x_cap_max, n_rules=mi.n_rules, hist_bins=mi.hist_bins,
                hist_lo=[mi.hist_lo[s] for s in range(S)], hist_width=[mi.hist_width[s] for s in range(S)],
                law=[mi.law[j] for j in range(M)], law_species=[mi.law_species[j] for j in range(M)],
                law_K=[mi.law_K[j] for j in range(M)], law_n=[mi.law_n[j] for j in range(M)],
                # reading R20 (dynamic compartments)
                gate_species=[mi.gate_species[j] for j in range(M)], gate_kind=[mi.gate_kind[j] for j in range(M)],
                place=[[(mi.place_alive[p], [(mi.add_species[e], mi.add_count[e])
                                              for e in range(mi.add_off[p], mi.add_off[p + 1])])
                        for p in range(mi.place_off[j], mi.place_off[j + 1])] for j in range(M)],
                transfer=[[(mi.xfer_src[e], mi.xfer_dst[e]) for e in range(mi.xfer_off[j], mi.xfer_off[j + 1])]
                          for j in range(M)],
                sentinel=mi.sentinel, flag=[bool(mi.flag[s]) for s in range(S)],
            )
        return self._info_cache

    @property
    def n_species(self) -> int:
        return len(self.info()["names"])

    def compile(self):
        """NVRTC-compile the model's kernel for sm_100a (no GPU needed); returns (source, log)."""
        src, log = ctypes.c_char_p(), ctypes.c_char_p()
        check(lib.cwc_model_compile(self._h, ctypes.byref(src), ctypes.byref(log)))
        return src.value.decode(), log.value.decode()

    def kernel_attributes(self) -> dict:
        r, l, t = ctypes.c_int32(), ctypes.c_int32(), ctypes.c_int32()
        check(lib.cwc_kernel_attributes(self._h, ctypes.byref(r), ctypes.byref(l), ctypes.byref(t)))
        return dict(registers=r.value, local_bytes=l.value, max_threads=t.value)

    def kernel_image_bytes(self) -> int:
        """Size of the compiled sm_100a cubin (uploaded to the device at module load)."""
        n = ctypes.c_size_t()
        check(lib.cwc_kernel_image(self._h, None, ctypes.byref(n)))
        return n.value

    def buffer_sizes(self, count: int, t_end: float, dt: float):
        a, b, c = ctypes.c_size_t(), ctypes.c_size_t(), ctypes.c_size_t()
        check(lib.cwc_buffer_sizes(self._h, int(count), float(t_end), float(dt), ctypes.byref(a), ctypes.byref(b),
                                   ctypes.byref(c)))
        return a.value, b.value, c.value

    # ---------------------------------------------------------------- simulation
    def simulate(self, n_instances: int, t_end: float, sample_dt: float, seed: int) -> EnsembleResult:
        """The public end-to-end call: simulate n instances, return host statistics.  With
        ``pool_auto`` (default) a run in which a compartment pool was full is repeated with doubled
        pool capacities (reading R20'), so the result has pool_full == 0 unless a pool reached 4096."""
        while True:
            check(lib.cwc_simulate(self._h, int(n_instances), float(t_end), float(sample_dt), int(seed)))
            res = self.stats()
            if res.pool_full == 0 or not self.pool_auto or not self.grow_pools():
                return res

    def simulate_range(self, n_total: int, first: int, count: int, t_end: float, sample_dt: float, seed: int,
                       stream=None) -> None:
        """Enqueue instances [first, first+count) on ``stream``: a torch.cuda.Stream, a raw
        cudaStream_t int, or None for torch's current stream.  Asynchronous."""
        stream = _stream_handle(stream)
        check(lib.cwc_simulate_range(self._h, int(n_total), int(first), int(count), float(t_end),
                                     float(sample_dt), int(seed), ctypes.c_void_p(stream)))

    def finalize(self, host_stats: Optional[np.ndarray] = None) -> EnsembleResult:
        if host_stats is not None:
            host_stats = np.ascontiguousarray(host_stats, dtype=np.int64)
            check(lib.cwc_stats_finalize(self._h, _ptr(host_stats)))
        else:
            check(lib.cwc_stats_finalize(self._h, None))
        return self.stats()

    def stats(self) -> EnsembleResult:
        st = _lib.Stats()
        check(lib.cwc_stats(self._h, ctypes.byref(st)))
        T, S, B, Q = st.T, st.S, st.B, st.n_q

        def arr(p, n, dt, shape):
            return np.ctypeslib.as_array(p, shape=(n,)).astype(dt, copy=True).reshape(shape)

        return EnsembleResult(
            times=arr(st.times, T, np.float64, (T,)), n=arr(st.n, T, np.int64, (T,)),
            sum=arr(st.sum, T * S, np.int64, (T, S)), sqlo=arr(st.sqlo, T * S, np.int64, (T, S)),
            sqhi=arr(st.sqhi, T * S, np.int64, (T, S)), sumsq=arr(st.sumsq, T * S, np.float64, (T, S)),
            mean=arr(st.mean, T * S, np.float64, (T, S)), var=arr(st.var, T * S, np.float64, (T, S)),
            hist=arr(st.hist, T * S * (B + 2), np.int64, (T, S, B + 2)),
            hist_lo=arr(st.hist_lo, S, np.int64, (S,)), hist_width=arr(st.hist_width, S, np.int64, (S,)),
            q=arr(st.q, Q, np.float64, (Q,)) if Q else np.zeros(0),
            quantile=arr(st.quantile, T * S * Q, np.float64, (T, S, Q)) if Q else np.zeros((T, S, 0)),
            reactions=st.reactions, absorbed=st.absorbed, overflowed=st.overflowed, finished=st.finished,
            kernel_ms=st.kernel_ms, species=[st.species_names[s].decode() for s in range(S)],
            cuts_final=st.cuts_final, pool_full=st.pool_full, launches=st.launches,
            raw_staged=st.raw_staged,
        )

    def snapshot(self):
        """Statistics of the running simulation ("stream" option): (cuts_final, items_done, result)."""
        cf, done = ctypes.c_int64(), ctypes.c_int64()
        check(lib.cwc_stats_snapshot(self._h, ctypes.byref(cf), ctypes.byref(done)))
        return cf.value, done.value, self.stats()

    def stats_host(self) -> np.ndarray:
        """Copy of the packed statistics behind the current views (last snapshot / finalize)."""
        p, n = ctypes.c_void_p(), ctypes.c_size_t()
        check(lib.cwc_stats_host(self._h, ctypes.byref(p), ctypes.byref(n)))
        return np.ctypeslib.as_array(ctypes.cast(p, ctypes.POINTER(ctypes.c_int64)), shape=(n.value,)).copy()

    def stats_load(self, packed: np.ndarray, cuts_final: int) -> "EnsembleResult":
        """Load a packed statistics buffer (e.g. summed over ranks) as the current result."""
        buf = np.ascontiguousarray(packed, dtype=np.int64)
        check(lib.cwc_stats_load(self._h, _ptr(buf), int(cuts_final)))
        return self.stats()

    def checkpoint(self) -> np.ndarray:
        """The last simulation as a host checkpoint (cwc_checkpoint_save; synchronises)."""
        n = ctypes.c_size_t()
        check(lib.cwc_checkpoint_bytes(self._h, ctypes.byref(n)))
        buf = np.empty(n.value, dtype=np.uint8)
        check(lib.cwc_checkpoint_save(self._h, _ptr(buf), n.value))
        return buf

    def restore(self, ckpt: np.ndarray) -> None:
        """Load a checkpoint of the same model / options into this handle (cwc_checkpoint_load)."""
        buf = np.ascontiguousarray(ckpt, dtype=np.uint8)
        check(lib.cwc_checkpoint_load(self._h, _ptr(buf), buf.size))

    def resume(self, stream=None) -> None:
        """Continue a terminated or restored run to its horizon (cwc_resume; asynchronous)."""
        stream = _stream_handle(stream)
        check(lib.cwc_resume(self._h, ctypes.c_void_p(stream)))

    def cancel(self):
        """Terminate the running streaming simulation (cwc_cancel)."""
        check(lib.cwc_cancel(self._h))

    def stream(self, n_instances: int, t_end: float, sample_dt: float, seed: int, poll_s: float = 0.02,
               stream=None, stop=None):
        """On-line streaming: launch, then yield (cuts_final, partial result) each
        time more cuts become final, and finally (cuts_final, finalised result) — cuts_final = T
        unless ``stop(cuts_final, partial_result)`` returned True, which terminates the running
        simulation (steering) and finalises the cuts completed so far."""
        import time
        self.set_option("stream", 1)
        self.simulate_range(n_instances, 0, n_instances, t_end, sample_dt, seed, stream=stream)
        last = -1
        T = int(round(t_end / sample_dt)) + 1
        while True:
            cf, _, res = self.snapshot()
            if cf > last:
                last = cf
                if cf < T:
                    yield cf, res
                    if stop is not None and stop(cf, res):
                        self.cancel()
                        break
            if cf >= T:
                break
            time.sleep(poll_s)
        res = self.finalize()
        yield res.cuts_final, res

    def period_stats(self) -> dict:
        """On-line period analysis of the last simulation (cwc_period_stats) as numpy arrays."""
        ps = _lib.PeriodStats()
        check(lib.cwc_period_stats(self._h, ctypes.byref(ps)))
        T = ps.T
        out = dict(species=ps.species, window=ps.window, lo=ps.lo, hi=ps.hi)
        for name in ("events", "pc_n", "pc_sum", "pc_sqlo", "pc_sqhi", "lp_n", "lp_sum", "lp_sqlo", "lp_sqhi"):
            out[name] = np.ctypeslib.as_array(getattr(ps, name), shape=(T,)).astype(np.int64, copy=True)
        for name in ("lp_mean", "lp_var", "moving_avg"):
            out[name] = np.ctypeslib.as_array(getattr(ps, name), shape=(T,)).astype(np.float64, copy=True)
        return out

    def stats_device(self):
        p, n = ctypes.c_void_p(), ctypes.c_size_t()
        check(lib.cwc_stats_device(self._h, ctypes.byref(p), ctypes.byref(n)))
        return p.value, n.value

    def samples(self, first: int, count: int) -> np.ndarray:
        info = self.info()
        n_t = self.stats_T()
        out = np.empty((n_t, len(info["names"]), count), dtype=np.int32)
        check(lib.cwc_samples(self._h, int(first), int(count), _ptr(out)))
        return out

    def stats_T(self) -> int:
        st = _lib.Stats()
        if lib.cwc_stats(self._h, ctypes.byref(st)) == 0:
            return st.T
        raise CWCError(6, "finalize before reading samples")

    def selftest_step(self, x, t, k, t_end: float, sample_dt: float, u_tau, u_sel, mode: int = 0) -> dict:
        """Injected-draw steps on the device (cwc_selftest_step): trajectory i starts from
        x[i], t[i], next cut k[i] and takes up to D steps with the uniforms u_tau[i][:D],
        u_sel[i][:D].  mode 0 = the SSA kernel's fast step + full step, 1 = full step only."""
        S = self.n_species
        x = np.ascontiguousarray(x, dtype=np.int32).reshape(-1, S)
        n = len(x)
        t = np.ascontiguousarray(t, dtype=np.float64).reshape(n)
        k = np.ascontiguousarray(k, dtype=np.int64).reshape(n)
        ut = np.ascontiguousarray(u_tau, dtype=np.float64).reshape(n, -1)
        us = np.ascontiguousarray(u_sel, dtype=np.float64).reshape(n, -1)
        D = ut.shape[1]
        if us.shape != ut.shape:
            raise ValueError("u_tau and u_sel must have the same shape")
        T = int(round(t_end / sample_dt)) + 1
        xo = np.empty_like(x)
        to = np.empty(n, dtype=np.float64)
        ko = np.empty(n, dtype=np.int64)
        st = np.empty(n, dtype=np.int32)
        nd = np.empty(n, dtype=np.int32)
        cuts = np.empty((n, T, S), dtype=np.int32)
        check(lib.cwc_selftest_step(self._h, n, D, _ptr(x), _ptr(t), _ptr(k), float(t_end), float(sample_dt),
                                    _ptr(ut), _ptr(us), int(mode), _ptr(xo), _ptr(to), _ptr(ko), _ptr(st), _ptr(nd),
                                    _ptr(cuts)))
        return {"x": xo, "t": to, "k": ko, "status": st, "n_done": nd, "cuts": cuts}

    def records(self, first: int, count: int):
        flags = np.empty(count, dtype=np.uint8)
        reactions = np.empty(count, dtype=np.int64)
        t_last = np.empty(count, dtype=np.float64)
        check(lib.cwc_instance_records(self._h, int(first), int(count), _ptr(flags), _ptr(reactions), _ptr(t_last)))
        return flags, reactions, t_last


class DeviceBuffers:
    """Torch-owned device buffers bound to a model for one (count, t_end, dt) geometry."""

    def __init__(self, model: Model, count: int, t_end: float, sample_dt: float, device=None):
        import torch
        n_stats, n_raw, n_scratch = model.buffer_sizes(count, t_end, sample_dt)
        dev = torch.device("cuda", torch.cuda.current_device()) if device is None else torch.device(device)
        self.stats = torch.empty(n_stats, dtype=torch.int64, device=dev)
        self.raw = torch.empty(max(n_raw, 1), dtype=torch.int32, device=dev) if n_raw else None
        self.scratch = torch.empty(n_scratch, dtype=torch.uint8, device=dev)
        # weak back-reference: the model holds its bound buffers (below), and a strong cycle would
        # keep both alive until a garbage-collector pass (device memory not returned on del)
        self._model = weakref.ref(model)
        model.set_option("device", dev.index)
        check(lib.cwc_bind_device_buffers(
            model.handle, ctypes.c_void_p(self.stats.data_ptr()), n_stats,
            ctypes.c_void_p(self.raw.data_ptr() if self.raw is not None else 0), n_raw,
            ctypes.c_void_p(self.scratch.data_ptr()), n_scratch))
        # the library keeps raw pointers into these tensors: the model holds the buffers alive
        # while they are bound (results, samples and records read them after the caller's
        # DeviceBuffers / ShardedRun object is gone)
        model._bound_buffers = self

    def unbind(self):
        model = self._model()
        if model is None or not model.handle:
            return
        check(lib.cwc_bind_device_buffers(model.handle, None, 0, None, 0, None, 0))
        if getattr(model, "_bound_buffers", None) is self:
            model._bound_buffers = None

    @property
    def model(self):
        return self._model()


def selftest_philox(ctr: np.ndarray, key: np.ndarray) -> np.ndarray:
    ctr = np.ascontiguousarray(ctr, dtype=np.uint32).reshape(-1, 4)
    key = np.ascontiguousarray(key, dtype=np.uint32).reshape(-1, 2)
    out = np.empty_like(ctr)
    check(lib.cwc_selftest_philox(len(ctr), _ptr(ctr), _ptr(key), _ptr(out)))
    return out


def selftest_log(x: np.ndarray) -> np.ndarray:
    x = np.ascontiguousarray(x, dtype=np.float64)
    out = np.empty_like(x)
    check(lib.cwc_selftest_log(len(x), _ptr(x), _ptr(out)))
    return out


def selftest_u01(words: np.ndarray) -> np.ndarray:
    w = np.ascontiguousarray(words, dtype=np.uint32).reshape(-1, 2)
    out = np.empty(len(w), dtype=np.float64)
    check(lib.cwc_selftest_u01(len(w), _ptr(w), _ptr(out)))
    return out


def selftest_div(num: np.ndarray, den: np.ndarray) -> np.ndarray:
    """The SSA kernel's branch-free IEEE division, evaluated on the GPU."""
    a = np.ascontiguousarray(num, dtype=np.float64)
    b = np.ascontiguousarray(den, dtype=np.float64)
    out = np.empty_like(a)
    check(lib.cwc_selftest_div(len(a), _ptr(a), _ptr(b), _ptr(out)))
    return out
