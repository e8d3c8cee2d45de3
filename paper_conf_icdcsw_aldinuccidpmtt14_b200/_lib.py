"""ctypes binding of libcwc.so (include/cwc.h).  Argument marshalling only.

The library is loaded from this package's lib/ directory (built in-tree by build.py).  There
is no fallback: if the shared library is missing or fails to load, import raises.
"""
from __future__ import annotations

import ctypes
import os

_HERE = os.path.dirname(os.path.abspath(__file__))
SO_PATH = os.path.join(_HERE, "lib", "libcwc.so")

CWC_OK = 0
STATUS_NAMES = {0: "CWC_OK", 1: "CWC_E_INVALID", 2: "CWC_E_PARSE", 3: "CWC_E_UNSUPPORTED",
                4: "CWC_E_CUDA", 5: "CWC_E_OOM", 6: "CWC_E_STATE"}
FLAG_ABSORBED = 1
FLAG_OVERFLOWED = 2
CTR_REACTIONS, CTR_ABSORBED, CTR_OVERFLOWED, CTR_FINISHED, N_CTR = 0, 1, 2, 3, 8


class CWCError(RuntimeError):
    def __init__(self, status: int, msg: str):
        super().__init__(f"{STATUS_NAMES.get(status, status)}: {msg}")
        self.status = status


c_i32, c_i64, c_u64, c_dbl, c_sz = ctypes.c_int32, ctypes.c_int64, ctypes.c_uint64, ctypes.c_double, ctypes.c_size_t
P = ctypes.POINTER
c_vp, c_cp = ctypes.c_void_p, ctypes.c_char_p


class ModelInfo(ctypes.Structure):
    _fields_ = [("n_species", c_i32), ("n_reactions", c_i32), ("n_rules", c_i32),
                ("species_names", P(c_cp)), ("x0", P(c_i32)), ("rates", P(c_dbl)),
                ("n_reactants", P(c_i32)), ("reactant_species", P(c_i32)), ("reactant_order", P(c_i32)),
                ("delta", P(c_i32)), ("rule_of", P(c_i32)), ("x_cap", c_i64), ("x_cap_max", c_i64),
                ("hist_bins", c_i32), ("hist_lo", P(c_i64)), ("hist_width", P(c_i64)),
                ("law", P(c_i32)), ("law_species", P(c_i32)), ("law_K", P(c_dbl)), ("law_n", P(c_i32)),
                ("gate_species", P(c_i32)), ("gate_kind", P(c_i32)), ("place_off", P(c_i32)),
                ("place_alive", P(c_i32)), ("add_off", P(c_i32)), ("add_species", P(c_i32)),
                ("add_count", P(c_i32)), ("xfer_off", P(c_i32)), ("xfer_src", P(c_i32)), ("xfer_dst", P(c_i32)),
                ("sentinel", c_i32), ("flag", P(ctypes.c_uint8))]

MAX_REACTANTS = 8  # CWC_MAX_REACTANTS


class Stats(ctypes.Structure):
    _fields_ = [("T", c_i32), ("S", c_i32), ("B", c_i32), ("n_q", c_i32),
                ("times", P(c_dbl)), ("n", P(c_i64)), ("sum", P(c_i64)), ("sumsq", P(c_dbl)),
                ("sqlo", P(c_i64)), ("sqhi", P(c_i64)), ("mean", P(c_dbl)), ("var", P(c_dbl)),
                ("hist", P(c_i64)), ("hist_lo", P(c_i64)), ("hist_width", P(c_i64)), ("q", P(c_dbl)),
                ("quantile", P(c_dbl)), ("reactions", c_i64), ("absorbed", c_i64), ("overflowed", c_i64),
                ("finished", c_i64), ("kernel_ms", c_dbl), ("cuts_final", c_i64), ("species_names", P(c_cp)),
                ("pool_full", c_i64), ("launches", c_i64), ("raw_staged", c_i64)]


class PeriodStats(ctypes.Structure):
    _fields_ = [("T", c_i32), ("species", c_i32), ("window", c_i32), ("lo", c_i64), ("hi", c_i64),
                ("events", P(c_i64)), ("pc_n", P(c_i64)), ("pc_sum", P(c_i64)), ("pc_sqlo", P(c_i64)),
                ("pc_sqhi", P(c_i64)), ("lp_n", P(c_i64)), ("lp_sum", P(c_i64)), ("lp_sqlo", P(c_i64)),
                ("lp_sqhi", P(c_i64)), ("lp_mean", P(c_dbl)), ("lp_var", P(c_dbl)), ("moving_avg", P(c_dbl))]


# name -> (restype, argtypes)
SIGNATURES = {
    "cwc_version": (c_cp, []),
    "cwc_last_error": (c_cp, []),
    "cwc_model_load": (c_i32, [P(c_vp), c_i32, P(c_cp), c_i32, P(c_cp), P(c_dbl), c_cp]),
    "cwc_model_free": (None, [c_vp]),
    "cwc_model_info": (c_i32, [c_vp, P(ModelInfo)]),
    "cwc_set_option_i64": (c_i32, [c_vp, c_cp, c_i64]),
    "cwc_set_quantiles": (c_i32, [c_vp, c_i32, P(c_dbl)]),
    "cwc_model_compile": (c_i32, [c_vp, P(c_cp), P(c_cp)]),
    "cwc_kernel_attributes": (c_i32, [c_vp, P(c_i32), P(c_i32), P(c_i32)]),
    "cwc_kernel_image": (c_i32, [c_vp, P(c_vp), P(c_sz)]),
    "cwc_cancel": (c_i32, [c_vp]),
    "cwc_resume": (c_i32, [c_vp, c_vp]),
    "cwc_checkpoint_bytes": (c_i32, [c_vp, P(c_sz)]),
    "cwc_checkpoint_save": (c_i32, [c_vp, c_vp, c_sz]),
    "cwc_checkpoint_load": (c_i32, [c_vp, c_vp, c_sz]),
    "cwc_stats_host": (c_i32, [c_vp, P(c_vp), P(c_sz)]),
    "cwc_stats_load": (c_i32, [c_vp, c_vp, c_i64]),
    "cwc_buffer_sizes": (c_i32, [c_vp, c_i64, c_dbl, c_dbl, P(c_sz), P(c_sz), P(c_sz)]),
    "cwc_bind_device_buffers": (c_i32, [c_vp, c_vp, c_sz, c_vp, c_sz, c_vp, c_sz]),
    "cwc_simulate": (c_i32, [c_vp, c_i64, c_dbl, c_dbl, c_u64]),
    "cwc_simulate_range": (c_i32, [c_vp, c_i64, c_i64, c_i64, c_dbl, c_dbl, c_u64, c_vp]),
    "cwc_stats_device": (c_i32, [c_vp, P(c_vp), P(c_sz)]),
    "cwc_stats_finalize": (c_i32, [c_vp, c_vp]),
    "cwc_stats_snapshot": (c_i32, [c_vp, P(c_i64), P(c_i64)]),
    "cwc_stats": (c_i32, [c_vp, P(Stats)]),
    "cwc_samples": (c_i32, [c_vp, c_i64, c_i64, c_vp]),
    "cwc_period_stats": (c_i32, [c_vp, P(PeriodStats)]),
    "cwc_instance_records": (c_i32, [c_vp, c_i64, c_i64, c_vp, c_vp, c_vp]),
    "cwc_selftest_philox": (c_i32, [c_i64, c_vp, c_vp, c_vp]),
    "cwc_selftest_log": (c_i32, [c_i64, c_vp, c_vp]),
    "cwc_selftest_u01": (c_i32, [c_i64, c_vp, c_vp]),
    "cwc_selftest_div": (c_i32, [c_i64, c_vp, c_vp, c_vp]),
    "cwc_selftest_step": (c_i32, [c_vp, c_i64, c_i32, c_vp, c_vp, c_vp, c_dbl, c_dbl, c_vp, c_vp, c_i32, c_vp, c_vp,
                                  c_vp, c_vp, c_vp, c_vp]),
}


def _load():
    if not os.path.exists(SO_PATH):
        raise ImportError(f"{SO_PATH} is missing: build it with `python "
                          f"paper_conf_icdcsw_aldinuccidpmtt14_b200/build.py` (there is no fallback)")
    lib = ctypes.CDLL(SO_PATH)
    for name, (res, args) in SIGNATURES.items():
        fn = getattr(lib, name)
        fn.restype = res
        fn.argtypes = args
    return lib


lib = _load()


def check(status: int) -> None:
    if status != CWC_OK:
        raise CWCError(status, lib.cwc_last_error().decode(errors="replace"))
