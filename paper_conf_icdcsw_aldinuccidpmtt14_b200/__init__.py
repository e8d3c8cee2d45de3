"""B200-native CWC ensemble stochastic simulator (Aldinucci et al., ICDCS-W 2014 hot path).

C ABI: include/cwc.h, implemented by lib/libcwc.so (built in-tree by ``build.py``).
Python: ``Model`` (load / options / simulate / stats), ``DeviceBuffers`` (torch-owned device
memory), ``dist.simulate_sharded`` (one process per GPU, one NCCL all-reduce).
"""
from .api import DeviceBuffers, EnsembleResult, Model, selftest_div, selftest_log, selftest_philox, selftest_u01  # noqa: F401
from ._lib import CWCError, FLAG_ABSORBED, FLAG_OVERFLOWED, SO_PATH  # noqa: F401

__all__ = ["Model", "DeviceBuffers", "EnsembleResult", "CWCError", "selftest_philox", "selftest_log",
           "selftest_u01", "FLAG_ABSORBED", "FLAG_OVERFLOWED", "SO_PATH"]
