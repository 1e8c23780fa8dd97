"""B200-native hot path of HetExchange (Chrysogelos et al., PVLDB 2019): the fused GPU
pipeline that runs a Star Schema Benchmark query (scan -> filter -> probe x k -> group-by
aggregate), its router / mem-move / broadcast / union-router plumbing, as the C-ABI library
libhx.so (include/hx.h) with this thin ctypes binding.

Importing the package loads libhx.so and fails loudly if it is missing: there is no CPU or
PyTorch fallback for any step of the path.
"""
from . import _hx
from ._hx import HxError  # noqa: F401

_hx.lib()  # fail at import time, not at first use

from . import hx  # noqa: E402,F401
from . import ssb  # noqa: E402,F401
