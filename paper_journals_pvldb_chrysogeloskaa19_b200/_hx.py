"""ctypes binding of libhx (include/hx.h) — argument marshalling only.

Every step of the SSB hot path runs in libhx's CUDA kernels; this module only converts
Python values to the C-ABI's plain structs and pointers and raises HxError on a non-zero
status. There is no fallback: if libhx.so is missing or cannot load, importing the package
fails loudly.
"""
from __future__ import annotations

import ctypes
import os

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.environ.get("HX_LIB", os.path.join(_HERE, "libhx.so"))  # HX_LIB: tuning builds

HX_OK, HX_EINVAL, HX_ECUDA, HX_ENCCL, HX_ENOMEM, HX_ECAPACITY, HX_EDUPKEY, HX_EUNSUPPORTED = (
    0, -1, -2, -3, -4, -5, -6, -7)
HX_POLICY_RANGE, HX_POLICY_ROUND_ROBIN = 0, 1
HX_PLACE_COPY, HX_PLACE_VIEW, HX_PLACE_HOST_PINNED, HX_PLACE_HOST_MAPPED = 0, 1, 2, 3
HX_PRED_RANGE, HX_PRED_IN = 0, 1
HX_AGG_SUM, HX_AGG_SUM_MUL, HX_AGG_SUM_SUB = 0, 1, 2
HX_MAX_COLS, HX_MAX_PREDS, HX_MAX_JOINS, HX_MAX_GDIMS = 16, 3, 4, 3
HX_BUILD_IDENTITY_RANKS = 1
HX_MAX_PARTS = 64
HX_OPT_JOIN_LAYOUT, HX_OPT_L2_PERSIST = 1, 2
HX_JOIN_AUTO, HX_JOIN_HASH = 0, 1
(HX_COLL_ALLREDUCE, HX_COLL_REDUCE, HX_COLL_BROADCAST, HX_COLL_ALLGATHER, HX_COLL_SEND,
 HX_COLL_RECV) = 1, 2, 3, 4, 5, 6

_NAMES = {0: "HX_OK", -1: "HX_EINVAL", -2: "HX_ECUDA", -3: "HX_ENCCL", -4: "HX_ENOMEM",
          -5: "HX_ECAPACITY", -6: "HX_EDUPKEY", -7: "HX_EUNSUPPORTED"}


class HxError(RuntimeError):
    def __init__(self, code: int, fn: str, msg: str):
        super().__init__(f"{fn}: {_NAMES.get(code, code)}: {msg}")
        self.code = code


class hx_block(ctypes.Structure):
    _fields_ = [("row_begin", ctypes.c_int64), ("row_end", ctypes.c_int64),
                ("part", ctypes.c_int32), ("reserved", ctypes.c_int32)]


class hx_col(ctypes.Structure):
    _fields_ = [("col_id", ctypes.c_int32), ("reserved", ctypes.c_int32),
                ("data", ctypes.c_void_p), ("n_rows", ctypes.c_int64)]


class hx_pred(ctypes.Structure):
    _fields_ = [("col_id", ctypes.c_int32), ("kind", ctypes.c_int32), ("lo", ctypes.c_int32),
                ("hi", ctypes.c_int32), ("n_in", ctypes.c_int32), ("in_", ctypes.c_int32 * 4)]


class hx_query_shape(ctypes.Structure):
    _fields_ = [("n_preds", ctypes.c_int32), ("preds", hx_pred * HX_MAX_PREDS),
                ("n_joins", ctypes.c_int32), ("join_fk_col", ctypes.c_int32 * HX_MAX_JOINS),
                ("join_ht", ctypes.c_int32 * HX_MAX_JOINS), ("agg_op", ctypes.c_int32),
                ("agg_a", ctypes.c_int32), ("agg_b", ctypes.c_int32),
                ("n_gdims", ctypes.c_int32), ("gdim_join", ctypes.c_int32 * HX_MAX_GDIMS)]


class hx_build_spec(ctypes.Structure):
    _fields_ = [("dim", ctypes.c_int32), ("key_col", ctypes.c_int32), ("n_preds", ctypes.c_int32),
                ("preds", hx_pred * HX_MAX_PREDS), ("group_col", ctypes.c_int32),
                ("group_lo", ctypes.c_int32), ("group_hi", ctypes.c_int32)]


class hx_coll_rec(ctypes.Structure):
    _fields_ = [("op", ctypes.c_int32), ("root_or_peer", ctypes.c_int32), ("count", ctypes.c_int64),
                ("elem_bytes", ctypes.c_int32), ("reserved", ctypes.c_int32), ("buf", ctypes.c_uint64)]


_P = ctypes.c_void_p
_PP = ctypes.POINTER(ctypes.c_void_p)
_I = ctypes.c_int
_I32 = ctypes.c_int32
_I64 = ctypes.c_int64
_PI64 = ctypes.POINTER(ctypes.c_int64)
_PI32 = ctypes.POINTER(ctypes.c_int32)

_SIGS = {
    "hx_last_error": ([], ctypes.c_char_p),
    "hx_init": ([_I, _P, _PP], _I),
    "hx_finalize": ([_P], _I),
    "hx_ctx_stream": ([_P, _PP], _I),
    "hx_ctx_info": ([_P, ctypes.POINTER(_I), ctypes.POINTER(_I)], _I),
    "hx_ctx_set_option": ([_P, _I, _I], _I),
    "hx_comm_unique_id": ([_P], _I),
    "hx_comm_init": ([_P, _I, _I, _P], _I),
    "hx_comm_info": ([_P, ctypes.POINTER(_I), ctypes.POINTER(_I)], _I),
    "hx_comm_trace": ([_P, ctypes.POINTER(hx_coll_rec), _I, ctypes.POINTER(_I), _I], _I),
    "hx_router_partition": ([_I64, _I, _I64, _I, _PP], _I),
    "hx_partition_info": ([_P, _PI64, ctypes.POINTER(ctypes.POINTER(hx_block))], _I),
    "hx_partition_rows": ([_P, _I, _PI64], _I),
    "hx_partition_free": ([_P], _I),
    "hx_load_columns": ([_P, ctypes.POINTER(hx_col), _I, _P, _I, _I, _PP], _I),
    "hx_table_info": ([_P, _PI64, ctypes.POINTER(_I)], _I),
    "hx_table_slice": ([_P, _I64, _I64, _PP], _I),
    "hx_table_free": ([_P], _I),
    "hx_table_read": ([_P, _I32, _I64, _I64, _PI32], _I),
    "hx_table_write": ([_P, _I32, _I64, _I64, _P], _I),
    "hx_build_dim_ht": ([_P, _P, _I32, ctypes.POINTER(hx_pred), _I, _I32, _I32, _I32, _PP], _I),
    "hx_build_dim_ht_ex": ([_P, _P, _I32, ctypes.POINTER(hx_pred), _I, _I32, _I32, _I32, _I, _PP], _I),
    "hx_hash_partition": ([_P, _P, _I32, _I, _PP, _PI64], _I),
    "hx_exchange_partitions": ([_P, _P, _PI64, _I, _PP], _I),
    "hx_ht_info": ([_P, _PI64, _PI64, _PI32, _PI32], _I),
    "hx_ht_broadcast": ([_P, _P, _I], _I),
    "hx_ht_free": ([_P], _I),
    "hx_pipeline_probe_agg": ([_P, _P, ctypes.POINTER(hx_query_shape), _PP, _I, _PP], _I),
    "hx_pipeline_probe_agg_into": ([_P, _P, ctypes.POINTER(hx_query_shape), _PP, _I, _P], _I),
    "hx_merge_aggregates": ([_P, _P, _I, _PI64, _PI64, _PI32, _I64, _PI64], _I),
    "hx_agg_free": ([_P], _I),
    "hx_shared_router_open": ([ctypes.c_char_p, _I64, _I, _PP], _I),
    "hx_shared_router_next": ([_P, _PI64], _I),
    "hx_shared_router_reset": ([_P], _I),
    "hx_shared_router_close": ([_P, _I], _I),
    "hx_pipeline_probe_agg_routed": ([_P, _P, ctypes.POINTER(hx_query_shape), _PP, _I, _P, _I64, _PP,
                                      _PI64], _I),
    "hx_group_layout": ([_I, _PI32, _PI64, _PI64], _I),
    "hx_group_decode": ([_I, _PI32, ctypes.POINTER(_PI32), _PI64, _PI64, _I64, _PI32, _PI64, _PI64,
                         _I64, _PI64], _I),
    "hx_profile_enable": ([_P, _I], _I),
    "hx_profile_read": ([_P, ctypes.POINTER(ctypes.c_double), _PI64, _PI64, _I], _I),
    "hx_stats": ([_P, _PI64, _PI64, _PI64, _I], _I),
    "hx_plan_create": ([_P, _P, _PP, _I, ctypes.POINTER(hx_build_spec), _I,
                        ctypes.POINTER(hx_query_shape), _PP], _I),
    "hx_plan_enqueue": ([_P, _P], _I),
    "hx_plans_enqueue": ([_P, _PP, _I], _I),
    "hx_plan_result": ([_P, _PI64, _PI64, _PI32, _I64, _PI64], _I),
    "hx_plan_k1_time": ([_P, ctypes.POINTER(ctypes.c_float), _PI64], _I),
    "hx_plan_k1_span": ([_P, _P, ctypes.POINTER(ctypes.c_float)], _I),
    "hx_plan_info": ([_P, _PI64, ctypes.POINTER(_I)], _I),
    "hx_plan_free": ([_P], _I),
    "hx_graph_begin": ([_P], _I),
    "hx_graph_end": ([_P, _PP], _I),
    "hx_graph_launch": ([_P, _P], _I),
    "hx_graph_free": ([_P], _I),
}
EXPORTED = sorted(_SIGS)

_lib = None


def lib():
    """The loaded libhx.so (raises if it is missing: no fallback path exists)."""
    global _lib
    if _lib is None:
        if not os.path.exists(LIB_PATH):
            raise ImportError(f"{LIB_PATH} is missing: build it with `make` (or "
                              f"__graft_entry__.build()); there is no non-CUDA fallback")
        l = ctypes.CDLL(LIB_PATH)
        for name, (args, res) in _SIGS.items():
            if "HX_LIB" in os.environ and not hasattr(l, name):
                continue  # an older tuning build (A/B timing) may lack newer entry points
            f = getattr(l, name)
            f.argtypes = args
            f.restype = res
        _lib = l
    return _lib


def call(name: str, *args) -> None:
    rc = getattr(lib(), name)(*args)
    if rc != HX_OK:
        raise HxError(rc, name, lib().hx_last_error().decode(errors="replace"))


def pred(col_id: int, lo: int | None = None, hi: int | None = None,
         isin: tuple | list | None = None) -> hx_pred:
    """RANGE lo <= v <= hi (None = unbounded) or IN isin (1..4 values)."""
    p = hx_pred()
    p.col_id = col_id
    if isin is not None:
        assert 1 <= len(isin) <= 4
        p.kind = HX_PRED_IN
        p.n_in = len(isin)
        for i, v in enumerate(isin):
            p.in_[i] = v
    else:
        p.kind = HX_PRED_RANGE
        p.lo = -(2 ** 31) if lo is None else lo
        p.hi = 2 ** 31 - 1 if hi is None else hi
    return p
