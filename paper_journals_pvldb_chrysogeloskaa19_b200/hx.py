"""Thin Python binding of the libhx C-ABI with the same call names (include/hx.h).

Argument marshalling only. Objects own their C handles and free them on close()/__del__.
PyTorch, when used by a caller, only provides device memory (tensor data pointers) and
streams (`torch.cuda.current_stream().cuda_stream`); nothing here imports torch.
"""
from __future__ import annotations

import ctypes
import weakref
from typing import Dict, List, Optional, Sequence, Tuple

import numpy as np

from . import _hx
from ._hx import call, hx_col, hx_query_shape, pred  # noqa: F401  (re-exported)


class Context:
    """hx_init / hx_finalize: one GPU, one stream (cudaStream_t as int, 0 = library-owned)."""

    def __init__(self, device: int = 0, stream: int = 0):
        h = ctypes.c_void_p()
        call("hx_init", device, ctypes.c_void_p(stream or None), ctypes.byref(h))
        self.h = h
        self.device = device

    @property
    def stream(self) -> int:
        s = ctypes.c_void_p()
        call("hx_ctx_stream", self.h, ctypes.byref(s))
        return s.value or 0

    def info(self) -> Tuple[int, int]:
        a, b = ctypes.c_int(), ctypes.c_int()
        call("hx_ctx_info", self.h, ctypes.byref(a), ctypes.byref(b))
        return a.value, b.value

    def set_option(self, option: int, value: int) -> None:
        """hx_ctx_set_option (HX_OPT_JOIN_LAYOUT: HX_JOIN_AUTO | HX_JOIN_HASH; HX_OPT_L2_PERSIST)."""
        call("hx_ctx_set_option", self.h, option, value)

    def comm_init(self, nranks: int, rank: int, uid: bytes) -> None:
        buf = ctypes.create_string_buffer(uid, 128)
        call("hx_comm_init", self.h, nranks, rank, buf)

    def comm_info(self) -> Tuple[int, int]:
        """(rank, nranks); (0, 1) without a communicator."""
        a, b = ctypes.c_int(), ctypes.c_int()
        call("hx_comm_info", self.h, ctypes.byref(a), ctypes.byref(b))
        return a.value, b.value

    def comm_trace(self, reset: bool = True) -> List[dict]:
        """The NCCL data calls libhx issued on this context (hx_comm_trace), oldest first."""
        n = ctypes.c_int()
        call("hx_comm_trace", self.h, None, 0, ctypes.byref(n), 0)
        recs = (_hx.hx_coll_rec * max(1, n.value))()
        call("hx_comm_trace", self.h, recs, n.value, ctypes.byref(n), 1 if reset else 0)
        names = {_hx.HX_COLL_ALLREDUCE: "allreduce", _hx.HX_COLL_REDUCE: "reduce",
                 _hx.HX_COLL_BROADCAST: "broadcast", _hx.HX_COLL_ALLGATHER: "allgather",
                 _hx.HX_COLL_SEND: "send", _hx.HX_COLL_RECV: "recv"}
        return [{"op": names[r.op], "root_or_peer": r.root_or_peer, "count": r.count,
                 "elem_bytes": r.elem_bytes, "buf": r.buf} for r in recs[:n.value]]

    def profile_enable(self, on: bool = True) -> None:
        call("hx_profile_enable", self.h, int(on))

    def profile_read(self, reset: bool = True) -> Tuple[float, int, int]:
        ms, n, b = ctypes.c_double(), ctypes.c_int64(), ctypes.c_int64()
        call("hx_profile_read", self.h, ctypes.byref(ms), ctypes.byref(n), ctypes.byref(b),
             int(reset))
        return ms.value, n.value, b.value

    def stats(self, reset: bool = False) -> Tuple[int, int, int]:
        """(kernels launched, H2D bytes, D2H bytes) since the last reset."""
        a, b, c = ctypes.c_int64(), ctypes.c_int64(), ctypes.c_int64()
        call("hx_stats", self.h, ctypes.byref(a), ctypes.byref(b), ctypes.byref(c), int(reset))
        return a.value, b.value, c.value

    def close(self) -> None:
        if getattr(self, "h", None):
            # free every live library object of this context first (graphs before the plans
            # they replay, plans / aggs before the tables they reference)
            kids = list(getattr(self, "_children", ()))
            for cls in (Graph, Plan, Agg, HashTable, Table):
                for k in kids:
                    if isinstance(k, cls):
                        k.close()
            call("hx_finalize", self.h)
            self.h = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass


def _adopt(ctx: Context, obj) -> None:
    if not hasattr(ctx, "_children"):
        ctx._children = weakref.WeakSet()
    ctx._children.add(obj)


def comm_unique_id() -> bytes:
    buf = ctypes.create_string_buffer(128)
    call("hx_comm_unique_id", buf)
    return buf.raw


class Partition:
    """hx_router_partition: block handles {row_begin, row_end, part}."""

    def __init__(self, n_rows: int, n_parts: int, block_rows: int, policy: int = _hx.HX_POLICY_RANGE):
        h = ctypes.c_void_p()
        call("hx_router_partition", n_rows, n_parts, block_rows, policy, ctypes.byref(h))
        self.h = h
        self.n_parts = n_parts

    def blocks(self) -> List[Tuple[int, int, int]]:
        n = ctypes.c_int64()
        ptr = ctypes.POINTER(_hx.hx_block)()
        call("hx_partition_info", self.h, ctypes.byref(n), ctypes.byref(ptr))
        return [(ptr[i].row_begin, ptr[i].row_end, ptr[i].part) for i in range(n.value)]

    def rows(self, part: int) -> int:
        n = ctypes.c_int64()
        call("hx_partition_rows", self.h, part, ctypes.byref(n))
        return n.value

    def close(self):
        if getattr(self, "h", None):
            call("hx_partition_free", self.h)
            self.h = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass


def router_partition(n_rows: int, n_parts: int, block_rows: int,
                     policy: int = _hx.HX_POLICY_RANGE) -> Partition:
    return Partition(n_rows, n_parts, block_rows, policy)


class Table:
    def __init__(self, ctx: Context, h, keep=None, parent=None):
        self.ctx, self.h, self._keep, self._parent = ctx, h, keep, parent
        _adopt(ctx, self)

    @property
    def n_rows(self) -> int:
        n, c = ctypes.c_int64(), ctypes.c_int()
        call("hx_table_info", self.h, ctypes.byref(n), ctypes.byref(c))
        return n.value

    def slice(self, row_begin: int, row_end: int) -> "Table":
        h = ctypes.c_void_p()
        call("hx_table_slice", self.h, row_begin, row_end, ctypes.byref(h))
        return Table(self.ctx, h, parent=self)

    def read(self, col_id: int, row_begin: int = 0, n: Optional[int] = None) -> np.ndarray:
        """Rows of one column, copied to the host (synchronous)."""
        if n is None:
            n = self.n_rows - row_begin
        out = np.empty(n, dtype=np.int32)
        call("hx_table_read", self.h, col_id, row_begin, n,
             out.ctypes.data_as(ctypes.POINTER(ctypes.c_int32)))
        return out

    def write(self, col_id: int, src_ptr: int, n: int, row_begin: int = 0) -> None:
        """Copy n int32 values from `src_ptr` (pinned host or device memory) into a column
        (asynchronous, on the ctx stream)."""
        call("hx_table_write", self.h, col_id, row_begin, n, src_ptr)

    def close(self):
        if getattr(self, "h", None):
            call("hx_table_free", self.h)
            self.h = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass


def load_columns(ctx: Context, cols: Sequence[Tuple[int, int, int]],
                 part: Optional[Partition] = None, part_index: int = 0,
                 placement: int = _hx.HX_PLACE_COPY, keep=None) -> Table:
    """cols: (col_id, data pointer (host or device), n_rows). `keep` holds the buffers
    alive for views."""
    arr = (hx_col * len(cols))()
    for i, (cid, ptr, n) in enumerate(cols):
        arr[i].col_id, arr[i].data, arr[i].n_rows = cid, ptr, n
    h = ctypes.c_void_p()
    call("hx_load_columns", ctx.h, arr, len(cols), part.h if part else None, part_index,
         placement, ctypes.byref(h))
    return Table(ctx, h, keep=keep)


def load_numpy(ctx: Context, cols: Dict[int, np.ndarray], part: Optional[Partition] = None,
               part_index: int = 0) -> Table:
    """Copy host int32 numpy columns to the device (HX_PLACE_COPY, H2D on the ctx stream)."""
    keep = {k: np.ascontiguousarray(v, dtype=np.int32) for k, v in cols.items()}
    spec = [(k, v.ctypes.data if v.size else 0, v.size) for k, v in keep.items()]
    t = load_columns(ctx, spec, part, part_index, _hx.HX_PLACE_COPY, keep=keep)
    return t


class HashTable:
    def __init__(self, ctx: Context, h, dim: Table):
        self.ctx, self.h, self._dim = ctx, h, dim
        _adopt(ctx, self)

    def info(self, with_codes: bool = False):
        nk, ns, nr = ctypes.c_int64(), ctypes.c_int64(), ctypes.c_int32()
        call("hx_ht_info", self.h, ctypes.byref(nk), ctypes.byref(ns), ctypes.byref(nr), None)
        codes = None
        if with_codes:
            buf = (ctypes.c_int32 * max(1, nr.value))()
            call("hx_ht_info", self.h, None, None, None, buf)
            codes = list(buf)[: nr.value]
        return {"n_keys": nk.value, "n_slots": ns.value, "n_ranks": nr.value, "rank_to_code": codes}

    def broadcast(self, root: int = 0) -> None:
        call("hx_ht_broadcast", self.ctx.h, self.h, root)

    def close(self):
        if getattr(self, "h", None):
            call("hx_ht_free", self.h)
            self.h = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass


def build_dim_ht(ctx: Context, dim: Table, key_col: int, preds: Sequence[_hx.hx_pred] = (),
                 group_col: int = -1, group_lo: int = 0, group_hi: int = 0,
                 flags: int = 0) -> HashTable:
    arr = (_hx.hx_pred * max(1, len(preds)))(*preds)
    h = ctypes.c_void_p()
    if flags:
        call("hx_build_dim_ht_ex", ctx.h, dim.h, key_col, arr, len(preds), group_col, group_lo,
             group_hi, flags, ctypes.byref(h))
    else:
        call("hx_build_dim_ht", ctx.h, dim.h, key_col, arr, len(preds), group_col, group_lo,
             group_hi, ctypes.byref(h))
    return HashTable(ctx, h, dim)


def hash_partition(ctx: Context, t: Table, key_col: int, n_parts: int) -> Tuple[Table, List[int]]:
    """Hash-pack (K3): a new device table with t's rows grouped by part of `key_col`, and the
    part offsets (n_parts + 1)."""
    offs = (ctypes.c_int64 * (n_parts + 1))()
    h = ctypes.c_void_p()
    call("hx_hash_partition", ctx.h, t.h, key_col, n_parts, ctypes.byref(h), offs)
    return Table(ctx, h), list(offs)


def exchange_partitions(ctx: Context, parted: Table, offsets: Sequence[int]) -> Table:
    """Hash-routing exchange: part p to rank p (NCCL); the rows routed to this rank."""
    offs = (ctypes.c_int64 * len(offsets))(*offsets)
    h = ctypes.c_void_p()
    call("hx_exchange_partitions", ctx.h, parted.h, offs, len(offsets) - 1, ctypes.byref(h))
    return Table(ctx, h)


def query_shape(preds=(), joins=(), agg_op=_hx.HX_AGG_SUM, agg_a=0, agg_b=0,
                gdims=()) -> hx_query_shape:
    """joins: sequence of (fk_col_id, ht_index) in probe order; gdims: join indices."""
    s = hx_query_shape()
    s.n_preds = len(preds)
    for i, p in enumerate(preds):
        s.preds[i] = p
    s.n_joins = len(joins)
    for i, (fk, ht) in enumerate(joins):
        s.join_fk_col[i], s.join_ht[i] = fk, ht
    s.agg_op, s.agg_a, s.agg_b = agg_op, agg_a, agg_b
    s.n_gdims = len(gdims)
    for i, g in enumerate(gdims):
        s.gdim_join[i] = g
    return s


class Agg:
    def __init__(self, ctx: Context, h, n_gdims: int, deps):
        self.ctx, self.h, self.n_gdims, self._deps = ctx, h, n_gdims, deps
        _adopt(ctx, self)

    def close(self):
        if getattr(self, "h", None):
            call("hx_agg_free", self.h)
            self.h = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass


def _hts_array(hts: Sequence[HashTable]):
    arr = (ctypes.c_void_p * max(1, len(hts)))()
    for i, t in enumerate(hts):
        arr[i] = t.h.value
    return arr


def pipeline_probe_agg(ctx: Context, fact: Table, shape: hx_query_shape,
                       hts: Sequence[HashTable]) -> Agg:
    h = ctypes.c_void_p()
    call("hx_pipeline_probe_agg", ctx.h, fact.h, ctypes.byref(shape), _hts_array(hts), len(hts),
         ctypes.byref(h))
    return Agg(ctx, h, shape.n_gdims, (fact, list(hts)))


def pipeline_probe_agg_into(ctx: Context, fact: Table, shape: hx_query_shape,
                            hts: Sequence[HashTable], agg: Agg) -> None:
    call("hx_pipeline_probe_agg_into", ctx.h, fact.h, ctypes.byref(shape), _hts_array(hts),
         len(hts), agg.h)


class Plan:
    """hx_plan_*: one prepared query (builds + fused pipeline + merge + finalize)."""

    def __init__(self, ctx: Context, fact: Table, dims: Sequence[Table], builds, shape):
        dim_arr = (ctypes.c_void_p * max(1, len(dims)))(*[d.h.value for d in dims])
        b_arr = (_hx.hx_build_spec * max(1, len(builds)))(*builds)
        h = ctypes.c_void_p()
        call("hx_plan_create", ctx.h, fact.h, dim_arr, len(dims), b_arr, len(builds),
             ctypes.byref(shape), ctypes.byref(h))
        self.ctx, self.h, self._keep = ctx, h, (fact, list(dims))
        _adopt(ctx, self)
        ng, nd = ctypes.c_int64(), ctypes.c_int()
        call("hx_plan_info", h, ctypes.byref(ng), ctypes.byref(nd))
        self.n_groups, self.n_gdims = ng.value, nd.value
        cap = max(1, self.n_groups)
        self._sums = np.zeros(cap, np.int64)
        self._cnts = np.zeros(cap, np.int64)
        self._keys = np.zeros(cap * max(1, self.n_gdims), np.int32)

    def enqueue(self) -> None:
        call("hx_plan_enqueue", self.ctx.h, self.h)

    def result(self):
        """-> (keys int32[n, n_gdims], sums int64[n], counts int64[n]) of the last run."""
        n = ctypes.c_int64()
        call("hx_plan_result", self.h, self._sums.ctypes.data_as(_hx._PI64),
             self._cnts.ctypes.data_as(_hx._PI64), self._keys.ctypes.data_as(_hx._PI32),
             len(self._sums), ctypes.byref(n))
        k = n.value
        return (self._keys[: k * self.n_gdims].reshape(k, self.n_gdims).copy(),
                self._sums[:k].copy(), self._cnts[:k].copy())

    def k1_time(self) -> Tuple[float, int]:
        ms, b = ctypes.c_float(), ctypes.c_int64()
        call("hx_plan_k1_time", self.h, ctypes.byref(ms), ctypes.byref(b))
        return ms.value, b.value

    def k1_span(self, last: "Plan") -> float:
        """ms from this plan's K1 start to `last`'s K1 end (same enqueue)."""
        ms = ctypes.c_float()
        call("hx_plan_k1_span", self.h, last.h, ctypes.byref(ms))
        return ms.value

    def close(self):
        if getattr(self, "h", None):
            call("hx_plan_free", self.h)
            self.h = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass


def plans_enqueue(ctx: Context, plans: Sequence["Plan"]) -> None:
    """hx_plans_enqueue: all builds first (overlapping earlier pipelines), then pipelines."""
    arr = (ctypes.c_void_p * max(1, len(plans)))(*[p.h.value for p in plans])
    call("hx_plans_enqueue", ctx.h, arr, len(plans))


def build_spec(dim: int, key_col: int, preds=(), group_col: int = -1, group_lo: int = 0,
               group_hi: int = 0) -> _hx.hx_build_spec:
    s = _hx.hx_build_spec()
    s.dim, s.key_col, s.n_preds = dim, key_col, len(preds)
    for i, p in enumerate(preds):
        s.preds[i] = p
    s.group_col, s.group_lo, s.group_hi = group_col, group_lo, group_hi
    return s


class Graph:
    """hx_graph_*: CUDA graph of the plan executions enqueued inside `with capture(ctx)`."""

    def __init__(self, ctx: Context, h):
        self.ctx, self.h = ctx, h
        _adopt(ctx, self)

    def launch(self) -> None:
        call("hx_graph_launch", self.ctx.h, self.h)

    def close(self):
        if getattr(self, "h", None):
            call("hx_graph_free", self.h)
            self.h = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass


def capture(ctx: Context, fn) -> Graph:
    """Run fn() (plan enqueues) under stream capture and return the instantiated graph."""
    call("hx_graph_begin", ctx.h)
    try:
        fn()
    finally:
        h = ctypes.c_void_p()
        call("hx_graph_end", ctx.h, ctypes.byref(h))
    return Graph(ctx, h)


def merge_aggregates(ctx: Context, agg: Agg, root: int = -1, cap: int = 4096):
    """-> (keys int32[n, n_gdims], sums int64[n], counts int64[n]) for non-empty groups."""
    while True:
        sums = np.zeros(cap, np.int64)
        cnts = np.zeros(cap, np.int64)
        keys = np.zeros(cap * max(1, agg.n_gdims), np.int32)
        n = ctypes.c_int64()
        rc = getattr(_hx.lib(), "hx_merge_aggregates")(
            ctx.h, agg.h, root, sums.ctypes.data_as(_hx._PI64), cnts.ctypes.data_as(_hx._PI64),
            keys.ctypes.data_as(_hx._PI32), cap, ctypes.byref(n))
        if rc == _hx.HX_ECAPACITY and n.value > cap:
            cap = n.value
            continue
        if rc != _hx.HX_OK:
            raise _hx.HxError(rc, "hx_merge_aggregates", _hx.lib().hx_last_error().decode())
        k = n.value
        return keys[: k * agg.n_gdims].reshape(k, agg.n_gdims), sums[:k], cnts[:k]


# ---- the union router's group layout and host finalize (no GPU needed) --------------------
def group_layout(n_ranks: Sequence[int]) -> Tuple[List[int], int]:
    """hx_group_layout: (strides per grouping dimension, n_groups)."""
    n = len(n_ranks)
    nr = (ctypes.c_int32 * max(1, n))(*n_ranks)
    st = (ctypes.c_int64 * max(1, n))()
    ng = ctypes.c_int64()
    call("hx_group_layout", n, nr, st, ctypes.byref(ng))
    return list(st)[:n], ng.value


def group_decode(n_ranks: Sequence[int], rank_to_code: Sequence[Sequence[int]],
                 sums: np.ndarray, counts: np.ndarray):
    """hx_group_decode: (keys [rows x n_gdims] int32, sums int64, counts int64)."""
    n = len(n_ranks)
    nr = (ctypes.c_int32 * max(1, n))(*n_ranks)
    maps = [np.ascontiguousarray(m, dtype=np.int32) for m in rank_to_code]
    mp = (ctypes.POINTER(ctypes.c_int32) * max(1, n))(
        *[m.ctypes.data_as(ctypes.POINTER(ctypes.c_int32)) for m in maps])
    s = np.ascontiguousarray(sums, dtype=np.int64)
    c = np.ascontiguousarray(counts, dtype=np.int64)
    cap = max(1, len(s))
    keys = np.zeros((cap, max(1, n)), dtype=np.int32)
    os_, oc = np.zeros(cap, dtype=np.int64), np.zeros(cap, dtype=np.int64)
    rows = ctypes.c_int64()
    P64 = ctypes.POINTER(ctypes.c_int64)
    call("hx_group_decode", n, nr, mp, s.ctypes.data_as(P64), c.ctypes.data_as(P64), len(s),
         keys.ctypes.data_as(ctypes.POINTER(ctypes.c_int32)), os_.ctypes.data_as(P64),
         oc.ctypes.data_as(P64), cap, ctypes.byref(rows))
    r = rows.value
    return keys[:r, :n], os_[:r], oc[:r]


# ---- the router's dynamic load balancing across processes (hx_shared_router_*) --------------
class SharedRouter:
    """A block counter in POSIX shared memory drawn from by every process of the node."""

    def __init__(self, name: str, n_blocks: int, create: bool):
        h = ctypes.c_void_p()
        call("hx_shared_router_open", name.encode(), n_blocks, 1 if create else 0, ctypes.byref(h))
        self.h, self.name, self.n_blocks = h, name, n_blocks

    def next(self) -> int:
        b = ctypes.c_int64()
        call("hx_shared_router_next", self.h, ctypes.byref(b))
        return b.value

    def reset(self) -> None:
        call("hx_shared_router_reset", self.h)

    def close(self, unlink: bool = False) -> None:
        if self.h:
            call("hx_shared_router_close", self.h, 1 if unlink else 0)
            self.h = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass


def pipeline_probe_agg_routed(ctx: Context, fact: Table, shape: hx_query_shape,
                              hts: Sequence[HashTable], router: SharedRouter,
                              block_rows: int) -> Tuple["Agg", int]:
    """hx_pipeline_probe_agg_routed -> (agg, blocks this process ran)."""
    arr = _hts_array(hts)
    h = ctypes.c_void_p()
    nb = ctypes.c_int64()
    call("hx_pipeline_probe_agg_routed", ctx.h, fact.h, ctypes.byref(shape), arr, len(hts),
         router.h, block_rows, ctypes.byref(h), ctypes.byref(nb))
    return Agg(ctx, h, shape.n_gdims, (fact, list(hts))), nb.value
