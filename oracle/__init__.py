"""Oracle for the SSB hot path — TEST INFRASTRUCTURE ONLY.

Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline / `--impl reference` legs
may import this package. The product package (paper_journals_pvldb_chrysogeloskaa19_b200)
never imports it and shares no code with it; both only consume columns from `ssbgen`.

`liboracle.so` (ssb_oracle.cpp) is the plain single-threaded SQL-definition evaluator of
the 13 SSB queries; see DESIGN.md "Oracle" for its pins.
"""
from __future__ import annotations

import ctypes
import os
import threading
from typing import Dict, List, Tuple

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))

QUERIES = ["q1.1", "q1.2", "q1.3", "q2.1", "q2.2", "q2.3", "q3.1", "q3.2", "q3.3", "q3.4",
           "q4.1", "q4.2", "q4.3"]
N_KEYS = {"q1.1": 0, "q1.2": 0, "q1.3": 0, "q2.1": 2, "q2.2": 2, "q2.3": 2, "q3.1": 3,
          "q3.2": 3, "q3.3": 3, "q3.4": 3, "q4.1": 2, "q4.2": 3, "q4.3": 3}

_P = ctypes.POINTER(ctypes.c_int32)


class OracleDb(ctypes.Structure):
    _fields_ = ([("n_lo", ctypes.c_int64)] +
                [(c, _P) for c in ("lo_orderdate", "lo_custkey", "lo_partkey", "lo_suppkey",
                                   "lo_quantity", "lo_extendedprice", "lo_discount",
                                   "lo_revenue", "lo_supplycost")] +
                [("n_date", ctypes.c_int64)] +
                [(c, _P) for c in ("d_datekey", "d_year", "d_yearmonthnum", "d_weeknuminyear")] +
                [("n_cust", ctypes.c_int64)] +
                [(c, _P) for c in ("c_custkey", "c_city", "c_nation", "c_region")] +
                [("n_supp", ctypes.c_int64)] +
                [(c, _P) for c in ("s_suppkey", "s_city", "s_nation", "s_region")] +
                [("n_part", ctypes.c_int64)] +
                [(c, _P) for c in ("p_partkey", "p_mfgr", "p_category", "p_brand1")])


class OracleRow(ctypes.Structure):
    _fields_ = [("key", ctypes.c_int32 * 3), ("n_keys", ctypes.c_int32),
                ("sum", ctypes.c_int64), ("count", ctypes.c_int64)]


_lib = None


def lib():
    global _lib
    if _lib is None:
        path = os.path.join(_HERE, "liboracle.so")
        if not os.path.exists(path):
            raise RuntimeError(f"{path} missing: run `make -C {os.path.dirname(_HERE)}`")
        _lib = ctypes.CDLL(path)
        _lib.oracle_ssb_query.argtypes = [ctypes.c_char_p, ctypes.POINTER(OracleDb),
                                          ctypes.c_int64, ctypes.c_int64,
                                          ctypes.POINTER(OracleRow), ctypes.c_int64]
        _lib.oracle_ssb_query.restype = ctypes.c_int64
        _lib.oracle_encode.argtypes = [ctypes.c_int, ctypes.c_char_p]
        _lib.oracle_encode.restype = ctypes.c_int32
    return _lib


def _ptr(a: np.ndarray):
    assert a.dtype == np.int32 and a.flags.c_contiguous
    return a.ctypes.data_as(_P)


def make_db(db: Dict[str, Dict[str, np.ndarray]]) -> Tuple[OracleDb, list]:
    """Marshal host columns (dict of tables of int32 numpy arrays) into an OracleDb."""
    keep = []
    s = OracleDb()
    for table, nfield in (("lineorder", "n_lo"), ("date", "n_date"), ("customer", "n_cust"),
                          ("supplier", "n_supp"), ("part", "n_part")):
        cols = db[table]
        n = None
        for name, arr in cols.items():
            arr = np.ascontiguousarray(arr, dtype=np.int32)
            keep.append(arr)
            if n is None:
                n = arr.size
            assert arr.size == n, f"{table}.{name} length mismatch"
            setattr(s, name, _ptr(arr))
        setattr(s, nfield, n or 0)
    return s, keep


def encode(kind: str, literal: str) -> int:
    kinds = {"region": 0, "nation": 1, "city": 2, "mfgr": 3, "category": 4, "brand1": 5}
    return lib().oracle_encode(kinds[kind], literal.encode())


def run_query(q: str, db: Dict[str, Dict[str, np.ndarray]], row_begin: int = 0,
              row_end: int | None = None, _cdb=None) -> List[Tuple]:
    """Rows (key..., sum, count) in the query's ORDER BY order."""
    if _cdb is None:
        cdb, keep = make_db(db)
    else:
        cdb = _cdb
    n_lo = cdb.n_lo
    if row_end is None:
        row_end = n_lo
    cap = 1 << 16
    out = (OracleRow * cap)()
    n = lib().oracle_ssb_query(q.encode(), ctypes.byref(cdb), row_begin, row_end, out, cap)
    if n < 0:
        raise ValueError(f"oracle_ssb_query({q}) failed: {n}")
    nk = N_KEYS[q]
    return [tuple(out[i].key[:nk]) + (out[i].sum, out[i].count) for i in range(n)]


def as_dict(rows: List[Tuple]) -> Dict[Tuple, Tuple[int, int]]:
    """{group codes: (sum, count)}; a no-GROUP-BY query maps () to its single row."""
    return {tuple(r[:-2]): (r[-2], r[-1]) for r in rows}


def run_query_ranges(q: str, db: Dict[str, Dict[str, np.ndarray]], n_threads: int,
                     row_begin: int = 0, row_end: int | None = None) -> Dict[Tuple, Tuple[int, int]]:
    """The same oracle over n_threads disjoint row ranges (threads; ctypes drops the GIL),
    partial results merged by summation — the union-router merge PAPER.md:485-488."""
    cdb, keep = make_db(db)
    if row_end is None:
        row_end = cdb.n_lo
    bounds = np.linspace(row_begin, row_end, n_threads + 1).astype(np.int64)
    parts: List[Dict] = [None] * n_threads

    def work(i):
        parts[i] = as_dict(run_query(q, db, int(bounds[i]), int(bounds[i + 1]), _cdb=cdb))

    ts = [threading.Thread(target=work, args=(i,)) for i in range(n_threads)]
    for t in ts:
        t.start()
    for t in ts:
        t.join()
    merged: Dict[Tuple, Tuple[int, int]] = {}
    for p in parts:
        for k, (s, c) in p.items():
            s0, c0 = merged.get(k, (0, 0))
            merged[k] = (s0 + s, c0 + c)
    if N_KEYS[q] > 0:
        merged = {k: v for k, v in merged.items() if v[1] > 0}
    return merged


def _lib_idx():
    L = lib()
    if not hasattr(L, "_idx_ready"):
        L.oracle_index_new.argtypes = [ctypes.POINTER(OracleDb)]
        L.oracle_index_new.restype = ctypes.c_void_p
        L.oracle_index_free.argtypes = [ctypes.c_void_p]
        L.oracle_index_free.restype = None
        L.oracle_ssb_query_idx.argtypes = [ctypes.c_char_p, ctypes.c_void_p, ctypes.POINTER(OracleDb),
                                           ctypes.c_int64, ctypes.c_int64,
                                           ctypes.POINTER(OracleRow), ctypes.c_int64]
        L.oracle_ssb_query_idx.restype = ctypes.c_int64
        L._idx_ready = True
    return L


class DimIndex:
    """The oracle's dimension maps built once (oracle_index_new), evaluated against many
    lineorder chunks — the same per-row SQL evaluation as run_query, without rebuilding the
    SF1000 customer map (30 M rows) for every chunk."""

    def __init__(self, db: Dict[str, Dict[str, np.ndarray]]):
        dims = {t: db[t] for t in ("date", "customer", "supplier", "part")}
        dims["lineorder"] = {}
        cdb, self._keep = make_db(dims)
        self._h = _lib_idx().oracle_index_new(ctypes.byref(cdb))
        if not self._h:
            raise RuntimeError("oracle_index_new failed")

    def query(self, q: str, lineorder: Dict[str, np.ndarray], row_begin: int = 0,
              row_end: int | None = None) -> Dict[Tuple, Tuple[int, int]]:
        cdb, keep = make_db({"lineorder": lineorder, "date": {}, "customer": {},
                             "supplier": {}, "part": {}})
        if row_end is None:
            row_end = cdb.n_lo
        cap = 1 << 16
        out = (OracleRow * cap)()
        n = _lib_idx().oracle_ssb_query_idx(q.encode(), self._h, ctypes.byref(cdb), row_begin,
                                            row_end, out, cap)
        if n < 0:
            raise ValueError(f"oracle_ssb_query_idx({q}) failed: {n}")
        nk = N_KEYS[q]
        return as_dict([tuple(out[i].key[:nk]) + (out[i].sum, out[i].count) for i in range(n)])

    def close(self):
        if self._h:
            _lib_idx().oracle_index_free(self._h)
            self._h = None


def merge(parts) -> Dict[Tuple, Tuple[int, int]]:
    """Σ of partial results (the union-router merge); empty groups of
    grouped queries dropped."""
    merged: Dict[Tuple, Tuple[int, int]] = {}
    for p in parts:
        for k, (s, c) in p.items():
            s0, c0 = merged.get(k, (0, 0))
            merged[k] = (s0 + s, c0 + c)
    return merged


def run_queries_generated(queries: List[str], dims_db, gen_lineorder, ranges, n_threads: int,
                          chunk_rows: int = 120_000_000) -> Dict[str, Dict[Tuple, Tuple[int, int]]]:
    """The oracle over lineorder rows that do not fit host memory at once (SF1000: 6e9 rows):
    for each (begin, end) in `ranges`, chunks of `chunk_rows` rows are generated by
    `gen_lineorder(begin, n) -> {column: int32 array}` (the seeded ssbgen fill, OpenMP) and
    every query is evaluated on n_threads row sub-ranges of the chunk (threads; ctypes drops
    the GIL); all partials are summed."""
    idx = DimIndex(dims_db)
    acc: Dict[str, List] = {q: [] for q in queries}
    try:
        for b, e in ranges:
            for c0 in range(b, e, chunk_rows):
                n = min(chunk_rows, e - c0)
                lo = gen_lineorder(c0, n)
                bounds = np.linspace(0, n, n_threads + 1).astype(np.int64)
                res: List = [None] * n_threads

                def work(i):
                    res[i] = {q: idx.query(q, lo, int(bounds[i]), int(bounds[i + 1])) for q in queries}

                ts = [threading.Thread(target=work, args=(i,)) for i in range(n_threads)]
                for t in ts:
                    t.start()
                for t in ts:
                    t.join()
                for q in queries:
                    acc[q].extend(r[q] for r in res)
    finally:
        idx.close()
    out = {}
    for q in queries:
        m = merge(acc[q])
        if N_KEYS[q] > 0:
            m = {k: v for k, v in m.items() if v[1] > 0}
        out[q] = m
    return out
