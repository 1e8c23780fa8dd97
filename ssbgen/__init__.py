"""Seeded SSB input generator shared by the oracle and the CUDA path.

This module produces INPUTS only (columns and the dictionary that encodes SSB strings as
order-preserving int32 codes). It holds none of the method's arithmetic: no filter, join,
group-by or aggregation. See ssbgen.h for the distributions; DESIGN.md "Input recipe".

The dictionary encodings are [SSB-spec] (PAPER.md cites SSB [26] at PAPER.md:1124-1125 and
never prints the schema): regions and nations alphabetical, city = nation*10 + digit,
mfgr = m-1, category = (m-1)*5 + (c-1), brand1 = category*40 + (bb-1).
"""
from __future__ import annotations

import ctypes
import os
from typing import Dict

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))

COLS: Dict[str, int] = {
    "lo_orderdate": 0, "lo_custkey": 1, "lo_partkey": 2, "lo_suppkey": 3, "lo_quantity": 4,
    "lo_extendedprice": 5, "lo_discount": 6, "lo_revenue": 7, "lo_supplycost": 8,
    "d_datekey": 16, "d_year": 17, "d_yearmonthnum": 18, "d_weeknuminyear": 19,
    "d_daynuminyear": 20, "d_monthnuminyear": 21,
    "c_custkey": 32, "c_city": 33, "c_nation": 34, "c_region": 35,
    "s_suppkey": 48, "s_city": 49, "s_nation": 50, "s_region": 51,
    "p_partkey": 64, "p_mfgr": 65, "p_category": 66, "p_brand1": 67,
    # §6.4 micro-benchmarks (ssbgen.h MB_*): fact value / probe-key columns, build keys
    "mb_value": 9, "mb_probekey": 10, "mb_buildkey": 68,
}
TABLE_COLS = {
    "lineorder": [c for c in COLS if c.startswith("lo_")],
    "date": ["d_datekey", "d_year", "d_yearmonthnum", "d_weeknuminyear"],
    "customer": ["c_custkey", "c_city", "c_nation", "c_region"],
    "supplier": ["s_suppkey", "s_city", "s_nation", "s_region"],
    "part": ["p_partkey", "p_mfgr", "p_category", "p_brand1"],
}
N_DATE = 2557

REGIONS = ["AFRICA", "AMERICA", "ASIA", "EUROPE", "MIDDLE EAST"]
NATIONS = ["ALGERIA", "ARGENTINA", "BRAZIL", "CANADA", "CHINA", "EGYPT", "ETHIOPIA", "FRANCE",
           "GERMANY", "INDIA", "INDONESIA", "IRAN", "IRAQ", "JAPAN", "JORDAN", "KENYA",
           "MOROCCO", "MOZAMBIQUE", "PERU", "ROMANIA", "RUSSIA", "SAUDI ARABIA",
           "UNITED KINGDOM", "UNITED STATES", "VIETNAM"]
# TPC-H nation -> region (by name), the map ssbgen.h's ssbgen_nation_region() encodes.
NATION_REGION = {
    "ALGERIA": "AFRICA", "ARGENTINA": "AMERICA", "BRAZIL": "AMERICA", "CANADA": "AMERICA",
    "CHINA": "ASIA", "EGYPT": "MIDDLE EAST", "ETHIOPIA": "AFRICA", "FRANCE": "EUROPE",
    "GERMANY": "EUROPE", "INDIA": "ASIA", "INDONESIA": "ASIA", "IRAN": "MIDDLE EAST",
    "IRAQ": "MIDDLE EAST", "JAPAN": "ASIA", "JORDAN": "MIDDLE EAST", "KENYA": "AFRICA",
    "MOROCCO": "AFRICA", "MOZAMBIQUE": "AFRICA", "PERU": "AMERICA", "ROMANIA": "EUROPE",
    "RUSSIA": "EUROPE", "SAUDI ARABIA": "MIDDLE EAST", "UNITED KINGDOM": "EUROPE",
    "UNITED STATES": "AMERICA", "VIETNAM": "ASIA",
}


def region(name: str) -> int:
    return REGIONS.index(name)


def nation(name: str) -> int:
    return NATIONS.index(name)


def city(name: str) -> int:
    """'UNITED KI1' -> nation code of the nation whose 9-char prefix matches, *10 + digit."""
    prefix, digit = name[:-1], int(name[-1])
    matches = [i for i, n in enumerate(NATIONS) if n.ljust(9)[:9] == prefix.ljust(9)[:9]]
    if len(matches) != 1:
        raise ValueError(f"ambiguous or unknown city {name!r}")
    return matches[0] * 10 + digit


def mfgr(name: str) -> int:
    assert name.startswith("MFGR#") and len(name) == 6
    return int(name[5]) - 1


def category(name: str) -> int:
    assert name.startswith("MFGR#") and len(name) == 7
    return (int(name[5]) - 1) * 5 + (int(name[6]) - 1)


def brand1(name: str) -> int:
    assert name.startswith("MFGR#") and len(name) in (8, 9)
    return category(name[:7]) * 40 + (int(name[7:]) - 1)


def sizes(sf: float) -> Dict[str, int]:
    """[SSB-spec] cardinalities: N = 6e6*SF, C = 3e4*SF, S = 2e3*SF,
    P = 2e5*floor(1+log2 SF) (SF >= 1; linear below 1), 2,557 dates."""
    import math
    if sf >= 1:
        n_part = 200_000 * int(math.floor(1 + math.log2(sf)))
    else:
        n_part = max(1, int(round(200_000 * sf)))
    return {
        "n_lineorder": int(round(6_000_000 * sf)),
        "n_customer": max(1, int(round(30_000 * sf))),
        "n_supplier": max(1, int(round(2_000 * sf))),
        "n_part": n_part,
        "n_date": N_DATE,
    }


# PAPER.md:1364-1366 §6.4: "a single column of 23GB" (sum; the join's probe side) and "a
# 7.7MB column" (the join's build side), as int32 values.
MICRO_PAPER_ROWS = 23_000_000_000 // 4
MICRO_PAPER_BUILD = 7_700_000 // 4


def micro_sizes(n_rows: int, n_build: int = MICRO_PAPER_BUILD) -> Dict[str, int]:
    """Sizes of the §6.4 micro-benchmark tables: n_rows fact rows (mb_value, mb_probekey),
    n_build build keys (mb_buildkey)."""
    return {"n_lineorder": int(n_rows), "n_customer": 1, "n_supplier": 1,
            "n_part": max(1, int(n_build)), "n_date": N_DATE}


class _Sizes(ctypes.Structure):
    _fields_ = [("n_lineorder", ctypes.c_int64), ("n_customer", ctypes.c_int64),
                ("n_supplier", ctypes.c_int64), ("n_part", ctypes.c_int64),
                ("n_date", ctypes.c_int64)]


def _csizes(sz: Dict[str, int]) -> _Sizes:
    return _Sizes(sz["n_lineorder"], sz["n_customer"], sz["n_supplier"], sz["n_part"],
                  sz["n_date"])


_host = None
_dev = None


def _host_lib():
    global _host
    if _host is None:
        path = os.path.join(_HERE, "libssbgen.so")
        if not os.path.exists(path):
            raise RuntimeError(f"{path} missing: run `make -C {os.path.dirname(_HERE)}`")
        _host = ctypes.CDLL(path)
        _host.ssbgen_fill.argtypes = [ctypes.c_uint64, ctypes.POINTER(_Sizes), ctypes.c_int,
                                      ctypes.c_int64, ctypes.c_int64, ctypes.c_void_p]
        _host.ssbgen_fill.restype = ctypes.c_int
    return _host


def _dev_lib():
    global _dev
    if _dev is None:
        path = os.path.join(_HERE, "libssbgen_cuda.so")
        if not os.path.exists(path):
            raise RuntimeError(f"{path} missing: run `make -C {os.path.dirname(_HERE)}`")
        _dev = ctypes.CDLL(path)
        _dev.ssbgen_fill_device.argtypes = [ctypes.c_uint64, ctypes.POINTER(_Sizes),
                                            ctypes.c_int, ctypes.c_int64, ctypes.c_int64,
                                            ctypes.c_void_p, ctypes.c_void_p]
        _dev.ssbgen_fill_device.restype = ctypes.c_int
    return _dev


def table_rows(sz: Dict[str, int], col: str) -> int:
    c = COLS[col]
    if c < 16:
        return sz["n_lineorder"]
    if c < 32:
        return sz["n_date"]
    if c < 48:
        return sz["n_customer"]
    if c < 64:
        return sz["n_supplier"]
    return sz["n_part"]


def column(seed: int, sz: Dict[str, int], col: str, row_begin: int = 0,
           n: int | None = None, out: np.ndarray | None = None) -> np.ndarray:
    """Host column `col` rows [row_begin, row_begin+n) as int32."""
    if n is None:
        n = table_rows(sz, col) - row_begin
    if out is None:
        out = np.empty(n, dtype=np.int32)
    assert out.dtype == np.int32 and out.flags.c_contiguous and out.size >= n
    cs = _csizes(sz)
    rc = _host_lib().ssbgen_fill(seed, ctypes.byref(cs), COLS[col], row_begin, n,
                                 out.ctypes.data if n else None)
    if rc != 0:
        raise ValueError(f"ssbgen_fill({col}, {row_begin}, {n}) failed")
    return out


def column_device(seed: int, sz: Dict[str, int], col: str, out_ptr: int, row_begin: int = 0,
                  n: int | None = None, stream: int = 0) -> None:
    """Device column into the CUDA buffer at out_ptr (async on `stream`)."""
    if n is None:
        n = table_rows(sz, col) - row_begin
    cs = _csizes(sz)
    rc = _dev_lib().ssbgen_fill_device(seed, ctypes.byref(cs), COLS[col], row_begin, n,
                                       out_ptr, stream)
    if rc != 0:
        raise RuntimeError(f"ssbgen_fill_device({col}) failed: {rc}")


def database(seed: int, sz: Dict[str, int], lo_begin: int = 0,
             lo_n: int | None = None) -> Dict[str, Dict[str, np.ndarray]]:
    """All SSB tables on the host; lineorder restricted to rows [lo_begin, lo_begin+lo_n)."""
    db: Dict[str, Dict[str, np.ndarray]] = {}
    for t, cols in TABLE_COLS.items():
        db[t] = {}
        for c in cols:
            if t == "lineorder":
                db[t][c] = column(seed, sz, c, lo_begin, lo_n)
            else:
                db[t][c] = column(seed, sz, c)
    return db
