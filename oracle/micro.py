"""Oracle of the §6.4 micro-benchmark queries — TEST INFRASTRUCTURE ONLY (same rule as the
package: only tests/, __graft_entry__.smoke() and bench.py's baseline legs may use it).

PAPER.md:1350-1356 §6.4: "two queries: i) a sum over a column and ii) a count of the
results of a non-partitioned 1:N join". Plain definitions, numpy as the only primitive:

  sum_column(v)          = SELECT SUM(v), COUNT(*) FROM T                 (int64, exact)
  join_count(b, p, v)    = SELECT COUNT(*), SUM(v) FROM B JOIN P ON B.key = P.key
                           (every pair of equal keys counts once: SQL multiplicity)

The fact columns may be given as an iterator of chunks so the full 23 GB input streams
through host memory; the result is the sum over chunks (the union-router merge,
PAPER.md:485-488, applied to row ranges).
"""
from __future__ import annotations

from typing import Iterable, Tuple

import numpy as np


def sum_column(chunks: Iterable[np.ndarray]) -> Tuple[int, int]:
    """(SUM(v), COUNT(*)) over all chunks of the column, exact int64."""
    total, count = 0, 0
    for v in chunks:
        total += int(np.sum(v, dtype=np.int64))
        count += int(v.size)
    return total, count


def join_count(build_keys: np.ndarray, chunks: Iterable[Tuple[np.ndarray, np.ndarray]]
               ) -> Tuple[int, int]:
    """(COUNT(*), SUM(v)) of build ⋈ probe on key equality, for chunks of (probe_key, v):
    each probe row contributes (multiplicity of its key among the build keys) pairs."""
    build_keys = np.asarray(build_keys)
    if build_keys.size and build_keys.min() >= 0 and build_keys.max() < (1 << 28):
        # non-negative bounded keys: the multiplicity of key k is bincount(build)[k]
        mult_of = np.bincount(build_keys).astype(np.int64)
        count, total = 0, 0
        for pk, v in chunks:
            pk = np.asarray(pk, dtype=np.int64)
            ok = (pk >= 0) & (pk < mult_of.size)
            m = np.where(ok, mult_of[np.where(ok, pk, 0)], 0)
            count += int(m.sum())
            total += int(np.dot(m, np.asarray(v, dtype=np.int64)))
        return count, total
    keys, mult = np.unique(build_keys, return_counts=True)
    count, total = 0, 0
    for pk, v in chunks:
        pos = np.searchsorted(keys, pk)
        pos_c = np.minimum(pos, max(len(keys) - 1, 0))
        hit = (pos < len(keys)) & (keys[pos_c] == pk) if len(keys) else np.zeros(len(pk), bool)
        m = np.where(hit, mult[pos_c] if len(keys) else 0, 0).astype(np.int64)
        count += int(m.sum())
        total += int(np.sum(m * np.asarray(v, dtype=np.int64)))
    return count, total
