"""Pins of the §6.4 micro-benchmark oracle (oracle/micro.py) and of its inputs
(ssbgen mb_* columns): closed forms, brute force on tiny inputs, chunking invariance,
the probe match rate."""
import numpy as np
import pytest

import ssbgen
from oracle import micro


def test_sum_closed_form_and_chunking():
    n = 1_000_003
    v = np.arange(n, dtype=np.int32)
    assert micro.sum_column([v]) == (n * (n - 1) // 2, n)
    parts = np.array_split(v, 7)
    assert micro.sum_column(parts) == (n * (n - 1) // 2, n)   # union-router merge of ranges
    assert micro.sum_column([]) == (0, 0)


def test_sum_brute_force_tiny():
    rng = np.random.default_rng(3)
    v = rng.integers(-2**31, 2**31, size=500, dtype=np.int64).astype(np.int32)
    want = 0
    for x in v.tolist():
        want += x
    assert micro.sum_column([v]) == (want, 500)


def test_join_closed_form():
    # build = odd keys 1..2n-1, probe = every key 1..2n with v = key: the odd half matches,
    # COUNT = n and SUM = 1 + 3 + .. + (2n-1) = n^2
    n = 100_000
    build = 2 * np.arange(n, dtype=np.int32) + 1
    probe = np.arange(1, 2 * n + 1, dtype=np.int32)
    assert micro.join_count(build, [(probe, probe)]) == (n, n * n)


def test_join_brute_force_with_duplicates_and_misses():
    rng = np.random.default_rng(5)
    build = rng.integers(0, 40, size=60).astype(np.int32)          # duplicate keys
    probe = rng.integers(-5, 50, size=300).astype(np.int32)        # misses on both sides
    v = rng.integers(-1000, 1000, size=300).astype(np.int32)
    cnt, tot = 0, 0
    for p, x in zip(probe.tolist(), v.tolist()):
        for b in build.tolist():
            if b == p:
                cnt += 1
                tot += x
    chunks = [(probe[:100], v[:100]), (probe[100:], v[100:])]
    assert micro.join_count(build, chunks) == (cnt, tot)
    # the same through the sorted-key path (a negative build key disables the bincount path)
    build_neg = np.concatenate([build, np.array([-7], np.int32)])
    probe_neg = np.concatenate([probe, np.array([-7, -7], np.int32)])
    v_neg = np.concatenate([v, np.array([11, 13], np.int32)])
    assert micro.join_count(build_neg, [(probe_neg, v_neg)]) == (cnt + 2, tot + 24)
    assert micro.join_count(np.array([], np.int32), chunks) == (0, 0)


def test_micro_inputs():
    sz = ssbgen.micro_sizes(200_000, 5_000)
    b = ssbgen.column(9, sz, "mb_buildkey")
    assert np.array_equal(b, 2 * np.arange(5_000, dtype=np.int32) + 1)
    p = ssbgen.column(9, sz, "mb_probekey")
    assert p.min() >= 1 and p.max() <= 10_000
    # a probe key matches iff it is odd: rate 1/2 within 5 sigma
    rate = float(np.mean(p % 2 == 1))
    assert abs(rate - 0.5) < 5 * np.sqrt(0.25 / p.size)
    v = ssbgen.column(9, sz, "mb_value")
    assert v.min() >= 0 and v.max() < 2**20
    assert abs(v.mean() - (2**20 - 1) / 2) < 5 * (2**20 / np.sqrt(12)) / np.sqrt(v.size)
