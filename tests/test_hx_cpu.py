"""CPU-side checks of the product library (no GPU needed):

  * libhx.so loads and exports every entry point include/hx.h declares;
  * the router (hx_router_partition, host-only) produces disjoint block handles covering
    [0, n_rows), contiguous and balanced for RANGE, block b -> b % P for ROUND_ROBIN;
  * without a GPU the library fails loudly (HX_ECUDA) — there is no CPU fallback;
  * the multi-GPU data path (router partition -> per-rank partial aggregate -> union-router
    sum) is exercised with world_size 2 over torch.distributed gloo.
"""
import os
import re

import numpy as np
import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))

from paper_journals_pvldb_chrysogeloskaa19_b200 import _hx, hx  # noqa: E402


def header_functions():
    src = open(os.path.join(ROOT, "include", "hx.h")).read()
    src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
    return sorted(set(re.findall(r"\b(hx_[a-z0-9_]+)\s*\(", src)))


def test_header_symbols_exported():
    names = header_functions()
    assert "hx_pipeline_probe_agg" in names and "hx_merge_aggregates" in names
    lib = _hx.lib()
    for n in names:
        assert hasattr(lib, n), f"libhx.so does not export {n}"
    assert set(names) == set(_hx.EXPORTED), set(names) ^ set(_hx.EXPORTED)


def test_boundary_calls_named_in_north_star():
    names = header_functions()
    for n in ("hx_load_columns", "hx_build_dim_ht", "hx_pipeline_probe_agg",
              "hx_router_partition", "hx_merge_aggregates"):
        assert n in names


@pytest.mark.parametrize("n_rows,parts,block", [(0, 3, 5), (10, 3, 3), (1, 4, 1 << 22),
                                                (1000, 7, 64), (4097, 2, 4096)])
@pytest.mark.parametrize("policy", [_hx.HX_POLICY_RANGE, _hx.HX_POLICY_ROUND_ROBIN])
def test_router_partition(n_rows, parts, block, policy):
    p = hx.router_partition(n_rows, parts, block, policy)
    blocks = p.blocks()
    assert len(blocks) == (n_rows + block - 1) // block
    cover = np.zeros(n_rows, np.int32)
    for b, (r0, r1, part) in enumerate(blocks):
        assert r0 == b * block and r1 == min(n_rows, (b + 1) * block)
        assert 0 <= part < parts
        cover[r0:r1] += 1
        if policy == _hx.HX_POLICY_ROUND_ROBIN:
            assert part == b % parts
    assert (cover == 1).all()  # disjoint, union = [0, n_rows)
    assert sum(p.rows(i) for i in range(parts)) == n_rows
    if policy == _hx.HX_POLICY_RANGE:
        owners = [part for _, _, part in blocks]
        assert owners == sorted(owners)  # contiguous runs of whole blocks
        counts = np.bincount(owners, minlength=parts) if owners else np.zeros(parts)
        assert counts.max() - counts.min() <= 1  # balanced to within one block


def test_router_rejects_bad_arguments():
    with pytest.raises(_hx.HxError) as e:
        hx.router_partition(-1, 2, 10)
    assert e.value.code == _hx.HX_EINVAL
    with pytest.raises(_hx.HxError):
        hx.router_partition(10, 0, 10)
    with pytest.raises(_hx.HxError):
        hx.router_partition(10, 2, 0)


def test_no_gpu_fails_loudly():
    import torch
    if torch.cuda.is_available():
        pytest.skip("a GPU is present")
    with pytest.raises(_hx.HxError) as e:
        hx.Context(0)
    assert e.value.code in (_hx.HX_ECUDA, _hx.HX_EINVAL)


# ---- world_size 2 over gloo: router partition -> partials -> union-router merge -------------
def _rank_main(rank, world, port, out):
    """One rank of the union-router merge, driven through libhx's host logic: the router
    partition (hx_router_partition) gives this rank its blocks; its partial aggregate (the
    oracle over those rows, standing in for K1, which needs a GPU) is laid out in libhx's
    dense group layout (hx_group_layout: {sums[n_groups], counts[n_groups]}, the 2 x n_groups
    int64 the merge all-reduces), all-reduced over gloo in place of NCCL, and finalized by
    libhx (hx_group_decode). The rank -> code maps come from the tables (tests/ssb_groups.py),
    not from libhx."""
    import torch
    import torch.distributed as dist

    import oracle
    from ssb_groups import rank_maps
    from ssb_tiny import tiny_db

    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    db = tiny_db(17, n_lo=12007)
    n = len(db["lineorder"]["lo_orderdate"])
    part = hx.router_partition(n, world, 1000, _hx.HX_POLICY_ROUND_ROBIN)
    mine = [(b, e) for b, e, p in part.blocks() if p == rank]
    assert sum(e - b for b, e in mine) == part.rows(rank)
    results = {}
    for q in ("q1.1", "q2.1", "q3.1", "q4.2", "q4.3"):
        maps = rank_maps(db, q)
        strides, ng = hx.group_layout([len(m) for m in maps])
        arr = torch.zeros(2 * ng, dtype=torch.int64)
        for b, e in mine:
            for k, (s_, c_) in oracle.as_dict(oracle.run_query(q, db, b, e)).items():
                i = sum(int(np.searchsorted(m, code)) * st for m, code, st in zip(maps, k, strides))
                arr[i] += s_
                arr[ng + i] += c_
        dist.all_reduce(arr)  # the union router's global aggregation (NCCL on GPUs)
        keys, sums, cnts = hx.group_decode([len(m) for m in maps], maps, arr[:ng].numpy(),
                                           arr[ng:].numpy())
        results[q] = {tuple(int(x) for x in keys[i]): (int(sums[i]), int(cnts[i]))
                      for i in range(len(sums))}
        results[q + ":elements"] = int(arr.numel())
    out.put((rank, results))
    dist.destroy_process_group()


def test_two_rank_partition_merge_gloo():
    import multiprocessing as mp
    import socket
    import sys

    sys.path.insert(0, os.path.join(ROOT, "tests"))
    import oracle
    from ssb_tiny import tiny_db

    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    port = s.getsockname()[1]
    s.close()
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    procs = [ctx.Process(target=_rank_main, args=(r, 2, port, q)) for r in range(2)]
    for p in procs:
        p.start()
    got = [q.get(timeout=240) for _ in procs]
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    from ssb_groups import n_groups
    db = tiny_db(17, n_lo=12007)
    for rank, res in got:
        for qq, merged in res.items():
            if qq.endswith(":elements"):  # the merge moves 2 x n_groups int64 per rank
                assert merged == 2 * n_groups(db, qq.split(":")[0]), (rank, qq)
                continue
            want = oracle.as_dict(oracle.run_query(qq, db))
            if not oracle.N_KEYS[qq]:  # ungrouped: one row, also when empty
                assert merged == want, (rank, qq)
            else:
                assert merged == {k: v for k, v in want.items() if v[1] > 0}, (rank, qq)


# ---- world_size 2 over gloo: the hash-partitioned join's exchange (§8(f) NEXT-1) ----------
def _part_of(keys, n_parts):
    """include/hx.h part function: fmix32 (murmur3 finaliser), then ((uint64)h * n_parts) >> 32."""
    m = np.uint64(0xFFFFFFFF)
    h = keys.astype(np.int64).astype(np.uint64) & m
    h ^= h >> np.uint64(16)
    h = (h * np.uint64(0x85EBCA6B)) & m
    h ^= h >> np.uint64(13)
    h = (h * np.uint64(0xC2B2AE35)) & m
    h ^= h >> np.uint64(16)
    return ((h * np.uint64(n_parts)) >> np.uint64(32)).astype(np.int64)


def _hash_rank_main(rank, world, port, out):
    """Each rank owns round-robin router blocks of lineorder and a disjoint half of the
    customer rows; both are hash-packed on the customer key and exchanged (all_to_all over
    gloo, the host stand-in for hx_exchange_partitions' NCCL send/recv); each rank evaluates
    the query on what it received, with the other dimensions replicated; the partials merge
    by group codes (union router). The routing host logic is what libhx runs per rank."""
    import torch
    import torch.distributed as dist

    import oracle
    from ssb_tiny import tiny_db

    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    db = tiny_db(23, n_lo=15013)
    lo, cu = db["lineorder"], db["customer"]
    n = len(lo["lo_orderdate"])
    part = hx.router_partition(n, world, 997, _hx.HX_POLICY_ROUND_ROBIN)
    mine = np.concatenate([np.arange(b, e) for b, e, p in part.blocks() if p == rank])
    cmine = np.arange(rank, len(cu["c_custkey"]), world)  # this rank's customer rows

    def exchange(cols, key):
        dest = _part_of(key, world)
        order = np.argsort(dest, kind="stable")
        send_counts = np.bincount(dest, minlength=world)
        recv_counts = torch.zeros(world, dtype=torch.int64)
        dist.all_to_all_single(recv_counts, torch.from_numpy(send_counts.astype(np.int64)))
        got = {}
        for name, v in cols.items():
            buf = torch.empty(int(recv_counts.sum()), dtype=torch.int32)
            dist.all_to_all_single(buf, torch.from_numpy(np.ascontiguousarray(v[order])),
                                   recv_counts.tolist(), send_counts.tolist())
            got[name] = buf.numpy()
        return got

    lo_in = exchange({k: v[mine] for k, v in lo.items()}, lo["lo_custkey"][mine])
    cu_in = exchange({k: v[cmine] for k, v in cu.items()}, cu["c_custkey"][cmine])
    assert (_part_of(lo_in["lo_custkey"], world) == rank).all()
    assert (_part_of(cu_in["c_custkey"], world) == rank).all()
    local = dict(db, lineorder=lo_in, customer=cu_in)
    results = {}
    for q in ("q3.1", "q3.2", "q4.1", "q4.2"):
        parts = [None] * world
        dist.all_gather_object(parts, oracle.as_dict(oracle.run_query(q, local)))
        m = oracle.merge(parts)
        results[q] = {k: v for k, v in m.items() if v[1] > 0} if oracle.N_KEYS[q] else m
    out.put((rank, results))
    dist.destroy_process_group()


def test_two_rank_hash_partitioned_join_gloo():
    import multiprocessing as mp
    import socket
    import sys

    sys.path.insert(0, os.path.join(ROOT, "tests"))
    import oracle
    from ssb_tiny import tiny_db

    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    port = s.getsockname()[1]
    s.close()
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    procs = [ctx.Process(target=_hash_rank_main, args=(r, 2, port, q)) for r in range(2)]
    for p in procs:
        p.start()
    got = [q.get(timeout=240) for _ in procs]
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    db = tiny_db(23, n_lo=15013)
    for rank, res in got:
        for qq, merged in res.items():
            assert merged == oracle.as_dict(oracle.run_query(qq, db)), (rank, qq)


# ---- the router's dynamic load balancing across processes (hx_shared_router) ---------------
def _router_worker(name, n_blocks, out):
    from paper_journals_pvldb_chrysogeloskaa19_b200 import hx as hx_
    r = hx_.SharedRouter(name, n_blocks, create=False)
    got = []
    while True:
        b = r.next()
        if b < 0:
            break
        got.append(b)
    r.close()
    out.put(got)


def test_shared_router_hands_out_every_block_once_across_processes():
    """Four processes draw from one counter in POSIX shared memory: the blocks they get are
    disjoint and cover 0 .. n_blocks-1 (dynamic routing to consumers)."""
    import multiprocessing as mp
    name, n = f"/hx_test_router_{os.getpid()}", 20011
    r = hx.SharedRouter(name, n, create=True)
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    procs = [ctx.Process(target=_router_worker, args=(name, n, q)) for _ in range(4)]
    for p in procs:
        p.start()
    parts = [q.get(timeout=120) for _ in procs]
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    allb = sorted(b for part in parts for b in part)
    assert allb == list(range(n))
    assert all(part == sorted(part) for part in parts)  # each draws in increasing order
    assert r.next() == -1
    r.reset()
    assert r.next() == 0
    r.close(unlink=True)


def test_shared_router_rejects_bad_arguments():
    with pytest.raises(_hx.HxError):
        hx.SharedRouter("no_slash", 4, create=True)
    name = f"/hx_test_router_b{os.getpid()}"
    r = hx.SharedRouter(name, 8, create=True)
    with pytest.raises(_hx.HxError) as e:
        hx.SharedRouter(name, 9, create=False)  # created for another block count
    assert e.value.code == _hx.HX_EINVAL
    with pytest.raises(_hx.HxError):
        hx.SharedRouter("/hx_test_router_missing_x", 8, create=False)
    r.close(unlink=True)


# ---- the union router's host layout and finalize (hx_group_layout / hx_group_decode) -------
def test_group_layout_is_row_major_mixed_radix():
    """Independent restatement: index = sum_g r_g * prod_{h > g} n_h (the last dimension
    fastest), n_groups = prod n_g."""
    n = [7, 5, 3]
    strides, ng = hx.group_layout(n)
    assert ng == 105 and strides == [15, 3, 1]
    seen = set()
    for r0 in range(7):
        for r1 in range(5):
            for r2 in range(3):
                seen.add(r0 * strides[0] + r1 * strides[1] + r2 * strides[2])
    assert seen == set(range(ng))
    assert hx.group_layout([]) == ([], 1)
    with pytest.raises(_hx.HxError) as e:
        hx.group_layout([1 << 14, 1 << 14])  # 2^28 > HX_MAX_GROUPS
    assert e.value.code == _hx.HX_ECAPACITY
    with pytest.raises(_hx.HxError):
        hx.group_layout([3, 0])


def test_group_decode_drops_empty_groups_and_maps_codes():
    rng = np.random.default_rng(5)
    n = [4, 6]
    maps = [np.array([1992, 1993, 1995, 1998]), np.array([3, 7, 11, 12, 40, 41])]
    ng = 24
    cnt = rng.integers(0, 3, ng)
    sums = rng.integers(-50, 50, ng) * (cnt > 0)
    keys, s, c = hx.group_decode(n, maps, sums, cnt)
    want = [(int(maps[0][i // 6]), int(maps[1][i % 6]), int(sums[i]), int(cnt[i]))
            for i in range(ng) if cnt[i] > 0]
    assert [(int(k[0]), int(k[1]), int(x), int(y)) for k, x, y in zip(keys, s, c)] == want
    # ungrouped: the one row is kept even with count 0 (SQL NULL sum, R7)
    k0, s0, c0 = hx.group_decode([], [], np.array([0]), np.array([0]))
    assert len(s0) == 1 and int(c0[0]) == 0
    with pytest.raises(_hx.HxError):  # n_groups must match the layout
        hx.group_decode(n, maps, sums[:10], cnt[:10])


def test_ring_slot_reciprocal_is_exact():
    """K1 finds the ring slot and phase of a CTA's i-th tile with a multiply-high by
    floor(2^32 / stages) + 1 (hx_probe.cu, K1Params::stage_magic) instead of a runtime divide:
    exact for every ring depth K1 plans (2..16) over more tiles than one CTA ever gets
    (a launch is at most 2^20 tiles; checked to 2^22 and at the top of 32 bits / stages)."""
    for stages in range(2, 17):
        magic = (1 << 32) // stages + 1
        i = np.concatenate([np.arange(1 << 22, dtype=np.uint64),
                            np.arange((1 << 32) // stages - 4096, (1 << 32) // stages, dtype=np.uint64)])
        q = (i * np.uint64(magic)) >> np.uint64(32)
        assert np.array_equal(q, i // np.uint64(stages)), stages
