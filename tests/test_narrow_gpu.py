"""Narrow column encodings (hx_table_encode) on the GPU: lineorder
columns stored in 1 or 2 bytes (frame of reference) give the oracle's rows bit-exactly for all
13 queries — plain calls and prepared plans, ragged tails at every width, both K1 consumer-warp
instances — and the operators that read only int32 columns refuse narrow tables."""
import numpy as np
import pytest

import oracle
import ssbgen
from ssb_tiny import tiny_db

pytestmark = pytest.mark.gpu

torch = pytest.importorskip("torch")
if not torch.cuda.is_available():
    pytest.skip("needs a CUDA GPU", allow_module_level=True)

from paper_journals_pvldb_chrysogeloskaa19_b200 import _hx, hx, ssb  # noqa: E402

C = ssbgen.COLS


@pytest.fixture(scope="module")
def ctx():
    c = hx.Context(0)
    yield c
    c.close()


def _run(ctx, db, plans=True):
    dims, fact = ssb.load_db_numpy(ctx, db)
    enc = ssb.narrow_fact(fact)
    eng = ssb.SsbEngine(ctx, dims, fact)
    for q in ssb.QUERIES:
        want = oracle.run_query(q, db)
        assert eng.run(q) == want, (q, enc)
        if plans:
            pl = eng.plan(q)
            pl.enqueue()
            assert pl.rows() == want, (q, enc)
            pl.close()
    return enc


@pytest.mark.parametrize("sf,seed", [(0.01, 42), (0.05, 7)])
def test_narrow_parity_small_sf(ctx, sf, seed):
    enc = _run(ctx, ssbgen.database(seed, ssbgen.sizes(sf)))
    # quantity and discount in one byte, the order date (and the small-SF keys) in two
    assert enc["lo_quantity"] == 1 and enc["lo_discount"] == 1 and enc["lo_orderdate"] == 2


@pytest.mark.parametrize("n_lo", [1, 5, 15, 16, 17, 2561, 4096 * 3 + 7])
def test_narrow_ragged_tails(ctx, n_lo):
    """Tails that are not a multiple of 16 rows (the 1-byte columns' bulk-copy unit)."""
    _run(ctx, tiny_db(11, n_lo=n_lo), plans=False)


@pytest.mark.parametrize("w", ["20", "26"])
def test_narrow_both_warp_instances(ctx, monkeypatch, w):
    monkeypatch.setenv("HX_K1_W", w)
    _run(ctx, tiny_db(3, n_lo=30001))


def test_encode_rejects_what_does_not_fit_and_unsupported_ops(ctx):
    db = ssbgen.database(5, ssbgen.sizes(0.01))
    dims, fact = ssb.load_db_numpy(ctx, db)
    with pytest.raises(_hx.HxError) as e:  # revenue spans far more than 16 bits
        fact.encode(C["lo_revenue"], 2)
    assert e.value.code == _hx.HX_EINVAL
    with pytest.raises(_hx.HxError):
        fact.encode(C["lo_quantity"], 3)
    fact.encode(C["lo_quantity"], 1)
    with pytest.raises(_hx.HxError):  # already encoded
        fact.encode(C["lo_quantity"], 1)
    for call in (lambda: fact.read(C["lo_revenue"]),
                 lambda: fact.slice(0, 10),
                 lambda: hx.hash_partition(ctx, fact, C["lo_custkey"], 2)):
        with pytest.raises(_hx.HxError) as e:
            call()
        assert e.value.code == _hx.HX_EUNSUPPORTED
    # a narrow dimension cannot be built from (the builds read int32 columns)
    dims["supplier"].encode(C["s_region"], 1)
    with pytest.raises(_hx.HxError) as e:
        ssb.SsbEngine(ctx, dims, fact).run("q2.1")
    assert e.value.code == _hx.HX_EUNSUPPORTED
