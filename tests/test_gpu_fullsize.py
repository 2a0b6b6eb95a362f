"""Full-size parity (-m gpu): BASELINE.json configs at their real sizes, in the
launch configuration bench.py times (bulk build with degree hints, 2^24-edge
insert / query / delete batches, bucket_bytes 128, lf 0.7), compared with the
unsharded oracle IN FULL: every exported row (canonicalised), every degree, every
query answer, every n_added / n_removed, and every triangle count (SURVEY §8(d):
"bit-exact against the oracle on all five configs").  The oracle runs on the host's
threads (T threads partitioned by source vertex).

The GPU export is canonicalised on the device (sort of (row, dst) keys with torch:
test-side only) before it is compared on the host; the table invariants
(dg_check_invariants) are checked after every compared stage.
"""
import numpy as np
import pytest
import torch

import workloads as wl
from oracle import Oracle
from oracle.compare import Candidates, compare_export, compare_queries
from tests.gpu_util import assert_table_invariants, distinct_nonloop as _distinct_nonloop, gpu_invariants

pytestmark = pytest.mark.gpu


@pytest.fixture(autouse=True)
def _dev(cuda_ok):
    torch.cuda.set_device(0)
    yield
    torch.cuda.synchronize()


def _cu(a):
    return torch.from_numpy(np.ascontiguousarray(a)).to("cuda")


def canonical_export(g):
    """The graph's export with every row sorted by dst (sorted on the device)."""
    ro, d, w = g.export()
    assert not gpu_invariants(ro, d, g.degrees()), "export invariants"
    ro64 = ro.to(torch.int64)
    lens = ro64[1:] - ro64[:-1]
    del ro64
    rows = torch.repeat_interleave(torch.arange(lens.numel(), device="cuda"), lens)
    key = (rows << 32) | d.to(torch.int64)
    del rows
    key, order = torch.sort(key)
    del key
    d = d.view(torch.int32)[order].view(torch.uint32)
    w = w.view(torch.int32)[order].view(torch.uint32)
    return ro.cpu().numpy(), d.cpu().numpy(), w.cpu().numpy()


def assert_same_graph(g, o, where):
    errs = compare_export(canonical_export(g), o.export(), Candidates(*o.candidates()))
    assert not errs, f"{where}: {errs}"
    assert np.array_equal(g.degrees().cpu().numpy(), o.degrees()), f"{where}: degrees"
    assert_table_invariants(g, where)


def assert_same_answers(g, o, qs, qd, where):
    f, qw = g.query_edges(_cu(qs), _cu(qd))
    st, rf, rw = o.query_edges(qs, qd)
    assert st == 0
    errs = compare_queries(qs, qd, f.cpu().numpy(), qw.cpu().numpy(), rf, rw,
                           Candidates(*o.candidates()))
    assert not errs, f"{where}: {errs}"
    return int(rf.sum())


def _bulk(nv, bs, bd, bw, bucket_bytes=128, directed=True, set_variant=False):
    from paper_conf_ipps_awadapo20_b200 import Graph
    src = bs if directed else np.concatenate([bs, bd])
    hints = torch.bincount(_cu(src.astype(np.int64)), minlength=nv).to(torch.int32)
    g = Graph(nv, hints, bucket_bytes=bucket_bytes, directed=directed, set_variant=set_variant)
    added = g.insert_edges(_cu(bs), _cu(bd), None if bw is None else _cu(bw), count=True)
    return g, added


def _bench_step(g, o, nv, B, seed, base, where):
    """bench.py's step: insert B uniform edges, query B (half live, half uniform),
    delete B (half of the inserted edges, half uniform), every result compared."""
    s, d, w = wl.uniform_edges(seed, 1000, B, nv)
    got = g.insert_edges(_cu(s), _cu(d), _cu(w), count=True)
    assert got == o.insert_edges(s, d, w)[1], where
    bs, bd = base
    idx = wl.uniform_index(seed, 5000, B // 2, bs.size)
    us, ud, _ = wl.uniform_edges(seed, 7000, B // 2, nv, weights=False)
    qs, qd = np.concatenate([bs[idx], us]), np.concatenate([bd[idx], ud])
    hits = assert_same_answers(g, o, qs, qd, f"{where} queries")
    assert hits >= int((bs[idx] != bd[idx]).sum())  # every sampled base edge but self-loops
    ys, yd, _ = wl.uniform_edges(seed, 8000, B // 2, nv, weights=False)
    xs, xd = np.concatenate([s[: B // 2], ys]), np.concatenate([d[: B // 2], yd])
    got = g.delete_edges(_cu(xs), _cu(xd), count=True)
    assert got == o.delete_edges(xs, xd)[1], where


def test_config2_fullsize():
    """LJ-like R-MAT, |V| = 4,847,571, |E| = 68,993,773: the bulk build in generator
    (random) order and in src-sorted order, then one bench step of 2^24 batches."""
    nv, m = 4_847_571, 68_993_773
    bs, bd = wl.rmat_edges(2, 0, m, 23, wl.LJLIKE, nv=nv)
    bw = wl.weights(2, 0, m)
    o = Oracle(nv)
    _, want = o.insert_edges(bs, bd, bw)
    g, added = _bulk(nv, bs, bd, bw)
    assert added == want
    assert_same_graph(g, o, "cfg2 bulk build")
    # the same build from src-sorted input (one table filled by consecutive ops)
    order = np.argsort(bs, kind="stable")
    g2, added2 = _bulk(nv, bs[order], bd[order], bw[order])
    assert added2 == want
    assert_same_graph(g2, o, "cfg2 sorted bulk build")
    g2.close()
    _bench_step(g, o, nv, 1 << 24, 2, (bs, bd), "cfg2 step")
    assert_same_graph(g, o, "cfg2 after a step")
    g.close()


@pytest.mark.parametrize("bb", [128, 32, 0])
def test_config3_fullsize(bb):
    """Road-like grid 4,894 x 4,894 (23,951,236 V, 57.7M directed edges): uniform 128-B
    and 32-B buckets and the degree-adaptive layout (bb = 0); one step of 2^22 batches,
    then road growth (held-out lattice edges) in and out again."""
    bs, bd = wl.grid_edges(3, 4894, 4894, 0.6025)
    nv = 4894 * 4894
    bw = wl.weights(3, 0, bs.size)
    o = Oracle(nv)
    _, want = o.insert_edges(bs, bd, bw)
    g, added = _bulk(nv, bs, bd, bw, bucket_bytes=bb)
    assert added == want
    _bench_step(g, o, nv, 1 << 22, 3, (bs, bd), "cfg3 step")
    hs, hd = wl.grid_heldout_edges(3, 4894, 4894, 0.6025)
    idx = wl.uniform_index(3, 424242, 1 << 22, hs.size)
    hw = wl.weights(3, 525252, 1 << 22)
    assert g.insert_edges(_cu(hs[idx]), _cu(hd[idx]), _cu(hw), count=True) == \
        o.insert_edges(hs[idx], hd[idx], hw)[1]
    assert_same_graph(g, o, f"cfg3 bb={bb} growth")
    g.close()


def test_config4_fullsize_stream():
    """R-MAT scale 24 (268M generated edges, Graph500), the mixed stream of SURVEY §8(d)
    for 8 rounds: insert 2^22 new R-MAT edges, query 2^22 (half live, half uniform),
    delete 2^21 (half live, half uniform), delete 2^12 vertices (1/4 from the top-1%
    out-degree vertices), insert 2^16 edges leaving the deleted IDs.  Every count and
    query answer is compared every round; the full graph at rounds 1, 4 and 8."""
    nv, m = 1 << 24, 1 << 28
    bs, bd = wl.rmat_edges(4, 0, m, 24, wl.GRAPH500)
    bw = wl.weights(4, 0, m)
    o = Oracle(nv)
    _, want = o.insert_edges(bs, bd, bw)
    g, added = _bulk(nv, bs, bd, bw)
    assert added == want
    top = np.argsort(o.degrees(), kind="stable")[-(nv // 100):].astype(np.uint32)
    for r in range(1, 9):
        s1, d1 = wl.rmat_edges(4, r, 1 << 22, 24, wl.GRAPH500)
        w1 = wl.weights(4, r, 1 << 22)
        assert g.insert_edges(_cu(s1), _cu(d1), _cu(w1), count=True) == \
            o.insert_edges(s1, d1, w1)[1], f"round {r} insert"
        li = wl.uniform_index(4, 5000 + r, 1 << 21, m)
        us, ud, _ = wl.uniform_edges(4, 6000 + r, 1 << 21, nv, weights=False)
        qs, qd = np.concatenate([bs[li], us]), np.concatenate([bd[li], ud])
        assert_same_answers(g, o, qs, qd, f"round {r} queries")
        li = wl.uniform_index(4, 7000 + r, 1 << 20, m)
        ys, yd, _ = wl.uniform_edges(4, 8000 + r, 1 << 20, nv, weights=False)
        ds, dd = np.concatenate([bs[li], ys]), np.concatenate([bd[li], yd])
        assert g.delete_edges(_cu(ds), _cu(dd), count=True) == o.delete_edges(ds, dd)[1], \
            f"round {r} delete"
        ids = np.concatenate([top[wl.uniform_u32(4, 9000 + r, 1024, top.size)],
                              wl.uniform_u32(4, 9100 + r, 3072, nv)])
        g.delete_vertices(_cu(ids))
        assert g.batch_status() == 0
        o.delete_vertices(ids)
        rs_ = ids[wl.uniform_u32(4, 9200 + r, 1 << 16, ids.size)]
        rd_, _, rw_ = wl.uniform_edges(4, 9300 + r, 1 << 16, nv)
        assert g.insert_edges(_cu(rs_), _cu(rd_), _cu(rw_), count=True) == \
            o.insert_edges(rs_, rd_, rw_)[1], f"round {r} re-insert"
        if r in (1, 4, 8):
            assert_same_graph(g, o, f"cfg4 round {r}")
    g.close()


def test_config5_tc_fullsize():
    """R-MAT scale 22 symmetrised (set variant, 64-B buckets, as bench.py runs it):
    the triangle count equals the oracle's forward-algorithm count on the bulk-built
    graph and after each of the 5 dynamic iterations (insert 2^22 new edges in both
    directions, then count), and is independent of the part split."""
    nv = 1 << 22
    bs, bd = wl.rmat_edges(5, 0, 1 << 26, 22, wl.GRAPH500)
    o = Oracle(nv, directed=False)
    o.insert_edges(bs, bd)
    g, _ = _bulk(nv, bs, bd, None, bucket_bytes=64, directed=False, set_variant=True)
    want = o.triangle_count()
    assert g.triangle_count() == want and want > 10**8
    assert sum(g.triangle_count(p, 4) for p in range(4)) == want
    for it in range(1, 6):
        s1, d1 = wl.rmat_edges(5, it, 1 << 22, 22, wl.GRAPH500)
        assert g.insert_edges(_cu(s1), _cu(d1), count=True) == o.insert_edges(s1, d1)[1]
        assert g.triangle_count() == o.triangle_count(), f"TC iteration {it}"
    assert_same_graph(g, o, "cfg5 after 5 iterations")
    g.close()
