"""Full-size parity (-m gpu): BASELINE.json configs at their real sizes, in the
launch configuration bench.py times (bulk build with degree hints, 2^24-edge
insert / query / delete batches, bucket_bytes 128, lf 0.7).

The oracle cannot hold these graphs cheaply, so it computes SAMPLED outputs one
row at a time: every adjacency list is independent (A_u only ever receives ops
whose source is u), so feeding the oracle the ops restricted to a random row
sample R reproduces the exact rows R.  Size-independent properties are checked on
the whole export: no duplicate edges, no self-loops, degree == row length, and the
number of stored edges equals the number of distinct non-loop keys (checked with
torch on the GPU: test-side accounting, not the product path).
"""
import numpy as np
import pytest
import torch

import workloads as wl
from oracle import Oracle
from oracle.compare import Candidates, compare_queries
from tests.gpu_util import distinct_nonloop as _distinct_nonloop, gpu_invariants

pytestmark = pytest.mark.gpu


@pytest.fixture(autouse=True)
def _dev(cuda_ok):
    torch.cuda.set_device(0)
    yield
    torch.cuda.synchronize()


def _cu(a):
    return torch.from_numpy(np.ascontiguousarray(a)).to("cuda")


def _rows_equal(g_export, o, rows, where):
    """GPU export rows `rows` (global ids) == oracle rows (oracle fed only those rows)."""
    ro, d, w = g_export
    ro_o, d_o, w_o = o.export()
    cand = Candidates(*o.candidates())
    for u in rows[:200000]:
        a, b = int(ro[u]), int(ro[u + 1])
        oa, ob = int(ro_o[u]), int(ro_o[u + 1])
        gd, gw = d[a:b], w[a:b]
        order = np.argsort(gd, kind="stable")
        gd, gw = gd[order], gw[order]
        assert np.array_equal(gd, d_o[oa:ob]), f"{where}: row {u} dst differs"
        bad = np.nonzero(gw != w_o[oa:ob])[0]
        if bad.size:
            keys = (np.uint64(u) << np.uint64(32)) | gd[bad].astype(np.uint64)
            assert cand.allowed(keys, gw[bad]).all(), f"{where}: row {u} weight differs"
    return cand


def _run_config(nv, bs, bd, bw, B, seed, sample_frac=1 / 256, bucket_bytes=128):
    from paper_conf_ipps_awadapo20_b200 import Graph
    hints = torch.bincount(_cu(bs.astype(np.int64)), minlength=nv).to(torch.int32)
    g = Graph(nv, hints, bucket_bytes=bucket_bytes)
    added = g.insert_edges(_cu(bs), _cu(bd), _cu(bw), count=True)
    distinct = _distinct_nonloop(bs, bd)
    assert added == distinct
    rs = np.random.RandomState(seed)
    R = np.sort(rs.choice(nv, max(1, int(nv * sample_frac)), replace=False)).astype(np.uint32)
    inR = np.zeros(nv, bool)
    inR[R] = True
    o = Oracle(nv)
    m = inR[bs]
    o.insert_edges(bs[m], bd[m], bw[m])
    exd = g.export()
    assert not gpu_invariants(exd[0], exd[1], g.degrees())
    assert exd[1].numel() == distinct
    ex = [x.cpu().numpy() for x in exd]
    _rows_equal(ex, o, R, "bulk build")
    # one bench step
    s, d, w = wl.uniform_edges(seed, 1000, B, nv)
    g.insert_edges(_cu(s), _cu(d), _cu(w))
    m = inR[s]
    o.insert_edges(s[m], d[m], w[m])
    qs, qd, _ = wl.uniform_edges(seed, 7000, B // 2, nv, weights=False)
    qs = np.concatenate([bs[: B // 2], qs])
    qd = np.concatenate([bd[: B // 2], qd])
    f, qw = g.query_edges(_cu(qs), _cu(qd))
    mq = inR[qs]
    st, rf, rw = o.query_edges(qs[mq], qd[mq])
    cand = Candidates(*o.candidates())
    errs = compare_queries(qs[mq], qd[mq], f.cpu().numpy()[mq], qw.cpu().numpy()[mq], rf, rw, cand)
    assert not errs, errs
    g.delete_edges(_cu(s), _cu(d))
    o.delete_edges(s[m], d[m])
    exd = g.export()
    assert not gpu_invariants(exd[0], exd[1], g.degrees())
    ex = [x.cpu().numpy() for x in exd]
    _rows_equal(ex, o, R, "after insert+delete step")
    return g, o, R, inR


def test_config2_fullsize_sampled():
    """LJ-like R-MAT, |V| = 4,847,571, |E| = 68,993,773; step batch 2^24."""
    nv, m = 4_847_571, 68_993_773
    bs, bd = wl.rmat_edges(2, 0, m, 23, wl.LJLIKE, nv=nv)
    bw = wl.weights(2, 0, m)
    g, o, R, inR = _run_config(nv, bs, bd, bw, 1 << 24, 2)
    g.close()


@pytest.mark.parametrize("bb", [128, 0])
def test_config3_fullsize_sampled(bb):
    """Road-like grid 4,894 x 4,894 (23,951,236 V, 57.7M directed edges); uniform
    128-B buckets and the degree-adaptive layout (bb = 0)."""
    bs, bd = wl.grid_edges(3, 4894, 4894, 0.6025)
    nv = 4894 * 4894
    bw = wl.weights(3, 0, bs.size)
    g, o, R, inR = _run_config(nv, bs, bd, bw, 1 << 22, 3, bucket_bytes=bb)
    g.close()


def test_config4_fullsize_sampled_with_vertex_deletion():
    """R-MAT scale 24 (268M generated edges, Graph500): bulk build, one mixed-stream
    step including vertex deletion (streaming purge sweep) and re-insertion."""
    from paper_conf_ipps_awadapo20_b200 import Graph
    nv, m = 1 << 24, 1 << 28
    bs, bd = wl.rmat_edges(4, 0, m, 24, wl.GRAPH500)
    bw = wl.weights(4, 0, m)
    hints = torch.bincount(_cu(bs.astype(np.int64)), minlength=nv)
    top = torch.topk(hints, nv // 100).indices.cpu().numpy().astype(np.uint32)
    g = Graph(nv, hints.to(torch.int32))
    del hints
    assert g.insert_edges(_cu(bs), _cu(bd), _cu(bw), count=True) == _distinct_nonloop(bs, bd)
    rs = np.random.RandomState(4)
    R = np.sort(rs.choice(nv, nv // 512, replace=False)).astype(np.uint32)
    inR = np.zeros(nv, bool)
    inR[R] = True
    o = Oracle(nv)
    mm = inR[bs]
    o.insert_edges(bs[mm], bd[mm], bw[mm])
    # mixed step: insert 2^22 R-MAT edges, delete 2^21, delete 2^12 vertices (1/4 hubs)
    s1, d1 = wl.rmat_edges(4, 1, 1 << 22, 24, wl.GRAPH500)
    w1 = wl.weights(4, 1, 1 << 22)
    g.insert_edges(_cu(s1), _cu(d1), _cu(w1))
    mm = inR[s1]
    o.insert_edges(s1[mm], d1[mm], w1[mm])
    ds, dd, _ = wl.uniform_edges(4, 8000, 1 << 21, nv, weights=False)
    ds[: 1 << 20], dd[: 1 << 20] = bs[: 1 << 20], bd[: 1 << 20]
    g.delete_edges(_cu(ds), _cu(dd))
    mm = inR[ds]
    o.delete_edges(ds[mm], dd[mm])
    ids = np.concatenate([top[wl.uniform_u32(4, 9000, 1024, top.size)],
                          wl.uniform_u32(4, 9100, 3072, nv)])
    g.delete_vertices(_cu(ids))
    assert g.batch_status() == 0
    o.delete_vertices(ids)  # removes rows in R and incoming edges into every row of R
    rs_, rd_, rw_ = ids[wl.uniform_u32(4, 9200, 1 << 16, ids.size)], \
        wl.uniform_u32(4, 9300, 1 << 16, nv), wl.uniform_u32(4, 9400, 1 << 16, 0)
    g.insert_edges(_cu(rs_), _cu(rd_), _cu(rw_))
    mm = inR[rs_]
    o.insert_edges(rs_[mm], rd_[mm], rw_[mm])
    exd = g.export()
    assert not gpu_invariants(exd[0], exd[1], g.degrees())
    # no stored edge points at a deleted vertex unless it was re-inserted afterwards
    d64 = exd[1].to(torch.int64)
    dead = torch.isin(d64, _cu(ids.astype(np.int64)))
    if bool(dead.any()):
        lens = (exd[0][1:].to(torch.int64) - exd[0][:-1].to(torch.int64))
        rows = torch.repeat_interleave(torch.arange(nv, device="cuda"), lens)
        reins = set(zip(rs_.tolist(), rd_.tolist()))
        for u, v in zip(rows[dead][:1000].tolist(), d64[dead][:1000].tolist()):
            assert (u, v) in reins
    ex = [x.cpu().numpy() for x in exd]
    _rows_equal(ex, o, R, "cfg4 mixed step")
    g.close()


def test_config5_tc_fullsize_properties():
    """R-MAT scale 22 symmetrised: the triangle count is independent of the bucket
    geometry and of the part/nparts split (properties that hold at any size; the
    oracle comparison runs at scale 15 in test_gpu_parity)."""
    from paper_conf_ipps_awadapo20_b200 import Graph
    nv = 1 << 22
    bs, bd = wl.rmat_edges(5, 0, 1 << 26, 22, wl.GRAPH500)
    deg = torch.bincount(_cu(np.concatenate([bs, bd]).astype(np.int64)), minlength=nv).to(torch.int32)
    counts = []
    for bb in (128, 32):
        g = Graph(nv, deg, directed=False, bucket_bytes=bb)
        g.insert_edges(_cu(bs), _cu(bd))
        counts.append(g.triangle_count())
        if bb == 128:
            assert sum(g.triangle_count(p, 4) for p in range(4)) == counts[0]
        g.close()
    assert counts[0] == counts[1] and counts[0] > 10**8
