"""GPU-vs-oracle parity through the C ABI (-m gpu).

Bit-exact on exports (canonicalised), degrees, counts and query answers; a key
duplicated inside its most recent insert batch may hold any of that batch's
weights for it (Q1).  Sizes span many warp tiles with ragged tails.
"""
import os
import subprocess
import sys

import numpy as np
import pytest
import torch

import workloads as wl
from oracle import Oracle
from tests.golden_script import load, run_script
from tests.gpu_util import GpuAdapter, check_against_oracle, check_queries, cuda

pytestmark = pytest.mark.gpu

GEOMS = [32, 64, 128]
GEOMS_A = GEOMS + [0]  # 0 = degree-adaptive bucket sizes (DG_FLAG_ADAPTIVE)


@pytest.fixture(autouse=True)
def _dev(cuda_ok):
    torch.cuda.set_device(0)
    yield
    torch.cuda.synchronize()


@pytest.mark.parametrize("bb", GEOMS_A)
@pytest.mark.parametrize("name", ["edge_ops_directed.txt", "edge_ops_undirected.txt"])
def test_golden_scripts_on_gpu(name, bb):
    run_script(load(name), lambda n, directed: GpuAdapter(n, directed, bucket_bytes=bb))


def _config1_stream(bb, hints, directed, seed=1, reuse=True, set_variant=False):
    """Config 1 (BASELINE.json configs[0]; SURVEY §8(d) cfg 1): |V| = 1,024;
    16 insert batches of 1,024 (5% forced intra-batch duplicates with distinct
    weights), queries, deletes, vertex deletions, re-insertion, growth and an
    out-of-range batch — compared with the oracle after every batch."""
    from paper_conf_ipps_awadapo20_b200 import DGError, DG_ERR_VERTEX_OUT_OF_RANGE, Graph
    nv = 1024
    hint = wl.out_degrees(wl.uniform_edges(seed, 0, 16 * 1024, nv)[0], nv) if hints else None
    g = Graph(nv, hint, bucket_bytes=bb, directed=directed, reuse_tombstones=reuse,
              set_variant=set_variant)
    o = Oracle(nv, directed)

    def ow(w):  # the set variant stores no weights: the oracle sees 0
        return np.zeros_like(w) if set_variant else w

    stream = 1000
    for b in range(16):
        s, d, w = wl.uniform_edges(seed, stream + b, 1024, nv)
        k = 51  # 5%: repeat earlier keys of the same batch with distinct weights
        s[-k:], d[-k:] = s[:k], d[:k]
        st, added = o.insert_edges(s, d, ow(w))
        assert g.insert_edges(cuda(s), cuda(d), cuda(w), count=True) == added
        cand = check_against_oracle(g, o, f"insert batch {b}")
        # queries: half live (from the oracle's export), half uniform
        ro, dd, _ = o.export()
        rows = np.repeat(np.arange(nv, dtype=np.uint32), np.diff(ro).astype(np.int64))
        pick = wl.uniform_index(seed, 5000 + b, 512, max(dd.size, 1))
        qs = np.concatenate([rows[pick], wl.uniform_edges(seed, 6000 + b, 512, nv)[0]])
        qd = np.concatenate([dd[pick], wl.uniform_edges(seed, 6000 + b, 512, nv)[1]])
        check_queries(g, o, qs, qd, cand, f"query batch {b}")
    for b in range(4):
        ro, dd, _ = o.export()
        rows = np.repeat(np.arange(nv, dtype=np.uint32), np.diff(ro).astype(np.int64))
        pick = wl.uniform_index(seed, 7000 + b, 512, dd.size)
        us, ud, _ = wl.uniform_edges(seed, 8000 + b, 512, nv)
        s = np.concatenate([rows[pick], us]); d = np.concatenate([dd[pick], ud])
        assert g.delete_edges(cuda(s), cuda(d), count=True) == o.delete_edges(s, d)[1]
        check_against_oracle(g, o, f"delete batch {b}")
    for b in range(4):
        ids = wl.uniform_u32(seed, 9000 + b, 16, nv)
        g.delete_vertices(cuda(ids))
        assert g.batch_status() == 0
        o.delete_vertices(ids)
        check_against_oracle(g, o, f"vertex deletion {b}")
        # re-insert edges touching the deleted IDs (vertex re-insertion)
        s, d, w = wl.uniform_edges(seed, 9500 + b, 256, nv)
        s[:128] = ids[np.arange(128) % ids.size]
        d[128:] = ids[np.arange(128) % ids.size]
        st, added = o.insert_edges(s, d, ow(w))
        assert g.insert_edges(cuda(s), cuda(d), cuda(w), count=True) == added
        check_against_oracle(g, o, f"re-insert {b}")
    # growth: vertex insertion 1024..1279, then 1,024 edges over [0, 1280)
    new = np.arange(1024, 1280, dtype=np.uint32)
    g.insert_vertices(cuda(new), cuda(np.full(new.size, 20, np.uint32)))
    o.insert_vertices(new)
    assert g.num_vertices == 1280
    s, d, w = wl.uniform_edges(seed, 9900, 1024, 1280)
    st, added = o.insert_edges(s, d, ow(w))
    assert g.insert_edges(cuda(s), cuda(d), cuda(w), count=True) == added
    check_against_oracle(g, o, "after growth")
    # out-of-range batch: rejected, graph unchanged (Q7)
    s, d, w = wl.uniform_edges(seed, 9901, 1024, 1280)
    s[500] = 1280
    with pytest.raises(DGError) as e:
        g.insert_edges(cuda(s), cuda(d), cuda(w), count=True)
    assert e.value.status == DG_ERR_VERTEX_OUT_OF_RANGE
    with pytest.raises(DGError):
        g.delete_edges(cuda(s), cuda(d), count=True)
    g.delete_vertices(cuda(np.array([5, 5000], np.uint32)))
    assert g.batch_status() == DG_ERR_VERTEX_OUT_OF_RANGE
    check_against_oracle(g, o, "after rejected batches")
    st = g.stats()
    assert st["live_pairs"] == o.num_edges()
    g.close()


@pytest.mark.parametrize("bb", GEOMS_A)
@pytest.mark.parametrize("hints", [False, True])
def test_config1_directed(bb, hints):
    _config1_stream(bb, hints, True)


@pytest.mark.parametrize("bb", [32, 128, 0])
def test_config1_undirected(bb):
    _config1_stream(bb, False, False, seed=3)


@pytest.mark.parametrize("bb", [32, 128, 0])
def test_config1_append_only(bb):
    """The paper's default policy: tombstones are never reused."""
    _config1_stream(bb, False, True, seed=4, reuse=False)


@pytest.mark.parametrize("bb", GEOMS_A)
@pytest.mark.parametrize("directed", [True, False])
def test_config1_set_variant(bb, directed):
    """Set variant (keys only): the config-1 stream
    against the oracle with weights read as 0."""
    _config1_stream(bb, directed, directed, seed=11, set_variant=True)


@pytest.mark.parametrize("bb", GEOMS)
def test_set_variant_bucket_capacity(bb):
    """A set bucket holds 30 keys per 128 B, W/4-2 in general: one vertex
    without a hint (one bucket) takes exactly Bc neighbours before its
    first overflow bucket; hinted tables get ceil(hint / (0.7 Bc)) base buckets."""
    from oracle import initial_buckets
    from paper_conf_ipps_awadapo20_b200 import Graph
    bc = bb // 4 - 2
    nv = 4 * bc + 8
    g = Graph(nv, set_variant=True, bucket_bytes=bb)
    g.insert_edges(cuda(np.zeros(bc, np.uint32)), cuda(np.arange(1, bc + 1, dtype=np.uint32)))
    st = g.stats()
    assert st["overflow_buckets"] == 0 and st["live_pairs"] == bc
    g.insert_edges(cuda([0]), cuda([bc + 1]))
    assert g.stats()["overflow_buckets"] == 1
    hints = np.arange(nv, dtype=np.uint32) * 3
    h = Graph(nv, hints, set_variant=True, bucket_bytes=bb)
    assert h.stats()["base_buckets"] == sum(initial_buckets(int(x), 700, bc) for x in hints)
    g.close()
    h.close()


@pytest.mark.parametrize("reuse", [True, False])
def test_churn_tombstone_policy(reuse):
    """Insert/delete churn: identical results under both tombstone policies; with
    reuse the chains stop growing (two-stage insert), without it every
    deleted key keeps its slot."""
    from paper_conf_ipps_awadapo20_b200 import Graph
    nv = 50_000
    s0, d0, w0 = wl.uniform_edges(13, 0, 400_000, nv)
    if not reuse:
        os.environ["DG_HOT_STEPS"] = "0"  # pure append-only policy: no re-sizing compaction
    try:
        g = Graph(nv, wl.out_degrees(s0, nv), reuse_tombstones=reuse)
    finally:
        os.environ.pop("DG_HOT_STEPS", None)
    o = Oracle(nv)
    g.insert_edges(cuda(s0), cuda(d0), cuda(w0))
    o.insert_edges(s0, d0, w0)
    for r in range(6):
        s, d, w = wl.uniform_edges(13, 10 + r, 200_000, nv)
        assert g.insert_edges(cuda(s), cuda(d), cuda(w), count=True) == o.insert_edges(s, d, w)[1]
        assert g.delete_edges(cuda(s), cuda(d), count=True) == o.delete_edges(s, d)[1]
    check_against_oracle(g, o, "churn")
    st = g.stats()
    if reuse:  # bounded by the churn per vertex, not by the number of rounds
        assert st["tombstones"] < 3 * 200_000
    else:
        assert st["tombstones"] >= 6 * 190_000


@pytest.mark.parametrize("bb", GEOMS_A)
def test_large_random_ragged(bb):
    """|V| = 100,000; 3 insert batches of 700,001 (ragged tail), queries, deletes."""
    nv = 100_000
    g = __import__("paper_conf_ipps_awadapo20_b200").Graph(nv, bucket_bytes=bb)
    o = Oracle(nv)
    for b in range(3):
        s, d, w = wl.uniform_edges(11, b, 700_001, nv)
        assert g.insert_edges(cuda(s), cuda(d), cuda(w), count=True) == o.insert_edges(s, d, w)[1]
    cand = check_against_oracle(g, o, "inserted")
    qs, qd, _ = wl.uniform_edges(11, 50, 300_007, nv)
    s, d, _ = wl.uniform_edges(11, 1, 300_007, nv)  # live keys from batch 1
    check_queries(g, o, np.concatenate([qs, s]), np.concatenate([qd, d]), cand, "queries")
    assert g.delete_edges(cuda(s), cuda(d), count=True) == o.delete_edges(s, d)[1]
    check_against_oracle(g, o, "deleted")


@pytest.mark.parametrize("bb", [32, 128, 0])
def test_rmat_hubs_without_hints(bb):
    """Scale-free input with one bucket per vertex (Tab. VI-style incremental build):
    long chains, many concurrent chain extensions and same-key races."""
    scale = 16
    nv = 1 << scale
    s, d = wl.rmat_edges(5, 0, 1_000_000, scale, wl.GRAPH500)
    w = wl.weights(5, 0, s.size)
    g = __import__("paper_conf_ipps_awadapo20_b200").Graph(nv, bucket_bytes=bb, pool_bytes=1 << 20)
    o = Oracle(nv)
    assert g.insert_edges(cuda(s), cuda(d), cuda(w), count=True) == o.insert_edges(s, d, w)[1]
    cand = check_against_oracle(g, o, "rmat")
    st = g.stats()
    assert st["max_chain"] > 10 and st["live_pairs"] == o.num_edges()
    check_queries(g, o, s[::7], d[::7], cand, "rmat queries")
    # hub deletion frees chained buckets; re-insertion reuses them from the free stack
    deg = np.bincount(s, minlength=nv)
    hubs = np.argsort(deg)[-8:].astype(np.uint32)
    g.delete_vertices(cuda(hubs))
    o.delete_vertices(hubs)
    check_against_oracle(g, o, "hubs deleted")
    st2 = g.stats()
    assert st2["free_buckets"] > 0
    m = (np.isin(s, hubs))
    assert g.insert_edges(cuda(s[m]), cuda(d[m]), cuda(w[m]), count=True) == \
        o.insert_edges(s[m], d[m], w[m])[1]
    check_against_oracle(g, o, "hubs re-inserted")
    st3 = g.stats()
    assert st3["base_buckets"] + st3["overflow_buckets"] + st3["free_buckets"] <= st3["bump_buckets"]


@pytest.mark.parametrize("hints", [True, False])
@pytest.mark.parametrize("reuse", [True, False])
@pytest.mark.parametrize("bb,set_variant", [(128, False), (0, False), (32, False), (64, True),
                                            (32, True)])
def test_src_sorted_batches(bb, set_variant, reuse, hints):
    """Src-sorted R-MAT batches (the sorted bulk build) take the
    same-source grouped path (a3, k_insert_sorted): the warp owning a row's first op
    installs the whole row, a chain's new keys going to its next free slots in one
    pass; rows with many chains (hubs) stay on the per-op path.  Duplicates of one key
    sit next to each other with different weights (Q1 membership rule); a third is
    deleted and re-inserted (tombstones present); every layout incl. the set variant
    and 32-B buckets (chains overflow into several new buckets per group)."""
    from paper_conf_ipps_awadapo20_b200 import Graph
    scale = 15
    nv = 1 << scale
    s, d = wl.rmat_edges(17, 0, 600_000, scale, wl.GRAPH500)
    w = None if set_variant else wl.weights(17, 0, s.size)
    order = np.lexsort((d, s))
    s, d = s[order], d[order]
    if w is not None:
        w = w[order]
    h = torch.bincount(torch.from_numpy(s.astype(np.int64)), minlength=nv).to(torch.int32)
    g = Graph(nv, h.cuda() if hints else None, bucket_bytes=bb, reuse_tombstones=reuse,
              set_variant=set_variant)
    o = Oracle(nv)
    half = s.size // 2
    W = (lambda x: None) if w is None else (lambda x: w[x])
    for lo, hi in ((0, half), (half, s.size)):
        sl = slice(lo, hi)
        assert g.insert_edges(cuda(s[sl]), cuda(d[sl]), cuda(W(sl)), count=True) == \
            o.insert_edges(s[sl], d[sl], W(sl))[1]
    cand = check_against_oracle(g, o, "sorted insert")
    check_queries(g, o, s[::5], d[::5], cand, "sorted queries")
    # delete a sorted third, re-insert it sorted (tombstone reuse path when enabled)
    m = slice(0, s.size // 3)
    assert g.delete_edges(cuda(s[m]), cuda(d[m]), count=True) == o.delete_edges(s[m], d[m])[1]
    assert g.insert_edges(cuda(s[m]), cuda(d[m]), cuda(W(m)), count=True) == \
        o.insert_edges(s[m], d[m], W(m))[1]
    check_against_oracle(g, o, "sorted churn")
    # a sorted batch of keys that all exist already (replace path) plus new ones
    m2 = slice(s.size // 4, s.size // 2)
    assert g.insert_edges(cuda(s[m2]), cuda(d[m2]), cuda(W(m2)), count=True) == \
        o.insert_edges(s[m2], d[m2], W(m2))[1]
    check_against_oracle(g, o, "sorted replace")
    g.close()


@pytest.mark.parametrize("retry_cap", [None, 1000])
def test_src_sorted_pool_exhaustion(retry_cap):
    """The sorted path in retry mode: groups whose new buckets cannot be allocated
    hand their overflow ops to the retry list (re-run by k_edges after the pool grows)."""
    code = r"""
import numpy as np, sys
sys.path.insert(0, %r)
import workloads as wl
from oracle import Oracle
from tests.gpu_util import check_against_oracle, cuda
from paper_conf_ipps_awadapo20_b200 import Graph
nv = 4096
g = Graph(nv, pool_bytes=4096, bucket_bytes=32)
o = Oracle(nv)
for b in range(3):
    s, d, w = wl.uniform_edges(2, b, 300_000, nv)
    order = np.argsort(s, kind="stable")
    s, d, w = s[order], d[order], w[order]
    assert g.insert_edges(cuda(s), cuda(d), cuda(w), count=True) == o.insert_edges(s, d, w)[1]
check_against_oracle(g, o, "sorted retry")
print("OK", g.stats()["pool_buckets"])
""" % os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    env = dict(os.environ, DG_TEST_RETRY_PATH="1", DG_HOT_STEPS="0")
    if retry_cap:
        env["DG_TEST_RETRY_CAP"] = str(retry_cap)
    r = subprocess.run([sys.executable, "-c", code], env=env, capture_output=True, text=True,
                       timeout=600)
    assert r.returncode == 0 and "OK" in r.stdout, r.stderr[-3000:]


def test_freed_buckets_are_reused():
    """Vertex deletion returns chained buckets to the allocator; later
    chain growth pops them before touching never-used memory."""
    from paper_conf_ipps_awadapo20_b200 import Graph
    s = np.zeros(3000, np.uint32)
    d = (np.arange(3000) + 4).astype(np.uint32)
    os.environ["DG_HOT_STEPS"] = "0"  # keep the long chain (no re-sizing) for this check
    try:
        g2 = Graph(3100, bucket_bytes=32)  # 3 pairs per bucket, one base bucket per vertex
    finally:
        del os.environ["DG_HOT_STEPS"]
    g2.insert_edges(cuda(s), cuda(d))
    st1 = g2.stats()
    assert st1["overflow_buckets"] == 999 and st1["live_pairs"] == 3000
    g2.delete_vertices(cuda(np.array([0], np.uint32)))
    st2 = g2.stats()
    assert st2["free_buckets"] - st1["free_buckets"] == 999 and st2["live_pairs"] == 0
    for i in range(60):  # one op per launch: no chain-link races, no spare buckets
        g2.insert_edges(cuda(s[i:i + 1]), cuda(d[i:i + 1]))
    st3 = g2.stats()
    assert st3["overflow_buckets"] == 19 and st3["live_pairs"] == 60
    assert st3["bump_buckets"] == st2["bump_buckets"]  # nothing new taken from the pool
    assert st3["free_buckets"] == st2["free_buckets"] - 19
    g2.close()


def test_heavy_intra_batch_duplicates():
    nv = 64
    s = np.full(50_000, 7, np.uint32)
    d = (np.arange(50_000) % 5 + 1).astype(np.uint32)
    w = np.arange(50_000, dtype=np.uint32)
    g = __import__("paper_conf_ipps_awadapo20_b200").Graph(nv)
    o = Oracle(nv)
    assert g.insert_edges(cuda(s), cuda(d), cuda(w), count=True) == o.insert_edges(s, d, w)[1] == 5
    check_against_oracle(g, o, "dups")
    # deleting the same key many times removes it once
    assert g.delete_edges(cuda(s), cuda(d), count=True) == 5


def test_host_buffers_match_device_buffers():
    from paper_conf_ipps_awadapo20_b200 import Graph
    nv = 5000
    s, d, _ = wl.uniform_edges(21, 0, 100_000, nv)
    w = (s.astype(np.uint64) * 2654435761 ^ d).astype(np.uint32)  # duplicate keys: equal weights (Q1)
    a, b = Graph(nv), Graph(nv)
    assert a.insert_edges(s, d, w, count=True) == b.insert_edges(cuda(s), cuda(d), cuda(w), count=True)
    qs, qd, _ = wl.uniform_edges(21, 1, 50_000, nv)
    fa, wa = a.query_edges(qs, qd)
    fb, wb = b.query_edges(cuda(qs), cuda(qd))
    assert isinstance(fa, np.ndarray)
    assert np.array_equal(fa, fb.cpu().numpy()) and np.array_equal(wa, wb.cpu().numpy())
    ea, eb = a.export_numpy(), b.export()
    assert np.array_equal(ea[0], eb[0].cpu().numpy())


@pytest.mark.parametrize("bb", [128, 0])
@pytest.mark.parametrize("directed", [True, False])
def test_vertex_deletion_modes(directed, bb):
    """Directed: streaming purge sweep; undirected: Alg. 2."""
    from paper_conf_ipps_awadapo20_b200 import Graph
    nv = 20_000
    s, d = wl.rmat_edges(8, 0, 200_000, 15, wl.GRAPH500, nv=nv)
    g = Graph(nv, wl.out_degrees(np.concatenate([s, d]), nv), directed=directed, bucket_bytes=bb)
    o = Oracle(nv, directed)
    g.insert_edges(cuda(s), cuda(d))
    o.insert_edges(s, d)
    for r in range(3):
        ids = np.concatenate([wl.uniform_u32(8, 100 + r, 300, nv), s[:5]])  # hubs + duplicates
        g.delete_vertices(cuda(ids))
        o.delete_vertices(ids)
        check_against_oracle(g, o, f"round {r}")
        qs = np.repeat(ids[:50], 40)
        qd = wl.uniform_u32(8, 200 + r, qs.size, nv)
        check_queries(g, o, np.concatenate([qs, qd]), np.concatenate([qd, qs]), None, "incident")


def test_empty_batches():
    from paper_conf_ipps_awadapo20_b200 import Graph
    g = Graph(10)
    e = torch.empty(0, dtype=torch.uint32, device="cuda")
    assert g.insert_edges(e, e, count=True) == 0
    assert g.delete_edges(e, e, count=True) == 0
    f, w = g.query_edges(e, e)
    assert f.numel() == 0
    g.delete_vertices(e)
    g.insert_vertices(e)
    ro, d, w = g.export()
    assert d.numel() == 0 and ro.numel() == 11
    g0 = Graph(0)
    assert g0.export()[1].numel() == 0


def test_geometry_invariance():
    """Deterministic weights -> identical exports across bucket size, load factor and
    hints (hints/load factor affect only performance)."""
    from paper_conf_ipps_awadapo20_b200 import Graph
    nv = 30_000
    s, d = wl.rmat_edges(9, 0, 400_000, 15, wl.LJLIKE, nv=nv)
    w = (s.astype(np.uint64) * 2654435761 ^ d).astype(np.uint32)  # equal weights for equal keys
    hint = wl.out_degrees(s, nv)
    ref = None
    for bb in GEOMS_A:
        for lf in (0.35, 0.7, 2.0):
            for h in (None, hint):
                g = Graph(nv, h, bucket_bytes=bb, load_factor=lf)
                g.insert_edges(cuda(s), cuda(d), cuda(w))
                g.delete_edges(cuda(s[::3]), cuda(d[::3]))
                ro, dd, ww = g.export()
                from oracle.compare import canonical
                out = canonical(ro.cpu().numpy(), dd.cpu().numpy(), ww.cpu().numpy())
                if ref is None:
                    ref = out
                else:
                    assert all(np.array_equal(a, b) for a, b in zip(ref, out)), (bb, lf, h is None)
                g.close()


def test_initial_bucket_rule_matches_oracle():
    """dg_create's base-bucket count equals the paper's closed form
    as computed by the oracle, for every vertex."""
    from oracle import initial_buckets
    from paper_conf_ipps_awadapo20_b200 import Graph
    hints = np.array([0, 1, 10, 11, 100, 105, 106, 1000, 20000, 7, 3], np.uint32)
    for bb, bc in ((128, 15), (64, 7), (32, 3)):
        for lf in (0.7, 0.5, 1.0):
            g = Graph(hints.size, hints, bucket_bytes=bb, load_factor=lf)
            want = sum(initial_buckets(int(h), int(round(lf * 1000)), bc) for h in hints)
            assert g.stats()["base_buckets"] == want


@pytest.mark.parametrize("retry_cap", [None, 1000])
def test_pool_exhaustion_retry_path(retry_cap):
    """Pool exhaustion mid-kernel: failed ops are re-run after the pool grows
    (forced with DG_TEST_RETRY_PATH, which disables up-front growth).  With a retry
    list smaller than the failures (DG_TEST_RETRY_CAP) the whole batch runs again."""
    code = r"""
import numpy as np, torch, sys
sys.path.insert(0, %r)
import workloads as wl
from oracle import Oracle
from tests.gpu_util import check_against_oracle, cuda
from paper_conf_ipps_awadapo20_b200 import Graph
nv = 4096
g = Graph(nv, pool_bytes=4096)
o = Oracle(nv)
for b in range(3):
    s, d, w = wl.uniform_edges(2, b, 400_000, nv)
    assert g.insert_edges(cuda(s), cuda(d), cuda(w), count=True) == o.insert_edges(s, d, w)[1]
check_against_oracle(g, o, "retry")
print("OK", g.stats()["pool_buckets"])
""" % os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    env = dict(os.environ, DG_TEST_RETRY_PATH="1")
    if retry_cap:
        env["DG_TEST_RETRY_CAP"] = str(retry_cap)
    r = subprocess.run([sys.executable, "-c", code], env=env, capture_output=True, text=True,
                       timeout=600)
    assert r.returncode == 0 and "OK" in r.stdout, r.stderr[-3000:]


@pytest.mark.parametrize("bb", [128, 0])
@pytest.mark.parametrize("directed", [True, False])
@pytest.mark.parametrize("exchange", ["fused", "nccl"])
def test_routed_single_gpu(directed, exchange, bb, monkeypatch):
    """The multi-GPU batch router (partition -> exchange -> local probe -> answers
    back in caller order) on a 1-rank communicator: results identical to the oracle,
    through the fused partition + window stores (default) and the NCCL exchange.
    One batch outgrows the initial receive window (collective window re-setup)."""
    from paper_conf_ipps_awadapo20_b200 import Graph, DGError, DG_ERR_VERTEX_OUT_OF_RANGE
    if exchange == "nccl":
        monkeypatch.setenv("DG_ROUTER", "nccl")
    nv = 30_000
    g = Graph(nv, directed=directed, force_router=True, bucket_bytes=bb)
    assert g.stats()["exchange"] == (2 if exchange == "fused" else 1)
    o = Oracle(nv, directed)
    s, d, w = wl.uniform_edges(17, 1000, 1_300_000, nv)  # > the 2^20-op initial window
    assert g.insert_edges(cuda(s), cuda(d), cuda(w), count=True) == o.insert_edges(s, d, w)[1]
    for b in range(3):
        s, d, w = wl.uniform_edges(17, b, 200_003, nv)
        s[-500:], d[-500:] = s[:500], d[:500]
        assert g.insert_edges(cuda(s), cuda(d), cuda(w), count=True) == o.insert_edges(s, d, w)[1]
    cand = check_against_oracle(g, o, "routed inserts")
    qs, qd, _ = wl.uniform_edges(17, 1, 100_001, nv)
    us, ud, _ = wl.uniform_edges(17, 50, 100_001, nv)
    check_queries(g, o, np.concatenate([qs, us]), np.concatenate([qd, ud]), cand, "routed queries")
    assert g.delete_edges(cuda(qs), cuda(qd), count=True) == o.delete_edges(qs, qd)[1]
    ids = wl.uniform_u32(17, 99, 100, nv)
    g.delete_vertices(cuda(ids))
    o.delete_vertices(ids)
    check_against_oracle(g, o, "routed deletes")
    g.insert_vertices(cuda(np.array([nv + 5], np.uint32)))
    o.insert_vertices(np.array([nv + 5], np.uint32))
    s, d, w = wl.uniform_edges(17, 77, 10_000, nv + 6)
    assert g.insert_edges(cuda(s), cuda(d), cuda(w), count=True) == o.insert_edges(s, d, w)[1]
    check_against_oracle(g, o, "routed growth")
    s[3] = nv + 100
    with pytest.raises(DGError) as e:
        g.insert_edges(cuda(s), cuda(d), cuda(w), count=True)
    assert e.value.status == DG_ERR_VERTEX_OUT_OF_RANGE
    check_against_oracle(g, o, "routed rejected batch")


def test_multi_gpu_torchrun():
    """Sharding by source vertex over NCCL with one process per GPU (needs >= 2 GPUs)."""
    n = torch.cuda.device_count()
    if n < 2:
        pytest.skip("needs >= 2 GPUs (the single-GPU routed path is covered above)")
    P = min(n, 4)
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    r = subprocess.run([sys.executable, "-m", "torch.distributed.run", "--nnodes=1",
                        f"--nproc-per-node={P}", "--master-addr=127.0.0.1", "--master-port=29517",
                        os.path.join(root, "tests", "multigpu_worker.py")],
                       capture_output=True, text=True, timeout=900, cwd=root)
    assert r.returncode == 0 and "MULTIGPU OK" in r.stdout, r.stdout[-2000:] + r.stderr[-4000:]


# ------------------------------------------------------------- triangle count --
def _golden_triangles():
    from tests.golden_script import load as _load
    out = []
    for ln in _load("triangles.txt"):
        f = ln.split()
        out.append((f[0], int(f[1]), int(f[2]), [tuple(int(x) for x in e.split("-")) for e in f[3:]]))
    return out


@pytest.mark.parametrize("set_variant", [False, True])
@pytest.mark.parametrize("bb", GEOMS_A)
def test_tc_golden_and_closed_forms(bb, set_variant):
    import math
    from paper_conf_ipps_awadapo20_b200 import Graph
    for name, n, want, edges in _golden_triangles():
        g = Graph(n, directed=False, bucket_bytes=bb, set_variant=set_variant)
        g.insert_edges(cuda([e[0] for e in edges]), cuda([e[1] for e in edges]))
        assert g.triangle_count() == want, name
    for n in (3, 10, 47):
        iu, ju = np.triu_indices(n, 1)
        g = Graph(n, directed=False, bucket_bytes=bb, set_variant=set_variant)
        g.insert_edges(cuda(iu), cuda(ju))
        assert g.triangle_count() == math.comb(n, 3)


@pytest.mark.parametrize("set_variant", [False, True])
@pytest.mark.parametrize("bb", GEOMS_A)
def test_tc_matches_oracle_rmat(bb, set_variant):
    """Hash-intersection TC (GPU) vs the forward algorithm on sorted lists (oracle)
    on a symmetrised R-MAT graph; the part/nparts split sums to the total."""
    from paper_conf_ipps_awadapo20_b200 import Graph
    scale = 15
    nv = 1 << scale
    s, d = wl.rmat_edges(5, 0, 400_000, scale, wl.GRAPH500)
    g = Graph(nv, wl.out_degrees(np.concatenate([s, d]), nv), directed=False, bucket_bytes=bb,
              set_variant=set_variant)
    o = Oracle(nv, directed=False)
    g.insert_edges(cuda(s), cuda(d))
    o.insert_edges(s, d)
    check_against_oracle(g, o, "sym rmat")
    want = o.triangle_count()
    assert want > 1000
    assert g.triangle_count() == want
    assert sum(g.triangle_count(p, 3) for p in range(3)) == want
    # dynamic: insert a new batch, recount (config 5 iteration)
    s2, d2 = wl.rmat_edges(5, 1, 100_000, scale, wl.GRAPH500)
    g.insert_edges(cuda(s2), cuda(d2))
    o.insert_edges(s2, d2)
    assert g.triangle_count() == o.triangle_count()


def test_host_query_pipeline_large():
    """Host-buffer queries above 2^23 take the chunked upload/probe/download pipeline;
    answers must equal the device-buffer path and the oracle on a sample."""
    from paper_conf_ipps_awadapo20_b200 import Graph
    nv = 200_000
    s, d, _ = wl.uniform_edges(23, 0, 2_000_000, nv)
    w = (s.astype(np.uint64) * 2654435761 ^ d).astype(np.uint32)
    g = Graph(nv)
    g.insert_edges(cuda(s), cuda(d), cuda(w))
    n = (1 << 23) + 12345
    qs, qd, _ = wl.uniform_edges(23, 1, n, nv, weights=False)
    qs[: 1 << 20], qd[: 1 << 20] = s[: 1 << 20], d[: 1 << 20]
    fh = np.empty(n, np.uint8)
    wh = np.empty(n, np.uint32)
    g.query_edges(qs, qd, found_out=fh, weight_out=wh)
    fd, wd = g.query_edges(cuda(qs), cuda(qd))
    assert np.array_equal(fh, fd.cpu().numpy()) and np.array_equal(wh, wd.cpu().numpy())
    live = s[: 1 << 20] != d[: 1 << 20]  # self-loops are never stored (Alg1:L3)
    assert fh[: 1 << 20][live].all() and not fh[: 1 << 20][~live].any()
    o = Oracle(nv)
    o.insert_edges(s, d, w)
    idx = np.arange(0, n, 97)
    st, rf, rw = o.query_edges(qs[idx], qd[idx])
    assert np.array_equal(rf, fh[idx]) and np.array_equal(rw, wh[idx])


@pytest.mark.parametrize("bb", [32, 128, 0])
def test_rehash_long_chains_without_hints(bb):
    """Per-vertex re-sizing: an R-MAT graph built
    incrementally with one bucket per vertex grows hub chains; flagged tables are
    re-sized before the next batch.  Results stay identical to the oracle and the
    chains end short."""
    from paper_conf_ipps_awadapo20_b200 import Graph
    scale = 16
    nv = 1 << scale
    g = Graph(nv, bucket_bytes=bb)
    o = Oracle(nv)
    for b in range(8):
        s, d = wl.rmat_edges(7, b, 150_000, scale, wl.GRAPH500)
        w = wl.weights(7, b, s.size)
        assert g.insert_edges(cuda(s), cuda(d), cuda(w), count=True) == o.insert_edges(s, d, w)[1]
        check_against_oracle(g, o, f"batch {b}")
        if b == 0:
            first_chain = g.stats()["max_chain"]
    ds, dd = wl.rmat_edges(7, 0, 50_000, scale, wl.GRAPH500)
    assert g.delete_edges(cuda(ds), cuda(dd), count=True) == o.delete_edges(ds, dd)[1]
    e = torch.empty(0, dtype=torch.uint32, device="cuda")
    g.insert_edges(e, e)  # the re-sizing check runs at the start of an insert batch
    check_against_oracle(g, o, "after re-sizing")
    st = g.stats()
    assert first_chain > 20 and st["max_chain"] <= 8, (first_chain, st["max_chain"])
    assert st["live_pairs"] == o.num_edges() and st["tombstones"] < 50_000


@pytest.mark.parametrize("bb", [128, 0])
@pytest.mark.parametrize("set_variant", [False, True])
@pytest.mark.parametrize("hints", [False, True])
def test_hub_rows_export_stats_tc(hints, set_variant, bb):
    """Hub rows (more than 32 base buckets / 1,024 neighbours) are exported, counted
    and oriented by the block-per-row kernels: a wheel W_n (hub 0 joined to the cycle
    1..n) has exactly n triangles for n >= 4 and 4n directed entries."""
    from paper_conf_ipps_awadapo20_b200 import Graph
    n = 6000
    rim = np.arange(1, n + 1, dtype=np.uint32)
    s = np.concatenate([np.zeros(n, np.uint32), rim])
    d = np.concatenate([rim, np.roll(rim, -1)])
    nv = n + 1
    h = wl.out_degrees(np.concatenate([s, d]), nv) if hints else None
    g = Graph(nv, h, directed=False, set_variant=set_variant, bucket_bytes=bb)
    o = Oracle(nv, directed=False)
    g.insert_edges(cuda(s), cuda(d))
    o.insert_edges(s, d)
    check_against_oracle(g, o, "wheel")
    st = g.stats()
    assert st["live_pairs"] == 4 * n
    assert g.triangle_count() == n == o.triangle_count()
    assert sum(g.triangle_count(p, 2) for p in range(2)) == n
    g.close()


def test_async_host_batches():
    """Host-buffer inserts/deletes without a count return once the batch is uploaded
    and validated; the kernels run behind the next call.  The caller may overwrite
    its host arrays on return (reused here for every batch), later calls see every
    earlier batch (stream order), and a rejected batch still reports its status."""
    from paper_conf_ipps_awadapo20_b200 import DGError, DG_ERR_VERTEX_OUT_OF_RANGE, Graph
    nv = 50_000
    g = Graph(nv)
    o = Oracle(nv)
    n = 300_000
    hs = torch.empty(n, dtype=torch.int32).pin_memory()
    hd = torch.empty(n, dtype=torch.int32).pin_memory()
    hw = torch.empty(n, dtype=torch.int32).pin_memory()
    hf = torch.empty(n, dtype=torch.uint8).pin_memory()
    hq = torch.empty(n, dtype=torch.int32).pin_memory()
    for b in range(6):
        s, d, w = wl.uniform_edges(41, b, n, nv)
        hs.numpy().view(np.uint32)[:] = s
        hd.numpy().view(np.uint32)[:] = d
        hw.numpy().view(np.uint32)[:] = w
        if b % 3 == 2:  # delete the previous batch's first half
            g.delete_edges(hs[: n // 2], hd[: n // 2])
            o.delete_edges(s[: n // 2], d[: n // 2])
        else:
            g.insert_edges(hs, hd, hw)
            o.insert_edges(s, d, w)
        hs.fill_(0)  # overwritten right away: the library must hold its own copy
        hd.fill_(0)
        qs, qd, _ = wl.uniform_edges(41, 100 + b, n, nv)
        qs[: n // 2], qd[: n // 2] = s[: n // 2], d[: n // 2]
        hq.numpy().view(np.uint32)[:] = qd
        f, qw = g.query_edges(qs, hq, found_out=hf, weight_out=np.empty(n, np.uint32))
        _, rf, rw = o.query_edges(qs, qd)
        assert np.array_equal(hf.numpy(), rf), b
    s, d, w = wl.uniform_edges(41, 99, 1000, nv)
    s[7] = nv
    with pytest.raises(DGError) as e:
        g.insert_edges(s, d, w)
    assert e.value.status == DG_ERR_VERTEX_OUT_OF_RANGE
    check_against_oracle(g, o, "async host batches")
    g.close()


@pytest.mark.parametrize("bb", [64, 0])
@pytest.mark.parametrize("set_variant", [False, True])
@pytest.mark.parametrize("reuse", [False, True])
def test_flush_tombstones(reuse, set_variant, bb):
    """Tombstone flush: after insert/delete churn the
    tables hold tombstones; flushing rebuilds every such table compactly (several
    rounds: > 65,536 rows carry tombstones), the logical graph is unchanged, no
    tombstone is left and the freed buckets serve later inserts."""
    from paper_conf_ipps_awadapo20_b200 import Graph
    nv = 200_000
    g = Graph(nv, reuse_tombstones=reuse, set_variant=set_variant, bucket_bytes=bb)
    o = Oracle(nv)

    def ow(w):
        return np.zeros_like(w) if set_variant else w
    for b in range(4):
        s, d, w = wl.uniform_edges(61, b, 600_000, nv)
        assert g.insert_edges(cuda(s), cuda(d), cuda(w), count=True) == o.insert_edges(s, d, ow(w))[1]
        assert g.delete_edges(cuda(s[::2]), cuda(d[::2]), count=True) == o.delete_edges(s[::2], d[::2])[1]
    before = g.stats()
    assert before["tombstones"] > 100_000
    rebuilt = g.flush_tombstones()
    assert rebuilt > 65_536
    after = g.stats()
    assert after["tombstones"] == 0 and after["live_pairs"] == o.num_edges()
    assert after["overflow_buckets"] < before["overflow_buckets"]
    check_against_oracle(g, o, "after flush")
    assert g.flush_tombstones() == 0
    s, d, w = wl.uniform_edges(61, 99, 300_000, nv)
    assert g.insert_edges(cuda(s), cuda(d), cuda(w), count=True) == o.insert_edges(s, d, ow(w))[1]
    check_against_oracle(g, o, "inserts after flush")
    g.close()


def _class_bytes(h, lf_milli, set_variant):
    """Bytes of the base table the degree-adaptive layout gives a vertex with hint h
    (include/dg.h DG_FLAG_ADAPTIVE; reading R-ADAPT): the smallest bucket
    whose single instance holds h at the load factor — 32 B (3 pairs / 6 keys), 64 B
    (7 / 14) — else 128-B buckets (15 / 30) by the initial rule."""
    from oracle import initial_buckets
    for size in (32, 64):
        bc = size // 4 - 2 if set_variant else size // 8 - 1
        if h * 1000 <= lf_milli * bc:
            return size
    return 128 * initial_buckets(int(h), lf_milli, 30 if set_variant else 15)


@pytest.mark.parametrize("set_variant", [False, True])
def test_adaptive_size_classes(set_variant):
    """Degree-adaptive bucket sizes: the base tables
    of dg_create take exactly the bytes of the size-class rule for every hint, far
    less than uniform 128-B buckets on a low-degree graph, and a 32-B table overflows
    into a chained 32-B bucket after its 3 pairs (6 keys)."""
    from paper_conf_ipps_awadapo20_b200 import Graph
    hints = np.array([0, 1, 2, 3, 4, 5, 6, 9, 10, 11, 20, 21, 22, 100, 105, 106, 1000, 20000],
                     np.uint32)
    for lf in (0.7, 0.5, 1.0):
        g = Graph(hints.size, hints, bucket_bytes=0, load_factor=lf, set_variant=set_variant)
        st = g.stats()
        want = sum(_class_bytes(int(h), int(round(lf * 1000)), set_variant) for h in hints)
        assert st["table_bytes"] == want, (lf, st["table_bytes"], want)
        assert st["overflow_buckets"] == 0
        g.close()
    nv = 64
    g = Graph(nv, bucket_bytes=0, set_variant=set_variant)
    assert g.stats()["table_bytes"] == 32 * nv
    bc = 6 if set_variant else 3
    g.insert_edges(cuda(np.zeros(bc, np.uint32)), cuda(np.arange(1, bc + 1, dtype=np.uint32)))
    assert g.stats()["overflow_buckets"] == 0
    g.insert_edges(cuda([0]), cuda([bc + 1]))
    st = g.stats()
    assert st["overflow_buckets"] == 1 and st["table_bytes"] == 32 * (nv + 1)
    g.close()


def test_adaptive_promotion_and_memory():
    """Without hints every vertex starts with one 32-B bucket; the re-sizing pass moves
    rows whose chains grow to larger size classes (P:L309-313 + P:L947-955).  The graph
    equals the oracle throughout, chains end short, and the adaptive tables of an
    R-MAT graph (many low-degree vertices) take fewer bytes than uniform 128-B ones."""
    from paper_conf_ipps_awadapo20_b200 import Graph
    scale = 15
    nv = 1 << scale
    g = Graph(nv, bucket_bytes=0)
    o = Oracle(nv)
    for b in range(6):
        s, d = wl.rmat_edges(23, b, 100_000, scale, wl.GRAPH500)
        w = wl.weights(23, b, s.size)
        assert g.insert_edges(cuda(s), cuda(d), cuda(w), count=True) == o.insert_edges(s, d, w)[1]
    e = torch.empty(0, dtype=torch.uint32, device="cuda")
    g.insert_edges(e, e)  # re-sizing runs at the start of an insert batch
    cand = check_against_oracle(g, o, "adaptive promotion")
    st = g.stats()
    assert st["max_chain"] <= 8, st
    qs, qd, _ = wl.uniform_edges(23, 9, 50_000, nv)
    check_queries(g, o, qs, qd, cand, "adaptive queries")
    # same graph from exact hints: adaptive vs uniform 128-B memory
    ro, dd, _ = g.export()
    ro, dd = ro.cpu().numpy(), dd.cpu().numpy()
    src = np.repeat(np.arange(nv, dtype=np.uint32), np.diff(ro).astype(np.int64))
    hint = wl.out_degrees(src, nv)
    a = Graph(nv, hint, bucket_bytes=0)
    u = Graph(nv, hint, bucket_bytes=128)
    for x in (a, u):
        x.insert_edges(cuda(src), cuda(dd))
    sa, su = a.stats(), u.stats()
    assert sa["live_pairs"] == su["live_pairs"] == o.num_edges()
    assert sa["table_bytes"] < su["table_bytes"], (sa["table_bytes"], su["table_bytes"])
    for x in (g, a, u):
        x.close()
    # road-like grid (degree <= 4): every table fits one 32-B or 64-B bucket
    gs, gd = wl.grid_edges(3, 300, 300, 0.6025)
    nv = 300 * 300
    hint = wl.out_degrees(gs, nv)
    a = Graph(nv, hint, bucket_bytes=0)
    u = Graph(nv, hint, bucket_bytes=128)
    o = Oracle(nv)
    o.insert_edges(gs, gd)
    for x in (a, u):
        x.insert_edges(cuda(gs), cuda(gd))
        check_against_oracle(x, o, "grid")
    sa, su = a.stats(), u.stats()
    assert sa["overflow_buckets"] == 0
    assert sa["table_bytes"] == sum(_class_bytes(int(h), 700, False) for h in hint)
    assert sa["table_bytes"] <= su["table_bytes"] // 2
    a.close()
    u.close()


def test_src_sorted_batch_beyond_2_24_rows():
    """The sorted path's chain groups use a 32-bit (row, chain) key below 2^24 rows and
    the exact 64-bit key above: a src-sorted batch on a graph of 2^24 + 4096 vertices,
    rows on both sides of the boundary, with hub rows (> 256 chains: per-op path)."""
    from paper_conf_ipps_awadapo20_b200 import Graph
    nv = (1 << 24) + 4096
    rs = np.random.RandomState(24)
    rows = np.concatenate([rs.randint(0, nv, 300_000), np.full(60_000, nv - 7),
                           np.full(40_000, 5)]).astype(np.uint32)
    dst = rs.randint(0, nv, rows.size).astype(np.uint32)
    w = rs.randint(0, 1 << 32, rows.size, dtype=np.uint64).astype(np.uint32)
    order = np.argsort(rows, kind="stable")
    s, d, w = rows[order], dst[order], w[order]
    hints = np.zeros(nv, np.uint32)
    hints[nv - 7] = 60_000  # > 256 chains: the per-op path inside the sorted kernel
    g = Graph(nv, hints)
    o = Oracle(nv)
    assert g.insert_edges(cuda(s), cuda(d), cuda(w), count=True) == o.insert_edges(s, d, w)[1]
    check_against_oracle(g, o, "sorted batch, 2^24+ rows")
    g.close()


def test_concurrent_fused_small_batches():
    """Two handles on one GPU, each fed small mutating batches (one launch each: the
    validation runs inside the probe kernel before a grid barrier) on
    its own stream, enqueued interleaved so the two kernels can overlap.  The
    cooperative launch keeps every block of each grid resident, so neither barrier
    can wait on blocks the other kernel holds; both graphs end equal to their oracles
    (a rejected batch on one of them changes nothing)."""
    from paper_conf_ipps_awadapo20_b200 import Graph
    nv = 1 << 16
    B = 1 << 17  # a near-full grid per launch (the fused path is < 2^18 ops)
    graphs = [Graph(nv), Graph(nv)]
    oracles = [Oracle(nv), Oracle(nv)]
    streams = [torch.cuda.Stream(), torch.cuda.Stream()]
    batches = {}
    for b in range(6):
        for k in range(2):
            s, d, w = wl.uniform_edges(40 + k, b, B, nv)
            if k == 1 and b == 3:
                s = s.copy()
                s[777] = nv  # out of range: this batch is rejected on graph 1 only
            batches[(b, k)] = (s, d, w)
    dev = [[cuda(x) for x in batches[(b, k)]] for b in range(6) for k in range(2)]
    torch.cuda.synchronize()
    for b in range(6):
        for k in range(2):
            S, D, W = dev[2 * b + k]
            with torch.cuda.stream(streams[k]):
                if b % 2 == 0:
                    graphs[k].insert_edges(S, D, W)
                else:
                    graphs[k].delete_edges(S[: B // 2], D[: B // 2])
    torch.cuda.synchronize()
    for b in range(6):
        for k in range(2):
            s, d, w = batches[(b, k)]
            if b % 2 == 0:
                oracles[k].insert_edges(s, d, w)
            else:
                oracles[k].delete_edges(s[: B // 2], d[: B // 2])
    for k in range(2):
        check_against_oracle(graphs[k], oracles[k], f"graph {k}")
        graphs[k].close()
