"""Small end-to-end run of every kernel family of libdg.so, for compute-sanitizer
(memcheck / racecheck / synccheck; tests/test_gpu_sanitizer.py).  Host numpy buffers
only (the library stages them), tiny sizes, every layout: map/set, 32/64/128-B
buckets, degree-adaptive, directed/undirected, tombstone policies; insert with chain
growth and pool exhaustion retry, query, delete, re-sizing of long chains, tombstone
flush, vertex deletion (purge sweep and Alg. 2), vertex insertion, export, stats,
invariant check, triangle count, and the router through a 1-rank in-process group.
Results are checked against the oracle so a silent corruption also fails.

    compute-sanitizer --tool memcheck python tests/sanitize_script.py
"""
import os
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import workloads as wl  # noqa: E402
from oracle import Oracle  # noqa: E402
from oracle.compare import Candidates, compare_export, compare_queries  # noqa: E402
from paper_conf_ipps_awadapo20_b200 import Graph, RankGroup  # noqa: E402


def check(g, o, where):
    ro, d, w = g.export(device=False)
    errs = compare_export((ro, d, w), o.export(), Candidates(*o.candidates()))
    assert not errs, (where, errs)
    inv = g.check_invariants()
    assert inv["violations"] == 0, (where, inv)


def run(nv=600, directed=True, **kw):
    g = Graph(nv, directed=directed, device=0, **kw)
    o = Oracle(nv, directed=directed)
    keys_only = kw.get("set_variant", False)  # the set variant stores no weights
    for b in range(3):
        s, d, w = wl.uniform_edges(9, b, 1500, nv, weights=not keys_only)
        s[:300] = 7  # a hub: chain growth and re-sizing
        assert g.insert_edges(s, d, w, count=True) == o.insert_edges(s, d, w)[1]
    check(g, o, f"insert {kw}")
    qs, qd, _ = wl.uniform_edges(9, 10, 2000, nv)
    f, qw = g.query_edges(qs, qd)
    _, rf, rw = o.query_edges(qs, qd)
    errs = compare_queries(qs, qd, f, qw, rf, rw, Candidates(*o.candidates()))
    assert not errs, errs
    ds, dd, _ = wl.uniform_edges(9, 1, 1200, nv)
    assert g.delete_edges(ds, dd, count=True) == o.delete_edges(ds, dd)[1]
    ids = wl.uniform_u32(9, 11, 12, nv)
    g.delete_vertices(ids)
    o.delete_vertices(ids)
    check(g, o, f"delete {kw}")
    g.flush_tombstones()
    g.insert_vertices(np.arange(nv, nv + 40, dtype=np.uint32))
    o.insert_vertices(np.arange(nv, nv + 40, dtype=np.uint32))
    s, d, w = wl.uniform_edges(9, 12, 800, nv + 40, weights=not keys_only)
    assert g.insert_edges(s, d, w, count=True) == o.insert_edges(s, d, w)[1]
    check(g, o, f"growth {kw}")
    g.stats()
    if not directed:
        assert g.triangle_count() == o.triangle_count()
    g.close()


def main():
    os.environ.setdefault("DG_HOT_STEPS", "2")  # re-sizing triggers at these sizes
    for bb in (32, 64, 128):
        run(bucket_bytes=bb)
    run(set_variant=True, bucket_bytes=64)
    run(adaptive=True)
    run(directed=False, set_variant=True, bucket_bytes=64)
    run(directed=False)
    run(reuse_tombstones=False)
    # the router through a 1-rank in-process group: count / scan / fused scatter /
    # spin wait / return / unpermute kernels (no NCCL)
    grp = RankGroup(1)
    run(group=grp, force_router=True)
    run(group=grp, force_router=True, copy_exchange=True)
    print("SANITIZE SCRIPT OK", flush=True)


if __name__ == "__main__":
    main()
