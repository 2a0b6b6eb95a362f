"""Multi-rank scenario of the sharded graph (router rows a2 / a11) and its
oracle check — test infrastructure.

``run_rank`` is what ONE rank does: it feeds its own slice of every batch of a
seeded stream to its ``Graph`` handle (every call collective, owner(u) = u mod P) and
records what the library answered.  The same function drives P host threads of one
process on one GPU (``tests/test_gpu_multirank.py``, in-process rank group) and P
processes on P GPUs (``tests/multigpu_worker.py`` under torchrun, NCCL).  ``check``
replays the union of the slices on the unsharded oracle and compares every status,
count, query answer and the merged shard exports (local row r of rank k is global
vertex r*P + k).

The stream covers: uneven slices (rank r gets a share proportional to r+1, and a batch
held by rank 0 alone, so most ranks pass n = 0), intra-batch duplicate keys (Q1),
R-MAT hub rows (chain growth), a mutating batch rejected because ONE rank's slice
holds an out-of-range ID (Q7: no rank mutates), a query batch with out-of-range IDs
on one rank (Q7/Q19: those answer 0, the rest are answered, the batch reports the
rejection on every rank — as at P = 1), deletes (half live, half uniform), vertex
deletion with duplicate IDs (the IDs are all-gathered), vertex insertion
that grows the capacity and edges into the new and the deleted vertices.
"""
from __future__ import annotations

import numpy as np

import workloads as wl

NV0 = 20_000
GROW = 64
SEED = 41


def bounds(n: int, rank: int, P: int, alone: bool = False):
    """[lo, hi) of rank's slice: shares proportional to rank+1 (uneven on purpose)."""
    if alone:
        return (0, n) if rank == 0 else (0, 0)
    tot = P * (P + 1) // 2
    lo = n * (rank * (rank + 1) // 2) // tot
    hi = n * ((rank + 1) * (rank + 2) // 2) // tot
    return lo, hi


def stream(P: int):
    """The global batches (every rank and the checker build the same arrays)."""
    nv = NV0
    steps = []
    s, d, w = wl.uniform_edges(SEED, 0, 40_000, nv)
    # 5% forced duplicates of earlier keys with their own weights (Q1)
    k = 2_000
    s = np.concatenate([s, s[:k]])
    d = np.concatenate([d, d[:k]])
    w = np.concatenate([w, wl.weights(SEED, 50, k)])
    steps.append(dict(op="insert", src=s, dst=d, w=w))
    rs, rd = wl.rmat_edges(SEED, 1, 40_000, 15, wl.GRAPH500, nv=nv)
    steps.append(dict(op="insert", src=rs, dst=rd, w=wl.weights(SEED, 1, rs.size)))
    # rejected batch: an out-of-range ID in the LAST rank's slice only
    bs, bd, bw = wl.uniform_edges(SEED, 2, 9_000, nv)
    lo, hi = bounds(bs.size, P - 1, P)
    bd[(lo + hi) // 2] = nv + 5
    steps.append(dict(op="insert", src=bs, dst=bd, w=bw, rejected=True))
    # queries: half live (from the first batch), half uniform; out-of-range on rank 0
    qs = np.concatenate([s[:15_000], wl.uniform_edges(SEED, 3, 15_000, nv)[0]])
    qd = np.concatenate([d[:15_000], wl.uniform_edges(SEED, 3, 15_000, nv)[1]])
    qs = qs.copy()
    lo, hi = bounds(qs.size, 0, P)
    bad = np.arange(lo, hi, 97)
    qs[bad] = nv + 1 + (bad % 7).astype(np.uint32)
    steps.append(dict(op="query", src=qs, dst=qd, rejected=True))
    # deletes: half of the R-MAT batch, half uniform
    ds = np.concatenate([rs[:10_000], wl.uniform_edges(SEED, 4, 10_000, nv)[0]])
    dd = np.concatenate([rd[:10_000], wl.uniform_edges(SEED, 4, 10_000, nv)[1]])
    steps.append(dict(op="delete", src=ds, dst=dd))
    # vertex deletion: 40 IDs with duplicates, incl. the R-MAT hubs
    hubs = np.bincount(rs, minlength=nv).argsort()[-8:].astype(np.uint32)
    ids = np.concatenate([wl.uniform_u32(SEED, 5, 32, nv), hubs, hubs[:4]])
    steps.append(dict(op="delete_vertices", ids=ids))
    # vertex insertion: capacity grows to nv + GROW (hints for half of them)
    new = np.arange(nv, nv + GROW, dtype=np.uint32)
    hints = np.where(new % 2 == 0, 40, 0).astype(np.uint32)
    steps.append(dict(op="insert_vertices", ids=new, hints=hints))
    nv2 = nv + GROW
    # edges into the new vertices and into / out of the deleted ones (re-insertion)
    es, ed, ew = wl.uniform_edges(SEED, 6, 16_000, nv2)
    es[:2_000] = np.resize(new, 2_000)
    ed[2_000:4_000] = np.resize(ids, 2_000)
    es[4_000:6_000] = np.resize(ids, 2_000)
    steps.append(dict(op="insert", src=es, dst=ed, w=ew))
    # a batch held by rank 0 alone (every other rank joins with n = 0)
    a_s, a_d, a_w = wl.uniform_edges(SEED, 7, 3_000, nv2)
    steps.append(dict(op="insert", src=a_s, dst=a_d, w=a_w, alone=True))
    q2s = np.concatenate([es[:6_000], wl.uniform_edges(SEED, 8, 10_000, nv2)[0]])
    q2d = np.concatenate([ed[:6_000], wl.uniform_edges(SEED, 8, 10_000, nv2)[1]])
    steps.append(dict(op="query", src=q2s, dst=q2d))
    d2s, d2d, _ = wl.uniform_edges(SEED, 9, 8_000, nv2)
    d2s[:4_000], d2d[:4_000] = es[6_000:10_000], ed[6_000:10_000]
    steps.append(dict(op="delete", src=d2s, dst=d2d, alone=True))
    return steps


def run_rank(g, rank: int, P: int, to_dev):
    """One rank's side of the stream on handle ``g``; ``to_dev`` moves a numpy slice
    to the rank's device.  Returns the per-step records."""
    from paper_conf_ipps_awadapo20_b200 import DGError
    out = []
    for st in stream(P):
        key = "ids" if st["op"] in ("delete_vertices", "insert_vertices") else "src"
        lo, hi = bounds(st[key].size, rank, P, st.get("alone", False))
        sl = slice(lo, hi)
        rec = {"op": st["op"], "lo": lo, "hi": hi}
        try:
            if st["op"] == "insert":
                rec["count"] = g.insert_edges(to_dev(st["src"][sl]), to_dev(st["dst"][sl]),
                                              to_dev(st["w"][sl]), count=True)
                rec["status"] = 0
            elif st["op"] == "delete":
                rec["count"] = g.delete_edges(to_dev(st["src"][sl]), to_dev(st["dst"][sl]),
                                              count=True)
                rec["status"] = 0
            elif st["op"] == "query":
                f, w = g.query_edges(to_dev(st["src"][sl]), to_dev(st["dst"][sl]))
                rec["status"] = g.batch_status()
                rec["found"] = f.cpu().numpy()
                rec["weight"] = w.cpu().numpy()
            elif st["op"] == "delete_vertices":
                g.delete_vertices(to_dev(st["ids"][sl]))
                rec["status"] = g.batch_status()
            else:
                g.insert_vertices(to_dev(st["ids"][sl]), to_dev(st["hints"][sl]))
                rec["status"] = 0
        except DGError as e:
            rec["status"] = e.status
        out.append(rec)
    bad = [(i, r["op"], r["status"]) for i, r in enumerate(out) if r["status"] not in (0, 2)]
    if bad:  # a collective failed: report where (the handle is unusable now)
        raise AssertionError(f"rank {rank}: failed calls (step, op, status): {bad}")
    ro, dst, wt = g.export(device=False)
    deg = g.degrees(device=False)
    st = g.stats()
    out.append({"op": "export", "ro": ro, "dst": dst, "w": wt, "deg": deg,
                "exchange": st["exchange"], "nv": g.num_vertices})
    return out


def check(records, P: int, directed: bool = True):
    """records[k] = run_rank output of rank k.  Raises AssertionError on a mismatch."""
    from oracle import Oracle
    from oracle.compare import Candidates, compare_export, compare_queries
    OOR = 2
    o = Oracle(NV0, directed=directed)
    steps = stream(P)
    for i, st in enumerate(steps):
        recs = [records[k][i] for k in range(P)]
        where = f"P={P} step {i} ({st['op']})"
        if st["op"] == "insert":
            ost, added = o.insert_edges(st["src"], st["dst"], st["w"])
            for r in recs:
                assert r["status"] == ost, (where, r["status"], ost)
                if ost == 0:
                    assert r["count"] == added, (where, r["count"], added)
            assert (ost == OOR) == bool(st.get("rejected")), where
        elif st["op"] == "delete":
            ost, removed = o.delete_edges(st["src"], st["dst"])
            for r in recs:
                assert r["status"] == ost and r["count"] == removed, (where, r, removed)
        elif st["op"] == "query":
            ost, rf, rw = o.query_edges(st["src"], st["dst"])
            if ost == OOR:
                # the header's reading of a rejected query batch (include/dg.h
                # dg_query_edges, Q7/Q19): each out-of-range query answers 0, the
                # in-range ones are answered; the self-loop (0, 0) answers 0 too
                nvq = o.num_vertices
                bad = (st["src"] >= nvq) | (st["dst"] >= nvq)
                qs = np.where(bad, 0, st["src"]).astype(np.uint32)
                qd = np.where(bad, 0, st["dst"]).astype(np.uint32)
                _, rf, rw = o.query_edges(qs, qd)
            cand = Candidates(*o.candidates())
            for k, r in enumerate(recs):
                assert r["status"] == ost, (where, k, r["status"], ost)
                sl = slice(r["lo"], r["hi"])
                errs = compare_queries(st["src"][sl], st["dst"][sl], r["found"], r["weight"],
                                       rf[sl], rw[sl], cand)
                assert not errs, (where, k, errs)
            assert (ost == OOR) == bool(st.get("rejected")), where
        elif st["op"] == "delete_vertices":
            ost = o.delete_vertices(st["ids"])
            for r in recs:
                assert r["status"] == ost, (where, r["status"], ost)
        else:
            o.insert_vertices(st["ids"])
    ro_g, d_g, w_g = o.export()
    deg = np.diff(ro_g).astype(np.int64)
    nv = o.num_vertices
    cu_, cv_, cw_ = o.candidates()
    for k in range(P):
        ex = records[k][-1]
        assert ex["nv"] == nv, (k, ex["nv"], nv)
        rows = np.arange(k, nv, P)
        assert ex["ro"].size == rows.size + 1, (k, ex["ro"].size, rows.size)
        want_ro = np.concatenate([[0], np.cumsum(deg[rows])]).astype(np.uint64)
        sel = (np.concatenate([np.arange(ro_g[u], ro_g[u + 1]) for u in rows]).astype(np.int64)
               if rows.size else np.zeros(0, np.int64))
        m = (cu_ % P) == k
        errs = compare_export((ex["ro"], ex["dst"], ex["w"]), (want_ro, d_g[sel], w_g[sel]),
                              Candidates(cu_[m] // P, cv_[m], cw_[m]))
        assert not errs, (f"P={P} rank {k} export", errs)
        assert np.array_equal(ex["deg"].astype(np.int64), deg[rows]), f"P={P} rank {k} degrees"
    return [records[k][-1]["exchange"] for k in range(P)]
