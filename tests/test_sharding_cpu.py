"""Multi-rank host logic on CPU (gloo, world_size 2; -m "not gpu").

Pins the router's semantics before any GPU runs (SURVEY §8(c) "sharded ==
unsharded"): every edge op is executed only by owner(u) = u mod P, each rank feeds
its own slice of every batch, ops travel by an all-to-all exchange, vertex
deletions are all-gathered; the union of the P shards must equal the unsharded
oracle on the same stream.  Also checks the NCCL-id bootstrap the Python binding
uses (rank 0's dg_get_unique_id broadcast over the process group)."""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import workloads as wl


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _exchange(arrs, owner, P):
    """all-to-all of the SoA arrays by owner rank (gloo)."""
    order = np.argsort(owner, kind="stable")
    counts = np.bincount(owner, minlength=P)
    send_counts = torch.tensor(counts, dtype=torch.int64)
    recv_counts = torch.empty(P, dtype=torch.int64)
    dist.all_to_all_single(recv_counts, send_counts)
    out = []
    for a in arrs:
        src = torch.from_numpy(a[order].astype(np.int64))
        dst = torch.empty(int(recv_counts.sum()), dtype=torch.int64)
        dist.all_to_all_single(dst, src, recv_counts.tolist(), counts.tolist())
        out.append(dst.numpy().astype(np.uint32))
    return out


def _worker(rank, P, port, q):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=P)
    try:
        from oracle import Oracle
        # NCCL id bootstrap as done by bench.py / the binding
        from paper_conf_ipps_awadapo20_b200 import get_unique_id
        obj = [get_unique_id() if rank == 0 else None]
        dist.broadcast_object_list(obj, src=0)
        assert isinstance(obj[0], bytes) and len(obj[0]) == 128
        nv = 3000
        o = Oracle(nv)  # holds only rows u with u % P == rank
        for b in range(4):
            n = 20_000
            off, cnt = n * rank // P, n * (rank + 1) // P - n * rank // P
            s, d, w = wl.uniform_edges(41, b, cnt, nv, offset=off)
            rs, rd, rw = _exchange([s, d, w], s % P, P)
            assert (rs % P == rank).all()
            o.insert_edges(rs, rd, rw)
        ds, dd, _ = wl.uniform_edges(41, 1, 5000, nv, offset=rank * 5000)
        rs, rd = _exchange([ds, dd], ds % P, P)
        o.delete_edges(rs, rd)
        ids = wl.uniform_u32(41, 7, 20, nv, offset=rank * 20)
        allids = [None] * P
        dist.all_gather_object(allids, ids)
        o.delete_vertices(np.concatenate(allids))
        ro, dd_, ww = o.export()
        q.put((rank, ro, dd_, ww))
    finally:
        dist.destroy_process_group()


def test_sharded_oracle_equals_unsharded():
    from oracle import Oracle
    P = 2
    port = _free_port()
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    procs = [ctx.Process(target=_worker, args=(r, P, port, q)) for r in range(P)]
    for p in procs:
        p.start()
    res = {}
    for _ in range(P):
        r, ro, dd, ww = q.get(timeout=300)
        res[r] = (ro, dd, ww)
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    nv = 3000
    o = Oracle(nv)
    for b in range(4):
        s, d, w = wl.uniform_edges(41, b, 20_000, nv)
        o.insert_edges(s, d, w)
    ds, dd, _ = wl.uniform_edges(41, 1, 5000 * P, nv)
    o.delete_edges(ds, dd)
    o.delete_vertices(wl.uniform_u32(41, 7, 20 * P, nv))
    ro_g, d_g, w_g = o.export()
    for u in range(nv):
        k = u % P
        ro, dd_, ww = res[k]
        a, b = int(ro[u]), int(ro[u + 1])
        ga, gb = int(ro_g[u]), int(ro_g[u + 1])
        assert np.array_equal(dd_[a:b], d_g[ga:gb]), u
        assert np.array_equal(ww[a:b], w_g[ga:gb]), u
        # rows not owned by k are empty on k
        other = res[1 - k][0]
        assert other[u + 1] == other[u]


def _query_worker(rank, P, port, q):
    """a2 + a11 for queries: each rank routes its slice of the query batch to
    owner(u) = u mod P, the owner answers from its shard, and the answers travel back
    by the reverse all-to-all and are scattered to the slice's original positions."""
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=P)
    try:
        from oracle import Oracle
        nv = 2000
        o = Oracle(nv)
        n = 30_000
        off, cnt = n * rank // P, n * (rank + 1) // P - n * rank // P
        s, d, w = wl.uniform_edges(43, 0, cnt, nv, offset=off)
        rs, rd, rw = _exchange([s, d, w], s % P, P)
        o.insert_edges(rs, rd, rw)
        # a query slice with self-loops and out-of-shard sources mixed in
        qs, qd, _ = wl.uniform_edges(43, 1, 7_001 + rank, nv, offset=rank * 8_000)
        qd[::97] = qs[::97]
        owner = (qs % P).astype(np.int64)
        order = np.argsort(owner, kind="stable")
        counts = np.bincount(owner, minlength=P)
        rqs, rqd = _exchange([qs, qd], owner, P)
        assert (rqs % P == rank).all()
        _, f, wq = o.query_edges(rqs, rqd)
        recv_counts = torch.empty(P, dtype=torch.int64)
        dist.all_to_all_single(recv_counts, torch.tensor(counts, dtype=torch.int64))
        back = []
        for a in (np.asarray(f, np.int64), np.asarray(wq, np.int64)):
            out = torch.empty(int(counts.sum()), dtype=torch.int64)
            # reverse exchange: send what was received, receive what was sent
            dist.all_to_all_single(out, torch.from_numpy(a), counts.tolist(), recv_counts.tolist())
            res = np.empty(len(qs), np.int64)
            res[order] = out.numpy()  # scatter to the original positions
            back.append(res)
        q.put((rank, qs, qd, back[0], back[1]))
    finally:
        dist.destroy_process_group()


def test_sharded_query_return_matches_unsharded():
    from oracle import Oracle
    P = 2
    port = _free_port()
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    procs = [ctx.Process(target=_query_worker, args=(r, P, port, q)) for r in range(P)]
    for p in procs:
        p.start()
    res = [q.get(timeout=300) for _ in range(P)]
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    nv = 2000
    o = Oracle(nv)
    s, d, w = wl.uniform_edges(43, 0, 30_000, nv)
    o.insert_edges(s, d, w)
    hits = 0
    for _, qs, qd, f, wq in res:
        _, ef, ew = o.query_edges(qs, qd)
        assert np.array_equal(np.asarray(ef, np.int64), f)
        assert np.array_equal(np.asarray(ew, np.int64), wq)
        assert not f[qs == qd].any()  # self-loops are never stored (Alg1:L3)
        hits += int(f.sum())
    assert hits > 0


class _ShardedOracleRank:
    """A CPU stand-in for one rank's ``Graph`` in ``tests/multirank.py``: the rank's
    shard is an oracle holding only the rows it owns (owner(u) = u mod P); every call
    is collective over gloo — the slices are all-gathered, each owner applies the ops
    of its rows, counts are summed and query answers travel back to the askers.  It
    pins the scenario and its checker (what the GPU router tests assert) on CPU."""

    def __init__(self, nv, rank, P, directed=True):
        from oracle import Oracle
        self.rank, self.P, self.directed = rank, P, directed
        self.o = Oracle(nv, directed=True)
        self.nv = nv
        self._status = 0

    def _union(self, *arrs):
        mine = [np.asarray(a, np.uint32) for a in arrs]
        allp = [None] * self.P
        dist.all_gather_object(allp, mine)
        return [np.concatenate([p[i] for p in allp]) for i in range(len(arrs))], \
            [p[0].size for p in allp]

    def _sum(self, x):
        t = torch.tensor([x], dtype=torch.int64)
        dist.all_reduce(t)
        return int(t.item())

    def _oob(self, *arrs):
        return any(bool((a >= self.nv).any()) for a in arrs)

    def _mirror(self, s, d, w=None):
        if self.directed:
            return s, d, w
        return (np.concatenate([s, d]), np.concatenate([d, s]),
                None if w is None else np.concatenate([w, w]))

    def insert_edges(self, s, d, w, count=True):
        from paper_conf_ipps_awadapo20_b200 import DGError
        (s, d, w), _ = self._union(s, d, w)
        if self._oob(s, d):
            raise DGError(2, "insert")
        s, d, w = self._mirror(s, d, w)
        m = (s % self.P) == self.rank
        return self._sum(self.o.insert_edges(s[m], d[m], w[m])[1])

    def delete_edges(self, s, d, count=True):
        from paper_conf_ipps_awadapo20_b200 import DGError
        (s, d), _ = self._union(s, d)
        if self._oob(s, d):
            raise DGError(2, "delete")
        s, d, _ = self._mirror(s, d)
        m = (s % self.P) == self.rank
        return self._sum(self.o.delete_edges(s[m], d[m])[1])

    def query_edges(self, s, d):
        (us, ud), sizes = self._union(s, d)
        bad = (us >= self.nv) | (ud >= self.nv)
        self._status = self._sum(int(bad.any())) and 2
        m = ((us % self.P) == self.rank) & ~bad
        f = np.zeros(us.size, np.int64)
        w = np.zeros(us.size, np.int64)
        _, f[m], w[m] = self.o.query_edges(us[m], ud[m])
        ft, wt = torch.from_numpy(f), torch.from_numpy(w)
        dist.all_reduce(ft)
        dist.all_reduce(wt)
        lo = sum(sizes[:self.rank])
        sl = slice(lo, lo + sizes[self.rank])

        class _T:  # .cpu().numpy() like a tensor
            def __init__(self, a):
                self.a = a

            def cpu(self):
                return self

            def numpy(self):
                return self.a
        return _T(ft.numpy()[sl].astype(np.uint8)), _T(wt.numpy()[sl].astype(np.uint32))

    def batch_status(self):
        st, self._status = self._status, 0
        return st

    def delete_vertices(self, ids):
        (ids,), _ = self._union(ids)
        self._status = 2 if self._oob(ids) else self.o.delete_vertices(ids)

    def insert_vertices(self, ids, hints=None):
        (ids,), _ = self._union(ids)
        self.o.insert_vertices(ids)
        self.nv = self.o.num_vertices

    def export(self, device=False):
        ro, d, w = self.o.export()
        rows = np.arange(self.rank, self.nv, self.P)
        deg = np.diff(ro)[rows].astype(np.int64)
        sel = (np.concatenate([np.arange(ro[u], ro[u + 1]) for u in rows]).astype(np.int64)
               if rows.size else np.zeros(0, np.int64))
        return np.concatenate([[0], np.cumsum(deg)]).astype(np.uint64), d[sel], w[sel]

    def degrees(self, device=False):
        return np.diff(self.export()[0]).astype(np.uint32)

    def stats(self):
        return {"exchange": 0}

    @property
    def num_vertices(self):
        return self.nv


def _scenario_worker(rank, P, port, directed, q):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=P)
    try:
        from tests import multirank
        g = _ShardedOracleRank(multirank.NV0, rank, P, directed)
        recs = multirank.run_rank(g, rank, P, lambda a: np.ascontiguousarray(a, np.uint32))
        out = [None] * P if rank == 0 else None
        dist.gather_object(recs, out, dst=0)
        if rank == 0:
            multirank.check(out, P, directed=directed)
        q.put((rank, "ok"))
    except BaseException as e:  # noqa: BLE001
        q.put((rank, repr(e)))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("P,directed", [(2, True), (3, False)])
def test_multirank_scenario_on_sharded_oracles(P, directed):
    """The stream and checker of the GPU router tests (tests/multirank.py), run by P
    gloo ranks whose shards are oracles: the union of the shards equals the unsharded
    oracle, rejected batches are rejected on every rank, out-of-range queries answer 0."""
    port = _free_port()
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    procs = [ctx.Process(target=_scenario_worker, args=(r, P, port, directed, q))
             for r in range(P)]
    for p in procs:
        p.start()
    res = [q.get(timeout=300) for _ in range(P)]
    for p in procs:
        p.join(timeout=60)
    assert all(r[1] == "ok" for r in res), res
