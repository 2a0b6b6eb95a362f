"""Pins for the CPU oracle (-m "not gpu").

The oracle is checked against things other than itself:
  * the hand-worked fixtures in tests/golden/ (each line cites its passage);
  * a dense |V|x|V| adjacency-matrix model (the textbook representation the paper
    calls "trivial to update") on random op sequences, compared after
    every batch — brute force on tiny inputs;
  * the north-star invariants (no duplicate edges, degree = unique out-neighbours,
    insert-then-delete restores, vertex deletion removes all incident edges);
  * triangle counts against closed forms (K_n -> C(n,3), bipartite -> 0), an O(n^3)
    brute force, and numpy's integer trace(A^3)/6;
  * the comparator detects seeded corruptions.
"""
import itertools
import math

import numpy as np
import pytest

import workloads as wl
from oracle import Oracle, initial_buckets, ERR_VERTEX_OUT_OF_RANGE
from oracle.compare import Candidates, compare_export, compare_queries, check_invariants
from tests.golden_script import GOLDEN, load, run_script

import os


# ----------------------------------------------------------------- golden ---
def test_golden_initial_buckets():
    n = 0
    for ln in load("initial_buckets.txt"):
        hint, lf, bc, want = (int(x) for x in ln.split())
        assert initial_buckets(hint, lf, bc) == want, ln
        n += 1
    assert n >= 10


@pytest.mark.parametrize("name", ["edge_ops_directed.txt", "edge_ops_undirected.txt"])
def test_golden_scripts(name):
    run_script(load(name), lambda n, directed: Oracle(n, directed))


def _golden_triangles():
    out = []
    for ln in load("triangles.txt"):
        f = ln.split()
        name, n, want = f[0], int(f[1]), int(f[2])
        edges = [tuple(int(x) for x in e.split("-")) for e in f[3:]]
        out.append((name, n, want, edges))
    return out


@pytest.mark.parametrize("case", _golden_triangles(), ids=lambda c: c[0])
def test_golden_triangles(case):
    name, n, want, edges = case
    g = Oracle(n, directed=False)
    s = np.array([e[0] for e in edges], np.uint32)
    d = np.array([e[1] for e in edges], np.uint32)
    assert g.insert_edges(s, d)[0] == 0
    assert g.triangle_count() == want


# ------------------------------------------------------------- dense model ---
class Dense:
    """|V|x|V| (present, weight) matrices — P:L138-140.  Sequential 'latest wins'."""

    def __init__(self, n, directed=True):
        self.P = np.zeros((n, n), bool)
        self.W = np.zeros((n, n), np.uint64)
        self.directed = directed
        # Q1: key -> the weights its most recent insert batch wrote, for
        # keys that batch wrote >= 2 times; a single write, a delete or the deletion
        # of an endpoint drops the entry
        self.cand = {}

    @property
    def n(self):
        return self.P.shape[0]

    def _expand(self, s, d, w):
        s = list(map(int, s)); d = list(map(int, d))
        w = [0] * len(s) if w is None else list(map(int, w))
        if not self.directed:
            s, d, w = s + d, d + s, w + w
        return s, d, w

    def insert(self, s, d, w):
        if any(x >= self.n for x in list(s) + list(d)):
            return 2, 0
        added = 0
        writes = {}
        for u, v, x in zip(*self._expand(s, d, w)):
            if u == v:
                continue
            writes.setdefault((u, v), []).append(x)
            if not self.P[u, v]:
                added += 1
            self.P[u, v] = True
            self.W[u, v] = x
        for k, ws in writes.items():
            if len(ws) >= 2:
                self.cand[k] = ws
            else:
                self.cand.pop(k, None)
        return 0, added

    def delete(self, s, d):
        if any(x >= self.n for x in list(s) + list(d)):
            return 2, 0
        removed = 0
        for u, v, _ in zip(*self._expand(s, d, None)):
            if u != v and self.P[u, v]:
                self.P[u, v] = False
                self.W[u, v] = 0
                removed += 1
                self.cand.pop((u, v), None)
        return 0, removed

    def query(self, s, d):
        f = np.array([1 if (u != v and self.P[u, v]) else 0 for u, v in zip(s, d)], np.uint8)
        w = np.array([self.W[u, v] if (u != v and self.P[u, v]) else 0 for u, v in zip(s, d)],
                     np.uint32)
        return f, w

    def delete_vertices(self, ids):
        if any(x >= self.n for x in ids):
            return 2
        for u in ids:
            self.P[u, :] = False
            self.P[:, u] = False
            self.W[u, :] = 0
            self.W[:, u] = 0
        D = set(int(x) for x in ids)
        self.cand = {k: v for k, v in self.cand.items() if k[0] not in D and k[1] not in D}
        return 0

    def candidates(self):
        return sorted((u, v, int(x)) for (u, v), ws in self.cand.items() for x in ws)

    def insert_vertices(self, ids):
        m = max([self.n] + [int(x) + 1 for x in ids])
        if m > self.n:
            P = np.zeros((m, m), bool); W = np.zeros((m, m), np.uint64)
            P[: self.n, : self.n] = self.P; W[: self.n, : self.n] = self.W
            self.P, self.W = P, W
        return 0

    def export(self):
        deg = self.P.sum(axis=1)
        ro = np.concatenate([[0], np.cumsum(deg)]).astype(np.uint64)
        rows, cols = np.nonzero(self.P)  # row-major, cols ascending within a row
        return ro, cols.astype(np.uint32), self.W[rows, cols].astype(np.uint32)


def _random_sequence_check(seed, directed, n0=48, steps=40):
    rs = np.random.RandomState(seed)
    g = Oracle(n0, directed, threads=1)
    m = Dense(n0, directed)
    for step in range(steps):
        op = rs.choice(["ins", "ins", "del", "qry", "dv", "iv", "bad"], p=[.3, .15, .2, .15, .08, .05, .07])
        n = m.n
        k = int(rs.randint(0, 64))
        # small vertex range + few distinct weights so in-batch duplicates occur
        s = rs.randint(0, n, k).astype(np.uint32)
        d = rs.randint(0, n, k).astype(np.uint32)
        w = rs.randint(0, 1 << 32, k, dtype=np.uint64).astype(np.uint32)
        if op == "ins":
            assert g.insert_edges(s, d, w) == m.insert(s, d, w)
        elif op == "del":
            assert g.delete_edges(s, d) == m.delete(s, d)
        elif op == "qry":
            st, f, ww = g.query_edges(s, d)
            f2, w2 = m.query(s, d)
            assert st == 0 and np.array_equal(f, f2) and np.array_equal(ww, w2)
        elif op == "dv":
            ids = rs.randint(0, n, rs.randint(0, 4)).astype(np.uint32)
            assert g.delete_vertices(ids) == m.delete_vertices(ids)
        elif op == "iv":
            ids = np.array([n + rs.randint(0, 3)], np.uint32)
            assert g.insert_vertices(ids) == m.insert_vertices(ids)
        elif op == "bad":
            s2 = s.copy()
            if k:
                s2[rs.randint(0, k)] = n + rs.randint(0, 5)
                before = g.export()
                assert g.insert_edges(s2, d, w)[0] == ERR_VERTEX_OUT_OF_RANGE
                assert g.delete_edges(s2, d)[0] == ERR_VERTEX_OUT_OF_RANGE
                after = g.export()
                assert all(np.array_equal(a, b) for a, b in zip(before, after))
        ro, dd, ww = g.export()
        mro, mdd, mww = m.export()
        assert np.array_equal(ro, mro), f"step {step} op {op}"
        assert np.array_equal(dd, mdd), f"step {step} op {op}"
        assert np.array_equal(ww, mww), f"step {step} op {op}"
        assert np.array_equal(g.degrees(), np.diff(ro).astype(np.uint32))
        assert check_invariants(ro, dd, g.degrees()) == []
        cu, cv, cw = g.candidates()
        assert sorted(zip(cu.tolist(), cv.tolist(), cw.tolist())) == m.candidates(), \
            f"step {step} op {op}: Q1 candidate sets"


@pytest.mark.parametrize("seed", range(6))
def test_dense_model_directed(seed):
    _random_sequence_check(seed, True)


@pytest.mark.parametrize("seed", range(3))
def test_dense_model_undirected(seed):
    _random_sequence_check(100 + seed, False)


def test_threads_do_not_change_results():
    """T threads, thread t owns the vertices u % T == t, so every
    vertex's ops keep their batch order — the graph, counts, answers, Q1 candidate
    sets and triangle count are those of one thread (batches above the oracle's
    one-thread cutoff of 2^15 ops, with duplicates, misses and vertex deletions)."""
    nv = 3000
    res = []
    for T in (1, 3, 8):
        g = Oracle(nv, directed=(T != 3), threads=T)
        out = []
        for b in range(3):
            s, d, w = wl.uniform_edges(21, b, 60_000, nv)
            s[:6000], d[:6000] = s[6000:12000], d[6000:12000]  # 10% duplicate keys (Q1)
            out.append(g.insert_edges(s, d, w))
        qs, qd, _ = wl.uniform_edges(21, 9, 50_000, nv)
        out.append(g.query_edges(qs, qd))
        ds, dd, _ = wl.uniform_edges(21, 1, 40_000, nv)
        out.append(g.delete_edges(ds, dd))
        out.append(g.delete_vertices(wl.uniform_u32(21, 5, 50, nv)))
        out.append(g.export())
        cu, cv, cw = g.candidates()
        out.append(sorted(zip(cu.tolist(), cv.tolist(), cw.tolist())))
        out.append(g.triangle_count() if T == 3 else None)
        res.append((T, out))
    # T = 1 and T = 8 (both directed) agree on everything
    a, b = res[0][1], res[2][1]
    for x, y in zip(a, b):
        if isinstance(x, tuple):
            for p, q in zip(x, y):
                assert np.array_equal(np.asarray(p), np.asarray(q))
        else:
            assert x == y
    assert len(a[-2]) > 1000  # duplicates were exercised
    # undirected T = 3 against one thread
    g1 = Oracle(nv, directed=False, threads=1)
    for b in range(3):
        s, d, w = wl.uniform_edges(21, b, 60_000, nv)
        s[:6000], d[:6000] = s[6000:12000], d[6000:12000]
        g1.insert_edges(s, d, w)
    ds, dd, _ = wl.uniform_edges(21, 1, 40_000, nv)
    g1.delete_edges(ds, dd)
    g1.delete_vertices(wl.uniform_u32(21, 5, 50, nv))
    for p, q in zip(g1.export(), res[1][1][6]):
        assert np.array_equal(p, q)
    assert g1.triangle_count() == res[1][1][8]


# --------------------------------------------------------------- invariants ---
def _rand_graph(seed, nv, m):
    s, d, w = wl.uniform_edges(seed, 1, m, nv)
    g = Oracle(nv)
    g.insert_edges(s, d, w)
    return g, (s, d, w)


def test_insert_then_delete_restores():
    """delete(insert(G, B), B) == G minus keys(B); == G when keys(B) ∩ G = ∅
    (key semantics P:L182-192)."""
    nv = 500
    g, _ = _rand_graph(7, nv, 3000)
    before = g.export()
    s, d, w = wl.uniform_edges(7, 2, 2000, nv)
    st, f, _ = g.query_edges(s, d)
    fresh = f == 0
    s2, d2, w2 = s[fresh], d[fresh], w[fresh]
    g.insert_edges(s2, d2, w2)
    g.delete_edges(s2, d2)
    after = g.export()
    for a, b in zip(before, after):
        assert np.array_equal(a, b)
    # general form: keys that existed before are removed too
    g.insert_edges(s, d, w)
    g.delete_edges(s, d)
    ro, dd, ww = g.export()
    bro, bdd, bww = before
    deg = np.diff(bro).astype(np.int64)
    rows = np.repeat(np.arange(nv), deg)
    removed = set(zip(s.tolist(), d.tolist()))
    keep = np.array([(int(r), int(x)) not in removed for r, x in zip(rows, bdd)], bool)
    assert np.array_equal(dd, bdd[keep]) and np.array_equal(ww, bww[keep])


def test_vertex_deletion_removes_incident_edges():
    nv = 300
    g, _ = _rand_graph(11, nv, 4000)
    ids = np.array([3, 17, 17, 250], np.uint32)
    assert g.delete_vertices(ids) == 0
    ro, dd, ww = g.export()
    D = set(ids.tolist())
    for u in D:
        assert ro[u + 1] == ro[u]
    assert not np.isin(dd, list(D)).any()
    qs = np.array([3] * nv + list(range(nv)), np.uint32)
    qd = np.array(list(range(nv)) + [3] * nv, np.uint32)
    st, f, w = g.query_edges(qs, qd)
    assert st == 0 and f.sum() == 0 and w.sum() == 0
    # the ID stays valid and can gain edges again (Q10)
    assert g.insert_edges(np.array([3], np.uint32), np.array([5], np.uint32))[1] == 1


def test_candidate_sets_intra_batch_duplicates():
    g = Oracle(10)
    s = np.array([1, 1, 1, 2], np.uint32)
    d = np.array([2, 2, 2, 3], np.uint32)
    w = np.array([5, 6, 7, 9], np.uint32)
    assert g.insert_edges(s, d, w) == (0, 2)
    cu, cv, cw = g.candidates()
    assert sorted(zip(cu.tolist(), cv.tolist(), cw.tolist())) == [(1, 2, 5), (1, 2, 6), (1, 2, 7)]
    # a later single write clears the candidate set (Q2: deterministic replace)
    g.insert_edges(np.array([1], np.uint32), np.array([2], np.uint32), np.array([8], np.uint32))
    assert g.candidates()[0].size == 0
    assert g.query_edges(np.array([1], np.uint32), np.array([2], np.uint32))[2][0] == 8


# ---------------------------------------------------------- triangle count ---
@pytest.mark.parametrize("n", [3, 4, 5, 10, 23])
def test_tc_complete_graph(n):
    s, d = zip(*itertools.combinations(range(n), 2))
    g = Oracle(n, directed=False)
    g.insert_edges(np.array(s, np.uint32), np.array(d, np.uint32))
    assert g.triangle_count() == math.comb(n, 3)


def test_tc_bipartite_and_grid_zero():
    a, b = 7, 9
    s = [i for i in range(a) for j in range(b)]
    d = [a + j for i in range(a) for j in range(b)]
    g = Oracle(a + b, directed=False)
    g.insert_edges(np.array(s, np.uint32), np.array(d, np.uint32))
    assert g.triangle_count() == 0
    gs, gd = wl.grid_edges(3, 20, 20, 1.0)
    g = Oracle(400, directed=True)  # grid edges already come in both directions
    g.insert_edges(gs, gd)
    assert g.triangle_count() == 0


def _sym_random(seed, n, m):
    s, d, _ = wl.uniform_edges(seed, 9, m, n, weights=False)
    g = Oracle(n, directed=False)
    g.insert_edges(s, d)
    A = np.zeros((n, n), np.int64)
    ro, dd, _ = g.export()
    rows = np.repeat(np.arange(n), np.diff(ro).astype(np.int64))
    A[rows, dd.astype(np.int64)] = 1
    return g, A


def test_tc_brute_force_small():
    g, A = _sym_random(5, 40, 300)
    n = A.shape[0]
    brute = sum(1 for i in range(n) for j in range(i + 1, n) for k in range(j + 1, n)
                if A[i, j] and A[j, k] and A[i, k])
    assert g.triangle_count() == brute


def test_tc_trace_a_cubed():
    g, A = _sym_random(6, 400, 6000)
    assert (A == A.T).all()
    assert g.triangle_count() == int(np.trace(A @ A @ A)) // 6


# ---------------------------------------------------------------- comparator ---
def test_comparator_detects_corruptions():
    nv = 200
    g = Oracle(nv)
    s, d, w = wl.uniform_edges(21, 1, 3000, nv)
    # force intra-batch duplicates with distinct weights (Q1)
    s[100:120] = s[:20]; d[100:120] = d[:20]
    g.insert_edges(s, d, w)
    ref = g.export()
    cand = Candidates(*g.candidates())
    assert cand.keys.size > 0
    ro, dd, ww = (x.copy() for x in ref)
    # shuffle within rows: still equal after canonicalisation
    perm = np.arange(dd.size)
    for u in range(nv):
        a, b = int(ro[u]), int(ro[u + 1])
        perm[a:b] = perm[a:b][::-1]
    assert compare_export((ro, dd[perm], ww[perm]), ref, cand) == []
    rs = np.random.RandomState(0)
    nonc = np.nonzero(~cand.is_cand((np.repeat(np.arange(nv, dtype=np.uint64),
                                               np.diff(ro).astype(np.int64)) << np.uint64(32))
                                    | dd.astype(np.uint64)))[0]
    i = int(nonc[rs.randint(nonc.size)])
    corrupt = []
    # drop one edge
    r = int(np.searchsorted(ro, i, side="right") - 1)
    ro2 = ro.copy(); ro2[r + 1:] -= 1
    corrupt.append((ro2, np.delete(dd, i), np.delete(ww, i)))
    # duplicate dst in a row
    d2 = dd.copy(); j = int(ro[r]); d2[j + 1 if ro[r + 1] > j + 1 else j] = d2[j]
    if ro[r + 1] - ro[r] >= 2:
        corrupt.append((ro, d2, ww))
    # flip a weight bit on a non-candidate key
    w2 = ww.copy(); w2[i] ^= np.uint32(1 << 7)
    corrupt.append((ro, dd, w2))
    # move an edge to another row
    ro3 = ro.copy(); ro3[r + 1] += 1
    corrupt.append((ro3, dd, ww))
    for c in corrupt:
        assert compare_export(c, ref, cand) != []
    # non-candidate weight on a candidate key
    cpos = np.nonzero(cand.is_cand((np.repeat(np.arange(nv, dtype=np.uint64),
                                              np.diff(ro).astype(np.int64)) << np.uint64(32))
                                   | dd.astype(np.uint64)))[0]
    w4 = ww.copy(); w4[cpos[0]] = np.uint32(0xDEADBEEF)
    assert compare_export((ro, dd, w4), ref, cand) != []
    # query comparator: found=1 on a miss
    qs, qd, _ = wl.uniform_edges(21, 5, 500, nv)
    st, f, qw = g.query_edges(qs, qd)
    assert compare_queries(qs, qd, f, qw, f, qw, cand) == []
    f2 = f.copy(); miss = np.nonzero(f == 0)[0][0]; f2[miss] = 1
    assert compare_queries(qs, qd, f2, qw, f, qw, cand) != []


# ----------------------------------------------------------------- generators ---
def test_generators_deterministic_and_shaped():
    a = wl.uniform_edges(1, 3, 1000, 1024)
    b = wl.uniform_edges(1, 3, 1000, 1024)
    assert all(np.array_equal(x, y) for x, y in zip(a, b))
    # slices regenerate independently: first 100 of a 1000-batch == a 100-batch
    c = wl.uniform_edges(1, 3, 100, 1024)
    assert np.array_equal(a[0][:100], c[0])
    s, d = wl.rmat_edges(2, 0, 20000, 14, wl.GRAPH500)
    assert s.max() < (1 << 14) and d.max() < (1 << 14)
    deg = np.bincount(s, minlength=1 << 14)
    assert deg.max() > 20 * deg.mean()          # scale-free: hubs exist
    s, d = wl.rmat_edges(2, 0, 20000, 14, wl.LJLIKE, nv=10000)
    assert s.max() < 10000 and d.max() < 10000
    # permutation is a bijection
    perm = [wl.permute(x, 9, 4) for x in range(512)]
    assert sorted(perm) == list(range(512))
    # road-like: average degree ~2.41 at p = 0.6025 (Tab.I road_usa 2.4)
    gs, gd = wl.grid_edges(3, 300, 300, 0.6025)
    assert abs(gs.size / 90000 - 2.41) < 0.05
    assert np.bincount(gs).max() <= 4


def test_grid_heldout_is_the_lattice_complement():
    """workloads.grid_heldout_edges (cfg3 road growth) = the lattice edges grid_edges
    did not keep: disjoint from them, and together every directed lattice edge once."""
    import workloads as wl
    rows, cols = 37, 53
    s, d = wl.grid_edges(3, rows, cols, 0.6025)
    hs, hd = wl.grid_heldout_edges(3, rows, cols, 0.6025)
    kept = set(zip(s.tolist(), d.tolist()))
    held = set(zip(hs.tolist(), hd.tolist()))
    assert len(kept) == s.size and len(held) == hs.size and not (kept & held)
    lattice = set()
    for r in range(rows):
        for c in range(cols):
            u = r * cols + c
            if c + 1 < cols:
                lattice |= {(u, u + 1), (u + 1, u)}
            if r + 1 < rows:
                lattice |= {(u, u + cols), (u + cols, u)}
    assert kept | held == lattice
