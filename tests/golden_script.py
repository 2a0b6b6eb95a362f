"""Parser/runner for the hand-worked operation scripts in tests/golden/.

The runner is generic over a "graph" object with the methods of ``oracle.Oracle``
(``insert_edges``, ``delete_edges``, ``query_edges``, ``delete_vertices``,
``insert_vertices``, ``export``) so the same fixture pins the oracle (CPU) and is
replayed on the GPU path.
"""
from __future__ import annotations

import os

import numpy as np

GOLDEN = os.path.join(os.path.dirname(os.path.abspath(__file__)), "golden")


def _triples(text, width):
    out = []
    for part in text.split("|"):
        f = part.split()
        if f:
            assert len(f) == width, part
            out.append([int(x) for x in f])
    return np.array(out, dtype=np.uint64).reshape(-1, width)


def parse_adjacency(text):
    """'0: 1/11 2/21 ; 2: 3/30' -> {0: {1: 11, 2: 21}, 2: {3: 30}}"""
    adj = {}
    for part in text.split(";"):
        part = part.strip()
        if not part:
            continue
        u, rest = part.split(":")
        row = {}
        for tok in rest.split():
            v, w = tok.split("/")
            row[int(v)] = int(w)
        adj[int(u)] = row
    return adj


def load(name):
    lines = []
    with open(os.path.join(GOLDEN, name)) as f:
        for ln in f:
            ln = ln.split("#", 1)[0].strip()
            if ln:
                lines.append(ln)
    return lines


def export_to_adj(ro, d, w):
    adj = {}
    ro = np.asarray(ro, np.int64)
    for u in range(ro.size - 1):
        a, b = int(ro[u]), int(ro[u + 1])
        if b > a:
            adj[u] = {int(d[i]): int(w[i]) for i in range(a, b)}
    return adj


def run_script(lines, make_graph):
    """Replays a script; raises AssertionError at the first mismatch."""
    g = None
    last = None
    for ln in lines:
        op, _, rest = ln.partition(" ")
        if op == "V":
            n, mode = rest.split()
            g = make_graph(int(n), mode == "directed")
        elif op == "I":
            t = _triples(rest, 3)
            last = g.insert_edges(t[:, 0], t[:, 1], t[:, 2])
        elif op == "D":
            t = _triples(rest, 2)
            last = g.delete_edges(t[:, 0], t[:, 1])
        elif op == "Q":
            t = _triples(rest, 2)
            last = g.query_edges(t[:, 0], t[:, 1])
        elif op == "DV":
            ids = np.array([int(x) for x in rest.split()], np.uint32)
            last = (g.delete_vertices(ids),)
        elif op == "IV":
            ids = np.array([int(x) for x in rest.split()], np.uint32)
            last = (g.insert_vertices(ids),)
        elif op == "E":
            kind, _, vals = rest.partition(" ")
            if kind in ("added", "removed"):
                assert last[0] == 0, f"{ln}: status {last[0]}"
                assert last[1] == int(vals), f"{ln}: got {last[1]}"
            elif kind == "found":
                t = _triples(vals, 2)
                st, found, weight = last
                assert st == 0
                assert np.array_equal(np.asarray(found, np.int64), t[:, 0].astype(np.int64)), \
                    f"{ln}: found {list(found)}"
                assert np.array_equal(np.asarray(weight, np.int64), t[:, 1].astype(np.int64)), \
                    f"{ln}: weight {list(weight)}"
            else:
                raise ValueError(ln)
        elif op == "R":
            assert last[0] == int(rest), f"{ln}: status {last[0]}"
        elif op == "X":
            want = parse_adjacency(rest)
            ro, d, w = g.export()
            from oracle.compare import canonical
            ro, d, w = canonical(ro, d, w)
            got = export_to_adj(ro, d, w)
            assert got == want, f"{ln}: got {got}"
        else:
            raise ValueError(ln)
    return g
