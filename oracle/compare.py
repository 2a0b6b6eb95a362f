"""Canonicalising comparator (SURVEY.md §8(c) "Comparator") — test infrastructure.

* row_offsets and (row-sorted) dst arrays: bit-exact;
* weights: bit-exact, except a key duplicated inside its most recent insert batch,
  whose weight must be one of that batch's weights for it (Q1);
* query answers: ``found`` bit-exact, weights under the same rule.

The GPU export is unsorted within rows; ``canonical`` sorts each row by dst,
carrying weights.  The oracle export is already sorted.
"""
from __future__ import annotations

import numpy as np


def canonical(row_offsets, dst, w=None):
    """Rows sorted by dst, weights carried (a stable sort of the (row, dst) keys; rows
    are already grouped, so an export that is sorted already costs one linear pass)."""
    ro = np.asarray(row_offsets, np.uint64)
    dst = np.asarray(dst, np.uint32)
    deg = np.diff(ro).astype(np.int64)
    rows = np.repeat(np.arange(deg.size, dtype=np.uint64), deg)
    key = (rows << np.uint64(32)) | dst.astype(np.uint64)
    del rows
    if key.size > 1 and bool((key[1:] >= key[:-1]).all()):
        return ro, dst, (None if w is None else np.asarray(w, np.uint32))
    order = np.argsort(key, kind="stable")
    return ro, dst[order], (None if w is None else np.asarray(w, np.uint32)[order])


def _keys(u, v):
    return (np.asarray(u, np.uint64) << np.uint64(32)) | np.asarray(v, np.uint64)


class Candidates:
    """Q1 candidate sets from ``Oracle.candidates()``."""

    def __init__(self, cu, cv, cw):
        keys = _keys(cu, cv)
        self.keys = np.unique(keys)
        self.pairs = set(zip(keys.tolist(), np.asarray(cw, np.uint32).tolist()))

    def allowed(self, keys, weights):
        """bool mask: (key, weight) is an allowed pair for a candidate key."""
        return np.array([(int(k), int(x)) in self.pairs for k, x in zip(keys, weights)],
                        dtype=bool)

    def is_cand(self, keys):
        return np.isin(keys, self.keys)


def compare_export(gpu, ref, cand: Candidates | None = None, max_report: int = 8):
    """Return a list of mismatch descriptions (empty = identical)."""
    errs = []
    if int(np.asarray(gpu[0])[-1]) != np.asarray(gpu[1]).size:
        return [f"row_offsets end {int(np.asarray(gpu[0])[-1])} != dst length {np.asarray(gpu[1]).size}"]
    g_ro, g_d, g_w = canonical(*gpu)
    r_ro, r_d, r_w = ref
    r_ro = np.asarray(r_ro, np.uint64)
    if g_ro.shape != r_ro.shape:
        return [f"row_offsets length {g_ro.size} != {r_ro.size}"]
    bad = np.nonzero(g_ro != r_ro)[0]
    if bad.size:
        i = int(bad[0])
        errs.append(f"row_offsets differ at {bad.size} rows, first row {i}: "
                    f"gpu {int(g_ro[i])} ref {int(r_ro[i])}")
        return errs
    if g_d.size != np.asarray(r_d).size:
        return [f"edge count {g_d.size} != {np.asarray(r_d).size}"]
    bad = np.nonzero(g_d != r_d)[0]
    if bad.size:
        errs.append(f"dst differs at {bad.size} positions, first {bad[:max_report].tolist()}")
        return errs
    if g_w is not None and r_w is not None:
        bad = np.nonzero(g_w != np.asarray(r_w, np.uint32))[0]
        if bad.size:
            deg = np.diff(r_ro).astype(np.int64)
            rows = np.repeat(np.arange(deg.size, dtype=np.uint64), deg)
            keys = _keys(rows[bad], g_d[bad])
            ok = np.zeros(bad.size, bool)
            if cand is not None:
                ok = cand.allowed(keys, g_w[bad])
            if not ok.all():
                b = bad[~ok]
                errs.append(f"weights differ at {b.size} non-candidate positions, first "
                            f"{b[:max_report].tolist()}")
    return errs


def compare_queries(src, dst, g_found, g_w, r_found, r_w, cand: Candidates | None = None,
                    max_report: int = 8):
    errs = []
    g_found = np.asarray(g_found, np.uint8)
    r_found = np.asarray(r_found, np.uint8)
    bad = np.nonzero(g_found != r_found)[0]
    if bad.size:
        errs.append(f"found differs at {bad.size} queries, first {bad[:max_report].tolist()}")
        return errs
    if g_w is not None:
        bad = np.nonzero(np.asarray(g_w, np.uint32) != np.asarray(r_w, np.uint32))[0]
        if bad.size:
            keys = _keys(np.asarray(src)[bad], np.asarray(dst)[bad])
            ok = np.zeros(bad.size, bool)
            if cand is not None:
                ok = cand.allowed(keys, np.asarray(g_w)[bad])
            if not ok.all():
                b = bad[~ok]
                errs.append(f"query weights differ at {b.size} non-candidate positions, first "
                            f"{b[:max_report].tolist()}")
    return errs


def check_invariants(row_offsets, dst, degrees=None):
    """North-star invariants on a canonical export: no duplicate edges (rows
    strictly increasing, fn3 P:L235-236), no self-loops (Alg1:L3), degree equals
    row length."""
    errs = []
    ro, d, _ = canonical(row_offsets, dst)
    deg = np.diff(ro).astype(np.int64)
    rows = np.repeat(np.arange(deg.size, dtype=np.int64), deg)
    if d.size > 1:
        same_row = rows[1:] == rows[:-1]
        dup = same_row & (d[1:] <= d[:-1])
        if dup.any():
            errs.append(f"duplicate/unsorted dst in {int(dup.sum())} places")
    loops = rows == d.astype(np.int64)
    if loops.any():
        errs.append(f"{int(loops.sum())} self-loops stored")
    if degrees is not None:
        dg = np.asarray(degrees, np.int64)
        if dg.shape != deg.shape or (dg != deg).any():
            errs.append("degree != row length")
    return errs
