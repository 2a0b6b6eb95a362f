"""Helpers shared by the GPU parity tests (-m gpu)."""
from __future__ import annotations

import numpy as np
import torch

from oracle import Oracle
from oracle.compare import Candidates, check_invariants, compare_export, compare_queries


def cuda(a):
    if a is None:
        return None
    return torch.from_numpy(np.ascontiguousarray(a, np.uint32)).to("cuda")


class GpuAdapter:
    """Oracle-shaped facade over the CUDA path (for the golden-script runner)."""

    def __init__(self, n, directed=True, **kw):
        from paper_conf_ipps_awadapo20_b200 import Graph
        self.g = Graph(n, directed=directed, **kw)

    def _call(self, fn, *a, **k):
        from paper_conf_ipps_awadapo20_b200 import DGError
        try:
            return 0, fn(*a, **k)
        except DGError as e:
            return e.status, 0

    def insert_edges(self, s, d, w=None):
        return self._call(self.g.insert_edges, cuda(s), cuda(d), cuda(w), count=True)

    def delete_edges(self, s, d):
        return self._call(self.g.delete_edges, cuda(s), cuda(d), count=True)

    def query_edges(self, s, d):
        f, w = self.g.query_edges(cuda(s), cuda(d))
        st = self.g.batch_status()
        return st, f.cpu().numpy(), w.cpu().numpy()

    def delete_vertices(self, ids):
        self.g.delete_vertices(cuda(ids))
        return self.g.batch_status()

    def insert_vertices(self, ids):
        st, _ = self._call(self.g.insert_vertices, cuda(ids))
        return st

    def export(self):
        ro, d, w = self.g.export()
        return ro.cpu().numpy(), d.cpu().numpy(), w.cpu().numpy()


def check_against_oracle(g, o: Oracle, where=""):
    """Full export + degree + invariant comparison of a Graph with the oracle."""
    ro, d, w = g.export()
    ro, d, w = ro.cpu().numpy(), d.cpu().numpy(), w.cpu().numpy()
    ref = o.export()
    cand = Candidates(*o.candidates())
    errs = compare_export((ro, d, w), ref, cand)
    assert not errs, f"{where}: {errs}"
    deg = g.degrees().cpu().numpy()
    assert np.array_equal(deg, o.degrees()), f"{where}: degrees differ"
    errs = check_invariants(ro, d, deg)
    assert not errs, f"{where}: {errs}"
    assert_table_invariants(g, where)
    return cand


def assert_table_invariants(g, where=""):
    """dg_check_invariants: EMPTY-suffix chains, keys in their hash chain, no duplicate,
    owner words, degree == live keys, chains end."""
    inv = g.check_invariants()
    assert inv["violations"] == 0, f"{where}: table invariants violated: {inv}"
    return inv


def check_queries(g, o: Oracle, qs, qd, cand=None, where=""):
    f, w = g.query_edges(cuda(qs), cuda(qd))
    st, rf, rw = o.query_edges(qs, qd)
    if cand is None:
        cand = Candidates(*o.candidates())
    errs = compare_queries(qs, qd, f.cpu().numpy(), w.cpu().numpy(), rf, rw, cand)
    assert not errs, f"{where}: {errs}"


def gpu_invariants(ro, dst, deg):
    """Size-independent invariants on a full export, computed with torch on the GPU
    (test-side checking only): no duplicate (u, v), no self-loop, degree == row length.
    ro: uint64 [V+1], dst: uint32 [E], deg: uint32 [V] (device tensors)."""
    ro64 = ro.to(torch.int64)
    lens = ro64[1:] - ro64[:-1]
    errs = []
    if not torch.equal(lens, deg.to(torch.int64)):
        errs.append("degree != row length")
    rows = torch.repeat_interleave(torch.arange(lens.numel(), device=ro.device), lens)
    d64 = dst.to(torch.int64)
    if bool((rows == d64).any()):
        errs.append("self-loop stored")
    keys = torch.sort((rows << 32) | d64).values
    if keys.numel() > 1 and bool((keys[1:] == keys[:-1]).any()):
        errs.append("duplicate edge stored")
    return errs


def distinct_nonloop(s, d):
    """number of distinct (u, v) keys with u != v (torch.unique on the GPU)."""
    ts = torch.from_numpy(np.ascontiguousarray(s).astype(np.int64)).cuda()
    td = torch.from_numpy(np.ascontiguousarray(d).astype(np.int64)).cuda()
    k = (ts << 32) | td
    k = k[ts != td]
    return int(torch.unique(k).numel())
