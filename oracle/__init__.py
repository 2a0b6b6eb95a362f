"""CPU oracle — TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s ``cpu_baseline`` /
``--impl reference`` leg may import this package.  It shares no code with the CUDA
path (``paper_conf_ipps_awadapo20_b200``) and neither imports the other.

``Oracle`` wraps ``oracle.cpp`` (one ``std::unordered_map`` per vertex, the plain
definition of the paper's graph, §II-A) through ctypes.
``compare`` holds the canonicalising comparator.
"""
from __future__ import annotations

import ctypes
import os
import subprocess
import threading

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SO = os.path.join(_HERE, "liboracle.so")
_lock = threading.Lock()
_lib = None

OK = 0
ERR_INVALID_ARGUMENT = 1
ERR_VERTEX_OUT_OF_RANGE = 2

U8P = ctypes.POINTER(ctypes.c_uint8)
U32P = ctypes.POINTER(ctypes.c_uint32)
U64P = ctypes.POINTER(ctypes.c_uint64)
VP = ctypes.c_void_p


def build(force: bool = False) -> str:
    src = os.path.join(_HERE, "oracle.cpp")
    if force or not os.path.exists(_SO) or os.path.getmtime(_SO) < os.path.getmtime(src):
        tmp = _SO + f".tmp{os.getpid()}"
        subprocess.check_call(["g++", "-O2", "-std=c++17", "-pthread", "-fPIC", "-shared", "-o", tmp,
                               src])
        os.replace(tmp, _SO)
    return _SO


def _L():
    global _lib
    with _lock:
        if _lib is None:
            lib = ctypes.CDLL(build())
            lib.orc_create.restype = VP
            lib.orc_create.argtypes = [ctypes.c_uint64, ctypes.c_int]
            lib.orc_destroy.argtypes = [VP]
            lib.orc_set_threads.restype = ctypes.c_int
            lib.orc_set_threads.argtypes = [VP, ctypes.c_uint]
            lib.orc_num_vertices.restype = ctypes.c_uint64
            lib.orc_num_vertices.argtypes = [VP]
            lib.orc_insert_edges.restype = ctypes.c_int
            lib.orc_insert_edges.argtypes = [VP, U32P, U32P, U32P, ctypes.c_uint64, U64P]
            lib.orc_delete_edges.restype = ctypes.c_int
            lib.orc_delete_edges.argtypes = [VP, U32P, U32P, ctypes.c_uint64, U64P]
            lib.orc_query_edges.restype = ctypes.c_int
            lib.orc_query_edges.argtypes = [VP, U32P, U32P, ctypes.c_uint64, U8P, U32P]
            lib.orc_delete_vertices.restype = ctypes.c_int
            lib.orc_delete_vertices.argtypes = [VP, U32P, ctypes.c_uint64]
            lib.orc_insert_vertices.restype = ctypes.c_int
            lib.orc_insert_vertices.argtypes = [VP, U32P, ctypes.c_uint64]
            lib.orc_num_edges.restype = ctypes.c_uint64
            lib.orc_num_edges.argtypes = [VP]
            lib.orc_export.argtypes = [VP, U64P, U32P, U32P]
            lib.orc_degrees.argtypes = [VP, U32P]
            lib.orc_candidates.restype = ctypes.c_uint64
            lib.orc_candidates.argtypes = [VP, U32P, U32P, U32P, ctypes.c_uint64]
            lib.orc_triangle_count.restype = ctypes.c_uint64
            lib.orc_triangle_count.argtypes = [VP]
            lib.orc_initial_buckets.restype = ctypes.c_uint64
            lib.orc_initial_buckets.argtypes = [ctypes.c_uint64] * 3
            _lib = lib
    return _lib


def _u32(a):
    if a is None:
        return None, None
    a = np.ascontiguousarray(a, dtype=np.uint32)
    return a, a.ctypes.data_as(U32P)


def default_threads() -> int:
    env = os.environ.get("ORACLE_THREADS")
    if env:
        return max(1, int(env))
    try:
        n = len(os.sched_getaffinity(0))
    except AttributeError:
        n = os.cpu_count() or 1
    return max(1, min(n, 16))


def initial_buckets(hint: int, lf_milli: int = 700, bucket_capacity: int = 15) -> int:
    """ceil(|A_u| / (lf*Bc)), 1 if unknown — PAPER.md §IV-A2 P:L411-414."""
    return int(_L().orc_initial_buckets(hint, lf_milli, bucket_capacity))


class Oracle:
    """One ``std::unordered_map`` per vertex; batches applied in order."""

    def __init__(self, num_vertices: int, directed: bool = True, threads: int | None = None):
        """``threads``: host threads (thread t owns the vertices u with
        u % T == t, so every vertex's ops keep their batch order; results do not
        depend on T).  Default: $ORACLE_THREADS, else min(usable CPUs, 16)."""
        self._L = _L()
        self.h = self._L.orc_create(num_vertices, int(directed))
        if not self.h:
            raise ValueError("num_vertices out of range")
        self.directed = directed
        self.threads = default_threads() if threads is None else int(threads)
        if self._L.orc_set_threads(self.h, self.threads) != OK:
            raise ValueError("threads out of range")

    def __del__(self):
        h = getattr(self, "h", None)
        if h:
            self._L.orc_destroy(h)
            self.h = None

    @property
    def num_vertices(self) -> int:
        return int(self._L.orc_num_vertices(self.h))

    def insert_edges(self, src, dst, w=None):
        s, ps = _u32(src)
        d, pd = _u32(dst)
        ww, pw = _u32(w)
        out = ctypes.c_uint64(0)
        st = self._L.orc_insert_edges(self.h, ps, pd, pw, s.size, ctypes.byref(out))
        return st, int(out.value)

    def delete_edges(self, src, dst):
        s, ps = _u32(src)
        d, pd = _u32(dst)
        out = ctypes.c_uint64(0)
        st = self._L.orc_delete_edges(self.h, ps, pd, s.size, ctypes.byref(out))
        return st, int(out.value)

    def query_edges(self, src, dst):
        s, ps = _u32(src)
        d, pd = _u32(dst)
        found = np.zeros(s.size, np.uint8)
        weight = np.zeros(s.size, np.uint32)
        st = self._L.orc_query_edges(self.h, ps, pd, s.size, found.ctypes.data_as(U8P),
                                     weight.ctypes.data_as(U32P))
        return st, found, weight

    def delete_vertices(self, ids):
        a, p = _u32(ids)
        return self._L.orc_delete_vertices(self.h, p, a.size)

    def insert_vertices(self, ids):
        a, p = _u32(ids)
        return self._L.orc_insert_vertices(self.h, p, a.size)

    def num_edges(self) -> int:
        return int(self._L.orc_num_edges(self.h))

    def export(self):
        """(row_offsets u64[V+1], dst u32[E], w u32[E]) with rows sorted by dst."""
        nv = self.num_vertices
        m = self.num_edges()
        ro = np.zeros(nv + 1, np.uint64)
        d = np.zeros(m, np.uint32)
        w = np.zeros(m, np.uint32)
        self._L.orc_export(self.h, ro.ctypes.data_as(U64P), d.ctypes.data_as(U32P),
                           w.ctypes.data_as(U32P))
        return ro, d, w

    def degrees(self) -> np.ndarray:
        out = np.zeros(self.num_vertices, np.uint32)
        self._L.orc_degrees(self.h, out.ctypes.data_as(U32P))
        return out

    def candidates(self):
        """Q1 candidate triples (u, v, w) as three u32 arrays."""
        k = int(self._L.orc_candidates(self.h, None, None, None, 0))
        u = np.zeros(k, np.uint32)
        v = np.zeros(k, np.uint32)
        w = np.zeros(k, np.uint32)
        self._L.orc_candidates(self.h, u.ctypes.data_as(U32P), v.ctypes.data_as(U32P),
                               w.ctypes.data_as(U32P), k)
        return u, v, w

    def triangle_count(self) -> int:
        return int(self._L.orc_triangle_count(self.h))
