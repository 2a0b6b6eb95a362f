"""Seeded synthetic workload generators (input production only).

This module is shared by the oracle harness and the GPU path and holds none of the
method's arithmetic: it draws counter-based random numbers (``gen.c``) and shapes
them into edge batches with the structure of the paper's workloads
(§V-A1; Tab. I; SURVEY.md §8(d) generator spec).

Every function returns numpy arrays (u32 SoA).  The C code is built on first use.
"""
from __future__ import annotations

import ctypes
import os
import subprocess
import threading

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SO = os.path.join(_HERE, "libdggen.so")
_lock = threading.Lock()
_lib = None

U32P = ctypes.POINTER(ctypes.c_uint32)
U64P = ctypes.POINTER(ctypes.c_uint64)


def build(force: bool = False) -> str:
    src = os.path.join(_HERE, "gen.c")
    if force or not os.path.exists(_SO) or os.path.getmtime(_SO) < os.path.getmtime(src):
        tmp = _SO + f".tmp{os.getpid()}"
        subprocess.check_call(["gcc", "-O3", "-std=c11", "-fopenmp", "-fPIC", "-shared",
                               "-o", tmp, src])
        os.replace(tmp, _SO)
    return _SO


def _L():
    global _lib
    with _lock:
        if _lib is None:
            lib = ctypes.CDLL(build())
            lib.wl_rng.restype = ctypes.c_uint64
            lib.wl_rng.argtypes = [ctypes.c_uint64] * 3
            lib.wl_uniform_edges.argtypes = [ctypes.c_uint64] * 5 + [U32P, U32P, U32P]
            lib.wl_uniform_u32.argtypes = [ctypes.c_uint64] * 5 + [U32P]
            lib.wl_uniform_index.argtypes = [ctypes.c_uint64] * 4 + [U64P]
            lib.wl_permute.restype = ctypes.c_uint32
            lib.wl_permute.argtypes = [ctypes.c_uint32, ctypes.c_int, ctypes.c_uint64]
            lib.wl_rmat_edges.argtypes = [ctypes.c_uint64, ctypes.c_uint64, ctypes.c_uint64,
                                          U64P, ctypes.c_uint64,
                                          ctypes.c_int, ctypes.c_double, ctypes.c_double,
                                          ctypes.c_double, ctypes.c_int, ctypes.c_uint64,
                                          U32P, U32P]
            lib.wl_grid_edges.restype = ctypes.c_uint64
            lib.wl_grid_edges.argtypes = [ctypes.c_uint64, ctypes.c_uint64, ctypes.c_uint64,
                                          ctypes.c_double, U32P, U32P]
            lib.wl_grid_heldout_edges.restype = ctypes.c_uint64
            lib.wl_grid_heldout_edges.argtypes = lib.wl_grid_edges.argtypes
            lib.wl_out_degrees.argtypes = [U32P, ctypes.c_uint64, ctypes.c_uint64, U32P]
            _lib = lib
    return _lib


def _p32(a):
    return None if a is None else a.ctypes.data_as(U32P)


def rng(seed: int, stream: int, index: int) -> int:
    return int(_L().wl_rng(seed, stream, index))


def uniform_edges(seed: int, stream: int, n: int, nv: int, weights: bool = True,
                  offset: int = 0):
    """Edges offset..offset+n-1 of a stream: src, dst uniform on [0, nv); weights
    uniform u32.  Any slice regenerates bit-identically."""
    s = np.empty(n, np.uint32)
    d = np.empty(n, np.uint32)
    w = np.empty(n, np.uint32) if weights else None
    _L().wl_uniform_edges(seed, stream, offset, n, nv, _p32(s), _p32(d), _p32(w))
    return s, d, w


def uniform_u32(seed: int, stream: int, n: int, bound: int = 0, offset: int = 0) -> np.ndarray:
    out = np.empty(n, np.uint32)
    _L().wl_uniform_u32(seed, stream, offset, n, bound, _p32(out))
    return out


def uniform_index(seed: int, stream: int, n: int, bound: int) -> np.ndarray:
    out = np.empty(n, np.uint64)
    _L().wl_uniform_index(seed, stream, n, bound, out.ctypes.data_as(U64P))
    return out


def permute(x: int, scale: int, seed: int) -> int:
    return int(_L().wl_permute(x, scale, seed))


GRAPH500 = (0.57, 0.19, 0.19)
LJLIKE = (0.50, 0.20, 0.20)


def rmat_edges(seed: int, stream: int, n: int, scale: int, abc=GRAPH500,
               permute_ids: bool = True, nv: int = 0, offset: int = 0, index=None):
    """R-MAT edges offset..offset+n-1 (or the edge ids in ``index``) over 2^scale
    vertices, rejected to [0, nv) if nv > 0."""
    if index is not None:
        index = np.ascontiguousarray(index, np.uint64)
        n = index.size
    s = np.empty(n, np.uint32)
    d = np.empty(n, np.uint32)
    a, b, c = abc
    _L().wl_rmat_edges(seed, stream, offset,
                       None if index is None else index.ctypes.data_as(U64P), n, scale,
                       a, b, c, int(permute_ids), nv, _p32(s), _p32(d))
    return s, d


def grid_edges(seed: int, rows: int, cols: int, p: float):
    """road-like lattice: each undirected lattice edge kept with prob. p, both directions."""
    L = _L()
    m = int(L.wl_grid_edges(seed, rows, cols, p, None, None))
    s = np.empty(m, np.uint32)
    d = np.empty(m, np.uint32)
    L.wl_grid_edges(seed, rows, cols, p, _p32(s), _p32(d))
    return s, d


def grid_heldout_edges(seed: int, rows: int, cols: int, p: float):
    """The lattice edges grid_edges() did not keep (both directions): road growth."""
    L = _L()
    m = int(L.wl_grid_heldout_edges(seed, rows, cols, p, None, None))
    s = np.empty(m, np.uint32)
    d = np.empty(m, np.uint32)
    L.wl_grid_heldout_edges(seed, rows, cols, p, _p32(s), _p32(d))
    return s, d


def out_degrees(src: np.ndarray, nv: int) -> np.ndarray:
    """Out-degree counts of an edge list (capacity hints)."""
    src = np.ascontiguousarray(src, np.uint32)
    deg = np.empty(nv, np.uint32)
    _L().wl_out_degrees(_p32(src), src.size, nv, _p32(deg))
    return deg


def weights(seed: int, stream: int, n: int, offset: int = 0) -> np.ndarray:
    return uniform_u32(seed, stream ^ 0x77777777, n, 0, offset)


def symmetrise(src: np.ndarray, dst: np.ndarray):
    """Both directions of every edge (undirected input shaping)."""
    return np.concatenate([src, dst]), np.concatenate([dst, src])
