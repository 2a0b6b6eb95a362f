"""Python handle over the C ABI (include/dg.h).  Argument marshalling only: every
step of the path runs in libdg.so's sm_100a kernels.

Arrays may be CUDA torch tensors (the calls are then stream-ordered and return
immediately, like the C ABI with device buffers), CPU torch tensors or numpy arrays
(host buffers: the library stages them and the call is synchronous).  IDs and
weights are 32-bit (uint32 or int32 bit patterns).
"""
from __future__ import annotations

import ctypes

import numpy as np
import torch

from . import _lib
from ._lib import DGError, check, dg_config, dg_profile, dg_stats, lib

_U32_OK = (torch.int32, torch.uint32)


def _ptr(a, n_expected=None, dtype_bytes=4, what="array"):
    """-> (pointer int, length, is_cuda)"""
    if a is None:
        return None, 0, False
    if type(a) is torch.Tensor or isinstance(a, torch.Tensor):
        if a.element_size() != dtype_bytes:
            raise TypeError(f"{what}: expected {dtype_bytes}-byte elements, got {a.dtype}")
        if not a.is_contiguous():
            raise ValueError(f"{what}: tensor must be contiguous")
        n = a.numel()
        return (a.data_ptr() if n else None), n, a.is_cuda
    arr = np.asarray(a)
    if arr.dtype.itemsize != dtype_bytes or not arr.flags.c_contiguous:
        raise TypeError(f"{what}: expected a contiguous {dtype_bytes}-byte numpy array")
    n = arr.size
    return (arr.ctypes.data if n else None), n, False


def _as_u32(a):
    """torch tensors pass through (int32/uint32); anything else becomes contiguous uint32 numpy."""
    if a is None:
        return None
    if type(a) is torch.Tensor or isinstance(a, torch.Tensor):
        if a.dtype not in _U32_OK:
            raise TypeError(f"expected int32/uint32 tensor, got {a.dtype}")
        return a if a.is_contiguous() else a.contiguous()
    return np.ascontiguousarray(np.asarray(a).astype(np.uint32, copy=False))


_HAS_CUDA = None
_raw_stream = getattr(torch._C, "_cuda_getCurrentRawStream", None)
_cur_dev = getattr(torch._C, "_cuda_getDevice", None) or torch.cuda.current_device


def _stream(stream):
    """cudaStream_t handle of `stream`, else of torch's current stream (legacy 0 without CUDA)."""
    global _HAS_CUDA
    if stream is not None:
        return stream.cuda_stream if hasattr(stream, "cuda_stream") else int(stream)
    if _HAS_CUDA is None:
        _HAS_CUDA = torch.cuda.is_available()
    if not _HAS_CUDA:
        return 0
    if _raw_stream is not None:  # (the current stream without building a Stream object)
        return _raw_stream(_cur_dev())
    return torch.cuda.current_stream().cuda_stream


class Graph:
    """A dynamic graph: one hash table per vertex (§III-IV).

    Parameters mirror ``dg_config`` (include/dg.h).  ``degree_hints`` (length
    ``num_vertices``) sizes each vertex's initial table; ``None`` gives
    every vertex one bucket.  ``set_variant`` stores keys only (twice
    as many per bucket): weights are ignored on insert and read as 0.
    ``adaptive`` (or ``bucket_bytes=0``) gives each vertex a bucket size (32 / 64 /
    128 B) chosen from its degree (DG_FLAG_ADAPTIVE).
    """

    def __init__(self, num_vertices: int, degree_hints=None, *, load_factor: float = 0.7,
                 bucket_bytes: int = 128, directed: bool = True, pool_bytes: int = 0,
                 device: int | None = None, rank: int = 0, nranks: int = 1,
                 nccl_unique_id: bytes | None = None, reuse_tombstones: bool = True,
                 force_router: bool = False, set_variant: bool = False,
                 adaptive: bool = False, group: "RankGroup | None" = None,
                 copy_exchange: bool = False, stream=None):
        if bucket_bytes == 0:
            adaptive, bucket_bytes = True, 128
        cfg = dg_config()
        lib.dg_config_init(ctypes.byref(cfg))
        cfg.load_factor = float(load_factor)
        cfg.bucket_bytes = int(bucket_bytes)
        cfg.directed = 1 if directed else 0
        cfg.pool_bytes = int(pool_bytes)
        if device is None:
            device = torch.cuda.current_device() if torch.cuda.is_available() else -1
        cfg.device = int(device)
        cfg.rank = int(rank)
        cfg.nranks = int(nranks)
        cfg.flags = (0 if reuse_tombstones else _lib.DG_FLAG_NO_TOMBSTONE_REUSE) | \
            (_lib.DG_FLAG_FORCE_ROUTER if force_router else 0) | \
            (_lib.DG_FLAG_SET if set_variant else 0) | \
            (_lib.DG_FLAG_ADAPTIVE if adaptive else 0) | \
            (_lib.DG_FLAG_COPY_EXCHANGE if copy_exchange else 0)
        self._group = group  # keeps the group alive while the handle exists
        if group is not None:
            cfg.group = group.handle.value
        self._uid = None
        if nccl_unique_id is not None:
            self._uid = ctypes.create_string_buffer(bytes(nccl_unique_id), 128)
            cfg.nccl_unique_id = ctypes.cast(self._uid, ctypes.c_void_p)
        hints = _as_u32(degree_hints)
        hp, hn, _ = _ptr(hints, what="degree_hints")
        if hints is not None and hn != num_vertices:
            raise ValueError("degree_hints must have num_vertices entries")
        self.device = torch.device("cuda", int(device)) if device >= 0 else None
        self._h = ctypes.c_void_p()
        self.directed = directed
        self.bucket_bytes = bucket_bytes
        self.set_variant = set_variant
        self.adaptive = adaptive
        self.rank, self.nranks = rank, nranks
        check(lib.dg_create(ctypes.byref(cfg), int(num_vertices), hp, _stream(stream),
                            ctypes.byref(self._h)), "dg_create")

    # ------------------------------------------------------------------ admin --
    def close(self):
        if getattr(self, "_h", None) and self._h.value:
            lib.dg_destroy(self._h)
            self._h = ctypes.c_void_p()

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass

    def __enter__(self):
        return self

    def __exit__(self, *exc):
        self.close()

    @property
    def handle(self):
        return self._h

    @property
    def num_vertices(self) -> int:
        nv = ctypes.c_uint64()
        check(lib.dg_num_vertices(self._h, ctypes.byref(nv), None))
        return nv.value

    @property
    def local_rows(self) -> int:
        r = ctypes.c_uint64()
        check(lib.dg_num_vertices(self._h, None, ctypes.byref(r)))
        return r.value

    # ------------------------------------------------------------ edge batches --
    def insert_edges(self, src, dst, weight=None, *, count: bool = False, stream=None):
        """Alg. 1.  Returns the number of new keys if ``count``."""
        src, dst, weight = _as_u32(src), _as_u32(dst), _as_u32(weight)
        ps, n, _ = _ptr(src, what="src")
        pd, nd, _ = _ptr(dst, what="dst")
        pw, nw, _ = _ptr(weight, what="weight")
        if nd != n or (weight is not None and nw != n):
            raise ValueError("src/dst/weight lengths differ")
        out = ctypes.c_uint64(0)
        check(lib.dg_insert_edges(self._h, ps, pd, pw, n, ctypes.byref(out) if count else None,
                                  _stream(stream)), "dg_insert_edges")
        return out.value if count else None

    def delete_edges(self, src, dst, *, count: bool = False, stream=None):
        """Delete by key.  Returns the number removed if ``count``."""
        src, dst = _as_u32(src), _as_u32(dst)
        ps, n, _ = _ptr(src, what="src")
        pd, nd, _ = _ptr(dst, what="dst")
        if nd != n:
            raise ValueError("src/dst lengths differ")
        out = ctypes.c_uint64(0)
        check(lib.dg_delete_edges(self._h, ps, pd, n, ctypes.byref(out) if count else None,
                                  _stream(stream)), "dg_delete_edges")
        return out.value if count else None

    def query_edges(self, src, dst, *, weights: bool = True, found_out=None, weight_out=None,
                    stream=None):
        """edgeExist -> (found uint8, weight uint32 or None)."""
        src, dst = _as_u32(src), _as_u32(dst)
        ps, n, cuda = _ptr(src, what="src")
        pd, nd, _ = _ptr(dst, what="dst")
        if nd != n:
            raise ValueError("src/dst lengths differ")
        if found_out is None:
            if cuda:
                found_out = torch.empty(n, dtype=torch.uint8, device=src.device)
                if weights:
                    weight_out = torch.empty(n, dtype=torch.uint32, device=src.device)
            else:
                found_out = np.empty(n, np.uint8)
                if weights:
                    weight_out = np.empty(n, np.uint32)
        pf, _, _ = _ptr(found_out, dtype_bytes=1, what="found")
        pw, _, _ = _ptr(weight_out, what="weight_out")
        check(lib.dg_query_edges(self._h, ps, pd, n, pf, pw, _stream(stream)), "dg_query_edges")
        return found_out, weight_out

    # --------------------------------------------------------- vertex batches --
    def insert_vertices(self, ids, degree_hints=None, stream=None):
        ids, hints = _as_u32(ids), _as_u32(degree_hints)
        pi, n, _ = _ptr(ids, what="ids")
        ph, nh, _ = _ptr(hints, what="degree_hints")
        if hints is not None and nh != n:
            raise ValueError("ids/degree_hints lengths differ")
        check(lib.dg_insert_vertices(self._h, pi, n, ph, _stream(stream)), "dg_insert_vertices")

    def delete_vertices(self, ids, stream=None):
        ids = _as_u32(ids)
        pi, n, _ = _ptr(ids, what="ids")
        check(lib.dg_delete_vertices(self._h, pi, n, _stream(stream)), "dg_delete_vertices")

    # ------------------------------------------------------------------ reads --
    def export(self, device: bool = True, stream=None):
        """Adjacency lists of the local rows as CSR (row_offsets u64, dst u32, w u32).
        Rows are unsorted within themselves."""
        rows = self.local_rows
        m = ctypes.c_uint64()
        st = _stream(stream)
        if device and self.device is not None:
            ro = torch.empty(rows + 1, dtype=torch.uint64, device=self.device)
            pro = ro.data_ptr()
        else:
            ro = np.empty(rows + 1, np.uint64)
            pro = ro.ctypes.data
        check(lib.dg_export_adjacency(self._h, pro, None, None, 0, ctypes.byref(m), st),
              "dg_export_adjacency")
        n = m.value
        if device and self.device is not None:
            d = torch.empty(max(n, 1), dtype=torch.uint32, device=self.device)
            w = torch.empty(max(n, 1), dtype=torch.uint32, device=self.device)
            pd, pw = d.data_ptr(), w.data_ptr()
        else:
            d = np.empty(max(n, 1), np.uint32)
            w = np.empty(max(n, 1), np.uint32)
            pd, pw = d.ctypes.data, w.ctypes.data
        check(lib.dg_export_adjacency(self._h, pro, pd, pw, max(n, 1), ctypes.byref(m), st),
              "dg_export_adjacency")
        return ro, d[:n], w[:n]

    def export_numpy(self):
        ro, d, w = self.export(device=False)
        return ro, d, w

    def degrees(self, device: bool = True, stream=None):
        rows = self.local_rows
        if device and self.device is not None:
            out = torch.empty(max(rows, 1), dtype=torch.uint32, device=self.device)
            p = out.data_ptr()
        else:
            out = np.empty(max(rows, 1), np.uint32)
            p = out.ctypes.data
        check(lib.dg_degrees(self._h, p, _stream(stream)), "dg_degrees")
        return out[:rows]

    def stats(self, stream=None) -> dict:
        s = dg_stats()
        check(lib.dg_get_stats(self._h, ctypes.byref(s), _stream(stream)), "dg_get_stats")
        return {name: getattr(s, name) for name, _ in dg_stats._fields_}

    def batch_status(self, stream=None) -> int:
        """0, or DG_ERR_VERTEX_OUT_OF_RANGE if an async batch since the last call was rejected."""
        st = lib.dg_batch_status(self._h, _stream(stream))
        if st not in (_lib.DG_OK, _lib.DG_ERR_VERTEX_OUT_OF_RANGE):
            check(st, "dg_batch_status")
        return st

    VIOLATIONS = ("empty_not_suffix", "misplaced_keys", "duplicate_keys", "self_loops",
                  "keys_out_of_range", "owner_mismatch", "degree_mismatch", "broken_chains")

    def check_invariants(self, stream=None) -> dict:
        """Structural invariants of the tables (dg_check_invariants): violation counts
        plus what was walked.  ``violations`` sums the violation counters."""
        r = _lib.dg_invariants()
        check(lib.dg_check_invariants(self._h, ctypes.byref(r), _stream(stream)),
              "dg_check_invariants")
        out = {name: getattr(r, name) for name, _ in _lib.dg_invariants._fields_}
        out["violations"] = sum(out[k] for k in self.VIOLATIONS)
        return out

    # ------------------------------------------------------- instrumentation --
    PROFILE_KINDS = ("insert", "delete", "query", "vertex_purge", "tc")

    def profile_enable(self, enable: bool = True):
        check(lib.dg_profile_enable(self._h, 1 if enable else 0), "dg_profile_enable")

    def profile_read(self, stream=None) -> dict:
        p = dg_profile()
        check(lib.dg_profile_read(self._h, ctypes.byref(p), _stream(stream)), "dg_profile_read")
        return {"launches": p.launches, "last_count": p.last_count,
                "kernel_launches": dict(zip(self.PROFILE_KINDS, list(p.kernel_launches))),
                "kernel_ms": dict(zip(self.PROFILE_KINDS, list(p.kernel_ms)))}

    def flush_tombstones(self, stream=None) -> int:
        """Rebuild every table holding tombstones compactly; returns the
        number of tables rebuilt.  The logical graph is unchanged."""
        n = ctypes.c_uint64(0)
        check(lib.dg_flush_tombstones(self._h, ctypes.byref(n), _stream(stream)),
              "dg_flush_tombstones")
        return n.value

    def triangle_count(self, part: int = 0, nparts: int = 1, stream=None) -> int:
        """Triangles by hash intersection (§VI-C); part/nparts split the work by u mod nparts."""
        c = ctypes.c_uint64()
        check(lib.dg_triangle_count(self._h, part, nparts, ctypes.byref(c), _stream(stream)),
              "dg_triangle_count")
        return c.value


class RankGroup:
    """In-process rank group (``dg_group_create``): ``nranks`` host threads of this
    process act as the ranks of a sharded graph, each creating its own ``Graph(...,
    rank=r, nranks=nranks, group=grp)`` and calling every collective with its own slice
    on its own (non-blocking) stream.  ctypes releases the GIL during library calls, so
    Python threads run the ranks concurrently."""

    def __init__(self, nranks: int):
        self._h = ctypes.c_void_p()
        check(lib.dg_group_create(int(nranks), ctypes.byref(self._h)), "dg_group_create")
        self.nranks = int(nranks)

    @property
    def handle(self):
        return self._h

    def close(self):
        if getattr(self, "_h", None) and self._h.value:
            lib.dg_group_destroy(self._h)
            self._h = ctypes.c_void_p()

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass


def get_unique_id() -> bytes:
    buf = ctypes.create_string_buffer(128)
    check(lib.dg_get_unique_id(buf), "dg_get_unique_id")
    return buf.raw


__all__ = ["Graph", "RankGroup", "DGError", "get_unique_id"]
