"""ctypes binding of libdg.so (include/dg.h).  Argument marshalling only.

The library is built in-tree (``python -m paper_conf_ipps_awadapo20_b200.build`` or
``__graft_entry__.build()``).  There is no fallback: if libdg.so is missing or does not
export a symbol of include/dg.h, importing this module raises.
"""
from __future__ import annotations

import ctypes
import os

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.environ.get("DG_LIB_PATH") or os.path.join(_HERE, "libdg.so")

DG_OK = 0
DG_ERR_INVALID_ARGUMENT = 1
DG_ERR_VERTEX_OUT_OF_RANGE = 2
DG_ERR_OUT_OF_MEMORY = 3
DG_ERR_CUDA = 4
DG_ERR_NCCL = 5
DG_ERR_BAD_STATE = 6
DG_ERR_UNSUPPORTED = 7
DG_FLAG_NO_TOMBSTONE_REUSE = 1
DG_FLAG_FORCE_ROUTER = 2
DG_FLAG_SET = 4
DG_FLAG_ADAPTIVE = 8
DG_FLAG_COPY_EXCHANGE = 16

VP = ctypes.c_void_p
U64 = ctypes.c_uint64
U32 = ctypes.c_uint32
P_U64 = ctypes.POINTER(ctypes.c_uint64)


class dg_config(ctypes.Structure):
    _fields_ = [
        ("struct_size", ctypes.c_uint32),
        ("load_factor", ctypes.c_float),
        ("bucket_bytes", ctypes.c_uint32),
        ("directed", ctypes.c_uint32),
        ("pool_bytes", ctypes.c_uint64),
        ("device", ctypes.c_int32),
        ("rank", ctypes.c_int32),
        ("nranks", ctypes.c_int32),
        ("flags", ctypes.c_uint32),
        ("nccl_unique_id", ctypes.c_void_p),
        ("group", ctypes.c_void_p),
    ]


class dg_stats(ctypes.Structure):
    _fields_ = [
        ("local_rows", ctypes.c_uint64),
        ("base_buckets", ctypes.c_uint64),
        ("overflow_buckets", ctypes.c_uint64),
        ("free_buckets", ctypes.c_uint64),
        ("pool_buckets", ctypes.c_uint64),
        ("bump_buckets", ctypes.c_uint64),
        ("live_pairs", ctypes.c_uint64),
        ("tombstones", ctypes.c_uint64),
        ("max_chain", ctypes.c_uint64),
        ("pool_bytes", ctypes.c_uint64),
        ("load_factor", ctypes.c_double),
        ("utilization", ctypes.c_double),
        ("exchange", ctypes.c_uint64),
        ("table_bytes", ctypes.c_uint64),
        ("bump_bytes", ctypes.c_uint64),
    ]


class dg_profile(ctypes.Structure):
    _fields_ = [
        ("launches", ctypes.c_uint64),
        ("kernel_launches", ctypes.c_uint64 * 5),
        ("kernel_ms", ctypes.c_double * 5),
        ("last_count", ctypes.c_uint64),
    ]


class dg_invariants(ctypes.Structure):
    _fields_ = [(n, ctypes.c_uint64) for n in (
        "rows", "chains", "buckets", "live_pairs", "tombstones", "empty_not_suffix",
        "misplaced_keys", "duplicate_keys", "self_loops", "keys_out_of_range", "owner_mismatch",
        "degree_mismatch", "broken_chains", "dup_unchecked_chains", "first_bad_row")]


# (name, restype, argtypes) — every entry point declared in include/dg.h
SIGNATURES = [
    ("dg_config_init", None, [ctypes.POINTER(dg_config)]),
    ("dg_status_string", ctypes.c_char_p, [ctypes.c_int]),
    ("dg_get_unique_id", ctypes.c_int, [VP]),
    ("dg_group_create", ctypes.c_int, [ctypes.c_int32, ctypes.POINTER(VP)]),
    ("dg_group_destroy", ctypes.c_int, [VP]),
    ("dg_create", ctypes.c_int, [ctypes.POINTER(dg_config), U64, VP, VP, ctypes.POINTER(VP)]),
    ("dg_destroy", ctypes.c_int, [VP]),
    ("dg_num_vertices", ctypes.c_int, [VP, P_U64, P_U64]),
    ("dg_insert_edges", ctypes.c_int, [VP, VP, VP, VP, U64, P_U64, VP]),
    ("dg_delete_edges", ctypes.c_int, [VP, VP, VP, U64, P_U64, VP]),
    ("dg_query_edges", ctypes.c_int, [VP, VP, VP, U64, VP, VP, VP]),
    ("dg_insert_vertices", ctypes.c_int, [VP, VP, U64, VP, VP]),
    ("dg_delete_vertices", ctypes.c_int, [VP, VP, U64, VP]),
    ("dg_export_adjacency", ctypes.c_int, [VP, VP, VP, VP, U64, P_U64, VP]),
    ("dg_degrees", ctypes.c_int, [VP, VP, VP]),
    ("dg_get_stats", ctypes.c_int, [VP, ctypes.POINTER(dg_stats), VP]),
    ("dg_batch_status", ctypes.c_int, [VP, VP]),
    ("dg_triangle_count", ctypes.c_int, [VP, U32, U32, P_U64, VP]),
    ("dg_flush_tombstones", ctypes.c_int, [VP, P_U64, VP]),
    ("dg_check_invariants", ctypes.c_int, [VP, ctypes.POINTER(dg_invariants), VP]),
    ("dg_profile_enable", ctypes.c_int, [VP, ctypes.c_int]),
    ("dg_profile_read", ctypes.c_int, [VP, ctypes.POINTER(dg_profile), VP]),
]


def load(path: str = LIB_PATH):
    if not os.path.exists(path):
        raise ImportError(
            f"{path} not found: build it with __graft_entry__.build() or "
            "`python -m paper_conf_ipps_awadapo20_b200.build` (there is no CPU fallback)")
    lib = ctypes.CDLL(path)
    for name, res, args in SIGNATURES:
        fn = getattr(lib, name)  # AttributeError if the symbol is missing
        fn.restype = res
        fn.argtypes = args
    return lib


lib = load()


class DGError(RuntimeError):
    def __init__(self, status: int, what: str = ""):
        self.status = status
        name = lib.dg_status_string(status).decode()
        super().__init__(f"{what}: {name}" if what else name)


def check(status: int, what: str = ""):
    if status != DG_OK:
        raise DGError(status, what)
