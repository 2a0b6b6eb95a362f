"""C-ABI checks that need no GPU: libdg.so loads, exports every entry point that
include/dg.h declares, the ctypes structs match the C layout, and host-detectable
argument errors return before any device work."""
import ctypes
import os
import re
import subprocess

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
HEADER = os.path.join(ROOT, "include", "dg.h")


def _declared():
    txt = open(HEADER).read()
    return sorted(set(re.findall(r"DG_API\s+[\w\s\*]+?\b(dg_\w+)\s*\(", txt)))


def test_header_declares_the_boundary():
    names = _declared()
    for need in ["dg_create", "dg_destroy", "dg_insert_edges", "dg_delete_edges", "dg_query_edges",
                 "dg_insert_vertices", "dg_delete_vertices", "dg_export_adjacency"]:
        assert need in names


def test_library_exports_every_declared_symbol():
    from paper_conf_ipps_awadapo20_b200 import _lib
    lib = ctypes.CDLL(_lib.LIB_PATH)
    for name in _declared():
        assert hasattr(lib, name), name
    bound = {n for n, _, _ in _lib.SIGNATURES}
    assert bound == set(_declared())


def test_library_has_sm100a_code():
    from paper_conf_ipps_awadapo20_b200 import _lib
    out = subprocess.run(["/usr/local/cuda/bin/cuobjdump", "--list-elf", _lib.LIB_PATH],
                         capture_output=True, text=True).stdout
    assert "sm_100a" in out


def test_struct_layout_matches_c(tmp_path):
    from paper_conf_ipps_awadapo20_b200._lib import dg_config, dg_stats
    src = tmp_path / "sz.c"
    src.write_text('#include "dg.h"\n#include <stdio.h>\n#include <stddef.h>\n'
                   'int main(){printf("%zu %zu %zu %zu %zu\\n", sizeof(dg_config), sizeof(dg_stats),'
                   ' offsetof(dg_config, nccl_unique_id), offsetof(dg_stats, load_factor),'
                   ' offsetof(dg_config, group));}\n')
    exe = tmp_path / "sz"
    subprocess.check_call(["gcc", "-I", os.path.join(ROOT, "include"), str(src), "-o", str(exe)])
    c = [int(x) for x in subprocess.check_output([str(exe)]).split()]
    assert c == [ctypes.sizeof(dg_config), ctypes.sizeof(dg_stats),
                 dg_config.nccl_unique_id.offset, dg_stats.load_factor.offset,
                 dg_config.group.offset]


def test_config_defaults_and_status_strings():
    from paper_conf_ipps_awadapo20_b200._lib import dg_config, lib
    c = dg_config()
    lib.dg_config_init(ctypes.byref(c))
    assert c.struct_size == ctypes.sizeof(dg_config)
    assert abs(c.load_factor - 0.7) < 1e-6
    assert c.bucket_bytes == 128 and c.directed == 1 and c.nranks == 1
    for code in range(8):
        assert lib.dg_status_string(code).startswith(b"DG_")


def test_host_detectable_errors_without_gpu():
    from paper_conf_ipps_awadapo20_b200 import _lib
    lib = _lib.lib
    c = _lib.dg_config()
    lib.dg_config_init(ctypes.byref(c))
    h = ctypes.c_void_p()
    bad = _lib.dg_config()
    lib.dg_config_init(ctypes.byref(bad))
    bad.bucket_bytes = 48
    assert lib.dg_create(ctypes.byref(bad), 10, None, None, ctypes.byref(h)) == _lib.DG_ERR_INVALID_ARGUMENT
    bad.bucket_bytes = 128
    bad.load_factor = 0.0
    assert lib.dg_create(ctypes.byref(bad), 10, None, None, ctypes.byref(h)) == _lib.DG_ERR_INVALID_ARGUMENT
    bad.load_factor = 0.7
    bad.nranks = 2  # multi-rank without a NCCL id
    assert lib.dg_create(ctypes.byref(bad), 10, None, None, ctypes.byref(h)) == _lib.DG_ERR_INVALID_ARGUMENT
    assert lib.dg_create(ctypes.byref(c), 1 << 33, None, None, ctypes.byref(h)) == _lib.DG_ERR_INVALID_ARGUMENT
    assert lib.dg_insert_edges(None, None, None, None, 0, None, None) == _lib.DG_ERR_INVALID_ARGUMENT
    assert lib.dg_destroy(None) == _lib.DG_ERR_INVALID_ARGUMENT
    assert lib.dg_get_unique_id(None) == _lib.DG_ERR_INVALID_ARGUMENT


def test_product_has_no_oracle_dependency():
    """The CUDA path never imports or links the oracle (test infrastructure only)."""
    pkg = os.path.join(ROOT, "paper_conf_ipps_awadapo20_b200")
    for dirpath, _, files in os.walk(pkg):
        for f in files:
            if f.endswith((".py", ".cu", ".cuh", ".h", ".cpp")):
                txt = open(os.path.join(dirpath, f)).read()
                assert "oracle" not in txt.replace("Oracle-free", ""), f


def test_flag_values_match_header():
    """The binding's DG_FLAG_* constants are the header's (include/dg.h)."""
    import re
    from paper_conf_ipps_awadapo20_b200 import _lib
    hdr = open(os.path.join(ROOT, "include", "dg.h")).read()
    flags = dict(re.findall(r"#define (DG_FLAG_\w+) (\d+)u", hdr))
    assert set(flags) == {"DG_FLAG_NO_TOMBSTONE_REUSE", "DG_FLAG_FORCE_ROUTER", "DG_FLAG_SET",
                          "DG_FLAG_ADAPTIVE", "DG_FLAG_COPY_EXCHANGE"}
    for k, v in flags.items():
        assert getattr(_lib, k) == int(v), k


def test_rank_group_is_host_only():
    """dg_group_create / dg_group_destroy need no GPU; a sharded create needs a NCCL id
    or a group, and a group must have the handle's nranks"""
    from paper_conf_ipps_awadapo20_b200 import RankGroup, _lib
    lib = _lib.lib
    h = ctypes.c_void_p()
    assert lib.dg_group_create(0, ctypes.byref(h)) == _lib.DG_ERR_INVALID_ARGUMENT
    assert lib.dg_group_create(65, ctypes.byref(h)) == _lib.DG_ERR_INVALID_ARGUMENT
    assert lib.dg_group_destroy(None) == _lib.DG_ERR_INVALID_ARGUMENT
    g = RankGroup(4)
    assert g.handle.value
    g.close()
    assert not g.handle.value
