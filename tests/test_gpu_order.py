"""Locality-ordered batches (kernels_order.cu) against the oracle.

Delete batches of at least DG_ORDER_MIN_OPS ops (default 2^21), and insert batches of
that size with at most DG_ORDER_INSERT_PER_ROW ops per row (default 1), are
partitioned by row (and validated by the partition's count pass) before their probe;
the full-size tests exercise that at the real sizes (cfg3's inserts, every config's
2^24 deletes).  Here the thresholds are forced in a child process so every delete
(and, in the second set, every insert) batch of the small parity cases (directed and undirected config 1, set variant, vertex deletion, hubs,
host buffers, the routed P = 2..8 rank groups) runs the ordered path, element by
element against the oracle."""
import os
import subprocess
import sys

import pytest

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))

DEL = {"DG_ORDER_MIN_OPS": "1"}
INS = {"DG_ORDER_MIN_OPS": "1", "DG_ORDER_INSERT_PER_ROW": "1e12"}
CASES = [
    ("tests/test_gpu_parity.py", "config1 or large_random_ragged or rmat_hubs or heavy_intra or "
                                 "host_buffers or vertex_deletion or empty_batches or churn or "
                                 "host_query_pipeline or async_host", DEL),
    ("tests/test_gpu_multirank.py", "directed or undirected or small_buckets", DEL),
    ("tests/test_gpu_parity.py", "config1 or large_random_ragged or rmat_hubs or heavy_intra or "
                                 "host_buffers or churn or src_sorted or retry_path or "
                                 "async_host or flush_tombstones or rehash", INS),
]


@pytest.mark.parametrize("path,expr,env_extra", CASES)
def test_ordered_batches_match_oracle(cuda_ok, path, expr, env_extra):
    env = dict(os.environ, **env_extra)
    r = subprocess.run([sys.executable, "-m", "pytest", "-q", "-x", "-m", "gpu", "-p", "no:cacheprovider",
                        os.path.join(ROOT, path), "-k", expr],
                       capture_output=True, text=True, timeout=1500, cwd=ROOT, env=env)
    out = r.stdout + r.stderr
    assert r.returncode == 0, out[-6000:]
    assert " passed" in out and "failed" not in out, out[-3000:]
