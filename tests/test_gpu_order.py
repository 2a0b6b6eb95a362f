"""Locality-ordered delete batches (kernels_order.cu) against the oracle.

Delete batches of at least DG_ORDER_MIN_OPS ops (default 2^20) are partitioned by row
(and validated by the partition's count pass) before their probe; the full-size tests
exercise that at the real sizes.  Here the threshold is forced to 1 in a child process
so every delete batch of the small parity cases (directed and undirected config 1, set variant, vertex deletion, hubs,
host buffers, the routed P = 2..8 rank groups) runs the ordered path, element by
element against the oracle."""
import os
import subprocess
import sys

import pytest

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))

CASES = [
    ("tests/test_gpu_parity.py", "config1 or large_random_ragged or rmat_hubs or heavy_intra or "
                                 "host_buffers or vertex_deletion or empty_batches or churn or "
                                 "host_query_pipeline or async_host"),
    ("tests/test_gpu_multirank.py", "directed or undirected or small_buckets"),
]


@pytest.mark.parametrize("path,expr", CASES)
def test_ordered_batches_match_oracle(cuda_ok, path, expr):
    env = dict(os.environ, DG_ORDER_MIN_OPS="1")
    r = subprocess.run([sys.executable, "-m", "pytest", "-q", "-x", "-m", "gpu", "-p", "no:cacheprovider",
                        os.path.join(ROOT, path), "-k", expr],
                       capture_output=True, text=True, timeout=1500, cwd=ROOT, env=env)
    out = r.stdout + r.stderr
    assert r.returncode == 0, out[-6000:]
    assert " passed" in out and "failed" not in out, out[-3000:]
