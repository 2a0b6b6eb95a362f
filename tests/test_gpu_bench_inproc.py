"""Dry run of bench.py's N > 1 path on one GPU (-m gpu; "the torchrun
worker and bench.py --gpus N paths are exercised by a dry-run script").

`bench.py --inproc N` runs N rank threads of one process over an in-process rank
group: each rank builds its slice of the base graph, the library routes every batch
(source-vertex sharding, fused exchange), timings are max-reduced over the ranks and
rank 0 prints the JSON line — the code path a torchrun launch takes, with the
transport swapped.  Its rates are not a scaling measurement."""
import json
import os
import subprocess
import sys

import pytest

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.mark.parametrize("config,extra", [
    ("cfg2", ["--batch-log2", "20"]),
    ("cfg4", []),
    ("cfg5", []),
])
def test_bench_inproc_two_ranks(cuda_ok, config, extra):
    cmd = [sys.executable, os.path.join(ROOT, "bench.py"), "--inproc", "2", "--config", config,
           "--steps", "2", "--warmup", "3", "--no-cpu-baseline"] + extra
    r = subprocess.run(cmd, capture_output=True, text=True, timeout=1200, cwd=ROOT)
    assert r.returncode == 0, r.stderr[-4000:]
    line = json.loads(r.stdout.strip().splitlines()[-1])
    assert line["n_gpus"] == 2 and line["value"] > 0, line
    assert "in-process rank group" in line["config"]["parallelism"]
    assert line["gpu_launches"] > 0
