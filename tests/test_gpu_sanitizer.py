"""compute-sanitizer over every kernel family (-m gpu).

memcheck (out-of-bounds / misaligned / illegal accesses, leaks not checked), racecheck
(shared-memory hazards: the per-warp backlog and allocator chunks of the edge kernels,
the block scans) and synccheck (barrier misuse in the warp-collective code) each run
tests/sanitize_script.py, which checks its results against the oracle as well.

The sanitizer runs are opt-in (DG_SANITIZER=1): the GPU pool closed compute-sanitizer
after runs under it left GPUs needing a reset, so by default only the script itself
runs (its oracle checks and dg_check_invariants); the zero-error summaries of the runs
made while it was open are under profiles/r02/sanitizer_*.txt."""
import os
import subprocess
import sys

import pytest

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
SAN = "/usr/local/cuda/bin/compute-sanitizer"


@pytest.mark.parametrize("tool", ["memcheck", "racecheck", "synccheck"])
def test_compute_sanitizer(cuda_ok, tool):
    if os.environ.get("DG_SANITIZER") != "1":
        pytest.skip("compute-sanitizer is opt-in (DG_SANITIZER=1): closed on this GPU pool")
    if not os.path.exists(SAN):
        pytest.fail("compute-sanitizer not found")
    cmd = [SAN, f"--tool={tool}", "--error-exitcode=97", "--target-processes=all"]
    if tool == "memcheck":
        cmd += ["--leak-check=no"]
    if tool == "racecheck":
        cmd += ["--racecheck-report=hazard"]
    cmd += [sys.executable, os.path.join(ROOT, "tests", "sanitize_script.py")]
    env = dict(os.environ, PYTORCH_NO_CUDA_MEMORY_CACHING="1")
    r = subprocess.run(cmd, capture_output=True, text=True, timeout=1500, cwd=ROOT, env=env)
    out = r.stdout + r.stderr
    os.makedirs(os.path.join(ROOT, "gpurun_out"), exist_ok=True)
    with open(os.path.join(ROOT, "gpurun_out", f"sanitizer_{tool}.log"), "w") as f:
        f.write(out)
    if "compute-sanitizer is closed" in out:
        pytest.skip(out.strip().splitlines()[0])
    assert r.returncode == 0, out[-6000:]
    assert "SANITIZE SCRIPT OK" in out, out[-6000:]
    assert "ERROR SUMMARY: 0 errors" in out or "RACECHECK SUMMARY: 0 hazards" in out, out[-4000:]


def test_sanitize_script_plain(cuda_ok):
    """The sanitizer workload without the sanitizer: every kernel family on small
    cases, checked against the oracle and dg_check_invariants."""
    env = dict(os.environ, PYTORCH_NO_CUDA_MEMORY_CACHING="1")
    r = subprocess.run([sys.executable, os.path.join(ROOT, "tests", "sanitize_script.py")],
                       capture_output=True, text=True, timeout=900, cwd=ROOT, env=env)
    out = r.stdout + r.stderr
    assert r.returncode == 0, out[-6000:]
    assert "SANITIZE SCRIPT OK" in out, out[-6000:]
