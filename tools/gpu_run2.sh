bash tools/gpu_ab.sh "base nopf base nopf"
timeout 1200 python -m pytest tests -m gpu -x -q -k "set_variant or tc_ or config1 or vertex_deletion or rehash" > gpurun_out/pytest_set.log 2>&1; echo pytest rc=$?
tail -5 gpurun_out/pytest_set.log
