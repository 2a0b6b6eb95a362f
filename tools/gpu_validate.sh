D=gpurun_out/r2s3; mkdir -p $D
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > $D/smoke.log 2>&1; echo smoke rc=$?; tail -1 $D/smoke.log
timeout 2400 python -m pytest tests -m gpu -q -x --durations=10 > $D/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -15 $D/pytest_gpu.log
timeout 900 python bench.py > $D/bench_cfg2.json 2> $D/bench_cfg2.err; echo bench rc=$?; tail -c 600 $D/bench_cfg2.json
