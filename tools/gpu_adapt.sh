# adaptive layout: GPU suite + default bench (uniform regression check) + adaptive configs
set -x
D=gpurun_out/adapt; mkdir -p $D
python -c "import __graft_entry__ as g; g.build(); g.smoke()" > $D/smoke.log 2>&1; echo smoke rc=$?
timeout 1500 python -m pytest tests -m gpu -q > $D/pytest_gpu.log 2>&1; echo pytest rc=$?
tail -15 $D/pytest_gpu.log
timeout 600 python bench.py > $D/bench_cfg2.json 2> $D/bench_cfg2.err; echo bench rc=$?
timeout 600 python bench.py --bucket-bytes 0 --no-e2e --no-cpu-baseline > $D/bench_cfg2_adaptive.json 2> $D/bench_cfg2_adaptive.err
timeout 900 python bench.py --config cfg3 --no-e2e --no-cpu-baseline > $D/bench_cfg3.json 2> $D/bench_cfg3.err
timeout 900 python bench.py --config cfg3 --bucket-bytes 0 --no-e2e --no-cpu-baseline > $D/bench_cfg3_adaptive.json 2> $D/bench_cfg3_adaptive.err
timeout 900 python bench.py --config cfg4 --no-cpu-baseline > $D/bench_cfg4.json 2> $D/bench_cfg4.err
timeout 900 python bench.py --config cfg4 --bucket-bytes 0 --no-cpu-baseline > $D/bench_cfg4_adaptive.json 2> $D/bench_cfg4_adaptive.err
tail -3 $D/*.err
