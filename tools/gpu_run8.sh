python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build.log 2>&1 || exit 1
timeout 900 python -m pytest tests -m gpu -x -q -k "async_host or host_ or config1_directed" > gpurun_out/pytest_async.log 2>&1; echo pytest rc=$?; tail -15 gpurun_out/pytest_async.log
timeout 600 python bench.py --steps 5 --warmup 3 --no-cpu-baseline --no-vdel > gpurun_out/bench_e2e.json 2> gpurun_out/bench_e2e.err
python -c "import json; d=json.load(open('gpurun_out/bench_e2e.json')); print(d['value'], d['e2e'])"
