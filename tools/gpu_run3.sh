python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build.log 2>&1 || exit 1
timeout 300 python tools/bulk_probe.py > gpurun_out/bulk_probe.log 2>&1; cat gpurun_out/bulk_probe.log
for v in set map; do
  timeout 600 python bench.py --config cfg5 --steps 3 --warmup 3 --variant $v > gpurun_out/cfg5_$v.json 2> gpurun_out/cfg5_$v.err
  python -c "import json; d=json.load(open('gpurun_out/cfg5_$v.json')); print('$v', json.dumps(d['tc']), d['roofline']['achieved'])"
done
timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -3 gpurun_out/pytest_gpu.log
