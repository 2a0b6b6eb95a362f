python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build.log 2>&1 || exit 1
timeout 900 python -m pytest tests -m gpu -x -q -k "vertex or config1 or routed" 2>&1 | tail -3
timeout 600 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/b9_cfg2.json 2>/dev/null
python -c "import json; d=json.load(open('gpurun_out/b9_cfg2.json')); print('cfg2', d['value'], d['vertex_deletion'])"
timeout 900 python bench.py --config cfg4 > gpurun_out/b9_cfg4.json 2>/dev/null
python -c "import json; d=json.load(open('gpurun_out/b9_cfg4.json')); print('cfg4', d['value'], d['ops']['delete_vertices'], d['roofline']['achieved'], d['roofline']['frac'])"
