# round 2: home-bucket layout — full GPU suite, benches, full-size parity
D=gpurun_out/r2d; mkdir -p $D
timeout 1500 python -m pytest tests -m gpu -q -x --ignore=tests/test_gpu_fullsize.py > $D/gpu_all.log 2>&1; echo gpu_all rc=$?; tail -5 $D/gpu_all.log
for c in cfg2 cfg3; do
timeout 600 python bench.py --config $c --steps 10 --warmup 3 --no-e2e --no-cpu-baseline > $D/bench_$c.json 2> $D/bench_$c.err; echo bench $c rc=$?
python -c "
import json;d=json.loads(open('$D/bench_$c.json').read().strip().splitlines()[-1])
print('$c', round(d['value']), {k:(round(v['M_edges_s']),round(v['kernel_ms_per_batch'],3)) for k,v in d['ops'].items()}, 'frac', round(d['roofline']['frac'],3), d['roofline']['kernel'], 'bulk', {k:round(v,2) for k,v in d['bulk_build'].items() if 'ms' in k}, 'vdel', d['vertex_deletion'])" || tail -5 $D/bench_$c.err
done
timeout 3000 python -m pytest tests/test_gpu_fullsize.py -q --durations=0 > $D/fullsize.log 2>&1; echo fullsize rc=$?; tail -12 $D/fullsize.log
