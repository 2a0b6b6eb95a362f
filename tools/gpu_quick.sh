# quick check: adaptive + allocation-heavy GPU tests, cfg2/cfg3 benches (uniform and adaptive)
D=gpurun_out/quick; mkdir -p $D
timeout 900 python -m pytest tests -m gpu -x -q -k "${TESTK:-adaptive or 0] or rehash or retry or freed or config1}" > $D/pytest.log 2>&1; echo pytest rc=$?; tail -3 $D/pytest.log
for a in "" "--bucket-bytes 0"; do for c in cfg2 cfg3; do
timeout 600 python bench.py --config $c $a --no-e2e --no-cpu-baseline --steps 5 > $D/b.json 2>$D/b.err
python -c "
import json;d=json.loads(open('$D/b.json').read().strip().splitlines()[-1])
print('$c $a', round(d['value']), {k:(round(v['M_edges_s']),round(v['kernel_ms_per_batch'],3)) for k,v in d['ops'].items()}, 'bulk', round(d['bulk_build']['insert_ms'],2), 'vdel', d['vertex_deletion'])" || tail -3 $D/b.err
done; done
