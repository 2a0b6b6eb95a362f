D=gpurun_out/quick; mkdir -p $D
timeout 900 python -m pytest tests -m gpu -x -q -k "${TESTK:-rehash or retry or freed or config1 or large or exhaust or rmat or flush or churn or adaptive or 0]}" > $D/pytest.log 2>&1; echo pytest rc=$?; tail -2 $D/pytest.log
timeout 600 python bench.py --no-e2e --no-cpu-baseline --steps 5 > $D/b.json 2>$D/b.err
python -c "
import json;d=json.loads(open('$D/b.json').read().strip().splitlines()[-1])
print('cfg2', round(d['value']), {k:(round(v['M_edges_s']),round(v['kernel_ms_per_batch'],3)) for k,v in d['ops'].items()}, 'bulk', round(d['bulk_build']['insert_ms'],2))"
timeout 900 python bench.py --config cfg4 --no-e2e --no-cpu-baseline --steps 5 > $D/b4.json 2>$D/b4.err
python -c "
import json;d=json.loads(open('$D/b4.json').read().strip().splitlines()[-1])
print('cfg4', round(d['value']), {k:(round(v.get('M_edges_s') or v.get('M_vertices_s')),round(v['ms_per_step'],3)) for k,v in d['ops'].items()}, d.get('bulk_build'))"
for c in cfg2 cfg3; do
timeout 900 python bench.py --config $c --bucket-bytes 0 --no-e2e --no-cpu-baseline --steps 5 > $D/ba.json 2>$D/ba.err
python -c "
import json;d=json.loads(open('$D/ba.json').read().strip().splitlines()[-1])
print('$c adaptive', round(d['value']), {k:(round(v['M_edges_s']),round(v['kernel_ms_per_batch'],3)) for k,v in d['ops'].items()}, 'bulk', round(d['bulk_build']['insert_ms'],2))"
done
