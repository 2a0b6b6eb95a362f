D=gpurun_out/tc; mkdir -p $D
python -c "import __graft_entry__ as g; g.build()" > $D/build.log 2>&1 || exit 1
timeout 900 python -m pytest tests -m gpu -x -q -k "tc or triangle or config5 or hub" > $D/pytest.log 2>&1; echo pytest rc=$?; tail -2 $D/pytest.log
for o in 0 1; do
DG_TC_ORDER=$o timeout 900 python bench.py --config cfg5 --steps 3 --warmup 1 --no-cpu-baseline > $D/b$o.json 2>$D/b$o.err
python -c "
import json;d=json.loads(open('$D/b$o.json').read().strip().splitlines()[-1])
print('order=$o', round(d['value']), d['tc']['tc_ms_per_step'], d['tc']['triangles_per_step'], round(d['roofline']['frac'],3))" || tail -3 $D/b$o.err
done
