# TC probe order (entries sorted by the probed vertex): parity + cfg5 A/B + ncu of the wedge kernel
D=gpurun_out/tcord; mkdir -p $D
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -x -k "tc or hub_rows" > $D/pytest.log 2>&1; echo pytest rc=$?; tail -2 $D/pytest.log
for v in 0 1; do
  DG_TC_ORDER=$v timeout 900 python bench.py --config cfg5 --steps 3 --warmup 1 > $D/cfg5_$v.json 2> $D/cfg5_$v.err
  python -c "
import json; d=json.loads(open('$D/cfg5_$v.json').read().strip().splitlines()[-1]); print('order=$v', round(d['value']), d['tc']['tc_ms_per_step'], d['tc']['wedge_G_per_s'], d['tc']['triangles_per_step'])" || tail -3 $D/cfg5_$v.err
done
timeout 600 ncu --set full --clock-control none -k regex:"k_tc_wedges" -c 1 -o $D/tc1 -f python bench.py --config cfg5 --steps 1 --warmup 0 > $D/ncu.log 2>&1; echo ncu rc=$?
python tools/ncu_summary.py $D/tc1.ncu-rep > $D/summary.txt 2>&1; cat $D/summary.txt | head -16
