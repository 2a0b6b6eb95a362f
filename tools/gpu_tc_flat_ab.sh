# flat wedge kernel: parity + cfg5 A/B (per-entry kernel, flat, flat + probe order)
D=gpurun_out/tcflat; mkdir -p $D
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -x -k "tc or hub_rows" > $D/pytest.log 2>&1; echo pytest rc=$?; tail -2 $D/pytest.log
for v in ${TC_VARIANTS:-"DG_TC_FLAT=0" "DG_TC_FLAT=1" "DG_TC_FLAT=1 DG_TC_ORDER=1"}; do
  env $v timeout 900 python bench.py --config cfg5 --steps 3 --warmup 1 > $D/cfg5.json 2> $D/cfg5.err
  python -c "
import json; d=json.loads(open('$D/cfg5.json').read().strip().splitlines()[-1]); print('$v', round(d['value']), d['tc']['tc_ms_per_step'], d['tc']['wedge_G_per_s'], d['tc']['triangles_per_step'])" || tail -3 $D/cfg5.err
done
timeout 600 ncu --set full --clock-control none -k regex:"k_tc_wedges" -c 1 -o $D/flat -f python bench.py --config cfg5 --steps 1 --warmup 0 > $D/ncu.log 2>&1; echo ncu rc=$?
python tools/ncu_summary.py $D/flat.ncu-rep > $D/summary.txt 2>&1; head -16 $D/summary.txt
