# quick GPU check of a change: parity suite, cfg2 + cfg3 full-size parity, default bench line
D=gpurun_out/${1:-quick}; mkdir -p $D
timeout 1200 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fullsize.py -m gpu -q -x -k "not config4 and not config5" > $D/pytest.log 2>&1; echo pytest rc=$?; tail -4 $D/pytest.log
timeout 900 python bench.py --no-cpu-baseline > $D/bench_cfg2.json 2> $D/bench_cfg2.err; echo bench rc=$?
python - $D/bench_cfg2.json <<'PY'
import json,sys
d=json.loads(open(sys.argv[1]).read().strip().splitlines()[-1])
print({k:d.get(k) for k in ("value","ms_per_step")}, d.get("roofline"), d.get("ops"), d.get("bulk_build"))
PY
