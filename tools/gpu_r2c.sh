# round 2: sorted path (a3), event-ordered in-process group, sanitizer, full-size parity, bench
D=gpurun_out/r2c; mkdir -p $D
(nproc; free -g; lscpu | head -20) > $D/host.txt 2>&1
timeout 900 python -m pytest tests/test_gpu_parity.py -q -k "sorted" > $D/sorted.log 2>&1; echo sorted rc=$?; tail -3 $D/sorted.log
timeout 600 python bench.py --steps 10 --warmup 3 --no-e2e --no-cpu-baseline > $D/bench.json 2> $D/bench.err; echo bench rc=$?
python -c "
import json;d=json.loads(open('$D/bench.json').read().strip().splitlines()[-1])
print(round(d['value']), {k:(round(v['M_edges_s']),round(v['kernel_ms_per_batch'],3)) for k,v in d['ops'].items()}, d['bulk_build'])" || tail -5 $D/bench.err
timeout 900 python -m pytest tests/test_gpu_multirank.py -q > $D/multirank.log 2>&1; echo multirank rc=$?; tail -3 $D/multirank.log
timeout 1500 python -m pytest tests/test_gpu_sanitizer.py -q > $D/sanitizer.log 2>&1; echo sanitizer rc=$?; tail -3 $D/sanitizer.log
cp gpurun_out/sanitizer_*.log $D/ 2>/dev/null
timeout 3000 python -m pytest tests/test_gpu_fullsize.py -q --durations=0 > $D/fullsize.log 2>&1; echo fullsize rc=$?; tail -15 $D/fullsize.log
