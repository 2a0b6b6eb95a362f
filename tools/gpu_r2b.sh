# round 2: multirank (quiesce fix), sanitizer, full GPU suite with invariants, bench
D=gpurun_out/r2b; mkdir -p $D
timeout 900 python -m pytest tests/test_gpu_multirank.py -q > $D/multirank.log 2>&1; echo multirank rc=$?; tail -3 $D/multirank.log
timeout 1500 python -m pytest tests/test_gpu_sanitizer.py -q > $D/sanitizer.log 2>&1; echo sanitizer rc=$?; tail -3 $D/sanitizer.log
cp gpurun_out/sanitizer_*.log $D/ 2>/dev/null
timeout 1500 python -m pytest tests -m gpu -q --deselect tests/test_gpu_sanitizer.py > $D/gpu_all.log 2>&1; echo gpu_all rc=$?; tail -3 $D/gpu_all.log
timeout 600 python bench.py --steps 10 --warmup 3 > $D/bench.json 2> $D/bench.err; echo bench rc=$?; tail -c 300 $D/bench.json
