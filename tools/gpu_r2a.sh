# round 2: P>=2 router on one GPU (in-process rank group) + full GPU suite + bench
D=gpurun_out/r2a; mkdir -p $D
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv > $D/smi.txt 2>&1
timeout 900 python -m pytest tests/test_gpu_multirank.py -x -q > $D/multirank.log 2>&1; echo multirank rc=$?; tail -3 $D/multirank.log
timeout 1200 python -m pytest tests -m gpu -q > $D/gpu_all.log 2>&1; echo gpu_all rc=$?; tail -3 $D/gpu_all.log
timeout 600 python bench.py --steps 10 --warmup 3 > $D/bench.json 2> $D/bench.err; echo bench rc=$?; tail -c 600 $D/bench.json
