D=gpurun_out/dbg; mkdir -p $D
CUDA_LAUNCH_BLOCKING=1 DG_DEBUG=1 timeout 300 python tools/dbg1.py > $D/plain.log 2>&1; echo plain rc=$?; tail -5 $D/plain.log
timeout 600 /usr/local/cuda/bin/compute-sanitizer --tool memcheck --show-backtrace device python tools/dbg1.py > $D/memcheck.log 2>&1; echo memcheck rc=$?; grep -v "^=========     " $D/memcheck.log | head -40
