python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build.log 2>&1 || exit 1
timeout 300 python tools/tc_probe.py 22 128 map 4
timeout 300 python tools/tc_probe.py 22 128 set 4
timeout 300 python tools/tc_probe.py 22 64 set 4
timeout 300 python tools/tc_probe.py 22 64 map 4
timeout 300 python tools/tc_probe.py 22 32 set 4
