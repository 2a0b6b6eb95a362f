python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build.log 2>&1 || exit 1
timeout 300 python tools/tc_probe.py 22 128 map 4
timeout 300 python tools/tc_probe.py 22 128 set 4
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/tc_launches.csv python tools/tc_probe.py 22 128 map 2 > /dev/null 2>&1
python tools/launch_share.py gpurun_out/tc_launches.csv | head -20
