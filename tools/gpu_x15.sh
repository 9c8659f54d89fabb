mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_emu8r3_x15.csv python tools/emulate_strong.py --config C4 --points 2e9 --ranks 8 --only-rank 3 --steps 3 > gpurun_out/emu8r3_x15.log 2>&1; echo "ncu rc=$?"
timeout 300 python tools/emulate_strong.py --config C4 --points 2e9 --ranks 8 --only-rank 3 --steps 10 2>/dev/null | tail -1 | cut -c1-600
