mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_x5.log 2>&1 || { tail -20 gpurun_out/build_x5.log; exit 1; }
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_emu8_x5.csv python tools/emulate_strong.py --config C2 --ranks 8 --only-rank 0 --steps 5 --points 1e9 > gpurun_out/emu8_x5.log 2>&1; echo "ncu rc=$?"
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_c3_x5.csv python bench.py --config C3 --steps 3 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "ncu rc=$?"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_point_pass -s 2 -c 1 -o gpurun_out/prof_C5b_x5 -f python bench.py --config C5 --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "ncu C5 rc=$?"
