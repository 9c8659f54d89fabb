mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_x9.log 2>&1 || { tail -20 gpurun_out/build_x9.log; exit 1; }
timeout 1500 python -m pytest tests -m gpu -q -x > gpurun_out/pytest_x9.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pytest_x9.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke_x9.log 2>&1; echo "smoke rc=$?"; tail -1 gpurun_out/smoke_x9.log
timeout 900 python bench.py > gpurun_out/bench_x9.json 2> gpurun_out/bench_x9.err; echo "bench rc=$?"; tail -c 400 gpurun_out/bench_x9.json
timeout 300 python bench.py --impl reference --steps 3 --warmup 3 > gpurun_out/bench_ref_x9.json 2>&1; echo "ref rc=$?"
: > gpurun_out/bench_lines_x9.jsonl
for spec in "C3 --mode bounded" "C3 --mode accurate" "C4" "C5" "C5 --mode accurate"; do
  timeout 600 python bench.py --config $spec --steps 10 --warmup 3 --no-cpu-baseline --e2e-steps 1 2>/dev/null | tail -1 >> gpurun_out/bench_lines_x9.jsonl
done
python tools/bench_table.py gpurun_out/bench_lines_x9.jsonl
timeout 1200 python tools/sweep_c5.py > gpurun_out/sweep_c5_x9.jsonl 2> gpurun_out/sweep_c5_x9.err; echo "sweep rc=$?"; tail -3 gpurun_out/sweep_c5_x9.err
timeout 1200 python tools/emulate_strong.py --config C4 --points 2e9 > gpurun_out/emu_C4_x9.jsonl 2> gpurun_out/emu_C4_x9.err; echo "emu C4 rc=$?"; head -3 gpurun_out/emu_C4_x9.jsonl | cut -c1-300
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 600 --csv --log-file gpurun_out/launches_x9.csv python bench.py --steps 3 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "ncu list rc=$?"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_point_pass -s 2 -c 1 -o gpurun_out/prof_C2_x9 -f python bench.py --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "ncu full rc=$?"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_point_pass -s 2 -c 1 -o gpurun_out/prof_C3b_x9 -f python bench.py --config C3 --mode bounded --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "ncu C3b rc=$?"
