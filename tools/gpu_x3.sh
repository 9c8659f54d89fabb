mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_x3.log 2>&1 || { tail -20 gpurun_out/build_x3.log; exit 1; }
timeout 1500 python -m pytest tests -m gpu -q -x > gpurun_out/pytest_x3.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pytest_x3.log
: > gpurun_out/bench_x3.jsonl
for spec in "C2" "C3 --mode accurate" "C3 --mode bounded" "C4" "C5" "C5 --mode accurate"; do
  timeout 600 python bench.py --config $spec --steps 10 --warmup 3 --no-cpu-baseline --e2e-steps 0 2>/dev/null | tail -1 >> gpurun_out/bench_x3.jsonl
done
python tools/bench_table.py gpurun_out/bench_x3.jsonl
timeout 900 python tools/emulate_strong.py --config C2 > gpurun_out/emu_C2_x3.jsonl 2> gpurun_out/emu_C2_x3.err; echo "emu C2 rc=$?"; head -3 gpurun_out/emu_C2_x3.jsonl | cut -c1-400
timeout 900 python tools/emulate_strong.py --config C3 > gpurun_out/emu_C3_x3.jsonl 2> gpurun_out/emu_C3_x3.err; echo "emu C3 rc=$?"; head -3 gpurun_out/emu_C3_x3.jsonl | cut -c1-400
