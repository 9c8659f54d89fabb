mkdir -p gpurun_out
free -g | head -2; nproc
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_x6.log 2>&1 || { tail -20 gpurun_out/build_x6.log; exit 1; }
timeout 1500 python -m pytest tests -m gpu -q -x > gpurun_out/pytest_x6.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pytest_x6.log
: > gpurun_out/bench_x6.jsonl
for spec in "C2" "C3 --mode accurate" "C4" "C5"; do
  timeout 600 python bench.py --config $spec --steps 10 --warmup 3 --no-cpu-baseline --e2e-steps 0 2>/dev/null | tail -1 >> gpurun_out/bench_x6.jsonl
done
python tools/bench_table.py gpurun_out/bench_x6.jsonl
timeout 1200 python tools/emulate_strong.py --config C4 --points 2e9 > gpurun_out/emu_C4_x6.jsonl 2> gpurun_out/emu_C4_x6.err; echo "emu C4 rc=$?"; head -3 gpurun_out/emu_C4_x6.jsonl | cut -c1-400; tail -3 gpurun_out/emu_C4_x6.err
