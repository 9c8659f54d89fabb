mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_x2.log 2>&1 || { tail -20 gpurun_out/build_x2.log; exit 1; }
timeout 600 python -m pytest tests/test_gpu_dist.py -q -x 2>&1 | tail -5
timeout 900 python tools/emulate_strong.py --config C3 > gpurun_out/emu_C3.jsonl 2> gpurun_out/emu_C3.err; echo "emu C3 rc=$?"; head -3 gpurun_out/emu_C3.jsonl | cut -c1-600
timeout 900 python tools/emulate_strong.py --config C2 > gpurun_out/emu_C2.jsonl 2> gpurun_out/emu_C2.err; echo "emu C2 rc=$?"; head -3 gpurun_out/emu_C2.jsonl | cut -c1-600
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_point_pass -s 2 -c 1 -o gpurun_out/prof_C3b_x2 -f python bench.py --config C3 --mode bounded --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "ncu C3b rc=$?"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k_point_pass|k_pip" -s 2 -c 2 -o gpurun_out/prof_C3a_x2 -f python bench.py --config C3 --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "ncu C3a rc=$?"
