mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_x14.log 2>&1 || { tail -20 gpurun_out/build_x14.log; exit 1; }
timeout 600 ncu --set full --clock-control none --import-source on -k regex:"k_point_pass|k_pip" -s 2 -c 2 -o gpurun_out/prof_C3a_x14 -f python bench.py --config C3 --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "ncu C3a rc=$?"
timeout 600 ncu --set full --clock-control none --import-source on -k regex:"k_point_pass" -s 2 -c 1 -o gpurun_out/prof_C4_x14 -f python bench.py --config C4 --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "ncu C4 rc=$?"
timeout 1200 python tools/emulate_strong.py --config C4 --points 2e9 > gpurun_out/emu_C4_x14.jsonl 2> gpurun_out/emu_C4_x14.err; echo "emu C4 rc=$?"; head -3 gpurun_out/emu_C4_x14.jsonl | cut -c1-300
timeout 1200 python tools/emulate_strong.py --config C3 > gpurun_out/emu_C3_x14.jsonl 2> gpurun_out/emu_C3_x14.err; echo "emu C3 rc=$?"; head -3 gpurun_out/emu_C3_x14.jsonl | cut -c1-300
