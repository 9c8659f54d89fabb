#!/bin/bash
tag=r2e
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$tag.log 2>&1 || { echo build failed; tail -20 gpurun_out/build_$tag.log; exit 1; }
timeout 1500 python -m pytest tests -m gpu -q -x -p no:cacheprovider > gpurun_out/pytest_gpu_$tag.log 2>&1; echo "pytest rc=$?"; tail -4 gpurun_out/pytest_gpu_$tag.log
tools/perf_quick.sh $tag C2 C3:accurate C3:bounded C4 C5 C5:accurate
timeout 600 python tools/emulate_strong.py --config C4 --points 2e9 --ranks 8 --spatial-only --poly-weight 0.1 > gpurun_out/emul_$tag.jsonl 2>gpurun_out/emul_$tag.err; echo "emul rc=$?"; tail -3 gpurun_out/emul_$tag.jsonl
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_point_pass -s 4 -c 1 -o gpurun_out/prof_C3a_$tag -f \
   python bench.py --config C3 --mode accurate --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "ncu C3a rc=$?"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_point_pass -s 4 -c 1 -o gpurun_out/prof_C5b_$tag -f \
   python bench.py --config C5 --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "ncu C5b rc=$?"
