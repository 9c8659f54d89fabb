#!/bin/bash
# ncu captures of the two kernels VERDICT r1 names (C3 accurate label + PIP
# queue, C5 32768^2 bounded tile kernel) with source lines, plus the raw C2
# launch list.   tools/prof_two.sh TAG
tag=${1:-r2b}
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$tag.log 2>&1 || exit 1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k_point_pass|k_pip" -s 4 -c 2 -o gpurun_out/prof_C3a_$tag -f \
   python bench.py --config C3 --mode accurate --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > gpurun_out/prof_C3a_$tag.log 2>&1; echo "ncu C3a rc=$?"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k_point_pass" -s 2 -c 1 -o gpurun_out/prof_C5b_$tag -f \
   python bench.py --config C5 --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > gpurun_out/prof_C5b_$tag.log 2>&1; echo "ncu C5b rc=$?"
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 600 --csv --log-file gpurun_out/launches_C2_$tag.csv \
   python bench.py --steps 3 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "list rc=$?"
for r in C3a C5b; do python tools/ncu_summary.py gpurun_out/prof_${r}_$tag.ncu-rep > gpurun_out/ncu_${r}_$tag.md 2>&1; done
python tools/ncu_lines.py gpurun_out/prof_C3a_$tag.ncu-rep 40 k_point_pass > gpurun_out/lines_C3a_$tag.txt 2>&1
python tools/ncu_lines.py gpurun_out/prof_C3a_$tag.ncu-rep 25 k_pip > gpurun_out/lines_C3pip_$tag.txt 2>&1
python tools/ncu_lines.py gpurun_out/prof_C5b_$tag.ncu-rep 40 > gpurun_out/lines_C5b_$tag.txt 2>&1
