#!/bin/bash
tag=${1:-c5}
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$tag.log 2>&1 || exit 1
P="python bench.py --config C5 --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline"
$P > gpurun_out/plain_$tag.log 2>&1 && \
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k_point_pass" -s 2 -c 1 -o gpurun_out/prof_C5_$tag -f $P > /dev/null 2>&1; echo "ncu rc=$?"
python tools/ncu_summary.py gpurun_out/prof_C5_$tag.ncu-rep > gpurun_out/ncu_C5_$tag.md 2>&1
python tools/ncu_lines.py gpurun_out/prof_C5_$tag.ncu-rep 40 > gpurun_out/lines_C5_$tag.txt 2>&1
