#!/bin/bash
# ncu --set full (source lines) of one config's point-pass kernels -- ONE
# profiler tool per GPU call (B200_PROFILING.md).   tools/prof_kernels.sh TAG CONFIG [bench args...]
#   e.g. tools/prof_kernels.sh c5 C5 ;  tools/prof_kernels.sh c3a C3 --mode accurate
tag=${1:?tag}; cfg=${2:?config}; shift 2
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$tag.log 2>&1 || exit 1
P="python bench.py --config $cfg $* --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline"
$P > gpurun_out/plain_$tag.log 2>&1 && \
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k_point_pass|k_pip" -s 2 -c 2 -o gpurun_out/prof_$tag -f $P > /dev/null 2>&1; echo "ncu rc=$?"
python tools/ncu_summary.py gpurun_out/prof_$tag.ncu-rep > gpurun_out/ncu_$tag.md 2>&1
python tools/ncu_lines.py gpurun_out/prof_$tag.ncu-rep 40 k_point_pass > gpurun_out/lines_$tag.txt 2>&1
