#!/bin/bash
# compute-sanitizer over every librj kernel variant (tools/sanitize.py), ONE
# tool per GPU call (B200_PROFILING.md: several sanitizer tools in one call
# have left a GPU unusable).
#   tools/sanitize.sh TAG TOOL      TOOL in memcheck | racecheck | synccheck | initcheck
tag=${1:-r2}; tool=${2:?tool}
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_san.log 2>&1 || { tail gpurun_out/build_san.log; exit 1; }
python tools/sanitize.py --quick > gpurun_out/sanitize_plain_$tag.log 2>&1 || { echo "plain run failed"; tail gpurun_out/sanitize_plain_$tag.log; exit 1; }
extra=""; [ $tool = memcheck ] && extra="--leak-check full"
quick=""; [ $tool = racecheck ] && quick="--quick"
timeout ${SAN_TIMEOUT:-1500} compute-sanitizer --tool $tool $extra --error-exitcode 99 --target-processes all \
   python tools/sanitize.py $quick > gpurun_out/sanitize_${tag}_$tool.txt 2>&1
echo "$tool rc=$?" | tee -a gpurun_out/sanitize_${tag}_$tool.txt
tail -3 gpurun_out/sanitize_${tag}_$tool.txt
