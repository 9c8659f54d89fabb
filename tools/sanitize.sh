#!/bin/bash
# compute-sanitizer over every librj kernel variant (tools/sanitize.py).
# Usage: tools/sanitize.sh TAG   -> gpurun_out/sanitize_TAG_<tool>.txt
tag=${1:-r2}
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_san.log 2>&1 || { tail gpurun_out/build_san.log; exit 1; }
for tool in memcheck synccheck initcheck racecheck; do
  extra=""
  [ $tool = memcheck ] && extra="--leak-check full"
  quick=""; [ $tool = racecheck ] && quick="--quick"
  timeout ${SAN_TIMEOUT:-1500} compute-sanitizer --tool $tool $extra --error-exitcode 99 --target-processes all \
     python tools/sanitize.py $quick > gpurun_out/sanitize_${tag}_$tool.txt 2>&1
  echo "$tool rc=$?" | tee -a gpurun_out/sanitize_${tag}_$tool.txt
  tail -3 gpurun_out/sanitize_${tag}_$tool.txt
done
