mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_p.log 2>&1 || exit 1
CFG=${CFG:-C3}; MODE=${MODE:-accurate}; TAG=${TAG:-C3a_r1s4}
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k_point_pass|k_pip" -s ${SKIP:-4} -c ${COUNT:-3} -o gpurun_out/prof_$TAG -f \
   python bench.py --config $CFG --mode $MODE --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > gpurun_out/prof_c3a.log 2>&1; echo "ncu rc=$?"
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 600 --csv --log-file gpurun_out/launches_$TAG.csv \
   python bench.py --config $CFG --mode $MODE --steps 3 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "list rc=$?"
