mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_x11.log 2>&1 || { tail -20 gpurun_out/build_x11.log; exit 1; }
timeout 600 python -m pytest tests/test_gpu_random.py -q 2>&1 | tail -15
