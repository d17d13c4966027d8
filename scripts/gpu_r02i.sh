mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_flow_waw.py -x -q > gpurun_out/pytest_waw.log 2>&1; echo pytest_waw=$?; tail -3 gpurun_out/pytest_waw.log
timeout 120 ./scripts/ubench/rand_l2 > gpurun_out/rand_l2.log 2>&1; echo ubench=$?; cat gpurun_out/rand_l2.log
timeout 300 python scripts/waw_time.py > gpurun_out/waw_time.log 2>&1; echo waw=$?; cat gpurun_out/waw_time.log | tail -12
timeout 1200 python bench.py > gpurun_out/bench.json 2> gpurun_out/bench.err; echo bench=$?
