mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_deferred_static.py -x -q > gpurun_out/pytest_def.log 2>&1; echo pytest_def=$?; tail -15 gpurun_out/pytest_def.log
timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo pytest=$?; tail -3 gpurun_out/pytest_gpu.log
timeout 300 python scripts/sched3_time.py > gpurun_out/sched3.log 2>&1; echo t=$?; cat gpurun_out/sched3.log
timeout 300 python scripts/waw_time.py > gpurun_out/waw_time.log 2>&1; echo waw=$?; cat gpurun_out/waw_time.log | tail -8
python scripts/timeline.py config3 0.01 2>/dev/null
