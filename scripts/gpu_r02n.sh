mkdir -p gpurun_out
timeout 300 python scripts/doall_phase_time.py; JP_DOALL_PHASED=0 timeout 300 python scripts/doall_phase_time.py
timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo pytest=$?; tail -3 gpurun_out/pytest_gpu.log
