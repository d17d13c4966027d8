mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_flow_waw.py -x -q > gpurun_out/pytest_waw.log 2>&1; echo pytest_waw=$?; tail -15 gpurun_out/pytest_waw.log
timeout 300 python scripts/waw_time.py > gpurun_out/waw_time.log 2>&1; echo waw=$?; cat gpurun_out/waw_time.log | tail -12
timeout 300 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k regex:"k_" --csv --log-file gpurun_out/launches_waw.csv python -c "
import sys; sys.path.insert(0,'.')
import torch, synth, paper_conf_icpp_hanzlw13_b200 as jp
wl=synth.config3_waw(0.01, device='cuda'); L=jp.Loop.from_workload(wl); ws=jp.workspace(L)
print(jp.jp_schedule(L, ws)); torch.cuda.synchronize()" > gpurun_out/ncu_waw.log 2>&1; echo ncu=$?
timeout 1800 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo pytest=$?; tail -5 gpurun_out/pytest_gpu.log
