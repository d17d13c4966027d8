import time, statistics, torch, ctypes as C, sys
sys.path.insert(0, '/root/repo')
import paper_conf_icpp_hanzlw13_b200 as jp
import synth
x = torch.zeros(1, device="cuda")
def t(fn, k=200):
    for _ in range(20): fn()
    ts=[]
    for _ in range(k):
        a=time.perf_counter(); fn(); ts.append((time.perf_counter()-a)*1e6)
    return round(statistics.median(ts),1), round(min(ts),1)
print("torch add_ + sync", t(lambda: (x.add_(1), torch.cuda.synchronize())))
print("sync only", t(lambda: torch.cuda.synchronize()))
wl = synth.config1(0.0, device="cuda"); L = jp.Loop.from_workload(wl); ws = jp.workspace(L)
cfg = jp.sched_cfg()
print("jp_schedule tiny", t(lambda: jp.jp_schedule(L, ws, cfg=cfg)))
lib = jp.lib(); res = jp._abi.jp_sched_result(); st = torch.cuda.current_stream().cuda_stream
p, nb = ws.data_ptr(), ws.numel()
print("raw C jp_schedule", t(lambda: lib.jp_schedule(L.ref, C.byref(cfg), p, nb, C.byref(res), st)))
import oracle as O

