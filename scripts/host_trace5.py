import sys; sys.path.insert(0,'.')
import torch, synth, paper_conf_icpp_hanzlw13_b200 as jp
wl=synth.config5(device='cuda'); A0=wl.A.clone(); L=jp.Loop.from_workload(wl); ws=jp.workspace(L)
for k in range(4):
    wl.A.copy_(A0); torch.cuda.synchronize()
    print("call", k, file=sys.stderr, flush=True)
    jp.jp_schedule(L, ws, scheme=jp.JP_SCHED_STEALING, chunk_iters=1<<16); torch.cuda.synchronize()
