"""PCIe bounds for the config-2 e2e step: pinned H2D of 2 GiB, D2H of 1 GiB,
and both at once on two streams (CUDA events)."""
import torch

h_in = torch.empty(1 << 29, dtype=torch.float32).pin_memory()
h_out = torch.empty(1 << 28, dtype=torch.float32).pin_memory()
d_in = torch.empty(1 << 29, dtype=torch.float32, device="cuda")
d_out = torch.empty(1 << 28, dtype=torch.float32, device="cuda")
s1, s2 = torch.cuda.Stream(), torch.cuda.Stream()


def timed(fn):
    for _ in range(2):
        fn()
    torch.cuda.synchronize()
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    a.record()
    fn()
    torch.cuda.synchronize()
    b.record()
    torch.cuda.synchronize()
    return a.elapsed_time(b)


def both():
    with torch.cuda.stream(s1):
        d_in.copy_(h_in, non_blocking=True)
    with torch.cuda.stream(s2):
        h_out.copy_(d_out, non_blocking=True)


t_h2d = timed(lambda: d_in.copy_(h_in, non_blocking=True))
t_d2h = timed(lambda: h_out.copy_(d_out, non_blocking=True))
t_both = timed(both)
print({"h2d_2GiB_ms": round(t_h2d, 2), "h2d_GBps": round(2 ** 31 / t_h2d / 1e6, 1), "d2h_1GiB_ms": round(t_d2h, 2),
       "d2h_GBps": round(2 ** 30 / t_d2h / 1e6, 1), "both_ms": round(t_both, 2),
       "e2e_bound_G_iter_per_s": round(2 ** 28 / (t_both * 1e-3) / 1e9, 2)})
