import sys; sys.path.insert(0, '/root/repo')
import torch, bench, paper_conf_icpp_hanzlw13_b200 as jp
print(bench.exchange_cost(jp, torch.device("cuda"), torch.cuda.current_stream()))
