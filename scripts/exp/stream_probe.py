import os, sys; sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import torch, paper_conf_cidr_appuswamykpa17_b200 as h
e=h.h2tap_open(0)
for nbytes in (720_000_000, 1_440_000_000, 4<<30):
    n=nbytes//4
    col=torch.ones(n,dtype=torch.int32,device='cuda'); torch.cuda.synchronize()
    best=min(h.h2tap_layout_sum(e,col,h.H2TAP_DSM,n,1,[0])[1] for _ in range(7))
    print(f"DSM read {nbytes/1e6:.0f} MB: {best*1e3:.1f} us -> {nbytes/best/1e6:.0f} GB/s")
    del col; torch.cuda.empty_cache()
