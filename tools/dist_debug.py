"""Debug driver: P ranks on one GPU (gloo, host-staged exchange), prints progress; dumps stacks if stuck."""
import faulthandler
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch.distributed as dist  # noqa: E402
import torch.multiprocessing as mp  # noqa: E402


def worker(rank, P, name):
    faulthandler.dump_traceback_later(60, exit=True)
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = "29533"
    dist.init_process_group("gloo", rank=rank, world_size=P)
    import torch
    torch.cuda.set_device(0)
    import oracle as O
    import paper_conf_sigmod_shalt19_b200 as G
    from paper_conf_sigmod_shalt19_b200.dist import DistBFS, GraphOps
    import synth
    import numpy as np
    cfg = synth.CONFIGS[name]
    ro, co = cfg.make()
    P3 = (cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)
    cgr = G.encode(ro, co, *P3)
    inc = None if cfg.symmetric else G.encode_transpose(ro, co, *P3)
    g = G.load(cgr, device=0, stream="torch", rank=rank, nranks=P, in_cgr=inc, symmetric=cfg.symmetric)
    print(rank, "loaded", g.range(), flush=True)
    d = DistBFS(GraphOps(g, "cuda:0"), exchange_on_host=True)
    print(rank, "driver", flush=True)
    lv, nl = d.bfs(0)
    print(rank, "bfs", nl, d.directions, np.array_equal(lv, O.bfs(ro, co, 0)), flush=True)
    lab, rounds = d.cc()
    print(rank, "cc", rounds, d.cc_modes, np.array_equal(lab, O.cc(ro, co)), flush=True)
    dist.destroy_process_group()


if __name__ == "__main__":
    name = sys.argv[1] if len(sys.argv) > 1 else "c1"
    P = int(sys.argv[2]) if len(sys.argv) > 2 else 2
    mp.spawn(worker, args=(P, name), nprocs=P)
