"""Multi-rank paths (§8 e).

CPU (-m "not gpu"): the DistBFS driver's exchange logic on world_size 2 / 3 with gloo, over a numpy double of the
per-rank steps, against the oracle.  GPU (-m gpu): two processes sharing cuda:0, real partitioned libgcgt graphs,
collectives through gloo with host staging (NCCL cannot put two ranks on one GPU), against the oracle.
"""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import oracle as O
import synth
from graphs import random_graph


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


class NumpyOps:
    """Test double of the per-rank device steps (the same contract as include/gcgt.h's gcgt_dist_*)."""

    def __init__(self, ro, co, lo, hi):
        self.ro, self.co, self.lo, self.hi = ro.astype(np.int64), co.astype(np.int64), lo, hi
        self.n = ro.size - 1
        self.nwf = (self.n + 31) // 32
        self.device = "cpu"

    def range(self):
        return self.lo, self.hi

    def _bits(self, words, v):
        return (words[v >> 5] >> (v & 31)) & 1

    def begin(self, s):
        self.V = np.zeros(self.nwf, np.uint32)
        self.F = np.zeros(self.nwf, np.uint32)
        self.lv = np.full(self.n, -1, np.int32)
        self.V[s >> 5] |= np.uint32(1 << (s & 31))
        self.F[s >> 5] |= np.uint32(1 << (s & 31))
        self.lv[s] = 0

    def expand(self, level, cand):
        c = np.zeros(cand.numel(), np.uint32)
        for u in range(self.lo, self.hi):
            if self._bits(self.F, u):
                for v in self.co[self.ro[u]:self.ro[u + 1]]:
                    if not self._bits(self.V, v):
                        c[v >> 5] |= np.uint32(1 << (v & 31))
        cand.copy_(torch.from_numpy(c.view(np.int32)))

    def commit(self, level, recv, P, fslice):
        r = recv.numpy().view(np.uint32).reshape(P, -1)
        w0 = self.lo // 32
        b = np.bitwise_or.reduce(r, axis=0) & ~self.V[w0:w0 + r.shape[1]]
        fslice[: b.size].copy_(torch.from_numpy(b.view(np.int32)))
        for i, word in enumerate(b):
            for k in range(32):
                if (int(word) >> k) & 1:
                    self.lv[(w0 + i) * 32 + k] = level + 1
        return int(sum(bin(int(x)).count("1") for x in b))

    def absorb(self, frontier):
        f = frontier.numpy().view(np.uint32)[: self.nwf]
        self.F = f.copy()
        self.V |= f

    def levels(self, out):
        out.copy_(torch.from_numpy(self.lv[self.lo:self.hi]))

    def cc_hook(self, parent):
        p = parent.numpy()
        hooks = 0

        def find(x):
            while p[x] != x:
                x = p[x]
            return x
        for u in range(self.lo, self.hi):
            for v in self.co[self.ro[u]:self.ro[u + 1]]:
                ru, rv = find(u), find(v)
                if ru != rv:
                    p[max(ru, rv)] = min(ru, rv)
                    hooks += 1
        return hooks

    def cc_jump(self, parent):
        p = parent.numpy()
        for v in range(self.n):
            x = v
            while p[x] != x:
                x = p[x]
            p[v] = x


def _bounds(n, P):
    step = ((n + P - 1) // P + 31) // 32 * 32
    return [min(n, r * step) for r in range(P)] + [n]


def _worker_cpu(rank, P, port, seed, q):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=P)
    from paper_conf_sigmod_shalt19_b200.dist import DistBFS
    ro, co = random_graph(300, 2400, seed=seed)
    b = _bounds(ro.size - 1, P)
    ops = NumpyOps(ro, co, b[rank], b[rank + 1])
    d = DistBFS(ops)
    out = {}
    for s in (0, 7, 299):
        lv, _ = d.bfs(s)
        out[s] = lv
    out["cc"] = d.cc()[0]
    q.put((rank, out))
    dist.destroy_process_group()


@pytest.mark.parametrize("P", [2, 3])
def test_dist_driver_gloo_cpu(P):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _port()
    procs = [ctx.Process(target=_worker_cpu, args=(r, P, port, P, q)) for r in range(P)]
    for p in procs:
        p.start()
    res = dict(q.get(timeout=300) for _ in range(P))
    for p in procs:
        p.join(60)
    ro, co = random_graph(300, 2400, seed=P)
    for r in range(P):
        for s in (0, 7, 299):
            assert np.array_equal(res[r][s], O.bfs(ro, co, s)), (r, s)
        assert np.array_equal(res[r]["cc"], O.cc(ro, co)), r


def _worker_gpu(rank, P, port, name, q):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=P)
    torch.cuda.set_device(0)
    import paper_conf_sigmod_shalt19_b200 as G
    from paper_conf_sigmod_shalt19_b200.dist import DistBFS, GraphOps, bc_sharded
    cfg = synth.CONFIGS[name]
    ro, co = cfg.make()
    cgr = G.encode(ro, co, cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)
    g = G.load(cgr, device=0, rank=rank, nranks=P)
    d = DistBFS(GraphOps(g, "cuda:0"), exchange_on_host=True)
    out = {"range": g.range()}
    roots = [0] + synth.pick_roots(ro, 2)
    for s in roots:
        out[s] = d.bfs(s)[0]
    out["cc"] = d.cc()[0]
    full = G.load(cgr, device=0)
    out["bc"] = bc_sharded(full, synth.bc_sources(ro, 4))
    q.put((rank, out))
    dist.destroy_process_group()


@pytest.mark.gpu
@pytest.mark.parametrize("name,P", [("web_s", 2), ("social_s", 3), ("c1", 2)])
def test_dist_partitioned_on_one_gpu(name, P):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _port()
    procs = [ctx.Process(target=_worker_gpu, args=(r, P, port, name, q)) for r in range(P)]
    for p in procs:
        p.start()
    res = dict(q.get(timeout=600) for _ in range(P))
    for p in procs:
        p.join(60)
    cfg = synth.CONFIGS[name]
    ro, co = cfg.make()
    ranges = [res[r]["range"] for r in range(P)]
    assert ranges[0][0] == 0 and ranges[-1][1] == ro.size - 1
    roots = [0] + synth.pick_roots(ro, 2)
    bc_ref = O.bc(ro, co, synth.bc_sources(ro, 4))
    for r in range(P):
        for s in roots:
            assert np.array_equal(res[r][s], O.bfs(ro, co, s)), (name, r, s)
        assert np.array_equal(res[r]["cc"], O.cc(ro, co)), (name, r)
        np.testing.assert_allclose(res[r]["bc"], bc_ref, rtol=1e-9, atol=0)
