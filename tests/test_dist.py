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

    def __init__(self, ro, co, lo, hi, with_in=True):
        self.ro, self.co, self.lo, self.hi = ro.astype(np.int64), co.astype(np.int64), lo, hi
        self.n = ro.size - 1
        self.nwf = (self.n + 31) // 32
        self.device = "cpu"
        self.has_in = with_in
        src = np.repeat(np.arange(self.n), np.diff(self.ro))
        order = np.argsort(self.co, kind="stable")
        self.tco = src[order]
        self.tro = np.zeros(self.n + 1, np.int64)
        np.add.at(self.tro, self.co + 1, 1)
        self.tro = np.cumsum(self.tro)

    def range(self):
        return self.lo, self.hi

    def _bits(self, words, v):
        return (int(words[v >> 5]) >> (v & 31)) & 1

    def begin(self, s):
        self.V = np.zeros(self.nwf, np.uint32)
        self.F = np.zeros(self.nwf, np.uint32)
        self.lv = np.full(self.n, -1, np.int32)
        self.V[s >> 5] |= np.uint32(1 << (s & 31))
        self.F[s >> 5] |= np.uint32(1 << (s & 31))
        self.lv[s] = 0

    def expand(self, level, cand, fslice, bottom_up):
        if bottom_up:
            w0 = self.lo // 32
            f = np.zeros(fslice.numel(), np.uint32)
            for v in range(self.lo, self.hi):
                if not self._bits(self.V, v):
                    for u in self.tco[self.tro[v]:self.tro[v + 1]]:
                        if self._bits(self.F, u):
                            f[(v >> 5) - w0] |= np.uint32(1 << (v & 31))
                            break
            fslice.copy_(torch.from_numpy(f.view(np.int32)))
            return
        c = np.zeros(cand.numel(), np.uint32)
        for u in range(self.lo, self.hi):
            if self._bits(self.F, u):
                for v in self.co[self.ro[u]:self.ro[u + 1]]:
                    if not self._bits(self.V, v):
                        c[v >> 5] |= np.uint32(1 << (v & 31))
        cand.copy_(torch.from_numpy(c.view(np.int32)))

    def commit(self, level, recv, P, fslice, keep):
        w0 = self.lo // 32
        nlw = (self.hi + 31) // 32 - w0
        b = fslice.numpy().view(np.uint32)[:nlw].copy() if keep else np.zeros(nlw, np.uint32)
        if P:
            b |= np.bitwise_or.reduce(recv.numpy().view(np.uint32).reshape(P, -1), axis=0)[:nlw]
        b &= ~self.V[w0:w0 + nlw]
        fslice[:nlw].copy_(torch.from_numpy(b.view(np.int32)))
        for i, word in enumerate(b):
            for k in range(32):
                if (int(word) >> k) & 1:
                    self.lv[(w0 + i) * 32 + k] = level + 1

    def absorb(self, frontier):
        f = frontier.numpy().view(np.uint32)[: self.nwf]
        self.F = f.copy()
        self.V |= f
        return int(sum(bin(int(x)).count("1") for x in f))

    def levels(self, out):
        out.copy_(torch.from_numpy(self.lv[self.lo:self.hi]))

    def cc_hook(self, parent, pairs):
        p = parent.numpy()
        pr = pairs.numpy()
        cap = pr.size // 2
        hooks = 0

        def find(x):  # no path halving (the partitioned contract)
            while p[x] != x:
                x = p[x]
            return x
        for u in range(self.lo, self.hi):
            for v in self.co[self.ro[u]:self.ro[u + 1]]:
                ru, rv = find(u), find(v)
                if ru != rv:
                    hi, lo = max(ru, rv), min(ru, rv)
                    p[hi] = lo
                    if hooks < cap:
                        pr[2 * hooks], pr[2 * hooks + 1] = hi, lo
                    hooks += 1
        return hooks

    def cc_merge(self, parent, pairs, npairs):
        p, pr = parent.numpy(), pairs.numpy()
        for i in range(npairs):
            p[pr[2 * i]] = min(p[pr[2 * i]], pr[2 * i + 1])

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
    try:
        _worker_cpu_body(rank, P, port, seed, q)
    except BaseException:
        import traceback
        q.put((rank, {"error": traceback.format_exc()}))
        raise


def _worker_cpu_body(rank, P, port, seed, q):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=P)
    from paper_conf_sigmod_shalt19_b200.dist import DistBFS
    ro, co = random_graph(300, 2400, seed=seed)
    b = _bounds(ro.size - 1, P)
    ops = NumpyOps(ro, co, b[rank], b[rank + 1])
    out = {"modes": set(), "dirs": set()}
    # default thresholds, bottom-up forced early and kept (alpha huge, beta 1), top-down only
    for alpha, beta, dopt in [(4, 128, True), (10**6, 1, True), (4, 128, False)]:
        d = DistBFS(ops, alpha=alpha, beta=beta)
        for s in (0, 7, 299):
            lv, _ = d.bfs(s, direction_optimizing=dopt)
            out[(alpha, dopt, s)] = lv
            out["dirs"] |= set(d.directions)
    d = DistBFS(ops)
    out["cc"] = d.cc()[0]
    out["modes"] |= set(d.cc_modes)
    d = DistBFS(ops, sparse_cc_frac=1.0)  # every round through the sparse delta exchange
    out["cc_sparse"] = d.cc()[0]
    out["modes"] |= set(d.cc_modes)
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
    res = {}
    for _ in range(P):
        r, out = q.get(timeout=300)
        res[r] = out
        if "error" in out:
            for p in procs:
                p.kill()
            pytest.fail(f"rank {r}: {out['error']}")
    for p in procs:
        p.join(60)
    ro, co = random_graph(300, 2400, seed=P)
    for r in range(P):
        for key, lv in res[r].items():
            if isinstance(key, tuple):
                assert np.array_equal(lv, O.bfs(ro, co, key[2])), (r, key)
        assert res[r]["dirs"] == {0, 1}  # both level kinds ran
        assert np.array_equal(res[r]["cc"], O.cc(ro, co)), r
        assert np.array_equal(res[r]["cc_sparse"], O.cc(ro, co)), r
        assert res[r]["modes"] == {"dense", "sparse"}, res[r]["modes"]


def _worker_gpu(rank, P, port, name, q, slices=False):
    try:
        _worker_gpu_body(rank, P, port, name, q, slices)
    except BaseException as e:  # report instead of leaving the other ranks (and the parent) waiting
        import traceback
        q.put((rank, {"error": traceback.format_exc()}))
        raise


def _worker_gpu_body(rank, P, port, name, q, slices):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=P)
    torch.cuda.set_device(0)
    import paper_conf_sigmod_shalt19_b200 as G
    from paper_conf_sigmod_shalt19_b200.dist import DistBFS, GraphOps, bc_sharded
    cfg = synth.CONFIGS[name]
    ro, co = cfg.make()
    P3 = (cfg.min_interval_len, cfg.residual_segment_len, cfg.zeta_k)
    cgr = G.encode(ro, co, *P3)
    inc = None if cfg.symmetric else G.encode_transpose(ro, co, *P3)
    if slices:  # C5's pipeline: this rank generates and encodes only its own vertex range, then loads that slice
        sc, ef, seed = cfg.args
        b = synth.rmat_slices(sc, ef, seed, P)
        sro, sco = synth.rmat_slice(sc, ef, seed, b[rank], b[rank + 1])
        g = G.load(G.encode_slice(sro, sco, b[rank], ro.size - 1, *P3), device=0, stream="torch", symmetric=True)
        assert g.range() == (b[rank], b[rank + 1])
    else:
        g = G.load(cgr, device=0, stream="torch", rank=rank, nranks=P, in_cgr=inc, symmetric=cfg.symmetric)
    out = {"range": g.range(), "dirs": set()}
    roots = [0] + synth.pick_roots(ro, 2)
    for alpha, beta in [(4, 128), (10**6, 1)]:
        d = DistBFS(GraphOps(g, "cuda:0"), exchange_on_host=True, alpha=alpha, beta=beta)
        for s in roots:
            out[(alpha, s)] = d.bfs(s)[0]
            out["dirs"] |= set(d.directions)
    d = DistBFS(GraphOps(g, "cuda:0"), exchange_on_host=True)
    out["cc"] = d.cc()[0]
    d = DistBFS(GraphOps(g, "cuda:0"), exchange_on_host=True, sparse_cc_frac=1.0)
    out["cc_sparse"] = d.cc()[0]
    full = G.load(cgr, device=0)
    out["bc"] = bc_sharded(full, synth.bc_sources(ro, 4))
    q.put((rank, out))
    dist.destroy_process_group()


@pytest.mark.gpu
@pytest.mark.parametrize("name,P,slices", [("web_s", 2, False), ("social_s", 3, False), ("c1", 2, False),
                                           ("rmat_s", 3, True)])
def test_dist_partitioned_on_one_gpu(name, P, slices):
    """slices=True: every rank generates, encodes and loads only its own R-MAT vertex range (the C5 pipeline)."""
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _port()
    procs = [ctx.Process(target=_worker_gpu, args=(r, P, port, name, q, slices)) for r in range(P)]
    for p in procs:
        p.start()
    res = {}
    for _ in range(P):
        r, out = q.get(timeout=600)
        res[r] = out
        if "error" in out:
            for p in procs:
                p.kill()
            pytest.fail(f"rank {r}: {out['error']}")
    for p in procs:
        p.join(60)
    cfg = synth.CONFIGS[name]
    ro, co = cfg.make()
    ranges = [res[r]["range"] for r in range(P)]
    assert ranges[0][0] == 0 and ranges[-1][1] == ro.size - 1
    roots = [0] + synth.pick_roots(ro, 2)
    bc_ref = O.bc(ro, co, synth.bc_sources(ro, 4))
    for r in range(P):
        for key, lv in res[r].items():
            if isinstance(key, tuple):
                assert np.array_equal(lv, O.bfs(ro, co, key[1])), (name, r, key)
        assert res[r]["dirs"] == {0, 1}
        assert np.array_equal(res[r]["cc"], O.cc(ro, co)), (name, r)
        assert np.array_equal(res[r]["cc_sparse"], O.cc(ro, co)), (name, r)
        np.testing.assert_allclose(res[r]["bc"], bc_ref, rtol=1e-9, atol=0)
