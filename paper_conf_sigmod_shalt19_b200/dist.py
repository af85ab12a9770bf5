"""Multi-GPU BFS / CC / BC over a 1-D vertex-range partition.

One process per GPU.  Every device step runs in libgcgt (``gcgt_dist_*``, include/gcgt.h); this module only moves
bitmaps between ranks with ``torch.distributed`` (NCCL over NVLink in production; gloo for CPU tests, or with
``exchange_on_host=True`` when several ranks share one GPU):

BFS level d (top-down):
    expand   (lib)  owned frontier -> candidate bitmap of all n vertices
    all-to-all      slice q of every rank's candidates -> rank q          (the OR-reduce-scatter's transport)
    commit   (lib)  OR of the received slices & ~visited -> owned next-frontier slice, levels, count
    all-gather      owned slices -> global next frontier
    absorb   (lib)  frontier := gathered, visited |= frontier
    all-reduce      new-vertex count (termination)
CC round: hook owned arcs into the replicated parent array (lib) | all-reduce(MIN) | pointer jump (lib) | stop when
no rank hooked.  BC: sources sharded over full replicas, one all-reduce(SUM) of the fp64 scores.

The paper is single-GPU and names multi-GPU only as orthogonal future work.
"""
from __future__ import annotations

import numpy as np
import torch
import torch.distributed as dist


class GraphOps:
    """Device steps of a partitioned ``Graph`` (torch int32 tensors carry the uint32 bitmaps bit for bit)."""

    def __init__(self, graph, device):
        self.g = graph
        self.device = device
        self.n = graph.n
        self.lo, self.hi = graph.range()

    def range(self):
        return self.lo, self.hi

    def begin(self, source):
        self.g.dist_bfs_begin(source)

    def expand(self, level, cand):
        self.g.dist_bfs_expand(level, cand.data_ptr())

    def commit(self, level, recv, nparts, fslice):
        return self.g.dist_bfs_commit(level, recv.data_ptr(), nparts, fslice.data_ptr())

    def absorb(self, frontier):
        self.g.dist_bfs_absorb(frontier.data_ptr())

    def levels(self, out):
        self.g.dist_bfs_levels(out)

    def cc_hook(self, parent):
        return self.g.dist_cc_hook(parent.data_ptr())

    def cc_jump(self, parent):
        self.g.dist_cc_jump(parent.data_ptr())


def word_range(lo, hi):
    return lo // 32, (hi + 31) // 32


class DistBFS:
    """Partitioned BFS / CC driver.  ``ops`` provides the per-rank steps (GraphOps, or a test double)."""

    def __init__(self, ops, group=None, exchange_on_host=False):
        self.ops = ops
        self.group = group
        self.P = dist.get_world_size(group)
        self.rank = dist.get_rank(group)
        self.host = exchange_on_host
        self.n = ops.n
        self.nwf = (self.n + 31) // 32
        lo, hi = ops.range()
        # every rank's owned range (gathered once)
        rng = self._x(torch.tensor([lo, hi], dtype=torch.int64))
        allr = [torch.zeros_like(rng) for _ in range(self.P)]
        dist.all_gather(allr, rng, group=group)
        self.ranges = [(int(r[0]), int(r[1])) for r in allr]
        self.wranges = [word_range(a, b) for a, b in self.ranges]
        for q in range(1, self.P):  # contiguous, ordered, word-aligned partition
            assert self.wranges[q][0] == self.wranges[q - 1][1], self.wranges
        self.my_w = self.wranges[self.rank][1] - self.wranges[self.rank][0]
        self.max_w = max(b - a for a, b in self.wranges)
        self.max_v = max(b - a for a, b in self.ranges)

    # -- helpers -------------------------------------------------------------------------------------------------
    def _dev_coll(self):
        return getattr(self.ops, "device", None) is not None and str(getattr(self.ops, "device")).startswith("cuda")

    def _x(self, t):
        """Tensor placement for collectives: the ops device, or host memory when exchanging on the host."""
        if self.host or not self._dev_coll():
            return t.cpu()
        return t.to(self.ops.device)

    def _dev(self):
        return getattr(self.ops, "device", "cpu")

    def _all_to_all(self, cand):
        sizes = [b - a for a, b in self.wranges]
        send = self._x(cand[: self.nwf])
        recv = torch.empty(self.P * self.my_w, dtype=torch.int32, device=send.device)
        dist.all_to_all_single(recv, send, output_split_sizes=[self.my_w] * self.P, input_split_sizes=sizes,
                               group=self.group)
        return recv

    def _all_gather_words(self, fslice):
        pad = torch.zeros(self.max_w, dtype=torch.int32, device=fslice.device)
        pad[: self.my_w] = fslice[: self.my_w]
        parts = [torch.empty_like(pad) for _ in range(self.P)]
        dist.all_gather(parts, pad, group=self.group)
        return torch.cat([p[: b - a] for p, (a, b) in zip(parts, self.wranges)])

    # -- BFS ------------------------------------------------------------------------------------------------------
    def bfs(self, source: int):
        """Returns the full levels array (int32 numpy, -1 = unreached) on every rank, and the level count."""
        dev = self._dev()
        ops = self.ops
        cand = torch.zeros(self.nwf + 1, dtype=torch.int32, device=dev)
        fslice = torch.zeros(max(self.my_w, 1), dtype=torch.int32, device=dev)
        ops.begin(source)
        level = 0
        while True:
            ops.expand(level, cand)
            recv = self._all_to_all(cand).to(dev)
            cnt = ops.commit(level, recv, self.P, fslice)
            frontier = self._all_gather_words(self._x(fslice)).to(dev)
            ops.absorb(frontier)
            tot = torch.tensor([cnt], dtype=torch.int64)
            tot = self._x(tot)
            dist.all_reduce(tot, op=dist.ReduceOp.SUM, group=self.group)
            level += 1
            if int(tot.item()) == 0:
                break
        lo, hi = ops.range()
        own = torch.empty(hi - lo, dtype=torch.int32, device=dev)
        ops.levels(own)
        pad = torch.full((self.max_v,), -1, dtype=torch.int32)
        pad[: hi - lo] = own.cpu()
        pad = self._x(pad)
        parts = [torch.empty_like(pad) for _ in range(self.P)]
        dist.all_gather(parts, pad, group=self.group)
        full = torch.cat([p.cpu()[: b - a] for p, (a, b) in zip(parts, self.ranges)])
        return full.numpy(), level

    # -- CC -------------------------------------------------------------------------------------------------------
    def cc(self):
        """Weakly connected components, min-id labels (uint32 numpy) on every rank; returns (labels, rounds)."""
        dev = self._dev()
        parent = torch.arange(self.n, dtype=torch.int32, device=dev)
        rounds = 0
        while True:
            hooks = self.ops.cc_hook(parent)
            xp = self._x(parent)
            dist.all_reduce(xp, op=dist.ReduceOp.MIN, group=self.group)
            if xp.data_ptr() != parent.data_ptr():
                parent.copy_(xp.to(dev))
            self.ops.cc_jump(parent)
            tot = self._x(torch.tensor([hooks], dtype=torch.int64))
            dist.all_reduce(tot, op=dist.ReduceOp.SUM, group=self.group)
            rounds += 1
            if int(tot.item()) == 0:
                break
        return parent.cpu().numpy().astype(np.uint32), rounds


def bc_sharded(graph, sources, group=None, device=None):
    """BC with sources sharded over ranks (each rank holds a full replica); one all-reduce(SUM) of the scores."""
    P, r = dist.get_world_size(group), dist.get_rank(group)
    mine = list(sources)[r::P]
    part = graph.bc(mine) if mine else np.zeros(graph.n)
    t = torch.from_numpy(np.ascontiguousarray(part, dtype=np.float64))
    if device is not None and str(device).startswith("cuda") and dist.get_backend(group) == "nccl":
        t = t.to(device)
    dist.all_reduce(t, op=dist.ReduceOp.SUM, group=group)
    return t.cpu().numpy()


def nccl_init_from_env(device_index: int):
    """One process per GPU: init the NCCL process group from torchrun's environment (MASTER_ADDR=127.0.0.1)."""
    import os
    os.environ.setdefault("MASTER_ADDR", "127.0.0.1")
    torch.cuda.set_device(device_index)
    dist.init_process_group("nccl", device_id=torch.device("cuda", device_index))
