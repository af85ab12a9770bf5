"""Multi-GPU BFS / CC / BC over a 1-D vertex-range partition.

One process per GPU.  Every device step runs in libgcgt (``gcgt_dist_*``, include/gcgt.h); this module only moves
bitmaps between ranks with ``torch.distributed`` (NCCL over NVLink in production; gloo for CPU tests, or with
``exchange_on_host=True`` when several ranks share one GPU).  The library enqueues its steps on the graph's stream,
which must be torch's current stream (load with ``stream="torch"``), so the collectives are ordered after them.

BFS level d, direction chosen identically on every rank from replicated counts (Beamer's vertex-count rule, the same
as the single-GPU contraction's):
  top-down   expand (lib)  owned frontier -> candidate bitmap of all n vertices
             all-to-all    slice q of every rank's candidates -> rank q           (the OR-reduce-scatter's transport)
             commit (lib)  OR of the received slices & ~visited -> owned next-frontier slice, levels
  bottom-up  expand (lib)  owned unvisited vertices scan their in-records against the replicated frontier; finds
                           land in the owned next-frontier slice (no exchange)
             commit (lib)  slice & ~visited -> levels
  both       all-gather    owned slices -> global next frontier
             absorb (lib)  frontier := gathered, visited |= frontier, count (identical on every rank: the only host
                           synchronisation of the level, and the termination test without another collective)
Bytes per rank and level: top-down n/8·(P-1)/P out + n/8·(P-1)/P in (all-to-all) + n/8·(P-1)/P in (all-gather);
bottom-up only the all-gather.

CC round: hook owned arcs into the replicated parent array (lib; no path halving, so the only parent writes are the
hooks) | exchange: all-reduce(MIN) of the whole array in the first round (nearly every vertex hooks), afterwards only
the (index, value) pairs of this round's hooks (all-gather of the pair lists, then a MIN-merge in the lib) | pointer
jump (lib) | stop when no rank hooked.  BC: sources sharded over full replicas, one all-reduce(SUM) of the scores.

The paper is single-GPU and names multi-GPU only as orthogonal future work.
"""
from __future__ import annotations

import numpy as np
import torch
import torch.distributed as dist


class GraphOps:
    """Device steps of a partitioned ``Graph`` (torch int32 tensors carry the uint32 bitmaps bit for bit)."""

    def __init__(self, graph, device):
        if getattr(graph, "stream_kind", "torch") != "torch":
            raise ValueError("GraphOps needs a graph loaded with stream='torch' (steps and collectives share a stream)")
        self.g = graph
        self.device = device
        self.n = graph.n
        self.lo, self.hi = graph.range()
        self.has_in = getattr(graph, "has_in", False)

    def range(self):
        return self.lo, self.hi

    def begin(self, source):
        self.g.dist_bfs_begin(source)

    def expand(self, level, cand, fslice, bottom_up):
        self.g.dist_bfs_expand(level, cand.data_ptr() if cand is not None else 0,
                               fslice.data_ptr() if fslice is not None else 0, bottom_up)

    def commit(self, level, recv, nparts, fslice, keep):
        self.g.dist_bfs_commit(level, recv.data_ptr() if recv is not None else 0, nparts, fslice.data_ptr(), keep)

    def absorb(self, frontier):
        return self.g.dist_bfs_absorb(frontier.data_ptr())

    def levels(self, out):
        self.g.dist_bfs_levels(out)

    def cc_hook(self, parent, pairs):
        return self.g.dist_cc_hook(parent.data_ptr(), pairs.data_ptr() if pairs is not None else 0,
                                   pairs.numel() // 2 if pairs is not None else 0)

    def cc_merge(self, parent, pairs, npairs):
        self.g.dist_cc_merge(parent.data_ptr(), pairs.data_ptr(), npairs)

    def cc_jump(self, parent):
        self.g.dist_cc_jump(parent.data_ptr())


def word_range(lo, hi):
    return lo // 32, (hi + 31) // 32


class DistBFS:
    """Partitioned BFS / CC driver.  ``ops`` provides the per-rank steps (GraphOps, or a test double)."""

    def __init__(self, ops, group=None, exchange_on_host=False, alpha=4.0, beta=128, sparse_cc_frac=0.02):
        self.ops = ops
        self.group = group
        self.P = dist.get_world_size(group)
        self.rank = dist.get_rank(group)
        self.host = exchange_on_host
        self.n = ops.n
        self.nwf = (self.n + 31) // 32
        self.alpha10, self.beta = int(round(alpha * 10)), beta
        self.sparse_cap = max(64, int(self.n * sparse_cc_frac))  # hook pairs per rank below which CC goes sparse
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
        self.bytes_moved = 0  # per-rank collective payload of the last bfs() / cc() (sent + received)

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
        self.bytes_moved += 4 * (self.nwf - self.my_w) + 4 * (self.P - 1) * self.my_w
        return recv

    def _all_gather_words(self, fslice):
        pad = torch.zeros(self.max_w, dtype=torch.int32, device=fslice.device)
        pad[: self.my_w] = fslice[: self.my_w]
        parts = [torch.empty_like(pad) for _ in range(self.P)]
        dist.all_gather(parts, pad, group=self.group)
        self.bytes_moved += 4 * self.max_w * (self.P - 1)
        return torch.cat([p[: b - a] for p, (a, b) in zip(parts, self.wranges)])

    def _decide(self, dirn, nf, prev, visited, can_bu):
        """Next direction (Beamer et al.): the rule of the single-GPU contraction (contract.cuh decide_body)."""
        if not can_bu or nf == 0:
            return 0
        nu = self.n - visited
        if dirn == 0 and nf * self.alpha10 > nu * 10 and nf > prev:
            return 1
        if dirn == 1 and nf * self.beta < self.n and nf < prev:
            return 0
        return dirn

    # -- BFS ------------------------------------------------------------------------------------------------------
    def bfs(self, source: int, direction_optimizing: bool = True):
        """Returns the full levels array (int32 numpy, -1 = unreached) on every rank, and the level count.
        Direction-optimizing when the ops hold in-records (``ops.has_in``)."""
        dev = self._dev()
        ops = self.ops
        can_bu = direction_optimizing and bool(getattr(ops, "has_in", False))
        cand = torch.zeros(self.nwf + 1, dtype=torch.int32, device=dev)
        fslice = torch.zeros(max(self.my_w, 1), dtype=torch.int32, device=dev)
        ops.begin(source)
        self.bytes_moved = 0
        self.directions = []
        level, dirn, prev, visited, nf = 0, 0, 1, 1, 1
        while True:
            self.directions.append(dirn)
            if dirn == 0:
                ops.expand(level, cand, None, False)
                recv = self._all_to_all(cand).to(dev)
                ops.commit(level, recv, self.P, fslice, False)
            else:
                ops.expand(level, None, fslice, True)
                ops.commit(level, None, 0, fslice, True)
            frontier = self._all_gather_words(self._x(fslice)).to(dev)
            nf = ops.absorb(frontier)
            level += 1
            if nf == 0:
                break
            visited += nf
            dirn = self._decide(dirn, nf, prev, visited, can_bu)
            prev = nf
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
        pairs = torch.empty(2 * self.sparse_cap, dtype=torch.int32, device=dev)
        rounds = 0
        self.bytes_moved = 0
        self.cc_modes = []
        while True:
            hooks = self.ops.cc_hook(parent, pairs)
            cnt = self._x(torch.tensor([hooks], dtype=torch.int64))
            allc = [torch.zeros_like(cnt) for _ in range(self.P)]
            dist.all_gather(allc, cnt, group=self.group)
            counts = [int(c.item()) for c in allc]
            if sum(counts) == 0:
                rounds += 1
                break
            if max(counts) > self.sparse_cap:  # dense: all-reduce(MIN) of the whole parent array
                self.cc_modes.append("dense")
                xp = self._x(parent)
                dist.all_reduce(xp, op=dist.ReduceOp.MIN, group=self.group)
                self.bytes_moved += 2 * 4 * self.n
                if xp.data_ptr() != parent.data_ptr():
                    parent.copy_(xp.to(dev))
            else:  # sparse delta: every rank's hook pairs, MIN-merged
                self.cc_modes.append("sparse")
                m = max(counts)
                mine = self._x(pairs[: 2 * m].clone())
                if hooks < m:
                    mine[2 * hooks:] = 0  # padding pairs (0, 0) merge as no-ops
                parts = [torch.empty_like(mine) for _ in range(self.P)]
                dist.all_gather(parts, mine, group=self.group)
                self.bytes_moved += 8 * m * self.P
                for q, part in enumerate(parts):
                    if q != self.rank and counts[q]:
                        self.ops.cc_merge(parent, part.to(dev), counts[q])
            self.ops.cc_jump(parent)
            rounds += 1
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
