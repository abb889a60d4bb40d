"""Distributed sample sort across GPUs (one process per GPU).

The method is the paper's sample sort (Algorithm 1) applied
across ranks, the setting the paper names as sample sort's home (P:24-25,
P:195-196): large random samples give splitters that balance the ranks
(P:228-233).  One call on every rank of the process group:

1. sample S keys of the local shard at hashed positions (level tag 255,
   lo = the shard's global start) -- gss_sample (kernel);
2. all-gather the samples (torch.distributed / NCCL);
3. sort the gathered sample -- gss_sort (kernel); every rank now holds the
   identical sorted sample and takes the identical P-1 splitters
   S[(i+1) * S_total/P - 1] (R1);
4. stable partition of the shard by the splitters, ties go left (R3) --
   gss_partition_by (kernels);
5. exchange the P bucket sizes, then the keys (and values): all-to-all-v over
   NCCL (NVLink) -- the path's one exchange step;
6. sort the received keys -- gss_sort (kernels).

Rank r ends with the r-th contiguous range of the global sorted order.  The
GPU work is in libgss.so; this module only orchestrates collectives and
buffers.  `ops` can be replaced (tests run the orchestration with gloo on CPU).
"""
from __future__ import annotations

import torch
import torch.distributed as dist

from . import partition_by, sample, sort

__all__ = ["DistSorter", "GpuOps", "splitter_positions"]


def splitter_positions(total_samples: int, nranks: int) -> list[int]:
    """Indices of the P-1 global splitters in the sorted gathered sample (R1)."""
    per = total_samples // nranks
    return [per * (i + 1) - 1 for i in range(nranks - 1)]


def _as_signed(t: torch.Tensor) -> torch.Tensor:
    """Same bytes, a dtype NCCL/gloo collectives accept."""
    if t.dtype == torch.uint64:
        return t.view(torch.int64)
    if t.dtype == torch.uint32:
        return t.view(torch.int32)
    return t


class GpuOps:
    """The kernels of libgss.so (the product path).  With `counting` set, the
    calls synchronise to count the kernels they launch (not for timing)."""

    PARTITION_BY_LAUNCHES = 7       # init, set_splitters, classify, scan x2, scatter, partition_out

    def __init__(self, **params):
        self.params = params
        self.counting = False
        self.launches = 0

    def sample(self, keys, s, lo_global, seed):
        self.launches += 1
        return sample(keys, s, lo_global=lo_global, level_tag=255, seed=seed)

    def sort(self, keys, vals=None):
        if self.counting:
            k, v, st = sort(keys, vals, stats=True, **self.params)
            self.launches += st.launches
            return k, v
        return sort(keys, vals, **self.params)

    def partition_by(self, keys, vals, splitters):
        self.launches += self.PARTITION_BY_LAUNCHES
        return partition_by(keys, vals, splitters)


class DistSorter:
    """Sorts a global array distributed as equal shards of n_local keys per rank."""

    def __init__(self, kind: str, n_local: int, pairs: bool = False, device=None, group=None,
                 samples_per_rank: int = 16384, seed: int = 5489, ops=None, **params):
        self.kind, self.n_local, self.pairs = kind, n_local, pairs
        self.device = torch.device(device) if device is not None else torch.device("cuda")
        self.group = group
        self.rank = dist.get_rank(group)
        self.world = dist.get_world_size(group)
        self.S = max(1, min(samples_per_rank, max(n_local, 1)))
        self.seed = seed
        self.ops = ops or GpuOps(**params)
        self.last_counts = None

    def _all_gather(self, t: torch.Tensor) -> torch.Tensor:
        out = torch.empty(self.world * t.numel(), dtype=t.dtype, device=t.device)
        dist.all_gather_into_tensor(_as_signed(out), _as_signed(t.contiguous()), group=self.group)
        return out

    def __call__(self, keys: torch.Tensor, vals: torch.Tensor | None = None):
        """Returns (sorted local range of keys, values or None, received count)."""
        P, r = self.world, self.rank
        lo_global = r * self.n_local
        # 1-3: identical global splitters on every rank
        smp = self.ops.sample(keys, self.S, lo_global, self.seed)
        gathered = self._all_gather(smp)
        sorted_smp, _ = self.ops.sort(gathered)
        pos = splitter_positions(gathered.numel(), P)
        spl = sorted_smp[torch.tensor(pos, dtype=torch.long, device=sorted_smp.device)] if pos else \
            sorted_smp[:0]
        # 4: stable partition of the shard into P destination ranges
        pk, pv, counts = self.ops.partition_by(keys, vals, spl.contiguous())
        # 5: exchange sizes, then data (all-to-all-v)
        send = counts.to(torch.int64)
        recv = torch.empty_like(send)
        dist.all_to_all_single(recv, send, group=self.group)
        send_l = [int(x) for x in send.cpu().tolist()]
        recv_l = [int(x) for x in recv.cpu().tolist()]
        self.last_counts = (send_l, recv_l)
        n_recv = sum(recv_l)
        rk = torch.empty(n_recv, dtype=keys.dtype, device=keys.device)
        dist.all_to_all_single(_as_signed(rk), _as_signed(pk), output_split_sizes=recv_l,
                               input_split_sizes=send_l, group=self.group)
        rv = None
        if vals is not None:
            rv = torch.empty(n_recv, dtype=vals.dtype, device=vals.device)
            dist.all_to_all_single(_as_signed(rv), _as_signed(pv), output_split_sizes=recv_l,
                                   input_split_sizes=send_l, group=self.group)
        # 6: local sort of the received range
        if n_recv == 0:
            return rk, rv, 0
        ok, ov = self.ops.sort(rk, rv)
        self.result = (ok, ov)
        return ok, ov, n_recv

    def count_launches(self, keys, vals=None) -> int:
        """Kernels of libgss.so one call launches on this rank (synchronising run)."""
        if not isinstance(self.ops, GpuOps):
            return 0
        self.ops.counting, self.ops.launches = True, 0
        try:
            self(keys, vals)
        finally:
            self.ops.counting = False
        return self.ops.launches

    # ------------------------------------------------------------------
    def verify(self, x_local_input) -> bool:
        """Global checks of the last result (not timed): every range sorted, ranges
        ordered across ranks, total count and a multiset fingerprint preserved."""
        import numpy as np
        ok_k, _ = self.result
        y = ok_k.cpu().numpy()
        good = bool(np.all(y[1:] >= y[:-1])) if y.size > 1 else True
        first = int(y[0]) if y.size else None
        last = int(y[-1]) if y.size else None
        objs = [None] * self.world
        dist.all_gather_object(objs, (first, last, int(y.size)), group=self.group)
        prev = None
        for f, l, cnt in objs:
            if cnt == 0:
                continue
            if prev is not None and f < prev:
                good = False
            prev = l

        def fp(a):
            z = a.astype(np.uint64) * np.uint64(0x9E3779B97F4A7C15)
            v = int(np.bitwise_xor.reduce(z ^ (z >> np.uint64(29)))) if a.size else 0
            return v - (1 << 64) if v >= (1 << 63) else v          # as a signed 64-bit value
        mine = torch.tensor([fp(np.asarray(x_local_input)), fp(y), len(x_local_input), y.size], dtype=torch.int64,
                            device=self.device)
        allv = [torch.zeros_like(mine) for _ in range(self.world)]
        dist.all_gather(allv, mine, group=self.group)
        fin = fout = 0
        nin = nout = 0
        for t in allv:
            fin ^= int(t[0]); fout ^= int(t[1]); nin += int(t[2]); nout += int(t[3])
        return good and fin == fout and nin == nout
