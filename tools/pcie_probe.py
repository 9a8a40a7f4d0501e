"""PCIe ceiling of the end-to-end skeleton step (bench.py e2e): pinned host <-> device
copy rates one direction at a time and both at once (two streams), 1 GiB buffers.
Prints one JSON line (GB/s)."""
import json
import torch

N = 1 << 28  # floats = 1 GiB
h_up = torch.empty(N, dtype=torch.float32, pin_memory=True)
h_dn = torch.empty(N, dtype=torch.float32, pin_memory=True)
d_up = torch.empty(N, dtype=torch.float32, device="cuda")
d_dn = torch.empty(N, dtype=torch.float32, device="cuda")
s1, s2 = torch.cuda.Stream(), torch.cuda.Stream()


def timed(fn, reps=5):
    fn()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(reps):
        fn()
    torch.cuda.synchronize()
    e1.record()
    torch.cuda.synchronize()
    return e0.elapsed_time(e1) / reps * 1e-3


def up():
    with torch.cuda.stream(s1):
        d_up.copy_(h_up, non_blocking=True)
    torch.cuda.current_stream().wait_stream(s1)


def down():
    with torch.cuda.stream(s2):
        h_dn.copy_(d_dn, non_blocking=True)
    torch.cuda.current_stream().wait_stream(s2)


def both():
    with torch.cuda.stream(s1):
        d_up.copy_(h_up, non_blocking=True)
    with torch.cuda.stream(s2):
        h_dn.copy_(d_dn, non_blocking=True)
    torch.cuda.current_stream().wait_stream(s1)
    torch.cuda.current_stream().wait_stream(s2)


B = N * 4
t_up, t_dn, t_both = timed(up), timed(down), timed(both)
print(json.dumps({"h2d_GBps": B / t_up / 1e9, "d2h_GBps": B / t_dn / 1e9,
                  "bidir_total_GBps": 2 * B / t_both / 1e9, "bytes": B}))
