"""Analyse a scan_lab trace (lab tool): where does a CTA wait for its slice prefix?

Events per (slice s, CTA c), globaltimer ns: 0 = P1 aggregate published,
1 = prefix ready (prefix warp), 2 = P2 start (consumers got the prefix),
3 = P2 outputs staged.
"""
import sys

import numpy as np

raw = np.fromfile(sys.argv[1], dtype=np.uint64)
LAG = int(sys.argv[2]) if len(sys.argv) > 2 else 1  # SKEL_SCAN_LAG of the traced build
G, S, SMAX, CMAX = (int(x) for x in raw[:4])
tr = raw[4:].reshape(-1, SMAX, CMAX)[:, :S, :G].astype(np.int64)
t0 = tr[0][tr[0] > 0].min()
pub, pre, p2s, p2e, pws, pwc = (tr[i] - t0 for i in range(6))
print(f"G={G} slices={S} kernel span ~{(p2e.max()) / 1e3:.1f} us, per slice {(p2e.max()) / S / 1e3:.2f} us")
ss = range(2, S - 1 - LAG)
need = np.array([[max(pub[s - 1].max(), pub[s, :c].max() if c else 0) for c in range(G)] for s in ss])
prev = np.array([pub[s + LAG] for s in ss])  # consumers reach the P2(s) wait after P1(s+LAG)
P2s = np.array([p2s[s] for s in ss]); PRE = np.array([pre[s] for s in ss])
stall = P2s - prev
print(f"consumer wait for the prefix (P2 start - own P1(s+LAG) publish): mean {stall.mean()/1e3:.2f} us, "
      f"p50 {np.median(stall)/1e3:.2f}, p90 {np.percentile(stall, 90)/1e3:.2f}")
print(f"prefix ready - inputs available: mean {(PRE - need).mean()/1e3:.2f} us, p50 {np.median(PRE-need)/1e3:.2f}, "
      f"p90 {np.percentile(PRE-need, 90)/1e3:.2f}")
print(f"inputs available - consumer reaches wait: mean {(need - prev).mean()/1e3:.2f} us "
      f"(>0: waiting on other CTAs' aggregates), frac>0 {(need > prev).mean():.2f}")
# skew: publish time of slice s relative to the slice's median
rel = np.array([pub[s] - np.median(pub[s]) for s in ss])
print(f"publish skew within a slice: p10 {np.percentile(rel,10)/1e3:.2f} p90 {np.percentile(rel,90)/1e3:.2f} "
      f"max-median mean {np.mean(rel.max(1))/1e3:.2f} us")
per_cta = rel.mean(0)
order = np.argsort(per_cta)
print("slowest CTAs (mean lag us):", [(int(c), round(per_cta[c] / 1e3, 2)) for c in order[-8:]])
print("fastest CTAs:", [(int(c), round(per_cta[c] / 1e3, 2)) for c in order[:5]])
# who gates need(s,c): the last publisher of slice s-1
last = np.array([pub[s - 1].argmax() for s in ss])
vals, cnt = np.unique(last, return_counts=True)
print("last publisher of slice s-1 (CTA: count):", sorted(zip(cnt.tolist(), vals.tolist()))[-8:])
dur = np.diff(np.median(pub[1:S - 1], axis=1))
print(f"median-publish period per slice: mean {dur.mean()/1e3:.2f} us")
PWS = np.array([pws[s] for s in ss]); PWC = np.array([pwc[s] for s in ss])
needc = np.array([pub[s - 1].max() for s in ss])[:, None]
needp = np.array([[pub[s, :c].max() if c else 0 for c in range(G)] for s in ss])
print(f"prefix warp: start(s) - prev prefix ready: {(PWS - np.array([pre[s-1] for s in ss])).mean()/1e3:.2f} us")
print(f"prefix warp: ready - max(start, window published): {(PRE - np.maximum(PWS, need)).mean()/1e3:.2f} us")
