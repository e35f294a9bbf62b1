"""Summarise tools/cw_exp JSON lines (one per distribution) from stdin."""
import sys, json
for l in sys.stdin:
    l = l.strip()
    if l.startswith('=='):
        print(l); continue
    try:
        d = json.loads(l)
    except Exception:
        continue
    if 'dist' in d:
        print(f"{d['dist']:18s} ref {d['ref_ms']:.3f} ({d['ref_frac']:.3f})  cw {d['cw_ms']:.3f} ({d['cw_frac']:.3f}) "
              f"fb {d['fallback_arrays']} mm {d['mismatched_words']}  S1 {d['s1_ms']:.3f} ({d['s1_frac']:.3f}) mm {d['s1_mismatched']}")
