"""Per-source-line instruction counts and stall samples of one kernel in an ncu report
(--page source --print-source cuda,sass). Usage: ncu_lines.py report.ncu-rep [units] [top]"""
import csv, io, subprocess, sys

def main(path, units=1.0, top=40):
    raw = subprocess.run(['ncu', '-i', path, '--page', 'source', '--csv', '--print-source', 'cuda,sass'],
                         capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(raw)))
    fname, hdr, out = None, None, []
    for r in rows:
        if r and r[0] == 'File Path':
            fname = r[1].split('/')[-1]
        elif r and r[0] == 'Line No':
            hdr = r
        elif hdr and r and r[0] not in ('', 'Function Name'):
            try:
                ie = float(r[hdr.index('Instructions Executed')] or 0)
                st = float(r[hdr.index('Warp Stall Sampling (All Samples)')] or 0)
            except (ValueError, IndexError):
                continue
            if ie or st:
                out.append((ie, st, f'{fname}:{r[0]}', r[1].strip()[:70]))
    tot_i = sum(o[0] for o in out); tot_s = sum(o[1] for o in out) or 1
    print(f'total warp-instr per unit {tot_i/units:.1f}')
    for ie, st, loc, src in sorted(out, key=lambda o: -o[0])[:top]:
        print(f'{ie/units:8.1f} {100*st/tot_s:5.1f}%  {loc:22s} {src}')

if __name__ == '__main__':
    main(sys.argv[1], float(sys.argv[2]) if len(sys.argv) > 2 else 1.0, int(sys.argv[3]) if len(sys.argv) > 3 else 40)
