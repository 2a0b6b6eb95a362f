"""Stall samples and executed instructions per CUDA source line for one launch of an
.ncu-rep (built with -lineinfo):  ncu_lines.py REP [SKIP] [TOP]"""
import csv, subprocess, sys
path = sys.argv[1]
skip = int(sys.argv[2]) if len(sys.argv) > 2 else 0
top = int(sys.argv[3]) if len(sys.argv) > 3 else 25
out = subprocess.run(['ncu', '-i', path, '--page', 'source', '--csv', '--print-source', 'cuda,sass',
                      '--launch-skip', str(skip), '--launch-count', '1'], capture_output=True, text=True).stdout
rows = list(csv.reader(out.splitlines()))
agg, fname, hdr, func = [], None, None, None
for r in rows:
    if len(r) == 2 and r[0] == 'File Path':
        fname = r[1].split('/')[-1]; continue
    if len(r) == 2 and r[0] == 'Function Name':
        func = r[1]; continue
    if r and r[0] == 'Line No':
        hdr = r; continue
    if hdr and len(r) == len(hdr) and r[0]:
        try:
            agg.append((fname, int(r[0]), r[1].strip(), float(r[4]), float(r[7])))
        except ValueError:
            pass
tot = sum(a[3] for a in agg)
print(func, f'total samples {tot:.0f}')
for f, ln, src, smp, ins in sorted(agg, key=lambda a: -a[3])[:top]:
    print(f'{100*smp/tot:5.1f}%  {f}:{ln:<5d} inst={ins:12.0f}  {src[:90]}')
