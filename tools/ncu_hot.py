"""Top SASS instructions by warp-stall samples for one launch of an .ncu-rep."""
import csv, subprocess, sys
path, skip = sys.argv[1], int(sys.argv[2]) if len(sys.argv) > 2 else 0
n = int(sys.argv[3]) if len(sys.argv) > 3 else 30
out = subprocess.run(['ncu', '-i', path, '--page', 'source', '--csv', '--print-source', 'sass',
                      '--launch-skip', str(skip), '--launch-count', '1'], capture_output=True, text=True).stdout
rows = list(csv.reader(out.splitlines()))
hdr = rows[1]
def num(x):
    try: return float(x.replace(',', ''))
    except Exception: return None
ie = hdr.index('Instructions Executed'); src = hdr.index('Source'); ss = hdr.index('Warp Stall Sampling (All Samples)')
data = [r for r in rows[2:] if len(r) == len(hdr) and num(r[ie]) is not None]
seen = set(); uniq = []
for r in data:
    if r[0] in seen: continue
    seen.add(r[0]); uniq.append(r)
tot_s = sum(num(r[ss]) or 0 for r in uniq); tot_i = sum(num(r[ie]) for r in uniq)
print(f'{rows[0][1]}  instructions {tot_i:.3e}  stall samples {tot_s:.0f}  sass lines {len(uniq)}')
for i, r in enumerate(uniq):
    r.append(i)
for r in sorted(uniq, key=lambda r: -(num(r[ss]) or 0))[:n]:
    print(f'{r[-1]:5d} {r[0][-5:]} {r[src][:60]:60s} inst={r[ie]:>10s} samples={r[ss]}')
