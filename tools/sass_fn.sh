#!/bin/bash
# Static SASS opcode histogram of one kernel: tools/sass_fn.sh lib.so <substring of mangled name>
cuobjdump -sass "$1" | awk -v pat="$2" '/Function :/ {on = index($0, pat) > 0} on' > /tmp/sass_fn.txt
echo "instructions: $(grep -cE '^\s+/\*[0-9a-f]{4}\*/' /tmp/sass_fn.txt)"
grep -E '^\s+/\*[0-9a-f]{4}\*/' /tmp/sass_fn.txt | sed -E 's/^\s+\/\*[0-9a-f]+\*\/\s+//; s/^@!?U?P[0-9T]+\s+//' | awk '{print $1}' | sort | uniq -c | sort -rn | head -${3:-45}
